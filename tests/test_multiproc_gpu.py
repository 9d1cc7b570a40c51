"""The one-process-per-GPU path (bench.py under torchrun, N > 1) run on one device: two ranks
in separate processes, linked by CUDA IPC handles exchanged through a gloo process group
(paper_conf_ppopp_mohantyc14_b200/dist.py), each sweeping its column slab; the slab-0 kernel
stores its east edge straight into slab 1's ring (same device here, a peer NVLink mapping on
the 8-GPU box -- same code).  Two processes share the GPU by time slicing, so the sizes are
small.  Output gathered on rank 0 and compared with the CPU oracle, bit-exact."""
from __future__ import annotations

import os
import socket

import numpy as np
import pytest

torch = pytest.importorskip("torch")
if not torch.cuda.is_available():
    pytest.skip("needs a CUDA device", allow_module_level=True)
import torch.distributed as dist  # noqa: E402
import torch.multiprocessing as mp  # noqa: E402

pytestmark = pytest.mark.gpu


def _free_port() -> int:
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, fn, dim, kw, reps, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import workloads
        from paper_conf_ppopp_mohantyc14_b200 import dist as wdist
        from paper_conf_ppopp_mohantyc14_b200.wf import Wavefront
        dev = torch.device("cuda", 0)
        staged = kw.get("transport") == "nccl"
        w = Wavefront(fn, dim, rank=rank, device=0, ngpus=world, watchdog_cycles=1 << 40, **kw)
        if not staged:
            wdist.connect_slab(w, rank, world)
        t = lambda a: torch.from_numpy(np.ascontiguousarray(a)).to(dev)  # noqa: E731
        if fn == "seqcmp":
            x, y = workloads.seqcmp_inputs(dim, dim)
            args = (t(x), t(y), None, None)   # col_in / top cover the whole grid (include/wf.h)
        elif fn == "nash":
            r_, c_, top, left = workloads.nash_inputs(dim)
            args = (t(r_), t(c_), [t(top[p]) for p in range(4)], [t(left[p]) for p in range(4)])
        else:
            u, v, top, left = workloads.synthetic_inputs(dim, dim, kw["dsize"])
            args = (t(u), t(v), [t(top[d]) for d in range(kw["dsize"])], [t(left[d]) for d in range(kw["dsize"])])
        outs = []
        for _ in range(reps):   # re-runs exercise the cross-run ack / the ring reset of the edge
            if staged:   # host-staged edges over the process group (gloo: CPU message buffers)
                out = wdist.staged_run(w, args, rank, world, comm_device="cpu")
            else:
                out = w.run(*args)
            w.sync()
            outs.append([o.cpu().numpy().copy() for o in out])
        gathered = [None] * world
        dist.all_gather_object(gathered, outs)
        w.close()
        q.put((rank, gathered if rank == 0 else None))
    except Exception as e:  # noqa: BLE001
        q.put((rank, repr(e)))
    finally:
        dist.destroy_process_group()


def _run(fn, dim, kw, reps=2, world=2):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, fn, dim, kw, reps, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = dict(q.get(timeout=600) for _ in range(world))
    for p in procs:
        p.join(timeout=120)
    for r in range(world):
        assert not isinstance(res[r], str), res[r]
    return res[0]


def test_two_process_ipc_slabs_seqcmp():
    import oracle
    import workloads
    dim = 1500
    gathered = _run("seqcmp", dim, dict(alphabet=4))
    x, y = workloads.seqcmp_inputs(dim, dim)
    H = oracle.seqcmp(x, y, 1, -1, -1)
    for rep in range(2):
        g = np.concatenate([gathered[r][rep][0] for r in range(2)], axis=1)
        assert np.array_equal(g, H)


def test_two_process_ipc_slabs_synthetic():
    import oracle
    import workloads
    dim = 700
    gathered = _run("synthetic", dim, dict(tsize=10, dsize=2))
    u, v, top, left = workloads.synthetic_inputs(dim, dim, 2)
    i0, i1, f = oracle.synthetic(u, v, top, left, 10)
    want = [i0, i1, f[0], f[1]]
    for rep in range(2):
        for p in range(4):
            g = np.concatenate([gathered[r][rep][p] for r in range(2)], axis=1)
            if want[p].dtype == np.float32:
                assert np.all(np.abs(g - want[p]) <= 1e-5 * np.abs(want[p]))
            else:
                assert np.array_equal(g, want[p])


# ---- transport = "nccl": the host-staged fallback (include/wf.h wf_edge_*; SURVEY.md §8(a) a8,
# §4.2-4c: "the NCCL fallback checked against the P2P path: grids must be identical")
def _gathered_grid(gathered, rep, plane, world=2):
    return np.concatenate([gathered[r][rep][plane] for r in range(world)], axis=1)


@pytest.mark.parametrize("kw", [dict(alphabet=4), dict(alphabet=4, kernel=4), dict(local=1)],
                         ids=["nw_gen8", "nw_gen4", "sw"])
def test_staged_transport_seqcmp_equals_p2p_and_oracle(kw):
    import oracle
    import workloads
    dim = 1100
    staged = _run("seqcmp", dim, dict(kw, transport="nccl"), reps=2)
    p2p = _run("seqcmp", dim, dict(kw), reps=1)
    x, y = workloads.seqcmp_inputs(dim, dim)
    H = oracle.seqcmp(x, y, 1, -1, -1, local=kw.get("local", 0))
    for rep in range(2):
        g = _gathered_grid(staged, rep, 0)
        assert np.array_equal(g, _gathered_grid(p2p, 0, 0))
        assert np.array_equal(g, H)


def test_staged_transport_synthetic_equals_p2p():
    import oracle
    import workloads
    dim = 600
    kw = dict(tsize=10, dsize=2)
    staged = _run("synthetic", dim, dict(kw, transport="nccl"), reps=2)
    p2p = _run("synthetic", dim, kw, reps=1)
    u, v, top, left = workloads.synthetic_inputs(dim, dim, 2)
    i0, i1, f = oracle.synthetic(u, v, top, left, 10)
    want = [i0, i1, f[0], f[1]]
    for rep in range(2):
        for p in range(4):
            g = _gathered_grid(staged, rep, p)
            assert np.array_equal(g.view(np.uint32), _gathered_grid(p2p, 0, p).view(np.uint32))
            assert np.array_equal(g.view(np.uint32), want[p].view(np.uint32))


def test_staged_transport_nash_equals_oracle():
    import oracle
    import workloads
    dim = 200
    staged = _run("nash", dim, dict(tsize=16, dsize=4, transport="nccl"), reps=2)
    r, c, top, left = workloads.nash_inputs(dim)
    ref = oracle.nash(r, c, top, left, nstrat=16)
    for rep in range(2):
        for p in range(4):
            assert np.array_equal(_gathered_grid(staged, rep, p), ref[p])
