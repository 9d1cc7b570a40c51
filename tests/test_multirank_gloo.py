"""World-size-2 tests of the multi-GPU host logic on CPU (gloo backend, 127.0.0.1).

The data path (P2P edge stores between slabs) needs GPUs and is covered by the -m gpu
virtual-slab tests; here: the slab partition seen from separate processes, the IPC-handle
exchange that links slab g to g+1, and the max-over-ranks timing reduction
(paper_conf_ppopp_mohantyc14_b200/dist.py)."""
from __future__ import annotations

import os
import socket

import pytest

torch = pytest.importorskip("torch")
import torch.distributed as dist  # noqa: E402
import torch.multiprocessing as mp  # noqa: E402


def _free_port() -> int:
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        from paper_conf_ppopp_mohantyc14_b200 import dist as wdist
        res = {}
        for fn, dim, kw in (("seqcmp", 32768, dict(alphabet=4)), ("seqcmp", 1000, {}),
                            ("synthetic", 16384, dict(tsize=10, dsize=1)), ("nash", 4096, dict(tsize=16, dsize=4))):
            c0, c1 = wdist.slab_bounds(fn, dim, rank, world, **kw)
            allb = [None] * world
            dist.all_gather_object(allb, (c0, c1))
            res[(fn, dim)] = allb
        prev, nxt = wdist.neighbour_handles(f"handle-of-rank-{rank}".encode(), rank, world)
        res["handles"] = (prev, nxt)
        # connect-time validation: the same problem / tuning on every rank, consecutive slabs
        prob = (2, 1000, 0, 0, 0, 0, 1, -1, -1, 0, world)
        bounds = wdist.slab_bounds("seqcmp", 1000, rank, world)
        ok = wdist.exchange_handles(b"h%d" % rank, (prob, (2, 4, 1, 16, 0), bounds), rank, world)
        res["fp_ok"] = ok
        verdicts = []
        for bad in ("strip", "bounds"):
            tun = (2, 4, 1, 32 if (bad == "strip" and rank == 1) else 16, 0)
            b = (bounds[0] + (1 if bad == "bounds" and rank == 1 else 0), bounds[1])
            try:
                wdist.exchange_handles(b"h%d" % rank, (prob, tun, b), rank, world)
                verdicts.append("accepted")
            except ValueError as e:
                verdicts.append(str(e)[:40])
        res["fp_bad"] = verdicts
        res["max"] = wdist.max_over_ranks(1.5 * rank + 0.25)
        q.put((rank, res))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world", [2])
def test_two_rank_slab_partition_handles_and_max(world):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, q)) for r in range(world)]
    for p in procs:
        p.start()
    out = dict(q.get(timeout=120) for _ in range(world))
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    for rank in range(world):
        r = out[rank]
        for (fn, dim), bounds in ((k, v) for k, v in r.items() if isinstance(k, tuple)):
            # every rank sees the same partition; slabs tile [0, dim) in rank order
            assert bounds == out[0][(fn, dim)]
            assert bounds[0][0] == 0 and bounds[-1][1] == dim
            assert all(bounds[g][1] == bounds[g + 1][0] for g in range(world - 1))
        prev, nxt = r["handles"]
        assert prev == (None if rank == 0 else f"handle-of-rank-{rank - 1}".encode())
        assert nxt == (None if rank == world - 1 else f"handle-of-rank-{rank + 1}".encode())
        assert r["max"] == 1.5 * (world - 1) + 0.25
        assert r["fp_ok"] == ((None if rank == 0 else b"h%d" % (rank - 1)), (None if rank == world - 1 else b"h%d" % (rank + 1)))
        # every rank refuses (the same verdict on both sides of the link)
        assert r["fp_bad"][0].startswith("rank 1 uses a different tuning")
        assert r["fp_bad"][1].startswith("slab 0 ends at column")


def test_check_fingerprints_single_process():
    from paper_conf_ppopp_mohantyc14_b200.dist import check_fingerprints
    prob, tun = (2, 100, 0, 0, 0, 0, 1, -1, -1, 0, 3), (2, 4, 1, 16, 0)
    check_fingerprints([(prob, tun, (0, 40)), (prob, tun, (40, 80)), (prob, tun, (80, 100))])
    for fps, msg in (([(prob, tun, (0, 40)), (prob[:1] + (101,) + prob[2:], tun, (40, 100))], "problem"),
                     ([(prob, tun, (0, 40)), (prob, (2, 4, 1, 8, 0), (40, 100))], "tuning"),
                     ([(prob, tun, (0, 40)), (prob, tun, (50, 100))], "ends at column"),
                     ([(prob, tun, (5, 40)), (prob, tun, (40, 100))], "starts at column")):
        with pytest.raises(ValueError, match=msg):
            check_fingerprints(fps)


def _staged_worker(rank, world, port, q):
    """transport="nccl" host sequencing (dist.staged_sequence) over gloo: each rank's 'sweep' adds
    its rank to every byte of the message it imported, so the last rank sees the chain's sum only
    if every message was received, imported, run, exported and sent in order."""
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        from paper_conf_ppopp_mohantyc14_b200 import dist as wdist
        state = {"in": torch.zeros(64, dtype=torch.uint8), "ring": None, "log": []}

        def recv(n):
            m = torch.empty(n, dtype=torch.uint8)
            dist.recv(m, src=rank - 1)
            state["log"].append("recv")
            return m

        def edge_import(m):
            state["in"] = m.clone()
            state["log"].append("import")

        def run():   # a pure function of this run's inputs, like the sweep
            state["ring"] = state["in"] + (rank + 1)
            state["log"].append("run")
            return state["ring"].clone()

        def edge_export(n):
            state["log"].append("export")
            return state["ring"][:n].clone()

        def send(m):
            dist.send(m, dst=rank + 1)
            state["log"].append("send")

        outs = [wdist.staged_sequence(rank, world, 64, recv=recv, edge_import=edge_import, run=run,
                                      edge_export=edge_export, send=send) for _ in range(2)]
        q.put((rank, (state["log"], [int(o[0]) for o in outs])))
    except Exception as e:  # noqa: BLE001
        q.put((rank, repr(e)))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world", [2, 3])
def test_staged_transport_sequence_gloo(world):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_staged_worker, args=(r, world, port, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = dict(q.get(timeout=300) for _ in range(world))
    for p in procs:
        p.join(timeout=60)
    for r in range(world):
        assert not isinstance(res[r], str), res[r]
        log, vals = res[r]
        one = (["recv", "import"] if r > 0 else []) + ["run"] + (["export", "send"] if r < world - 1 else [])
        assert log == one * 2
        # run k of rank r sees the sum 1 + 2 + ... + (r + 1) (each run re-imports a fresh message)
        assert vals == [sum(range(1, r + 2))] * 2
