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
