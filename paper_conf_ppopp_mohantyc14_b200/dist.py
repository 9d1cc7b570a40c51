"""Multi-GPU plumbing of the column-slab pipeline.

One process per GPU; rank g owns column slab g (PAPER.md P:238-255 distributes the grid over
GPUs; here the slabs are consecutive column blocks and the only exchange is the west edge
g -> g+1, stored by the kernel straight into the successor's ring over NVLink).  torch's
process group carries only the setup traffic: the CUDA IPC handles of the edge rings and the
max-over-ranks reduction of the timings.  These helpers hold that host-side logic so it can
be exercised with the gloo backend on CPU (tests/test_multirank_gloo.py).
"""
from __future__ import annotations

import torch
import torch.distributed as dist

from .wf import query


def slab_bounds(fn: str, dim: int, rank: int, world: int, **kw) -> tuple[int, int]:
    """[c0, c1) interior columns of rank's slab (the library's wf_query partition)."""
    lay = query(fn, dim, rank=rank, ngpus=world, **kw)
    return lay.col_begin, lay.col_end


def neighbour_handles(my_handle: bytes, rank: int, world: int, group=None) -> tuple[bytes | None, bytes | None]:
    """All-gather every rank's edge-ring IPC handle; return (handle of rank-1, handle of rank+1)."""
    handles: list = [None] * world
    dist.all_gather_object(handles, bytes(my_handle), group=group)
    prev = handles[rank - 1] if rank > 0 else None
    nxt = handles[rank + 1] if rank < world - 1 else None
    return prev, nxt


def max_over_ranks(x: float, device=None, group=None) -> float:
    """Max of a per-rank time (ms) over all ranks (BASELINE timing rule: max over ranks)."""
    t = torch.tensor([float(x)], dtype=torch.float64, device=device)
    dist.all_reduce(t, op=dist.ReduceOp.MAX, group=group)
    return float(t.item())


def connect_slab(w, rank: int, world: int, group=None) -> None:
    """Link a rank's Wavefront context to its neighbours' edge rings (wf_connect)."""
    prev, nxt = neighbour_handles(w.ipc_handle(), rank, world, group)
    w.connect(prev, nxt)
