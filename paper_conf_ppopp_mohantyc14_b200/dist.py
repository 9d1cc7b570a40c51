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


def slab_fingerprint(w) -> tuple:
    """What every rank must agree on before wf_connect: the problem and the tuning (equal on all
    ranks) and this slab's column range (consecutive across ranks).  wf_link_local checks the same
    in C for slabs of one process; across processes the IPC handle carries only memory."""
    p, lay = w.params, w.layout
    problem = (int(p.fn), int(p.dim), int(p.cols), int(p.tsize), int(p.dsize), int(p.local), int(p.match),
               int(p.mismatch), int(p.gap), int(p.alphabet), int(p.ngpus))
    tuning = (int(lay.lane_cols), int(lay.warps), int(lay.skew), int(lay.strip), int(p.kernel))
    return problem, tuning, (int(lay.col_begin), int(lay.col_end))


def check_fingerprints(fps: list) -> None:
    """Raise ValueError unless all ranks describe the same problem and tuning and their slabs are
    consecutive column blocks covering [0, cols)."""
    for g, (prob, tun, _) in enumerate(fps):
        if prob != fps[0][0]:
            raise ValueError(f"rank {g} describes a different problem than rank 0: {prob} vs {fps[0][0]}")
        if tun != fps[0][1]:
            raise ValueError(f"rank {g} uses a different tuning than rank 0: {tun} vs {fps[0][1]}")
    if fps[0][2][0] != 0:
        raise ValueError(f"rank 0 starts at column {fps[0][2][0]}")
    for g in range(1, len(fps)):
        if fps[g][2][0] != fps[g - 1][2][1]:
            raise ValueError(f"slab {g - 1} ends at column {fps[g - 1][2][1]} but slab {g} starts at {fps[g][2][0]}")


def exchange_handles(my_handle: bytes, fingerprint: tuple, rank: int, world: int,
                     group=None) -> tuple[bytes | None, bytes | None]:
    """All-gather (handle, fingerprint) of every rank, validate the fingerprints
    (check_fingerprints, identical verdict on every rank), return (handle of rank-1, of rank+1)."""
    recs: list = [None] * world
    dist.all_gather_object(recs, (bytes(my_handle), fingerprint), group=group)
    check_fingerprints([r[1] for r in recs])
    prev = recs[rank - 1][0] if rank > 0 else None
    nxt = recs[rank + 1][0] if rank < world - 1 else None
    return prev, nxt


def max_over_ranks(x: float, device=None, group=None) -> float:
    """Max of a per-rank time (ms) over all ranks (BASELINE timing rule: max over ranks)."""
    t = torch.tensor([float(x)], dtype=torch.float64, device=device)
    dist.all_reduce(t, op=dist.ReduceOp.MAX, group=group)
    return float(t.item())


def connect_slab(w, rank: int, world: int, group=None) -> None:
    """Link a rank's Wavefront context to its neighbours' edge rings (wf_connect), after checking
    that all ranks agree on problem, tuning and slab adjacency (ValueError otherwise)."""
    prev, nxt = exchange_handles(w.ipc_handle(), slab_fingerprint(w), rank, world, group)
    w.connect(prev, nxt)


def staged_sequence(rank: int, world: int, nbytes: int, *, recv, edge_import, run, edge_export, send):
    """The host-staged slab chain of one run (transport="nccl"): rank g > 0 receives rank g-1's
    edge message (nbytes) and imports it before its sweep; rank g < G-1 exports its east edge
    after the sweep and sends it to g+1.  The callables carry the data movement, so the ordering
    is testable with gloo on CPU (tests/test_multirank_gloo.py).  Returns run()'s result."""
    if rank > 0:
        edge_import(recv(nbytes))
    out = run()
    if rank < world - 1:
        send(edge_export(nbytes))
    return out


def staged_run(w, args, rank: int, world: int, group=None, comm_device=None, stream=None, out=None):
    """One wf_run of a transport="nccl" slab (SURVEY.md §8(a) a8 fallback): receive
    rank-1's edge message, import it, sweep, export this slab's east edge and send it to rank+1.
    The slabs therefore run one after another -- the host-staged halo swap of P:247-253 over the
    process group (NCCL on the GPU box; gloo with CPU buffers in the tests), not pipelined.

    comm_device: where the message lives for send/recv (None = the slab's CUDA device, as NCCL
    needs; "cpu" for gloo).  Returns the output planes."""
    dev = torch.device("cuda", w.device)
    cdev = dev if comm_device is None else torch.device(comm_device)

    def recv(n):
        msg = torch.empty(n, dtype=torch.uint8, device=cdev)
        dist.recv(msg, src=rank - 1, group=group)
        return msg

    def edge_import(msg):
        w.edge_import(msg if msg.device == dev else msg.to(dev), stream)

    def edge_export(n):
        buf = torch.empty(n, dtype=torch.uint8, device=dev)
        w.edge_export(buf, stream)
        (torch.cuda.current_stream(dev) if stream is None else stream).synchronize()   # the send reads buf
        return buf

    def send(buf):
        dist.send(buf if cdev == dev else buf.to(cdev), dst=rank + 1, group=group)

    return staged_sequence(rank, world, w.edge_bytes(), recv=recv, edge_import=edge_import,
                           run=lambda: w.run(*args, out=out, stream=stream), edge_export=edge_export, send=send)
