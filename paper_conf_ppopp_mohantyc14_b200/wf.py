"""Python binding of libwf (include/wf.h): argument marshalling only.

Every step of the sweep runs in the CUDA library; this module turns torch tensors
(device memory, streams) into the C-ABI's plain pointers.  PAPER.md P:127-136: the
pattern's API "requires the programmer to code only application specific aspects" --
here the caller names the cell function and the Table 1 features (dim, tsize, dsize).
"""
from __future__ import annotations

import ctypes
from dataclasses import dataclass

import torch

from . import _abi
from ._abi import WfDist, WfIo, WfLayout, WfParams, check

_TRANSPORTS = {"p2p": _abi.WF_TRANSPORT_P2P, "nccl": _abi.WF_TRANSPORT_NCCL}


@dataclass
class Layout:
    nplanes: int
    plane_is_float: list
    nbound: int
    col_begin: int
    col_end: int
    min_pitch: int
    bytes_out: int
    lane_cols: int
    warps: int
    skew: int
    band_cols: int
    nbands: int
    strip: int = 0   # rows per hand-off block (generation 8); 0 = fixed by the generation

    @property
    def width(self) -> int:
        return self.col_end - self.col_begin


def make_params(fn, dim, *, cols=0, tsize=0, dsize=0, lane_cols=0, warps=0, skew=0, strip=0, ngpus=1,
                match=0, mismatch=0, gap=0, local=0, transport="p2p", max_ctas=0, watchdog_cycles=0,
                alphabet=0, kernel=0, halo=0) -> WfParams:
    p = WfParams()
    p.dim = int(dim)
    p.cols = int(cols)
    p.fn = _abi.FN_IDS[fn] if isinstance(fn, str) else int(fn)
    p.tsize = int(tsize)
    p.dsize = int(dsize)
    p.lane_cols = int(lane_cols)
    p.warps = int(warps)
    p.skew = int(skew)
    p.strip = int(strip)
    p.ngpus = int(ngpus)
    p.match, p.mismatch, p.gap = int(match), int(mismatch), int(gap)
    p.local = int(local)
    p.transport = _TRANSPORTS[transport] if isinstance(transport, str) else int(transport)
    p.max_ctas = int(max_ctas)
    p.watchdog_cycles = int(watchdog_cycles)
    p.alphabet = int(alphabet)
    p.kernel = int(kernel)
    p.halo = int(halo)
    return p


def query(fn, dim, rank: int = 0, **kw) -> Layout:
    p = make_params(fn, dim, **kw)
    lay = WfLayout()
    check(_abi.lib().wf_query(ctypes.byref(p), int(rank), ctypes.byref(lay)))
    return Layout(lay.nplanes, [bool(lay.plane_is_float[i]) for i in range(lay.nplanes)], lay.nbound,
                  lay.col_begin, lay.col_end, lay.min_pitch, lay.bytes_out, lay.lane_cols, lay.warps,
                  lay.skew, lay.band_cols, lay.nbands, lay.strip)


def _stream_handle(stream) -> int:
    if stream is None:
        stream = torch.cuda.current_stream()
    return int(stream.cuda_stream)


class Wavefront:
    """One column slab of a wavefront instance on one GPU (a libwf context).

    fn: 'seqcmp' | 'synthetic' | 'nash'; dim, tsize, dsize: PAPER.md Table 1.
    Tunables replace the paper's Table 2: lane_cols, warps, skew, strip, ngpus.
    """

    def __init__(self, fn, dim, *, rank: int = 0, device: int | None = None, device_share: int = 1, **kw):
        self.fn = fn
        self.params = make_params(fn, dim, **kw)
        self.rank = int(rank)
        self.world = max(1, self.params.ngpus)
        self.device = torch.cuda.current_device() if device is None else int(device)
        self.layout = query(fn, dim, rank=self.rank, **kw)
        dist = WfDist(self.rank, self.world, self.device, int(device_share))
        ctx = ctypes.c_void_p()
        with torch.cuda.device(self.device):
            check(_abi.lib().wf_create(ctypes.byref(self.params), ctypes.byref(dist) if self.world > 1 or device is not None
                                       or device_share > 1 else None, ctypes.byref(ctx)))
        self._ctx = ctx

    # ---- buffers
    def alloc_out(self) -> list:
        """Output planes for this slab: (rows, width) views of (rows, min_pitch) allocations."""
        rows, pitch, width = self.params.dim, self.layout.min_pitch, self.layout.width
        dev = torch.device("cuda", self.device)
        planes = []
        for f in range(self.layout.nplanes):
            dt = torch.float32 if self.layout.plane_is_float[f] else torch.int32
            planes.append(torch.empty((rows, pitch), dtype=dt, device=dev)[:, :width])
        return planes

    def _io(self, row_in, col_in, top, left, out) -> WfIo:
        io = WfIo()
        io.row_in = row_in.data_ptr()
        io.col_in = col_in.data_ptr()
        for b in range(self.layout.nbound):
            io.top[b] = top[b].data_ptr()
            io.left[b] = left[b].data_ptr()
        pitch = None
        for f, t in enumerate(out):
            if t.stride(1) != 1:
                raise ValueError("output planes must be row-major with unit column stride")
            if pitch is None:
                pitch = t.stride(0)
            elif t.stride(0) != pitch:
                raise ValueError("all output planes must share one pitch")
            io.out[f] = t.data_ptr()
        io.out_pitch = int(pitch)
        return io

    def run(self, row_in: torch.Tensor, col_in: torch.Tensor, top=None, left=None, out=None, stream=None):
        """Enqueue one sweep (asynchronous).  Returns the output planes."""
        if out is None:
            out = self.alloc_out()
        for t in (row_in, col_in, *(top or []), *(left or []), *out):
            if not t.is_cuda or t.device.index != self.device:
                raise ValueError(f"all buffers must be CUDA tensors on device {self.device}")
        io = self._io(row_in, col_in, top, left, out)
        with torch.cuda.device(self.device):
            check(_abi.lib().wf_run(self._ctx, ctypes.byref(io), ctypes.c_void_p(_stream_handle(stream))), self._ctx)
        return out

    def sync(self) -> None:
        check(_abi.lib().wf_sync(self._ctx), self._ctx)

    def local_best(self) -> tuple[int, int, int]:
        """Smith-Waterman (local=1): (best score, 1-based row, 1-based global column) of the
        first cell in row-major order holding it, from the last run (wf_local_best)."""
        v, r, c = ctypes.c_int32(), ctypes.c_int32(), ctypes.c_int32()
        check(_abi.lib().wf_local_best(self._ctx, ctypes.byref(v), ctypes.byref(r), ctypes.byref(c)), self._ctx)
        return int(v.value), int(r.value), int(c.value)

    def last_run_ms(self) -> float:
        ms = ctypes.c_float()
        check(_abi.lib().wf_last_run_ms(self._ctx, ctypes.byref(ms)), self._ctx)
        return float(ms.value)

    def debug_trace(self):
        """(nbands, slots) uint64 timeline of the last run (needs WF_TRACE=1 at run time)."""
        import numpy as np
        buf = np.zeros((self.layout.nbands, 64), dtype=np.uint64)
        slots = ctypes.c_int32()
        check(_abi.lib().wf_debug_trace(self._ctx, buf.ctypes.data, buf.nbytes, ctypes.byref(slots)), self._ctx)
        buf = np.zeros((self.layout.nbands, slots.value), dtype=np.uint64)
        check(_abi.lib().wf_debug_trace(self._ctx, buf.ctypes.data, buf.nbytes, ctypes.byref(slots)), self._ctx)
        return buf

    # ---- multi-slab plumbing
    def link(self, nxt: "Wavefront") -> None:
        check(_abi.lib().wf_link_local(self._ctx, nxt._ctx), self._ctx)

    def ipc_handle(self) -> bytes:
        buf = ctypes.create_string_buffer(_abi.WF_IPC_HANDLE_BYTES)
        check(_abi.lib().wf_ipc_handle(self._ctx, buf), self._ctx)
        return buf.raw

    def connect(self, prev_handle: bytes | None, next_handle: bytes | None) -> None:
        """Open rank-1's and rank+1's exchange buffers (IPC handles from ipc_handle())."""
        bufs = [None if h is None else ctypes.create_string_buffer(bytes(h), _abi.WF_IPC_HANDLE_BYTES)
                for h in (prev_handle, next_handle)]
        with torch.cuda.device(self.device):
            check(_abi.lib().wf_connect(self._ctx, bufs[0], bufs[1]), self._ctx)

    # ---- transport = "nccl": host-staged slab edges (wf_edge_export / wf_edge_import)
    def edge_bytes(self) -> int:
        n = ctypes.c_size_t()
        check(_abi.lib().wf_edge_bytes(self._ctx, ctypes.byref(n)), self._ctx)
        return int(n.value)

    def edge_export(self, dst: torch.Tensor, stream=None) -> None:
        """Enqueue a copy of the east edge of this slab's last run into `dst` (>= edge_bytes())."""
        if dst.numel() * dst.element_size() < self.edge_bytes() or not dst.is_contiguous():
            raise ValueError("edge_export: dst must be contiguous and hold edge_bytes() bytes")
        with torch.cuda.device(self.device):
            check(_abi.lib().wf_edge_export(self._ctx, ctypes.c_void_p(dst.data_ptr()),
                                            ctypes.c_void_p(_stream_handle(stream))), self._ctx)

    def edge_import(self, src: torch.Tensor, stream=None) -> None:
        """Enqueue a copy of the predecessor's exported edge `src` into this slab's inbound ring."""
        if src.numel() * src.element_size() < self.edge_bytes() or not src.is_contiguous():
            raise ValueError("edge_import: src must be contiguous and hold edge_bytes() bytes")
        with torch.cuda.device(self.device):
            check(_abi.lib().wf_edge_import(self._ctx, ctypes.c_void_p(src.data_ptr()),
                                            ctypes.c_void_p(_stream_handle(stream))), self._ctx)

    def close(self) -> None:
        if getattr(self, "_ctx", None) is not None and self._ctx.value:
            _abi.lib().wf_destroy(self._ctx)
            self._ctx = ctypes.c_void_p()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def __enter__(self):
        return self

    def __exit__(self, *a):
        self.close()


def to_device(arrays, device) -> list:
    """numpy arrays -> contiguous CUDA tensors (input staging; not part of the sweep)."""
    out = []
    for a in arrays:
        out.append(torch.from_numpy(a).to(device=device, non_blocking=False).contiguous())
    return out


class LocalSlabs:
    """G slabs in ONE process: one context per slab, linked slab g -> g+1.

    devices: list of CUDA ordinals (len G).  Several slabs may share one device ("virtual
    GPUs"): they run concurrently on separate streams, each with 1/share of the
    resident CTAs, and exchange edges through the same rings as real GPUs.  Slabs are launched
    in slab order, so when streams share a hardware queue a slab can only wait behind a LOWER
    slab, which never waits on it -- no deadlock; but with 8 or more slabs per device set
    CUDA_DEVICE_MAX_CONNECTIONS=32 before CUDA initialises, or a slab may start only after an
    earlier slab's whole run (C4, 8 virtual slabs: 2.71 vs 2.01 ms)."""

    def __init__(self, fn, dim, ngpus: int, devices=None, **kw):
        devices = list(devices) if devices is not None else [torch.cuda.current_device()] * ngpus
        assert len(devices) == ngpus
        share = {d: devices.count(d) for d in devices}
        self.slabs = [Wavefront(fn, dim, rank=g, device=devices[g], device_share=share[devices[g]], ngpus=ngpus, **kw)
                      for g in range(ngpus)]
        for g in range(ngpus - 1):
            self.slabs[g].link(self.slabs[g + 1])
        self.streams = [torch.cuda.Stream(device=d) for d in devices]

    def run(self, inputs_per_device, outs=None):
        """inputs_per_device[g] = (row_in, col_in, top, left) on slab g's device."""
        outs = outs or [s.alloc_out() for s in self.slabs]
        for g, s in enumerate(self.slabs):
            self.streams[g].wait_stream(torch.cuda.current_stream(s.device))
        for g, s in enumerate(self.slabs):
            row_in, col_in, top, left = inputs_per_device[g]
            s.run(row_in, col_in, top, left, out=outs[g], stream=self.streams[g])
        return outs

    def sync(self):
        for s in self.slabs:
            s.sync()

    def close(self):
        for s in self.slabs:
            s.close()
