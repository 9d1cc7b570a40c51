"""Shared helpers of the GPU tests: run the CUDA path through the C ABI on numpy inputs.

These helpers only marshal data (numpy <-> torch CUDA tensors); they hold none of the
method's arithmetic and never call the oracle."""
from __future__ import annotations

import numpy as np
import torch

from paper_conf_ppopp_mohantyc14_b200.wf import LocalSlabs, Wavefront


def dev_inputs(fn, inputs, device):
    """inputs: seqcmp (x, y); synthetic (u, v, top, left); nash (r, c, top, left)."""
    def t(a):
        return torch.from_numpy(np.ascontiguousarray(a)).to(device)
    if fn == "seqcmp":
        x, y = inputs
        return t(x), t(y), None, None
    row, col, top, left = inputs
    tops = [t(top[p]) for p in range(top.shape[0])]
    lefts = [t(left[p]) for p in range(left.shape[0])]
    return t(row), t(col), tops, lefts


def run_gpu(fn, dim, inputs, cols=0, **kw):
    """One slab (or G local slabs when ngpus > 1) -> list of numpy planes (rows x cols)."""
    ngpus = kw.pop("ngpus", 1)
    devices = kw.pop("devices", None)
    dev = torch.device("cuda", torch.cuda.current_device())
    if ngpus == 1:
        with Wavefront(fn, dim, cols=cols, **kw) as w:
            row_in, col_in, top, left = dev_inputs(fn, inputs, dev)
            out = w.run(row_in, col_in, top, left)
            w.sync()
            return [o.cpu().numpy() for o in out]
    ls = LocalSlabs(fn, dim, ngpus, devices=devices, cols=cols, **kw)
    try:
        per = [dev_inputs(fn, inputs, torch.device("cuda", s.device)) for s in ls.slabs]
        outs = ls.run(per)
        ls.sync()
        planes = []
        for f in range(len(outs[0])):
            planes.append(np.concatenate([o[f].cpu().numpy() for o in outs], axis=1))
        return planes
    finally:
        ls.close()
