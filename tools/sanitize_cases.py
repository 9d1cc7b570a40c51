"""Small instances of every kernel family, each checked against the CPU oracle -- the workload of
the compute-sanitizer runs (profiles/r02_sanitizer.txt):

    compute-sanitizer --tool memcheck|racecheck|synccheck python tools/sanitize_cases.py CASE
    python tools/sanitize_cases.py --list

Each case prints "CASE ok" or raises.  Sizes are small (the sanitizers instrument every
shared / global access of spinning warps) but still span several bands and ring laps.
"""
from __future__ import annotations

import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tests"))

if os.environ.get("WF_PROBE_LIB"):   # the jitter / sanitizer build (tools/xbuild_jitter.sh)
    from paper_conf_ppopp_mohantyc14_b200 import _abi
    _abi.LIB_PATH = os.path.abspath(os.environ["WF_PROBE_LIB"])

CASES = {
    # name: (fn, dim, kwargs)
    "nw8": ("seqcmp", 300, {}),
    "nw8_sw": ("seqcmp", 300, {"local": 1}),
    "nw8_k4w2": ("seqcmp", 300, {"lane_cols": 4, "warps": 2, "kernel": 8}),
    "nw8_slabs2": ("seqcmp", 300, {"ngpus": 2}),
    "nw4": ("seqcmp", 300, {"lane_cols": 4, "warps": 2, "kernel": 4, "alphabet": 4}),
    "nw4_sw": ("seqcmp", 300, {"lane_cols": 4, "warps": 1, "skew": 2, "local": 1}),
    "syn_d1_t10": ("synthetic", 200, {"tsize": 10, "dsize": 1}),
    "syn_d5_t1000": ("synthetic", 80, {"tsize": 1000, "dsize": 5}),
    "syn_plane_split": ("synthetic", 150, {"tsize": 7, "dsize": 3, "kernel": 8, "lane_cols": 1, "warps": 1,
                                           "skew": 1}),
    "syn_generic": ("synthetic", 150, {"tsize": 5, "dsize": 2, "kernel": 4}),
    "syn_slabs2": ("synthetic", 150, {"tsize": 3, "dsize": 2, "ngpus": 2}),
    "nash": ("nash", 40, {"tsize": 16, "dsize": 4}),
    "nw8_halo": ("seqcmp", 1100, {"ngpus": 2, "halo": 256}),
    "nw8_staged": ("seqcmp", 600, {"ngpus": 2, "transport": "nccl"}),
    "syn_staged": ("synthetic", 150, {"tsize": 3, "dsize": 2, "ngpus": 2, "transport": "nccl"}),
}


def run_staged_in_process(fn, dim, inputs, **kw):
    """transport="nccl" slabs in ONE process: each slab's edge message is exported into a device
    buffer and imported by its successor (the copy the process group's send/recv makes between
    ranks), slabs run in order; returns the concatenated planes."""
    import torch
    from _gpu_helpers import dev_inputs
    from paper_conf_ppopp_mohantyc14_b200.wf import Wavefront
    G = kw.pop("ngpus")
    dev = torch.device("cuda", torch.cuda.current_device())
    slabs = [Wavefront(fn, dim, rank=g, device=dev.index, ngpus=G, **kw) for g in range(G)]
    try:
        args = dev_inputs(fn, inputs, dev)
        outs, msg = [], None
        for g, w in enumerate(slabs):
            if g > 0:
                w.edge_import(msg)
            outs.append(w.run(*args))
            if g < G - 1:
                msg = torch.empty(w.edge_bytes(), dtype=torch.uint8, device=dev)
                w.edge_export(msg)
        torch.cuda.synchronize()
        for w in slabs:
            w.sync()
        return [np.concatenate([o[f].cpu().numpy() for o in outs], axis=1) for f in range(len(outs[0]))]
    finally:
        for w in slabs:
            w.close()


def run(name):
    import oracle
    import workloads
    from _gpu_helpers import run_gpu
    fn, dim, kw = CASES[name]
    kw = dict(kw)
    runner = run_staged_in_process if kw.get("transport") == "nccl" else run_gpu
    if fn == "seqcmp":
        x, y = workloads.seqcmp_inputs(dim)
        want = [oracle.seqcmp(x, y, 1, -1, -1, local=bool(kw.get("local", 0)))]
        got = runner(fn, dim, (x, y), **kw)
    elif fn == "synthetic":
        u, v, top, left = workloads.synthetic_inputs(dim, dim, kw["dsize"])
        i0, i1, f = oracle.synthetic(u, v, top, left, kw["tsize"])
        want = [i0, i1] + [f[d] for d in range(f.shape[0])]
        got = runner(fn, dim, (u, v, top, left), **kw)
    else:
        r, c, top, left = workloads.nash_inputs(dim, dim)
        o = oracle.nash(r, c, top, left, nstrat=kw["tsize"])
        want = [o[p] for p in range(4)]
        got = runner(fn, dim, (r, c, top, left), **kw)
    for p, (g, o) in enumerate(zip(got, want)):
        o = np.asarray(o)
        g = np.asarray(g).view(o.dtype)
        assert np.array_equal(g.view(np.uint32), o.view(np.uint32)), f"{name}: plane {p} differs from the oracle"
    print(f"{name} ok", flush=True)


if __name__ == "__main__":
    if sys.argv[1] == "--list":
        print(" ".join(CASES))
    else:
        for n in sys.argv[1:]:
            run(n)
