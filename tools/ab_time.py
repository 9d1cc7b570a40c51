"""Interleaved A/B timing of libwf builds on one config (not a test): each round runs every build
once in a fresh process (median of N timed wf_runs after 3 warm-ups, CUDA events), rounds
alternate the order, so box-to-box and drift effects hit every build alike.

    python tools/ab_time.py [--config C4] [--rounds 3] [--runs 10] NAME=path/libwf.so ...
    (path '-' = the in-tree paper_conf_ppopp_mohantyc14_b200/libwf.so)
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))

CHILD = r'''
import json, os, statistics, sys
sys.path.insert(0, {root!r})
from paper_conf_ppopp_mohantyc14_b200 import _abi
if {lib!r} != "-":
    _abi.LIB_PATH = os.path.abspath({lib!r})
import numpy as np, torch, workloads
from paper_conf_ppopp_mohantyc14_b200.wf import Wavefront
cfg = workloads.CONFIGS[{cfg!r}]
dev = torch.device("cuda", 0)
if cfg.fn == "seqcmp":
    x, y = workloads.seqcmp_inputs(cfg.dim)
    ins = [torch.from_numpy(x).to(dev), torch.from_numpy(y).to(dev)]
    tops = lefts = None
    kw = dict(alphabet=4)
else:
    u, v, top, left = workloads.synthetic_inputs(cfg.dim, cfg.dim, cfg.dsize)
    ins = [torch.from_numpy(u).to(dev), torch.from_numpy(v).to(dev)]
    tops = [torch.from_numpy(np.ascontiguousarray(top[p])).to(dev) for p in range(cfg.dsize)]
    lefts = [torch.from_numpy(np.ascontiguousarray(left[p])).to(dev) for p in range(cfg.dsize)]
    kw = dict(tsize=cfg.tsize, dsize=cfg.dsize)
with Wavefront(cfg.fn, cfg.dim, **kw) as w:
    out = w.alloc_out()
    ms = []
    for i in range({runs} + 3):
        w.run(ins[0], ins[1], tops, lefts, out=out)
        w.sync()
        if i >= 3:
            ms.append(w.last_run_ms())
print(json.dumps(dict(median=statistics.median(ms), min=min(ms))))
'''


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--config", default="C4")
    ap.add_argument("--rounds", type=int, default=3)
    ap.add_argument("--runs", type=int, default=10)
    ap.add_argument("builds", nargs="+")
    a = ap.parse_args()
    builds = [b.split("=", 1) for b in a.builds]
    res = {n: [] for n, _ in builds}
    for rnd in range(a.rounds):
        order = builds if rnd % 2 == 0 else builds[::-1]
        for name, lib in order:
            code = CHILD.format(root=ROOT, lib=lib, cfg=a.config, runs=a.runs)
            out = subprocess.run([sys.executable, "-c", code], capture_output=True, text=True, timeout=600)
            try:
                res[name].append(json.loads(out.stdout.strip().splitlines()[-1])["median"])
            except Exception:
                print(name, "failed:", out.stderr[-500:], flush=True)
    for name, v in res.items():
        if v:
            print(f"{name:12s} median {statistics.median(v):.4f} ms  runs {' '.join(f'{x:.4f}' for x in v)}")


if __name__ == "__main__":
    main()
