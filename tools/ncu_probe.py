"""Tiny driver for ncu captures: a few wf_run launches of one config (no timing)."""
import os, sys
import numpy as np
import torch
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import workloads
from paper_conf_ppopp_mohantyc14_b200.wf import Wavefront

fn = sys.argv[1] if len(sys.argv) > 1 else "seqcmp"
dim = int(sys.argv[2]) if len(sys.argv) > 2 else 4096
k, w, d = (int(s) for s in (sys.argv[3] if len(sys.argv) > 3 else "4,2,2").split(","))
reps = int(sys.argv[4]) if len(sys.argv) > 4 else 3
tsize = int(sys.argv[5]) if len(sys.argv) > 5 else 0
dsize = int(sys.argv[6]) if len(sys.argv) > 6 else 0
cols = int(sys.argv[7]) if len(sys.argv) > 7 else 0
kernel = int(sys.argv[8]) if len(sys.argv) > 8 else 0
strip = int(sys.argv[9]) if len(sys.argv) > 9 else 0
dev = torch.device("cuda", 0)
t = lambda a: torch.from_numpy(np.ascontiguousarray(a)).to(dev)
if fn == "seqcmp":
    x, y = workloads.seqcmp_inputs(dim, cols or dim); ins = (t(x), t(y), None, None); kw = {}
elif fn == "nash":
    r, c, top, left = workloads.nash_inputs(dim, cols or dim)
    ins = (t(r), t(c), [t(top[i]) for i in range(4)], [t(left[i]) for i in range(4)])
    kw = dict(tsize=tsize or 16, dsize=4)
else:
    u, v, top, left = workloads.synthetic_inputs(dim, cols or dim, dsize)
    ins = (t(u), t(v), [t(top[i]) for i in range(dsize)], [t(left[i]) for i in range(dsize)])
    kw = dict(tsize=tsize, dsize=dsize)
wf = Wavefront(fn, dim, cols=cols, lane_cols=k, warps=w, skew=d, watchdog_cycles=1 << 42, kernel=kernel, strip=strip, **({"alphabet": 4} if fn == "seqcmp" else {}), **kw)
out = wf.alloc_out()
for _ in range(reps):
    wf.run(*ins, out=out)
wf.sync()
print("done", wf.last_run_ms())
