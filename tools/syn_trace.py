"""WF_TRACE timeline of a synthetic config (not a test): per band the time its first compute warp
had row 1 available (trace slot 0 / 44+w) and finished (slot 52+w); band hop statistics.

    WF_TRACE=1 python tools/syn_trace.py [C5a]
"""
import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
os.environ["WF_TRACE"] = "1"
import torch  # noqa: E402

import workloads  # noqa: E402
from paper_conf_ppopp_mohantyc14_b200.wf import Wavefront  # noqa: E402

cfg = workloads.CONFIGS[sys.argv[1] if len(sys.argv) > 1 else "C5a"]
dev = torch.device("cuda", 0)
u, v, top, left = workloads.synthetic_inputs(cfg.dim, cfg.dim, cfg.dsize)
t = lambda a: torch.from_numpy(np.ascontiguousarray(a)).to(dev)  # noqa: E731
with Wavefront("synthetic", cfg.dim, tsize=cfg.tsize, dsize=cfg.dsize) as w:
    args = (t(u), t(v), [t(top[d]) for d in range(cfg.dsize)], [t(left[d]) for d in range(cfg.dsize)])
    out = w.alloc_out()
    for _ in range(3):
        w.run(*args, out=out)
    w.sync()
    ms = w.last_run_ms()
    tr = w.debug_trace().astype(np.int64)
    lay = w.layout
start = tr[:, 0]
end = tr[:, 52]
t0 = start.min()
print(f"{cfg.name}: run {ms:.3f} ms, bands {lay.nbands}, band_cols {lay.band_cols}")
hop = np.diff(start) / 1e3
print(f"band start hop (us): median {np.median(hop):.3f}, mean {hop.mean():.3f}, p10 {np.percentile(hop, 10):.3f}, p90 {np.percentile(hop, 90):.3f}")
sweep = (end - start) / 1e3
print(f"band sweep (us): first {sweep[0]:.1f}, median {np.median(sweep):.1f}, last {sweep[-1]:.1f}")
print(f"last band starts at {(start[-1] - t0) / 1e3:.1f} us, ends at {(end[-1] - t0) / 1e3:.1f} us")
