"""Nash sweep timeline (WF_TRACE=1): west-value arrival at warp 0 of each band for every
(rows/32)-th row -> per-band lag at the start / middle / end of the sweep."""
import os, sys, json
import numpy as np, torch
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import workloads
from paper_conf_ppopp_mohantyc14_b200.wf import Wavefront
dev = torch.device("cuda", 0)
t = lambda a: torch.from_numpy(np.ascontiguousarray(a)).to(dev)
WARPS = int(os.environ.get("NASH_WARPS", "8"))
for cols in [int(x) for x in (sys.argv[1:] or ["64"])]:
    r, c, top, left = workloads.nash_inputs(4096, cols)
    ins = (t(r), t(c), [t(top[p]) for p in range(4)], [t(left[p]) for p in range(4)])
    wf = Wavefront("nash", 4096, cols=cols, tsize=16, dsize=4, warps=WARPS)
    out = wf.alloc_out()
    for _ in range(2): wf.run(*ins, out=out)
    wf.sync()
    tr = wf.debug_trace().astype(np.int64)
    arr = tr[:, :32] * 1.92                     # cycles (globaltimer ns * 1.92 GHz)
    lag = np.diff(arr, axis=0) if len(arr) > 1 else np.zeros((1, 32))
    rowstep = np.diff(arr, axis=1) / (4096 / 32)
    print(json.dumps({"cols": cols,
                      "lag_row1": [round(float(x)) for x in lag[:8, 0]],
                      "lag_row_mid": [round(float(x)) for x in lag[:8, 16]],
                      "lag_row_last": [round(float(x)) for x in lag[:8, 31]],
                      "rowstep_band0": [round(float(x)) for x in rowstep[0, ::4]],
                      "rowstep_band3": [round(float(x)) for x in rowstep[min(3, len(rowstep) - 1), ::4]]}))
    wf.close()
    if os.environ.get("WF_NASH_PROF_OUT"):
        print("phase cycles per row (prefix, wait, W-part+solve, out+handoff), band0 / band3:",
              [round(float(x) / 4096) for x in tr[0, 48:52]], [round(float(x) / 4096) for x in tr[min(3, len(tr) - 1), 48:52]])
