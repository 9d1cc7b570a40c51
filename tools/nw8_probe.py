"""Diagnostics for the generation-8 NW sweep on one GPU (not a test):

  * parity probes: run (dim, lane_cols, warps) cases against the oracle and print where the
    first mismatches sit (row, column, band / warp / lane of the column);
  * timeline: run C4 with WF_TRACE=1 and summarise per band / warp start lags, sweep cycles
    per step and slow-path counts (wf_nw8.cu trace slots).

    python tools/nw8_probe.py parity 777:2:2 777:2:4 ...
    WF_TRACE=1 python tools/nw8_probe.py trace [dim] [lane_cols] [warps] [strip] [kernel]
    WF_PROBE_LIB=tools/abl_out/libwf_X.so ...      (an A/B build of tools/xbuild8.sh)
"""
from __future__ import annotations

import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tests"))

if os.environ.get("WF_PROBE_LIB"):   # A/B builds from tools/xbuild8.sh (the product always loads its in-tree libwf.so)
    from paper_conf_ppopp_mohantyc14_b200 import _abi
    _abi.LIB_PATH = os.path.abspath(os.environ["WF_PROBE_LIB"])


def parity(specs, kernel=0):
    import oracle
    import workloads
    from _gpu_helpers import run_gpu
    for spec in specs:
        dim, k, w = (int(v) for v in spec.split(":")[:3])
        kern = int(spec.split(":")[3]) if spec.count(":") >= 3 else kernel
        x, y = workloads.seqcmp_inputs(dim, dim, seed_x=dim, seed_y=dim + 1)
        H = oracle.seqcmp(x, y, 1, -1, -1)
        (g,) = run_gpu("seqcmp", dim, (x, y), lane_cols=k, warps=w, skew=1, kernel=kern)
        bad = np.argwhere(H != g)
        bw = 32 * k * w
        print(f"dim={dim} K={k} W={w} kernel={kern}: {len(bad)} mismatches", flush=True)
        if len(bad):
            cols = np.unique(bad[:, 1])
            rows = np.unique(bad[:, 0])
            print("  first (row,col):", [tuple(int(v) + 1 for v in b) for b in bad[:5]])
            print("  rows", rows.min() + 1, "..", rows.max() + 1, "cols", cols.min() + 1, "..", cols.max() + 1)
            c0 = int(cols.min())
            print("  first bad col -> band", c0 // bw, "warp", (c0 % bw) // (32 * k), "lane", (c0 % (32 * k)) // k)
            r0 = int(bad[0][0])
            print("  H row", r0 + 1, "cols", c0 - 2, "..", c0 + 3, ":", H[r0, max(0, c0 - 3):c0 + 3], "gpu",
                  g[r0, max(0, c0 - 3):c0 + 3])


def trace(dim=32768, k=0, w=0, strip=0, kernel=0):
    import torch
    import workloads
    from paper_conf_ppopp_mohantyc14_b200.wf import Wavefront
    os.environ["WF_TRACE"] = "1"
    x, y = workloads.seqcmp_inputs(dim)
    dev = torch.device("cuda", 0)
    xd, yd = torch.from_numpy(x).to(dev), torch.from_numpy(y).to(dev)
    kw = {}
    if k:
        kw["lane_cols"] = k
    if w:
        kw["warps"] = w
    if strip:
        kw["strip"] = strip
    if kernel:
        kw["kernel"] = kernel
    with Wavefront("seqcmp", dim, **kw) as wf:
        out = wf.alloc_out()
        for _ in range(3):
            wf.run(xd, yd, out=out)
        wf.sync()
        ms = wf.last_run_ms()
        tr = wf.debug_trace()
        lay = wf.layout
    tr = np.asarray(tr, dtype=np.uint64).reshape(lay.nbands, -1)
    W = lay.warps
    t0 = int(tr[:, 0].min())
    print(f"dim={dim} K={lay.lane_cols} W={W} bands={lay.nbands} run {ms:.3f} ms")
    steps = (dim + 1) // 2 + 31 if kernel == 9 else dim + 31
    rows_out = []
    for b in range(lay.nbands):
        for w_ in range(W):
            s = tr[b, 8 * w_: 8 * w_ + 8].astype(np.int64)
            start, arrive, end, cyc, nslow, wcyc = s[0] - t0, s[1] - t0, s[2] - t0, s[3], s[4], s[5]
            rows_out.append((b, w_, start, arrive, end, cyc / steps, nslow, wcyc))
    arr = np.array([r[3] for r in rows_out], dtype=np.float64)
    print("row-1 arrival (us) of warps 0,1,2,3 of bands 0,1,2,64,127:")
    for b in (0, 1, 2, lay.nbands // 2, lay.nbands - 1):
        print("  band", b, [f"{rows_out[b * W + w_][3] / 1e3:.2f}" for w_ in range(W)],
              "end", f"{rows_out[b * W + W - 1][4] / 1e3:.1f}",
              "cyc/step", [f"{rows_out[b * W + w_][5]:.1f}" for w_ in range(W)],
              "slow bodies", [int(rows_out[b * W + w_][6]) for w_ in range(W)])
    d = np.diff(arr)
    print(f"mean lag per warp hop {d.mean() / 1e3:.3f} us; per band {W * d.mean() / 1e3:.3f} us;"
          f" intra-CTA hops {np.mean([d[i] for i in range(len(d)) if (i + 1) % W]) / 1e3:.3f} us,"
          f" CTA hops {np.mean([d[i] for i in range(len(d)) if (i + 1) % W == 0]) / 1e3:.3f} us")
    cyc = np.array([r[5] for r in rows_out])
    print(f"sweep cycles per step: median {np.median(cyc):.1f}, min {cyc.min():.1f}, max {cyc.max():.1f}")
    hs = tr[:, 8 * W + 4].astype(np.int64)
    print("helper slow-path blocks per band: bands 1,2,64,last:", [int(hs[b]) for b in (1, 2, lay.nbands // 2, lay.nbands - 1)],
          "mean", float(hs[1:].mean()) if lay.nbands > 1 else 0.0, "of", (dim + 31) // 16, "blocks")


if __name__ == "__main__":
    if sys.argv[1] == "parity":
        parity(sys.argv[2:])
    else:
        trace(*(int(v) for v in sys.argv[2:]))
