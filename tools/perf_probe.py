"""Quick timing / timeline probe of the sweep kernel (diagnostics, not the bench).

    WF_TRACE=1 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,2 2,2,2
Prints ms per run and GCUPS per variant; with WF_TRACE=1 also the per-band timeline
(band start lag, steady per-row time, end) and feeder poll counts.
"""
from __future__ import annotations

import argparse
import json
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import workloads  # noqa: E402
from paper_conf_ppopp_mohantyc14_b200.wf import Wavefront  # noqa: E402


def inputs(fn, dim, dsize, dev, cols=0):
    t = lambda a: torch.from_numpy(np.ascontiguousarray(a)).to(dev)  # noqa: E731
    if fn == "seqcmp":
        x, y = workloads.seqcmp_inputs(dim, cols or dim)
        return t(x), t(y), None, None
    if fn == "nash":
        r, c, top, left = workloads.nash_inputs(dim, cols or dim)
        return t(r), t(c), [t(top[p]) for p in range(4)], [t(left[p]) for p in range(4)]
    u, v, top, left = workloads.synthetic_inputs(dim, cols or dim, dsize)
    return t(u), t(v), [t(top[d]) for d in range(dsize)], [t(left[d]) for d in range(dsize)]


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--fn", default="seqcmp")
    ap.add_argument("--dim", type=int, nargs="+", default=[32768])
    ap.add_argument("--cols", type=int, default=0)
    ap.add_argument("--alphabet", type=int, default=4)
    ap.add_argument("--tsize", type=int, default=0)
    ap.add_argument("--dsize", type=int, default=0)
    ap.add_argument("--variants", nargs="+", default=["4,2,2"])
    ap.add_argument("--reps", type=int, default=10)
    a = ap.parse_args()
    dev = torch.device("cuda", 0)
    res = []
    for dim in a.dim:
        ins = inputs(a.fn, dim, a.dsize, dev, a.cols)
        for v in a.variants:
            parts = [int(s) for s in v.split(",")]   # k,w,d[,kernel]
            k, w, d = parts[:3]
            kw = dict(lane_cols=k, warps=w, skew=d)
            if len(parts) > 3:
                kw.update(kernel=parts[3])
            if a.fn == "seqcmp":
                kw.update(alphabet=a.alphabet)
            if a.fn == "synthetic":
                kw.update(tsize=a.tsize, dsize=a.dsize)
            if a.fn == "nash":
                kw.update(tsize=a.tsize or 16, dsize=4)
            try:
                wf = Wavefront(a.fn, dim, cols=a.cols, **kw)
            except Exception as e:  # noqa: BLE001
                print(json.dumps({"dim": dim, "variant": v, "error": str(e)}))
                continue
            out = wf.alloc_out()
            for _ in range(3):
                wf.run(*ins, out=out)
            wf.sync()
            ev = [torch.cuda.Event(enable_timing=True) for _ in range(2)]
            ev[0].record()
            for _ in range(a.reps):
                wf.run(*ins, out=out)
            ev[1].record()
            torch.cuda.synchronize()
            wf.sync()
            ms = ev[0].elapsed_time(ev[1]) / a.reps
            rec = {"dim": dim, "variant": v, "ms": round(ms, 4), "gcups": round(dim * (a.cols or dim) / ms / 1e6, 2),
                   "nbands": wf.layout.nbands}
            if os.environ.get("WF_TRACE") == "1":
                tr = wf.debug_trace().astype(np.int64)
                t0 = tr[0, 0]
                starts = (tr[:, 0] - t0) / 1e3
                ends = (tr[:, 32] - t0) / 1e3
                rows_per = (dim + 31) // 32
                steady = (tr[:, 31] - tr[:, 1]) / (30 * rows_per)  # ns per row
                rec.update({
                    "band_start_us": [round(float(x), 1) for x in starts[:: max(1, len(starts) // 16)]],
                    "band_end_us": [round(float(x), 1) for x in ends[:: max(1, len(ends) // 16)]],
                    "ns_per_row_median": float(np.median(steady)),
                    "ns_per_row_band0": float(steady[0]),
                    "sm_ghz_band0": float((tr[0, 43] - tr[0, 42]) / max(1, tr[0, 32] - tr[0, 0])),
                    "steady_entry_us_first_bands": [[round(float(tr[b, 33 + w] - t0) / 1e3, 2) for w in range(wf.layout.warps)]
                                                    for b in range(min(6, len(tr)))],
                    "io_fwd32_feed32_us": [[round(float(tr[b, 36] - t0) / 1e3, 2), round(float(tr[b, 37] - t0) / 1e3, 2)]
                                           for b in range(min(4, len(tr)))],
                    "steady_entry_us_band_step": round(float(tr[-1, 33] - tr[0, 33]) / 1e3 / max(1, len(tr) - 1), 2),
                    # NW: per warp (lane 0) SM cycles per row step in [west wait, west loads,
                    # free wait, compute, publish]; band 0 and the middle band
                    "nw_phase_cyc_per_row_band0": [[round(float(v) / dim, 1) for v in tr[0, 48 + 4 * w:52 + 4 * w]]
                                                   for w in range(min(4, wf.layout.warps))],
                    "nw_phase_cyc_per_row_mid": [[round(float(v) / dim, 1)
                                                  for v in tr[len(tr) // 2, 48 + 4 * w:52 + 4 * w]]
                                                 for w in range(min(4, wf.layout.warps))],
                    "nw_slow_west_entries_polls_band0": [int(tr[0, 43 + w])
                                                         for w in range(min(4, wf.layout.warps))],
                    "nw_slow_west_entries_polls_mid": [int(tr[len(tr) // 2, 43 + w])
                                                        for w in range(min(4, wf.layout.warps))],
                    "feeder_polls": [int(x) for x in tr[:: max(1, len(tr) // 8), 40]],
                    "feeder_empty": [int(x) for x in tr[:: max(1, len(tr) // 8), 41]],
                    # NW: end of the first 15 blocks of warps 0 / 1, us after the band's feed of 32 rows
                    "nw_block_ends_us_band1": [[round(float(tr[1, 1 + 15 * w + b] - tr[1, 37]) / 1e3, 2)
                                                for b in range(15)] for w in range(min(2, wf.layout.warps))]
                    if len(tr) > 1 else [],
                    "raw32_band0": [int(x) for x in tr[0, 32:64]],
                    "raw32_mid": [int(x) for x in tr[len(tr) // 2, 32:64]],
                })
            print(json.dumps(rec))
            res.append(rec)
            wf.close()


if __name__ == "__main__":
    main()
