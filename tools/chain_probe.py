"""Serial cost of one cell on the dependency chain, per cell function (bench.py latency roofs).

A one-column grid (cols=1) is a pure chain: row i needs row i-1.  Timing it at two heights and
taking the difference cancels launch and fill costs:
    cycles per cell = (T(2R) - T(R)) / R x sm clock.
This is the measured counterpart of the microbenchmark latencies (profiles/r01_microbench.txt):
for NW it is the in-lane DPX chain plus the kernel's per-row overhead, for the synthetic cell the
(tsize+3)-deep FMA chain, for Nash the whole warp-cooperative cell (no microbenchmark covers it).

    python tools/chain_probe.py > gpurun_out/chain.txt
"""
from __future__ import annotations

import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tests"))

import torch  # noqa: E402

import workloads  # noqa: E402
from paper_conf_ppopp_mohantyc14_b200.wf import Wavefront  # noqa: E402


def sm_mhz():
    try:
        import pynvml
        pynvml.nvmlInit()
        h = pynvml.nvmlDeviceGetHandleByIndex(torch.cuda.current_device())
        return pynvml.nvmlDeviceGetClockInfo(h, pynvml.NVML_CLOCK_SM), h, pynvml
    except Exception:
        return None, None, None


def time_chain(fn, rows, reps=5, **kw):
    dev = torch.device("cuda", 0)
    if fn == "seqcmp":
        x, y = workloads.seqcmp_inputs(rows, 1)
        tops = lefts = []
        row, col = x, y
    elif fn == "synthetic":
        row, col, top, left = workloads.synthetic_inputs(rows, 1, kw["dsize"])
    else:
        row, col, top, left = workloads.nash_inputs(rows, 1)
    if fn != "seqcmp":
        tops = [torch.from_numpy(np.ascontiguousarray(top[p])).to(dev) for p in range(top.shape[0])]
        lefts = [torch.from_numpy(np.ascontiguousarray(left[p])).to(dev) for p in range(left.shape[0])]
    r_d = torch.from_numpy(np.ascontiguousarray(row)).to(dev)
    c_d = torch.from_numpy(np.ascontiguousarray(col)).to(dev)
    with Wavefront(fn, rows, cols=1, **kw) as w:
        out = w.alloc_out()
        for _ in range(2):
            w.run(r_d, c_d, tops, lefts, out=out)
        w.sync()
        ts = []
        for _ in range(reps):
            a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            a.record()
            w.run(r_d, c_d, tops, lefts, out=out)
            b.record()
            torch.cuda.synchronize()
            ts.append(a.elapsed_time(b))
        w.sync()
    return float(np.median(ts))


CASES = [
    ("seqcmp", 16384, dict(alphabet=4)),
    ("synthetic", 2048, dict(tsize=10, dsize=1)),
    ("synthetic", 512, dict(tsize=1000, dsize=1)),
    ("nash", 1024, dict(tsize=16, dsize=4)),
]


def main():
    mhz, h, nv = sm_mhz()
    for fn, R, kw in CASES:
        t1 = time_chain(fn, R, **kw)
        t2 = time_chain(fn, 2 * R, **kw)
        clk = mhz
        if nv is not None:
            clk = nv.nvmlDeviceGetMaxClockInfo(h, nv.NVML_CLOCK_SM)
        cyc = (t2 - t1) * 1e-3 / R * (clk or 1965) * 1e6
        print(f"{fn} {kw}: T({R})={t1:.3f} ms T({2 * R})={t2:.3f} ms -> {cyc:.1f} cycles/cell on the chain "
              f"(at {clk} MHz)", flush=True)


if __name__ == "__main__":
    main()
