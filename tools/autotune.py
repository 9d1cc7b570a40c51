"""Exhaustive autotune of the sweep's tunables on the B200 (BASELINE.json north_star: "an
exhaustive autotune harness over tile size, strip size and GPU count ... stands in for the
paper's ML-tuned parameters"; Table 2, Sec. 3.1.2).

    python tools/autotune.py --config C5a [--reps 5] [--out profiles/autotune_C5a.json]
    python tools/autotune.py --all

The paper's tunables (cpu-tile, band, gpu-count, gpu-tile, halo) map onto this build's
(DESIGN.md §6-7):
  * tile      -> lane_cols K (columns per lane) x warps W (the CTA band is 32*K*W columns),
  * strip     -> wf_params.strip S: rows per hand-off block, i.e. per band-to-band and
                 slab-to-slab message (generation 8: 8 / 16 / 32), plus the lane skew D and the
                 kernel generation (wf_params.kernel 8 = lockstep lane pipeline, 4 = U-row block
                 hand-offs),
  * gpu-count -> column slabs (--slabs G...): G slabs linked by the per-row P2P hand-off.  On one
                 physical GPU they are virtual slabs sharing its SMs (device_share) -- a
                 correctness and hand-off-cost point, not a speed-up; with G visible GPUs each slab
                 gets its own device.
Every point is first checked against the CPU oracle on a small instance of the same
function (parity gate: a point that is wrong is discarded, never timed), then timed on the
config's full size with CUDA events (median of --reps runs after 3 warm-ups).  The winner
per config is written with all points to profiles/autotune_<config>.json; the library's
defaults (wf_api.cpp::defaults) follow those winners.
"""
from __future__ import annotations

import argparse
import itertools
import json
import os
import statistics
import sys
import time

import numpy as np

# G virtual slabs = G streams + the current stream; with the default 8 hardware queues a later
# slab's kernel can queue behind an earlier slab's whole run (measured: C4 at G = 8 2.71 vs
# 2.01 ms).  Must be set before the CUDA context exists.
os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
import torch  # noqa: E402

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import oracle  # noqa: E402  (parity gate only; the timed path never touches it)
import workloads  # noqa: E402
from paper_conf_ppopp_mohantyc14_b200.wf import LocalSlabs, Wavefront, query  # noqa: E402

# impl = wf_params.kernel: SEQCMP 8 = lockstep lane pipeline (wf_nw8.cu), 4 = block hand-offs (v4);
# SYNTHETIC 7 = wf_syn, 4 = generic sweep, 8 = plane-split wf_syn (dsize >= 2, k = w = d = 1);
# Nash has one kernel (0).  Combinations a generation does not compile are skipped (wf_query).
SEARCH = {
    "seqcmp": {"k": [1, 2, 4, 8], "w": [1, 2, 4, 8], "d": [1, 2], "impl": [8, 4], "s": [0, 8, 32]},
    "synthetic": {"k": [1, 2], "w": [1, 2, 4], "d": [1, 2], "impl": [7, 4, 8], "s": [0]},
    "nash": {"k": [1], "w": [1, 2, 4, 8], "d": [1], "impl": [0], "s": [0]},
}


def _dev(a, dev):
    return torch.from_numpy(np.ascontiguousarray(a)).to(dev)


def inputs_for(fn, dim, dsize, dev):
    if fn == "seqcmp":
        x, y = workloads.seqcmp_inputs(dim, dim)
        return (x, y), (_dev(x, dev), _dev(y, dev), None, None)
    if fn == "synthetic":
        u, v, top, left = workloads.synthetic_inputs(dim, dim, dsize)
        return (u, v, top, left), (_dev(u, dev), _dev(v, dev), [_dev(top[d], dev) for d in range(dsize)],
                                   [_dev(left[d], dev) for d in range(dsize)])
    r, c, top, left = workloads.nash_inputs(dim, dim)
    return (r, c, top, left), (_dev(r, dev), _dev(c, dev), [_dev(top[p], dev) for p in range(4)],
                               [_dev(left[p], dev) for p in range(4)])


def oracle_grid(fn, host, cfg):
    if fn == "seqcmp":
        return [oracle.seqcmp(host[0], host[1], 1, -1, -1)]
    if fn == "synthetic":
        u, v, top, left = host
        i0, i1, f = oracle.synthetic(u, v, top, left, cfg.tsize)
        return [i0, i1] + [f[d] for d in range(f.shape[0])]
    r, c, top, left = host
    out = oracle.nash(r, c, top, left, nstrat=cfg.tsize)
    return [out[p] for p in range(4)]


def fn_kw(cfg):
    if cfg.fn == "seqcmp":
        return dict(alphabet=4)
    if cfg.fn == "synthetic":
        return dict(tsize=cfg.tsize, dsize=cfg.dsize)
    return dict(tsize=cfg.tsize, dsize=4)


def parity_ok(cfg, k, w, d, impl, dev, small, strip=0):
    host, devin = inputs_for(cfg.fn, small, cfg.dsize, dev)
    small_cfg = workloads.Config(cfg.name, cfg.fn, small, tsize=cfg.tsize, dsize=cfg.dsize)
    want = oracle_grid(cfg.fn, host, small_cfg)
    with Wavefront(cfg.fn, small, lane_cols=k, warps=w, skew=d, kernel=impl, strip=strip, **fn_kw(cfg)) as wf:
        out = wf.run(*devin)
        wf.sync()
        got = [o.cpu().numpy() for o in out]
    if len(got) != len(want):
        return False
    for g, o in zip(got, want):
        o = np.asarray(o)
        if o.dtype.kind == "f":
            g = g.view(np.float32) if g.dtype != np.float32 else g
            if not np.all(np.abs(g - o) <= 1e-5 * np.abs(o)):   # BASELINE.json float bar
                return False
        elif not np.array_equal(g.view(o.dtype) if g.dtype != o.dtype else g, o):
            return False
    return True


def time_point(cfg, k, w, d, impl, devin, reps, strip=0):
    with Wavefront(cfg.fn, cfg.dim, lane_cols=k, warps=w, skew=d, kernel=impl, strip=strip, **fn_kw(cfg)) as wf:
        out = wf.alloc_out()
        for _ in range(3):
            wf.run(*devin, out=out)
        wf.sync()
        ms = []
        for _ in range(reps):
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record()
            wf.run(*devin, out=out)
            e1.record()
            torch.cuda.synchronize()
            wf.sync()
            ms.append(e0.elapsed_time(e1))
        return statistics.median(ms), wf.layout.nbands


def compiled(cfg, k, w, d, impl, strip=0):
    """Does the library build this (fn, tuning, generation, strip)?  (host-side wf_query; no GPU work)"""
    try:
        lay = query(cfg.fn, cfg.dim, lane_cols=k, warps=w, skew=d, kernel=impl, strip=strip, **fn_kw(cfg))
    except Exception:  # noqa: BLE001 -- WF_EUNSUPPORTED / WF_EINVAL
        return False
    return (lay.lane_cols, lay.warps, lay.skew) == (k, w, d)


def time_slabs(cfg, k, w, d, impl, host, G, reps, strip=0, **extra):
    """G column slabs of the same grid linked by the per-row P2P hand-off.  Virtual slabs (one
    GPU): device time between two events on the current stream, which gates every slab stream --
    a ~10 ms device-side sleep ahead of the start event holds the slabs back until the host has
    enqueued all G launches, so host launch latency is not timed.  One GPU per slab: wall clock."""
    ngpu = torch.cuda.device_count()
    devices = [g % ngpu for g in range(G)]
    ls = LocalSlabs(cfg.fn, cfg.dim, G, devices=devices, lane_cols=k, warps=w, skew=d, kernel=impl, strip=strip,
                    **fn_kw(cfg), **extra)
    virtual = len(set(devices)) == 1
    try:
        per = [inputs_for(cfg.fn, cfg.dim, cfg.dsize, torch.device("cuda", s.device))[1] for s in ls.slabs]
        outs = None
        for _ in range(3):
            outs = ls.run(per, outs)
        ls.sync()
        ms = []
        for _ in range(reps):
            for dv in set(devices):
                torch.cuda.synchronize(dv)
            if virtual:
                cur = torch.cuda.current_stream()
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                torch.cuda._sleep(20_000_000)
                e0.record(cur)
                outs = ls.run(per, outs)   # every slab stream waits on cur (LocalSlabs.run)
                for st in ls.streams:
                    cur.wait_stream(st)
                e1.record(cur)
                ls.sync()
                torch.cuda.synchronize()
                ms.append(e0.elapsed_time(e1))
            else:
                t0 = time.perf_counter()
                outs = ls.run(per, outs)
                ls.sync()
                ms.append((time.perf_counter() - t0) * 1e3)
        return statistics.median(ms)
    finally:
        ls.close()


# tunings tried per G on the gpu-count axis (the config default is always tried first)
SLAB_TUNINGS = {   # (lane_cols, warps, skew, kernel, strip)
    "seqcmp": [(2, 4, 1, 8, 8), (2, 4, 1, 8, 32), (4, 2, 1, 8, 0), (2, 2, 1, 8, 0), (1, 4, 1, 8, 0),
               (2, 1, 1, 8, 0), (4, 2, 1, 4, 0)],
    "synthetic": [(2, 1, 1, 0, 0), (1, 2, 1, 0, 0)],
    "nash": [(1, 1, 1, 0, 0), (1, 4, 1, 0, 0)],
}


def rect_inputs(fn, m, n, dsize, dev):
    if fn == "seqcmp":
        x, y = workloads.seqcmp_inputs(m, n)
        return (x, y), (_dev(x, dev), _dev(y, dev), None, None)
    if fn == "synthetic":
        u, v, top, left = workloads.synthetic_inputs(m, n, dsize)
        return (u, v, top, left), (_dev(u, dev), _dev(v, dev), [_dev(top[d], dev) for d in range(dsize)],
                                   [_dev(left[d], dev) for d in range(dsize)])
    r, c, top, left = workloads.nash_inputs(m, n)
    return (r, c, top, left), (_dev(r, dev), _dev(c, dev), [_dev(top[p], dev) for p in range(4)],
                               [_dev(left[p], dev) for p in range(4)])


def slab_parity_ok(cfg, k, w, d, impl, G, band_cols, strip=0, rows=64):
    """G linked slabs of a small rectangular instance (rows x (G bands + a ragged tail)) against
    the oracle (exact for integers, 1e-5 for floats)."""
    cols = max(300, G * band_cols + 77)
    host, _ = rect_inputs(cfg.fn, rows, cols, cfg.dsize, torch.device("cuda", 0))
    want = oracle_grid(cfg.fn, host, cfg)
    ngpu = torch.cuda.device_count()
    ls = LocalSlabs(cfg.fn, rows, G, devices=[g % ngpu for g in range(G)], cols=cols, lane_cols=k, warps=w, skew=d,
                    kernel=impl, strip=strip, **fn_kw(cfg))
    try:
        per = [rect_inputs(cfg.fn, rows, cols, cfg.dsize, torch.device("cuda", s.device))[1] for s in ls.slabs]
        outs = ls.run(per)
        ls.sync()
        got = [np.concatenate([o[p].cpu().numpy() for o in outs], axis=1) for p in range(len(want))]
    finally:
        ls.close()
    for g, o in zip(got, want):
        o = np.asarray(o)
        if o.dtype.kind == "f":
            g = g.view(np.float32)
            if not np.all(np.abs(g - o) <= 1e-5 * np.abs(o)):
                return False
        elif not np.array_equal(g.view(o.dtype), o):
            return False
    return True


def sweep_slabs(cfg, reps, slabs):
    """The gpu-count axis: for every G, the config default plus SLAB_TUNINGS[fn] on G linked column
    slabs, each point parity-gated on G slabs of a small instance, then timed (wall clock around the
    linked runs).  With fewer physical GPUs than G the slabs are virtual (one GPU, each slab 1/G of
    the resident CTAs): a point whose slabs together need more CTAs than the GPU holds at once is
    marked 'ctas_exceed_sms' -- for one-CTA-per-SM kernels its time is not a prediction of G real
    GPUs."""
    host, _ = inputs_for(cfg.fn, 16, cfg.dsize, torch.device("cuda", 0))
    sms = torch.cuda.get_device_properties(0).multi_processor_count
    recs = []
    for G in slabs:
        for tun in [(0, 0, 0, 0, 0)] + SLAB_TUNINGS[cfg.fn]:
            k, w, d, impl, st = tun
            rec = {"slabs": G, "lane_cols": k, "warps": w, "skew": d, "kernel": impl, "strip": st,
                   "visible_gpus": torch.cuda.device_count(),
                   "placement": "virtual (one GPU)" if torch.cuda.device_count() < G else "one GPU per slab"}
            try:
                lay = [query(cfg.fn, cfg.dim, rank=g, ngpus=G, lane_cols=k, warps=w, skew=d, kernel=impl, strip=st,
                             **fn_kw(cfg)) for g in range(G)]
                rec.update(lane_cols=lay[0].lane_cols, warps=lay[0].warps, skew=lay[0].skew, strip=lay[0].strip,
                           band_cols=lay[0].band_cols, bands_per_slab=[l_.nbands for l_ in lay])
                if k and (lay[0].lane_cols, lay[0].warps, lay[0].skew) != (k, w, d):
                    continue
                rec["ctas_total"] = sum(l_.nbands for l_ in lay)
                # virtual slabs share one GPU: with more bands than SMs, kernels that fit one CTA per
                # SM (generation 8: ~199 KB of shared memory) make bands wait for a CTA, so the point
                # does not predict G real GPUs (one-warp synthetic CTAs fit several per SM)
                rec["sms"] = sms
                rec["ctas_exceed_sms"] = rec["placement"].startswith("virtual") and rec["ctas_total"] > sms
                if not slab_parity_ok(cfg, k, w, d, impl, G, lay[0].band_cols, st):
                    rec["error"] = "parity"
                else:
                    ms = time_slabs(cfg, k, w, d, impl, host, G, reps, st)
                    rec.update(ms=round(ms, 4), gcups=round(cfg.dim * cfg.dim / ms / 1e6, 3))
            except Exception as e:  # noqa: BLE001
                rec["error"] = str(e)[:160]
            recs.append(rec)
            print(json.dumps(rec), flush=True)
    return recs


def tune(cfg, reps, small, budget_s):
    dev = torch.device("cuda", 0)
    _, devin = inputs_for(cfg.fn, cfg.dim, cfg.dsize, dev)
    sp = SEARCH[cfg.fn]
    points = []
    t_start = time.time()
    for impl, k, w, d, st in itertools.product(sp["impl"], sp["k"], sp["w"], sp["d"], sp["s"]):
        if not compiled(cfg, k, w, d, impl, st):
            continue
        rec = {"impl": impl, "k": k, "w": w, "d": d, "strip": st}
        if time.time() - t_start > budget_s:
            rec["skipped"] = "time budget"
            points.append(rec)
            continue
        try:
            if not parity_ok(cfg, k, w, d, impl, dev, small, st):
                rec["error"] = "parity mismatch vs oracle"
            else:
                ms, nb = time_point(cfg, k, w, d, impl, devin, reps, st)
                rec.update(ms=round(ms, 4), gcups=round(cfg.dim * cfg.dim / ms / 1e6, 3), nbands=nb)
        except Exception as e:  # noqa: BLE001 -- unsupported variants are part of the sweep
            rec["error"] = str(e)[:160]
        points.append(rec)
        print(json.dumps(rec), flush=True)
    ok = [p for p in points if "ms" in p]
    best = min(ok, key=lambda p: p["ms"]) if ok else None
    return {"config": cfg.name, "workload": cfg.note or cfg.name, "fn": cfg.fn, "dim": cfg.dim, "tsize": cfg.tsize,
            "dsize": cfg.dsize, "gpus": torch.cuda.device_count(), "device": torch.cuda.get_device_name(0),
            "parity_dim": small, "reps": reps, "best": best, "points": points}


# Problem design for the learned tuner (tools/train_tuner.py): the
# paper trained its models on sweeps over (dim, tsize, dsize); here the
# same features on B200 sizes.
GRID = ([("seqcmp", d, 0, 0) for d in (1024, 2048, 4096, 8192, 16384, 32768)]
        + [("synthetic", d, t, ds) for d in (1024, 4096, 16384) for t in (10, 100, 1000) for ds in (1, 3, 5)]
        + [("nash", d, 16, 4) for d in (1024, 2048, 4096)])


def sweep_grid(reps, out, only_fn=None):
    """Time every compiled variant on every GRID instance; with only_fn, re-sweep that function and
    keep the other functions' points of the existing file."""
    dev = torch.device("cuda", 0)
    recs = []
    if only_fn and os.path.exists(out):
        recs = [p for p in json.load(open(out))["points"] if p["fn"] != only_fn]
    for fn, dim, tsize, dsize in GRID:
        if only_fn and fn != only_fn:
            continue
        cfg = workloads.Config(f"{fn}-{dim}-{tsize}-{dsize}", fn, dim, tsize=tsize, dsize=dsize)
        _, devin = inputs_for(fn, dim, dsize, dev)
        sp = SEARCH[fn]
        for impl, k, w, d in itertools.product(sp["impl"], sp["k"], sp["w"], sp["d"]):
            if not compiled(cfg, k, w, d, impl):
                continue
            rec = {"fn": fn, "dim": dim, "tsize": tsize, "dsize": dsize, "impl": impl, "k": k, "w": w, "d": d}
            try:
                ms, nb = time_point(cfg, k, w, d, impl, devin, reps)
                rec.update(ms=round(ms, 5), nbands=nb)
            except Exception as e:  # noqa: BLE001
                rec["error"] = str(e)[:120]
            recs.append(rec)
            print(json.dumps(rec), flush=True)
        del devin
    with open(out, "w") as f:
        json.dump({"device": torch.cuda.get_device_name(0), "reps": reps, "points": recs}, f, indent=0)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--grid", action="store_true", help="sweep the tuner's problem design (GRID)")
    ap.add_argument("--config", default="C5a", choices=sorted(workloads.CONFIGS))
    ap.add_argument("--all", action="store_true")
    ap.add_argument("--reps", type=int, default=5)
    ap.add_argument("--small", type=int, default=300, help="parity-gate instance size")
    ap.add_argument("--budget-s", type=float, default=240.0, help="per-config time budget")
    ap.add_argument("--out", default="")
    ap.add_argument("--grid-fn", default=None, choices=[None, "seqcmp", "synthetic", "nash"],
                    help="with --grid: re-sweep one function, keep the others' points")
    ap.add_argument("--slabs", default="", help="gpu-count axis, e.g. 1,2,4,8 (column slabs of --config)")
    a = ap.parse_args()
    if a.grid:
        sweep_grid(a.reps, a.out or os.path.join(ROOT, "profiles", "tuner_sweep.json"), a.grid_fn)
        return
    if a.slabs:
        cfg = workloads.CONFIGS[a.config]
        res = {"config": cfg.name, "fn": cfg.fn, "dim": cfg.dim, "reps": a.reps,
               "device": torch.cuda.get_device_name(0), "points": sweep_slabs(cfg, a.reps, [int(g) for g in a.slabs.split(",")])}
        out = a.out or os.path.join(ROOT, "profiles", f"autotune_slabs_{cfg.name}.json")
        with open(out, "w") as f:
            json.dump(res, f, indent=1)
        return
    names = sorted(workloads.CONFIGS) if a.all else [a.config]
    for n in names:
        cfg = workloads.CONFIGS[n]
        res = tune(cfg, a.reps, a.small, a.budget_s)
        out = a.out if (a.out and not a.all) else os.path.join(ROOT, "profiles", f"autotune_{n}.json")
        with open(out, "w") as f:
            json.dump(res, f, indent=1)
        print(json.dumps({"config": n, "best": res["best"], "file": os.path.relpath(out, ROOT)}), flush=True)


if __name__ == "__main__":
    main()
