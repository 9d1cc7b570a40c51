"""Learned tuning parameters: evaluate the
regression tree trained by tools/train_tuner.py on this build's B200 sweep and return the
compiled variant with the smallest predicted run time for an instance.  Pure Python (no
scikit-learn at run time); host-side only -- it chooses parameters, the sweep itself always
runs in the CUDA library.

    from paper_conf_ppopp_mohantyc14_b200.tuner import suggest
    Wavefront("synthetic", 8192, tsize=100, dsize=3, **suggest("synthetic", 8192, 100, 3))
"""
from __future__ import annotations

import json
import math
import os

FNS = ("synthetic", "nash", "seqcmp")
_MODEL = os.path.join(os.path.dirname(os.path.abspath(__file__)), "tuner_model.json")
_cache = None


def features(fn, dim, tsize, dsize, k, w, d, impl):
    return [1.0 if fn == f else 0.0 for f in FNS] + [math.log2(dim), math.log10(1 + tsize), float(dsize),
                                                     float(k), float(w), float(d), float(impl)]


def _model():
    global _cache
    if _cache is None:
        with open(_MODEL) as f:
            _cache = json.load(f)
    return _cache


def predict_log_ms(x, tree=None) -> float:
    t = tree or _model()["tree"]
    n = 0
    while t["left"][n] != -1:
        n = t["left"][n] if x[t["feature"][n]] <= t["threshold"][n] else t["right"][n]
    return t["value"][n]


def suggest(fn: str, dim: int, tsize: int = 0, dsize: int = 0) -> dict:
    """Wavefront keyword arguments (lane_cols, warps, skew, kernel) of the predicted-fastest
    variant among those the model was trained on for this function that the library accepts
    for this instance (wf_query: compiled, fits shared memory -- e.g. a wide synthetic variant
    with many float items does not).  Falls back to the library defaults (all zero)."""
    from .wf import query   # host-side wf_query only
    m = _model()
    ranked = sorted((predict_log_ms(features(fn, dim, tsize, dsize, k, w, d, impl), m["tree"]), k, w, d, impl)
                    for k, w, d, impl in m["candidates"][fn])
    extra = {"tsize": tsize, "dsize": dsize} if fn != "seqcmp" else {}
    for _, k, w, d, impl in ranked:
        try:
            lay = query(fn, dim, lane_cols=k, warps=w, skew=d, kernel=impl, **extra)
        except Exception:   # noqa: BLE001 -- WF_EUNSUPPORTED / WF_EINVAL: not buildable here
            continue
        if (lay.lane_cols, lay.warps, lay.skew) == (k, w, d):
            return {"lane_cols": k, "warps": w, "skew": d, "kernel": impl}
    return {"lane_cols": 0, "warps": 0, "skew": 0, "kernel": 0}
