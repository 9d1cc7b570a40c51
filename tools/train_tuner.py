"""Learned tuner (the paper's contribution, Sec. 3.1.2 and
P:687-728 Sec. 4.1.5: machine-learned models map a wavefront instance's features to its tuning
parameters).  The paper trained M5P / REP regression trees in Weka on its CPU+GPU sweeps; here
a regression tree (scikit-learn DecisionTreeRegressor, the REP-tree analogue) is trained on
THIS build's B200 sweep (tools/autotune.py --grid -> profiles/tuner_sweep.json):

    features = (function one-hot, log2 dim, log10(1 + tsize), dsize,  K, W, D, kernel generation)
    target   = log(run time)

and the tuner picks, for a new instance, the compiled variant with the smallest predicted
time.  Evaluation is leave-one-instance-out: the instance's own timings are never in the
training set; the regret is t(chosen) / t(best) on that instance, reported next to the
regret of the library's fixed defaults.

    python tools/train_tuner.py [--sweep profiles/tuner_sweep.json]
writes paper_conf_ppopp_mohantyc14_b200/tuner_model.json (the tree, evaluated without
scikit-learn by paper_conf_ppopp_mohantyc14_b200/tuner.py) and profiles/tuner_eval.json.
"""
from __future__ import annotations

import argparse
import json
import math
import os
import sys

import numpy as np
from sklearn.tree import DecisionTreeRegressor

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
from paper_conf_ppopp_mohantyc14_b200.tuner import FNS, features  # noqa: E402


def default_choice(fn, dim, tsize, dsize):
    """The library's fixed defaults (wf_api.cpp::defaults) as a (k, w, d, impl) tuple."""
    if fn == "seqcmp":
        return (2, 4, 1, 8)   # generation 8, K = 2 x 4 warps
    if fn == "nash":
        return (1, 2, 1, 0)
    syn_pad_wins = dsize == 5 and tsize >= 1000
    heavy = not syn_pad_wins and ((dsize >= 3 and tsize >= 1000) or (dsize >= 5 and tsize >= 100))
    return (1, 4 if dsize >= 5 else 2, 1, 4) if heavy else (1, 1, 1, 7)


def fit(X, y, seed=0):
    return DecisionTreeRegressor(min_samples_leaf=2, random_state=seed).fit(X, y)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--sweep", default=os.path.join(ROOT, "profiles", "tuner_sweep.json"))
    ap.add_argument("--model", default=os.path.join(ROOT, "paper_conf_ppopp_mohantyc14_b200", "tuner_model.json"))
    ap.add_argument("--eval", default=os.path.join(ROOT, "profiles", "tuner_eval.json"))
    a = ap.parse_args()
    pts = [p for p in json.load(open(a.sweep))["points"] if "ms" in p]
    inst = sorted({(p["fn"], p["dim"], p["tsize"], p["dsize"]) for p in pts})
    X = np.array([features(p["fn"], p["dim"], p["tsize"], p["dsize"], p["k"], p["w"], p["d"], p["impl"]) for p in pts])
    y = np.array([math.log(p["ms"]) for p in pts])
    key = [(p["fn"], p["dim"], p["tsize"], p["dsize"]) for p in pts]
    rows = []
    for ins in inst:
        tr = np.array([k != ins for k in key])
        te = [i for i, k in enumerate(key) if k == ins]
        m = fit(X[tr], y[tr])
        pred = m.predict(X[te])
        best = min(pts[i]["ms"] for i in te)
        chosen = pts[te[int(np.argmin(pred))]]
        dflt = default_choice(*ins)
        dms = [pts[i]["ms"] for i in te if (pts[i]["k"], pts[i]["w"], pts[i]["d"], pts[i]["impl"]) == dflt]
        rows.append({"instance": list(ins), "best_ms": best,
                     "tuner": {"k": chosen["k"], "w": chosen["w"], "d": chosen["d"], "impl": chosen["impl"],
                               "ms": chosen["ms"], "regret": chosen["ms"] / best},
                     "default": {"choice": list(dflt), "ms": dms[0] if dms else None,
                                 "regret": (dms[0] / best) if dms else None}})
    tr_reg = [r["tuner"]["regret"] for r in rows]
    df_reg = [r["default"]["regret"] for r in rows if r["default"]["regret"] is not None]
    summary = {"instances": len(rows), "points": len(pts),
               "tuner_regret_geomean": float(np.exp(np.mean(np.log(tr_reg)))), "tuner_regret_max": max(tr_reg),
               "default_regret_geomean": float(np.exp(np.mean(np.log(df_reg)))), "default_regret_max": max(df_reg),
               "tuner_picks_best": sum(r < 1.0001 for r in tr_reg)}
    json.dump({"summary": summary, "leave_one_instance_out": rows}, open(a.eval, "w"), indent=1)
    full = fit(X, y)
    t = full.tree_
    cands = {}
    for p in pts:
        cands.setdefault(p["fn"], set()).add((p["k"], p["w"], p["d"], p["impl"]))
    model = {"kind": "regression tree on log(ms) (sklearn DecisionTreeRegressor, min_samples_leaf=2)",
             "features": ["fn=synthetic", "fn=nash", "fn=seqcmp", "log2 dim", "log10(1+tsize)", "dsize", "K", "W", "D",
                          "kernel"],
             "trained_on": os.path.relpath(a.sweep, ROOT), "n_points": len(pts),
             "candidates": {fn: sorted(list(c)) for fn, c in cands.items()},
             "tree": {"left": t.children_left.tolist(), "right": t.children_right.tolist(),
                      "feature": t.feature.tolist(), "threshold": t.threshold.tolist(),
                      "value": [float(v) for v in t.value.reshape(-1)]}}
    json.dump(model, open(a.model, "w"))
    print(json.dumps(summary))


if __name__ == "__main__":
    main()
