"""The learned tuner: the shipped tree evaluator reproduces the
regression tree scikit-learn fits on the committed B200 sweep, and every suggestion is a
compiled, valid variant (host-side logic only; no GPU)."""
from __future__ import annotations

import json
import math
import os

import numpy as np
import pytest

from paper_conf_ppopp_mohantyc14_b200 import tuner
from paper_conf_ppopp_mohantyc14_b200.wf import query

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
SWEEP = os.path.join(ROOT, "profiles", "tuner_sweep.json")


def test_tree_evaluator_matches_sklearn_fit_on_the_sweep():
    sk = pytest.importorskip("sklearn.tree")
    pts = [p for p in json.load(open(SWEEP))["points"] if "ms" in p]
    X = np.array([tuner.features(p["fn"], p["dim"], p["tsize"], p["dsize"], p["k"], p["w"], p["d"], p["impl"])
                  for p in pts])
    y = np.array([math.log(p["ms"]) for p in pts])
    ref = sk.DecisionTreeRegressor(min_samples_leaf=2, random_state=0).fit(X, y)
    mine = np.array([tuner.predict_log_ms(list(x)) for x in X])
    assert np.allclose(mine, ref.predict(X), rtol=0, atol=1e-9)


@pytest.mark.parametrize("fn,dim,tsize,dsize", [("seqcmp", 32768, 0, 0), ("seqcmp", 3000, 0, 0),
                                                ("synthetic", 16384, 10, 1), ("synthetic", 2048, 100, 1),
                                                ("synthetic", 8000, 500, 4), ("nash", 4096, 16, 4),
                                                ("synthetic", 16384, 100, 8), ("synthetic", 16384, 1000, 8),
                                                ("synthetic", 4096, 1000, 6), ("synthetic", 4096, 1000, 7)])
def test_suggestions_are_compiled_variants(fn, dim, tsize, dsize):
    kw = tuner.suggest(fn, dim, tsize, dsize)
    assert set(kw) == {"lane_cols", "warps", "skew", "kernel"}
    extra = {"tsize": tsize, "dsize": dsize} if fn != "seqcmp" else {}
    lay = query(fn, dim, **kw, **extra)
    assert (lay.lane_cols, lay.warps, lay.skew) == (kw["lane_cols"], kw["warps"], kw["skew"])


def test_leave_one_out_evaluation_is_recorded():
    ev = json.load(open(os.path.join(ROOT, "profiles", "tuner_eval.json")))
    s = ev["summary"]
    assert s["instances"] == len(ev["leave_one_instance_out"]) >= 30
    assert 1.0 <= s["tuner_regret_geomean"] < 2.0
