"""Write tests/golden/c5_rowhash_<config>.npy: per-row 64-bit hashes (tests/_rowhash.py) of the
ORACLE's full C5 grids (full-grid parity for C5 by per-row hashes precomputed
by the oracle; BASELINE.json config 5: synthetic dim=16384, tsize in {10, 1000}, dsize in {1, 5}).

Calls only oracle/ (the plain row-major CPU evaluator) and the seeded input
generators of workloads/ -- never the CUDA path.  One process per config; C5c/C5d take minutes
to tens of minutes on one core (tsize = 1000 FMA iterations per float item per cell).

    python tools/make_c5_golden.py C5a C5b C5c C5d      # all four, in parallel processes
"""
from __future__ import annotations

import multiprocessing as mp
import os
import sys
import time

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tests"))

import oracle  # noqa: E402
import workloads  # noqa: E402
from _rowhash import row_hashes  # noqa: E402

GOLDEN = os.path.join(ROOT, "tests", "golden")


def one(name: str) -> str:
    c = workloads.CONFIGS[name]
    t0 = time.time()
    u, v, top, left = workloads.synthetic_inputs(c.dim, c.dim, c.dsize)   # default seeds 3, 4, 5
    i0, i1, f = oracle.synthetic(u, v, top, left, c.tsize)
    planes = [i0, i1] + [f[d] for d in range(c.dsize)]
    h = row_hashes(planes)
    path = os.path.join(GOLDEN, f"c5_rowhash_{name}.npy")
    np.save(path, h)
    with open(os.path.join(GOLDEN, f"c5_rowhash_{name}.txt"), "w") as fh:
        fh.write(f"# {name}: synthetic dim={c.dim} tsize={c.tsize} dsize={c.dsize}, seeds (3, 4, 5)\n"
                 f"# per-row hashes of the oracle grid (planes i0, i1, f0..f{c.dsize - 1}), tests/_rowhash.py\n"
                 f"# written by tools/make_c5_golden.py (calls only oracle/), {time.time() - t0:.0f} s on one core\n"
                 f"# row 1: {int(h[0]):016x}  row {c.dim}: {int(h[-1]):016x}\n")
    return f"{name}: {time.time() - t0:.0f} s"


if __name__ == "__main__":
    names = sys.argv[1:] or ["C5a", "C5b", "C5c", "C5d"]
    oracle.build()
    with mp.Pool(len(names)) as pool:
        for msg in pool.imap_unordered(one, names):
            print(msg, flush=True)
