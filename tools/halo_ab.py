"""NEXT-4 A/B: C4 on G linked column slabs with the per-row P2P
hand-off alone (halo 0) against the halo-overlap variant (wf_params.halo = 1 or 2 bands: slab
g > 0 recomputes the last halo columns of slab g-1 and takes its west input halo columns earlier).
Virtual slabs on one GPU, device-timed (tools/autotune.py time_slabs), interleaved rounds; plus a
bitwise check of each halo grid against the single-slab grid.

    CUDA_DEVICE_MAX_CONNECTIONS=32 python tools/halo_ab.py [rounds] > profiles/r02_halo_ab.txt
"""
from __future__ import annotations

import os
import statistics
import sys

os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tools"))

import numpy as np  # noqa: E402
import torch  # noqa: E402

import workloads  # noqa: E402
from autotune import time_slabs  # noqa: E402
from paper_conf_ppopp_mohantyc14_b200.wf import LocalSlabs, Wavefront  # noqa: E402


def grid_check(dim, G, halo):
    x, y = workloads.seqcmp_inputs(dim, dim)
    dev = torch.device("cuda", 0)
    xd, yd = torch.from_numpy(x).to(dev), torch.from_numpy(y).to(dev)
    with Wavefront("seqcmp", dim, alphabet=4) as w:
        ref = w.run(xd, yd)[0]
        w.sync()
    ls = LocalSlabs("seqcmp", dim, G, alphabet=4, halo=halo)
    try:
        outs = ls.run([(xd, yd, None, None)] * G)
        ls.sync()
        got = torch.cat([o[0] for o in outs], dim=1)
        return bool(torch.equal(got, ref))
    finally:
        ls.close()


def main():
    rounds = int(sys.argv[1]) if len(sys.argv) > 1 else 3
    cfg = workloads.CONFIGS["C4"]
    points = [(G, h) for G in (2, 4) for h in (0, 256, 512)]
    res = {p: [] for p in points}
    for r in range(rounds):
        for p in (points if r % 2 == 0 else points[::-1]):
            G, h = p
            res[p].append(time_slabs(cfg, 2, 4, 1, 8, None, G, reps=5, halo=h))
    print("# C4 (NW dim 32768, generation 8, K=2 x 4 warps, 256-column bands) on G virtual slabs of one B200;")
    print("# device time per run (ms), median over rounds of the median of 5 runs; halo = overlap columns per slab")
    for (G, h), v in res.items():
        print(f"G={G} halo={h:4d} ({h // 256} band{'s' if h != 256 else ''}): {statistics.median(v):.4f} ms   rounds {' '.join(f'{x:.4f}' for x in v)}")
    for G, h in ((2, 256), (4, 512)):
        print(f"bitwise grid check vs one slab, C4, G={G} halo={h}: {grid_check(cfg.dim, G, h)}")


if __name__ == "__main__":
    main()
