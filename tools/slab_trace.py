"""Timeline of G virtual slabs of C4 on one GPU (WF_TRACE=1; not a test): per slab, when its
first band starts, when its band 0 gets row 1, and when its last band ends -- shows whether a
slab boundary costs more than a band boundary.

    WF_TRACE=1 python tools/slab_trace.py [G] [dim]
"""
from __future__ import annotations

import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
os.environ["WF_TRACE"] = "1"
os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")   # see LocalSlabs

import torch  # noqa: E402

import workloads  # noqa: E402
from paper_conf_ppopp_mohantyc14_b200.wf import LocalSlabs  # noqa: E402


def main(G=8, dim=32768):
    x, y = workloads.seqcmp_inputs(dim)
    dev = torch.device("cuda", 0)
    xd, yd = torch.from_numpy(x).to(dev), torch.from_numpy(y).to(dev)
    ls = LocalSlabs("seqcmp", dim, G, alphabet=4)
    per = [(xd, yd, None, None)] * G
    outs = None
    for _ in range(3):
        torch.cuda._sleep(4_000_000)
        outs = ls.run(per, outs)
        ls.sync()
    trs = [np.asarray(s.debug_trace(), dtype=np.uint64).reshape(s.layout.nbands, -1) for s in ls.slabs]
    t0 = min(int(t[:, 0].min()) for t in trs)
    print(f"G={G} dim={dim} bands/slab={[s.layout.nbands for s in ls.slabs]}")
    for g, t in enumerate(trs):
        W = ls.slabs[g].layout.warps
        st = (t[:, 0].astype(np.int64) - t0) / 1e3
        first = (t[:, 1].astype(np.int64) - t0) / 1e3          # warp 0 row 1
        end = (t[:, 8 * (W - 1) + 2].astype(np.int64) - t0) / 1e3
        hops = np.diff(first)
        print(f"slab {g}: CTA start {st.min():8.2f}..{st.max():8.2f} us; band0 row1 {first[0]:8.2f} us; "
              f"last band row1 {first[-1]:8.2f}; end {end.max():8.2f} us; band hop median {np.median(hops):.2f} us")
    ls.close()


if __name__ == "__main__":
    main(*(int(a) for a in sys.argv[1:]))
