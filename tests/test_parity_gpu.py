"""GPU parity: the CUDA path (through the C ABI) against the CPU oracle, element by element.

Bars (BASELINE.json north_star): integer planes bit-exact; fp32 planes
within |g - o| <= 1e-5 |o| per cell (and, by construction of the fixed op order, expected
bit-exact -- asserted separately).  Sizes span several bands and ragged tails; the full
BASELINE configs are covered at the end (C4 full grid; C2 full grid; C5 row prefix plus
any-size closed forms).
"""
from __future__ import annotations

import numpy as np
import pytest

torch = pytest.importorskip("torch")
if not torch.cuda.is_available():
    pytest.skip("needs a CUDA device", allow_module_level=True)

import oracle  # noqa: E402
import workloads  # noqa: E402
from paper_conf_ppopp_mohantyc14_b200 import _abi  # noqa: E402
from paper_conf_ppopp_mohantyc14_b200.wf import Wavefront  # noqa: E402

from _gpu_helpers import dev_inputs, run_gpu  # noqa: E402

pytestmark = pytest.mark.gpu

FTOL = 1e-5


def _seq(dim, cols=0, kind="random", scoring=(1, -1, -1), seed=(1, 2), **kw):
    n = cols or dim
    x, y = workloads.seqcmp_inputs(dim, n, kind=kind, seed_x=seed[0], seed_y=seed[1])
    M, X, G = scoring
    H = oracle.seqcmp(x, y, M, X, G)
    (g,) = run_gpu("seqcmp", dim, (x, y), cols=cols, match=M, mismatch=X, gap=G, **kw)
    return H, g


# ------------------------------------------------------------------ sequence comparison
@pytest.mark.parametrize("dim", [1, 2, 3, 7, 31, 32, 33, 63, 64, 65, 100, 127, 129, 255, 256, 257, 500, 512, 1100])
def test_seqcmp_dims_default_tiling(dim):
    H, g = _seq(dim)
    assert np.array_equal(H, g)


SEQ_VARIANTS = [(1, 1, 1), (1, 4, 1), (2, 1, 1), (2, 2, 2), (2, 2, 3), (2, 4, 1), (4, 1, 1), (4, 2, 1), (4, 3, 1), (4, 1, 2),
                (4, 1, 3), (8, 1, 1), (8, 1, 2)]


@pytest.mark.parametrize("k,w,d", SEQ_VARIANTS)
@pytest.mark.parametrize("dim", [97, 777, 1100])
@pytest.mark.parametrize("alphabet", [0, 4])
def test_seqcmp_variants(k, w, d, dim, alphabet):
    H, g = _seq(dim, lane_cols=k, warps=w, skew=d, seed=(dim, dim + 1), alphabet=alphabet)
    assert np.array_equal(H, g)


NW8_VARIANTS = [(2, 4), (2, 2), (1, 4), (1, 8), (4, 2), (4, 1), (2, 1)]


@pytest.mark.parametrize("k,w", NW8_VARIANTS)
@pytest.mark.parametrize("dim", [1, 33, 64, 97, 777, 1100, 3001])
def test_seqcmp_generation8_variants(k, w, dim):
    """Every compiled (lane_cols, warps) of the lockstep lane pipeline (wf_nw8.cu, kernel=8):
    one band, several bands, ragged last band, a ring lap (rows > 64) and ramp / drain blocks."""
    H, g = _seq(dim, lane_cols=k, warps=w, skew=1, kernel=8, seed=(dim + 5, dim + 6))
    assert np.array_equal(H, g)


@pytest.mark.parametrize("k,w", [(2, 4), (4, 2)])
@pytest.mark.parametrize("strip", [8, 32])
@pytest.mark.parametrize("dim", [1, 33, 97, 777, 3001])
def test_seqcmp_generation8_strips(k, w, strip, dim):
    """wf_params.strip: rows per hand-off block (8 / 32 besides the default 16)."""
    H, g = _seq(dim, lane_cols=k, warps=w, skew=1, kernel=8, strip=strip, seed=(dim + 1, dim + 2))
    assert np.array_equal(H, g)


@pytest.mark.parametrize("strip", [8, 32])
@pytest.mark.parametrize("G", [2, 3])
def test_seqcmp_strips_local_slabs(strip, G):
    H, g = _seq(1000, ngpus=G, strip=strip, seed=(5, 6))
    assert np.array_equal(H, g)


@pytest.mark.parametrize("G,halo,dim", [(2, 256, 1100), (2, 256, 3001), (3, 256, 3001), (2, 512, 3001), (4, 256, 4097)])
def test_seqcmp_halo_overlap_slabs(G, halo, dim):
    """NEXT-4 (wf_params.halo): slab g > 0 recomputes halo columns of slab g-1 into a scratch plane
    and takes its west input from slab g-1's column c0 - halo - 1; the grid is unchanged."""
    H, g = _seq(dim, ngpus=G, halo=halo, seed=(dim + 3, dim + 4), alphabet=4)
    assert np.array_equal(H, g)


@pytest.mark.parametrize("halo", [256, 512])
def test_seqcmp_halo_reruns_and_scoring(halo):
    x, y = workloads.seqcmp_inputs(2500, 2500, seed_x=11, seed_y=12)
    H = oracle.seqcmp(x, y, 2, -3, -2)
    for _ in range(2):
        (g,) = run_gpu("seqcmp", 2500, (x, y), ngpus=2, halo=halo, match=2, mismatch=-3, gap=-2)
        assert np.array_equal(H, g)


@pytest.mark.parametrize("k,w,d", [(4, 2, 1), (2, 4, 1), (4, 1, 2)])
@pytest.mark.parametrize("dim", [33, 777, 1100])
def test_seqcmp_generation4_kernel(k, w, d, dim):
    """The block hand-off generation (wf_nw.cuh, kernel=4) stays correct as the comparison kernel."""
    H, g = _seq(dim, lane_cols=k, warps=w, skew=d, kernel=4, seed=(dim + 7, dim + 8), alphabet=4)
    assert np.array_equal(H, g)


@pytest.mark.parametrize("G", [2, 3])
@pytest.mark.parametrize("kernel", [4, 8])
def test_seqcmp_generations_local_slabs(G, kernel):
    H, g = _seq(1000, ngpus=G, kernel=kernel, alphabet=4)
    assert np.array_equal(H, g)


def _sw_expect(H):
    """Best local score and its first cell in row-major order (1-based), by definition."""
    flat = int(np.argmax(H))
    r, c = divmod(flat, H.shape[1])
    return int(H.flat[flat]), r + 1, c + 1


def _sw_run(dim, cols=0, kind="random", scoring=(2, -1, -1), seed=(1, 2), **kw):
    n = cols or dim
    x, y = workloads.seqcmp_inputs(dim, n, kind=kind, seed_x=seed[0], seed_y=seed[1])
    M, X, G = scoring
    H = oracle.seqcmp(x, y, M, X, G, local=True)
    dev = torch.device("cuda", torch.cuda.current_device())
    with Wavefront("seqcmp", dim, cols=cols, match=M, mismatch=X, gap=G, local=1, **kw) as w:
        row_in, col_in, top, left = dev_inputs("seqcmp", (x, y), dev)
        (g,) = w.run(row_in, col_in, top, left)
        w.sync()
        best = w.local_best()
        g = g.cpu().numpy()
    return H, g, best


@pytest.mark.parametrize("dim", [1, 2, 7, 33, 64, 97, 300, 777, 1100])
@pytest.mark.parametrize("scoring", [(2, -1, -1), (1, -1, -1), (3, -2, -2), (-1, -1, -1)])
def test_smith_waterman_grid_and_best_cell(dim, scoring):
    H, g, best = _sw_run(dim, scoring=scoring, seed=(dim + 11, dim + 12), alphabet=4)
    assert np.array_equal(H, g)
    assert best == _sw_expect(H)


@pytest.mark.parametrize("k,w,d", [(4, 2, 1), (4, 1, 1), (2, 2, 1), (2, 4, 1), (8, 1, 1), (4, 1, 2), (2, 2, 2), (1, 2, 1)])
@pytest.mark.parametrize("alphabet", [0, 4])
def test_smith_waterman_variants(k, w, d, alphabet):
    for dim, cols in ((1000, 0), (513, 1200), (1300, 257)):
        H, g, best = _sw_run(dim, cols=cols, lane_cols=k, warps=w, skew=d, alphabet=alphabet, seed=(dim, cols + 3))
        assert np.array_equal(H, g)
        assert best == _sw_expect(H)


def test_smith_waterman_related_sequences_best_cell():
    # a 10%-mutated copy: a long diagonal of matches, best cell far from the start
    H, g, best = _sw_run(2000, kind="mutated", scoring=(1, -1, -1), alphabet=4)
    assert np.array_equal(H, g)
    assert best == _sw_expect(H) and best[0] > 1000


def test_smith_waterman_c4_size_best_cell():
    """C4 shape (dim 32768, 1 Gi cells) in the bench launch configuration: the best cell
    against the oracle's rows up to it (an exact row prefix), and the grid's last row."""
    dim = 32768
    x, y = workloads.seqcmp_inputs(dim, dim, kind="mutated")
    dev = torch.device("cuda", torch.cuda.current_device())
    with Wavefront("seqcmp", dim, match=1, mismatch=-1, gap=-1, local=1, alphabet=4) as w:
        row_in, col_in, top, left = dev_inputs("seqcmp", (x, y), dev)
        (g,) = w.run(row_in, col_in, top, left)
        w.sync()
        v, r, c = w.local_best()
        last = g[-1].cpu().numpy()
        assert int(g[r - 1, c - 1].item()) == v
        del g
    want = oracle.seqcmp(x, y, 1, -1, -1, local=True)
    assert np.array_equal(last, want[-1])
    assert (v, r, c) == _sw_expect(want)


@pytest.mark.parametrize("alphabet", [4, 8])
@pytest.mark.parametrize("scoring", [(1, -1, -1), (2, -3, -1), (-3, 2, -1), (64, -64, -64), (-64, 64, 64)])
def test_seqcmp_byte_permute_scores(alphabet, scoring):
    # the PRMT score lookup must sign-extend every int8 score and honour match < mismatch
    dim = 555
    rng = np.random.default_rng(alphabet)
    x = rng.integers(0, alphabet, size=dim).astype(np.uint8)
    y = rng.integers(0, alphabet, size=dim).astype(np.uint8)
    M, X, G = scoring
    H = oracle.seqcmp(x, y, M, X, G)
    (g,) = run_gpu("seqcmp", dim, (x, y), match=M, mismatch=X, gap=G, alphabet=alphabet)
    assert np.array_equal(H, g)


@pytest.mark.parametrize("kind", ["identical", "disjoint", "mutated"])
@pytest.mark.parametrize("scoring", [(1, -1, -1), (1, -1, -2), (2, -3, -1), (5, -4, -10), (64, -64, -64), (0, 0, 1)])
def test_seqcmp_input_kinds_and_scorings(kind, scoring):
    H, g = _seq(613, kind=kind, scoring=scoring)
    assert np.array_equal(H, g)


ASCII_KINDS = ["protein", "dna_ascii", "bytes"]


@pytest.mark.parametrize("kind", ASCII_KINDS)
@pytest.mark.parametrize("k,w,d,kernel", [(2, 4, 1, 8), (4, 2, 1, 8), (1, 4, 1, 8), (2, 1, 1, 8), (4, 2, 1, 4),
                                          (4, 1, 2, 4), (8, 1, 1, 4)])
def test_seqcmp_any_byte_residues(kind, k, w, d, kernel):
    """alphabet = 0 (include/wf.h: codes may be any byte value): ASCII amino-acid and DNA
    letters, and raw bytes 0..255 (codes >= 0x80 must not sign-extend into a false match)."""
    for dim, cols, scoring in ((1100, 0, (2, -1, -1)), (777, 1301, (5, -4, -10))):
        H, g = _seq(dim, cols=cols, kind=kind, scoring=scoring, seed=(dim + 3, cols + 5), lane_cols=k, warps=w, skew=d,
                    kernel=kernel, alphabet=0)
        assert np.array_equal(H, g), (kind, dim, cols)


@pytest.mark.parametrize("kind", ASCII_KINDS)
def test_smith_waterman_any_byte_residues(kind):
    for k, w, d in ((2, 4, 1), (4, 2, 1), (4, 1, 2)):
        H, g, best = _sw_run(1000, cols=1200, kind=kind, scoring=(2, -1, -1), lane_cols=k, warps=w, skew=d, alphabet=0)
        assert np.array_equal(H, g)
        assert best == _sw_expect(H)


@pytest.mark.parametrize("G", [2, 3])
def test_seqcmp_any_byte_residues_local_slabs(G):
    H, g = _seq(1000, kind="bytes", ngpus=G, alphabet=0)
    assert np.array_equal(H, g)


@pytest.mark.parametrize("dim,cols", [(300, 517), (517, 300), (1, 1000), (1000, 1), (2, 3), (33, 4097)])
def test_seqcmp_rectangular(dim, cols):
    H, g = _seq(dim, cols=cols)
    assert np.array_equal(H, g)


@pytest.mark.parametrize("max_ctas", [1, 2, 3])
def test_seqcmp_bands_outnumber_ctas(max_ctas):
    # persistent loop: CTA i takes bands i, i+grid, ...
    H, g = _seq(1500, lane_cols=2, warps=1, skew=1, max_ctas=max_ctas)
    assert np.array_equal(H, g)


@pytest.mark.parametrize("G", [2, 3, 4])
def test_seqcmp_local_slabs_on_one_gpu(G):
    # G column slabs ("virtual GPUs") on one device, linked through the LL edge rings
    H, g = _seq(1337, ngpus=G, lane_cols=2, warps=2, skew=2)
    assert np.array_equal(H, g)
    H, g = _seq(2900, ngpus=G, lane_cols=4, warps=2, skew=1, alphabet=4)
    assert np.array_equal(H, g)


def test_seqcmp_rerun_same_context_new_inputs():
    dim = 700
    dev = torch.device("cuda")
    with Wavefront("seqcmp", dim) as w:
        for seed in range(3):
            x, y = workloads.seqcmp_inputs(dim, seed_x=10 + seed, seed_y=20 + seed)
            row_in, col_in, _, _ = dev_inputs("seqcmp", (x, y), dev)
            out = w.run(row_in, col_in)
            w.sync()
            assert np.array_equal(out[0].cpu().numpy(), oracle.seqcmp(x, y))
        assert w.last_run_ms() > 0


def test_seqcmp_determinism_across_tunables():
    dim = 901
    x, y = workloads.seqcmp_inputs(dim, seed_x=5, seed_y=6)
    ref = None
    for k, w, d in [(1, 1, 1), (2, 2, 3), (4, 1, 2), (8, 1, 2)]:
        for G in (1, 2):
            (g,) = run_gpu("seqcmp", dim, (x, y), lane_cols=k, warps=w, skew=d, ngpus=G)
            if ref is None:
                ref = g
            assert np.array_equal(ref, g)


def test_watchdog_turns_a_missing_producer_into_a_timeout():
    # slab 1 of 2 run alone: its west ring is never written -> WF_ETIMEOUT, not a hang
    dim = 256
    x, y = workloads.seqcmp_inputs(dim)
    dev = torch.device("cuda")
    w = Wavefront("seqcmp", dim, rank=1, device=torch.cuda.current_device(), ngpus=2, lane_cols=1, warps=1,
                  skew=1, watchdog_cycles=20_000_000)
    try:
        row_in, col_in, _, _ = dev_inputs("seqcmp", (x, y), dev)
        w.run(row_in, col_in)
        with pytest.raises(_abi.WfError) as ei:
            w.sync()
        assert ei.value.status == _abi.WF_ETIMEOUT
    finally:
        w.close()


def test_seqcmp_c1_config():
    c = workloads.CONFIGS["C1"]
    H, g = _seq(c.dim)
    assert np.array_equal(H, g)


@pytest.mark.slow
def test_seqcmp_c4_full_grid():
    """C4 (dim=32768) in the launch configuration bench.py times: whole grid bit-exact."""
    c = workloads.CONFIGS["C4"]
    H, g = _seq(c.dim, alphabet=4)
    assert np.array_equal(H, g)


@pytest.mark.parametrize("kind,scoring", [("identical", (1, -1, -1)), ("disjoint", (1, -1, -1)),
                                          ("disjoint", (1, -1, -2))])
def test_seqcmp_maximum_dim_closed_forms(kind, scoring):
    """dim = 65535 (the ABI maximum; 4.3 G cells, 17 GB of output): closed forms of the
    recurrence checked on sampled rows -- identical sequences H = min(i,j) M + |i-j| G;
    disjoint alphabets H = min(i,j) X + |i-j| G when X >= 2G (else -max(i,j) for (1,-1,-1))."""
    dim = 65535
    x, y = workloads.seqcmp_inputs(dim, dim, kind=kind)
    M, X, G = scoring
    dev = torch.device("cuda", torch.cuda.current_device())
    with Wavefront("seqcmp", dim, match=M, mismatch=X, gap=G, alphabet=4) as w:
        row_in, col_in, top, left = dev_inputs("seqcmp", (x, y), dev)
        (g,) = w.run(row_in, col_in, top, left)
        w.sync()
        j = np.arange(1, dim + 1, dtype=np.int64)
        for i in (1, 2, 31, 32, 33, 1000, 32767, 32768, 65534, 65535):
            row = g[i - 1].cpu().numpy().astype(np.int64)
            lo, d = np.minimum(i, j), np.abs(i - j)
            if kind == "identical":
                want = lo * M + d * G
            elif X >= 2 * G:
                want = lo * X + d * G
            else:
                want = -np.maximum(i, j)
            assert np.array_equal(row, want), (kind, scoring, i)
        del g


# ------------------------------------------------------------------ synthetic
def _syn(dim, tsize, dsize, cols=0, seeds=(3, 4, 5), m_compute=None, **kw):
    n = cols or dim
    u, v, top, left = workloads.synthetic_inputs(dim, n, dsize, *seeds)
    i0, i1, f = oracle.synthetic(u, v, top, left, tsize, m_compute=m_compute)
    g = run_gpu("synthetic", dim, (u, v, top, left), cols=cols, tsize=tsize, dsize=dsize, **kw)
    return (i0, i1, f), g


def _check_syn(o, g, rows=None):
    i0, i1, f = o
    r = slice(0, rows)
    assert np.array_equal(i0[r], g[0][r])
    assert np.array_equal(i1[r], g[1][r])
    for d in range(f.shape[0]):
        ref, got = f[d][r], g[2 + d][r]
        assert np.all(np.abs(got - ref) <= FTOL * np.abs(ref)), f"plane f{d} exceeds 1e-5 relative"
        assert np.array_equal(ref.view(np.uint32), got.view(np.uint32)), f"plane f{d} not bit-exact"


@pytest.mark.parametrize("dim", [1, 2, 31, 33, 100, 257])
@pytest.mark.parametrize("tsize", [0, 1, 10, 100])
@pytest.mark.parametrize("dsize", [0, 1, 2, 5, 8])
def test_synthetic_grid(dim, tsize, dsize):
    o, g = _syn(dim, tsize, dsize)
    _check_syn(o, g)


@pytest.mark.parametrize("k,w,d", [(1, 1, 1), (1, 4, 1), (2, 1, 1), (2, 2, 1), (1, 2, 2), (2, 2, 2)])
def test_synthetic_variants(k, w, d):
    o, g = _syn(419, 7, 3, lane_cols=k, warps=w, skew=d)
    _check_syn(o, g)


@pytest.mark.parametrize("dim", [1, 33, 257, 419])
@pytest.mark.parametrize("tsize", [0, 7, 100])
@pytest.mark.parametrize("dsize", [2, 3, 5, 8])
def test_synthetic_plane_split(dim, tsize, dsize):
    """kernel=8: one warp per float item on the same columns (R5: the items of a cell are
    independent given its inputs) -- same grid as the oracle, bit-exact."""
    o, g = _syn(dim, tsize, dsize, kernel=8, lane_cols=1, warps=1, skew=1)
    _check_syn(o, g)


@pytest.mark.parametrize("tsize", [100, 1000])
def test_synthetic_plane_split_compiled_tsize(tsize):
    o, g = _syn(300, tsize, 5, kernel=8, lane_cols=1, warps=1, skew=1)
    _check_syn(o, g)


@pytest.mark.parametrize("G", [2, 3])
def test_synthetic_plane_split_slabs_and_rect(G):
    o, g = _syn(333, 9, 5, kernel=8, lane_cols=1, warps=1, skew=1, ngpus=G)
    _check_syn(o, g)
    o, g = _syn(129, 9, 3, cols=300, kernel=8, lane_cols=1, warps=1, skew=1)
    _check_syn(o, g)


def test_synthetic_plane_split_rejects_single_item():
    with pytest.raises(_abi.WfError) as ei:
        _syn(64, 5, 1, kernel=8, lane_cols=1, warps=1, skew=1)
    assert ei.value.status == _abi.WF_EUNSUPPORTED


@pytest.mark.parametrize("G", [2, 3])
def test_synthetic_local_slabs(G):
    o, g = _syn(333, 5, 2, ngpus=G)
    _check_syn(o, g)


def test_synthetic_rectangular():
    o, g = _syn(129, 3, 2, cols=300)
    _check_syn(o, g)


def test_synthetic_c2_full_grid():
    c = workloads.CONFIGS["C2"]
    o, g = _syn(c.dim, c.tsize, c.dsize)
    _check_syn(o, g)


@pytest.mark.slow
@pytest.mark.parametrize("name,prefix,kw", [("C5a", 64, {}), ("C5b", 32, {}), ("C5c", 8, {}), ("C5d", 4, {}),
                                            ("C5d", 4, {"kernel": 8, "lane_cols": 1, "warps": 1, "skew": 1})])
def test_synthetic_c5_prefix_and_closed_forms(name, prefix, kw):
    """C5 at full size: exact parity on a row prefix (a true prefix of the grid), plus the
    closed forms i0 = (i-1)+(j-1), i1 = i*j and the value range on EVERY cell."""
    c = workloads.CONFIGS[name]
    o, g = _syn(c.dim, c.tsize, c.dsize, m_compute=prefix, **kw)
    _check_syn(o, g, rows=prefix)
    i = np.arange(1, c.dim + 1, dtype=np.int64)[:, None]
    j = np.arange(1, c.dim + 1, dtype=np.int64)[None, :]
    assert np.array_equal(g[0], (i - 1) + (j - 1))
    assert np.array_equal(g[1], (i * j).astype(np.int64).astype(np.int32))
    for d in range(c.dsize):
        assert g[2 + d].min() >= 0.25 and g[2 + d].max() < 1.0


@pytest.mark.parametrize("dsize", [1, 5])
def test_synthetic_default_kernel_tsize1000_full_grid(dsize):
    """The shipped default kernels at tsize = 1000 (syn_kernel<1|5,1,1,1000>, the only users of the
    UB = 4 hand-off block): full grid, bit-exact.  dim 333 = 11 one-warp bands with a ragged last
    band, 333 > 128 rows so the staging and hand-off rings wrap."""
    o, g = _syn(333, 1000, dsize)
    _check_syn(o, g)


@pytest.mark.slow
@pytest.mark.parametrize("name", ["C5a", "C5b", "C5c", "C5d"])
def test_synthetic_c5_full_grid_row_hashes(name):
    """C5 at full size in the bench's launch configuration: every row of every plane against the
    oracle's full grid through per-row 64-bit hashes (tests/golden/c5_rowhash_<C>.npy, written
    by tools/make_c5_golden.py from oracle/ only)."""
    import os
    from _rowhash import row_hashes
    c = workloads.CONFIGS[name]
    want = np.load(os.path.join(os.path.dirname(__file__), "golden", f"c5_rowhash_{name}.npy"))
    u, v, top, left = workloads.synthetic_inputs(c.dim, c.dim, c.dsize)
    g = run_gpu("synthetic", c.dim, (u, v, top, left), tsize=c.tsize, dsize=c.dsize)
    got = row_hashes(g)
    bad = np.flatnonzero(got != want)
    assert bad.size == 0, f"{name}: {bad.size} rows differ from the oracle, first row {bad[:5] + 1}"


# ------------------------------------------------------------------ Nash stand-in
def _nash(dim, n=16, cols=0, seeds=(6, 7, 8), m_compute=None, **kw):
    nc = cols or dim
    r, c, top, left = workloads.nash_inputs(dim, nc, *seeds)
    o = oracle.nash(r, c, top, left, nstrat=n, m_compute=m_compute)
    g = run_gpu("nash", dim, (r, c, top, left), cols=cols, tsize=n, dsize=4, **kw)
    return o, g


def _check_nash(o, g, rows=None):
    r = slice(0, rows)
    for p in range(4):
        assert np.array_equal(o[p][r], g[p][r]), f"plane p{p} differs"


@pytest.mark.parametrize("dim", [1, 2, 7, 8, 9, 33, 100, 130])
def test_nash_dims(dim):
    o, g = _nash(dim)
    _check_nash(o, g)


@pytest.mark.parametrize("n", [1, 2, 3, 5, 7, 16, 31, 32, 33, 64])
def test_nash_strategy_counts(n):
    # n spans: single entry, sub-warp, not dividing 32, exactly one round, > 32 columns
    o, g = _nash(41, n=n, seeds=(n, n + 1, n + 2))
    _check_nash(o, g)


@pytest.mark.parametrize("w", [1, 2, 4, 8])
def test_nash_band_widths(w):
    o, g = _nash(75, warps=w)
    _check_nash(o, g)


def test_nash_rectangular_and_band_loop():
    o, g = _nash(20, cols=203, max_ctas=2)
    _check_nash(o, g)
    o, g = _nash(203, cols=20)
    _check_nash(o, g)


@pytest.mark.parametrize("G", [2, 3])
def test_nash_local_slabs(G):
    o, g = _nash(150, ngpus=G)
    _check_nash(o, g)


def test_nash_outputs_are_valid_equilibria():
    # property check independent of the oracle: p1 indexes an entry whose payoffs are p2, p3
    o, g = _nash(64)
    cnt, first, pa, pb = g
    assert np.all((first == -1) == (cnt == 0))
    assert np.all((pa == -1) == (first == -1)) and np.all((pb == -1) == (first == -1))
    assert np.all((first >= -1) & (first < 256)) and np.all((pa >= -1) & (pa < 256))


@pytest.mark.slow
def test_nash_c3_prefix():
    """C3 (dim=4096, n=16) at full size in the bench's launch configuration: exact parity
    on a row prefix (a true prefix of the grid) and the validity properties on every cell."""
    c = workloads.CONFIGS["C3"]
    o, g = _nash(c.dim, n=c.tsize, m_compute=48)
    _check_nash(o, g, rows=48)
    cnt, first = g[0], g[1]
    assert np.all((first == -1) == (cnt == 0)) and cnt.max() <= 16 * 16


# ---- transport = "nccl" in one process (the message moved by a device copy instead of send/recv)
@pytest.mark.parametrize("case", ["nw8_staged", "syn_staged"])
def test_staged_transport_in_process(case):
    import sys
    import os
    sys.path.insert(0, os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "tools"))
    import sanitize_cases
    sanitize_cases.run(case)


@pytest.mark.parametrize("G", [2, 3])
def test_staged_transport_in_process_nw_three_slabs(G):
    import sys
    import os
    sys.path.insert(0, os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "tools"))
    from sanitize_cases import run_staged_in_process
    x, y = workloads.seqcmp_inputs(1500, 1500, seed_x=21, seed_y=22)
    H = oracle.seqcmp(x, y, 1, -1, -1)
    (g,) = run_staged_in_process("seqcmp", 1500, (x, y), ngpus=G, transport="nccl", alphabet=4)
    assert np.array_equal(g, H)
