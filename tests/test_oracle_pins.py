"""Pins of the CPU oracle against things other than itself.

Each test pins the oracle to a value or property fixed by a textbook, the paper or
mathematics -- never to a re-typing of the oracle's own formula.  CPU only.
"""
from __future__ import annotations

import itertools
import math
import os

import numpy as np
import pytest

import oracle
import workloads

GOLDEN = os.path.join(os.path.dirname(__file__), "golden")
DNA = {c: i for i, c in enumerate("ACGT")}


def _read_golden(name):
    rec = {"align": [], "game": []}
    with open(os.path.join(GOLDEN, name)) as f:
        for line in f:
            line = line.strip()
            if not line or line.startswith("#"):
                continue
            key, *rest = line.split()
            if key in ("align", "game"):
                rec[key].append(rest)
            else:
                rec[key] = rest if len(rest) > 1 else rest[0]
    return rec


def _codes(s):
    return np.array([DNA[c] for c in s], dtype=np.uint8)


def _score_alignment(a, b, match, mismatch, gap):
    """Score of an explicit alignment (gap columns are '-'); independent of any DP."""
    assert len(a) == len(b)
    s = 0
    for p, q in zip(a, b):
        if p == "-" or q == "-":
            s += gap
        else:
            s += match if p == q else mismatch
    return s


# ---------------------------------------------------------------- sequence comparison
@pytest.mark.parametrize("golden", ["nw_wikipedia.txt", "nw_setubal_meidanis.txt"])
def test_nw_textbook_worked_examples(golden):
    g = _read_golden(golden)
    M, X, G = int(g["match"]), int(g["mismatch"]), int(g["gap"])
    H = oracle.seqcmp(_codes(g["x"]), _codes(g["y"]), M, X, G)
    assert H[-1, -1] == int(g["score"])
    for a, b in g["align"]:
        # the printed optimal alignments really are alignments of x, y with that score
        assert a.replace("-", "") == g["x"] and b.replace("-", "") == g["y"]
        assert _score_alignment(a, b, M, X, G) == int(g["score"])


def _all_global_alignment_scores(x, y, M, X, G):
    """Enumerate every global alignment of x and y (move sequences D/U/L) -> list of scores."""
    out = []

    def rec(i, j, s):
        if i == len(x) and j == len(y):
            out.append(s)
            return
        if i < len(x) and j < len(y):
            rec(i + 1, j + 1, s + (M if x[i] == y[j] else X))
        if i < len(x):
            rec(i + 1, j, s + G)
        if j < len(y):
            rec(i, j + 1, s + G)

    rec(0, 0, 0)
    return out


def test_alignment_enumeration_counts_delannoy():
    # number of global alignments of lengths (m, n) is the Delannoy number D(m, n)
    def delannoy(m, n):
        return sum(math.comb(m, k) * math.comb(n, k) * 2 ** k for k in range(min(m, n) + 1))
    assert delannoy(6, 6) == 8989
    assert len(_all_global_alignment_scores([0] * 6, [1] * 6, 1, -1, -1)) == 8989
    assert len(_all_global_alignment_scores([0] * 3, [1] * 5, 1, -1, -1)) == delannoy(3, 5)


@pytest.mark.parametrize("scoring", [(1, -1, -1), (1, -1, -2), (2, -3, -1)])
def test_nw_brute_force_all_prefixes(scoring):
    """H[i][j] == max over ALL alignments of x[:i], y[:j] (m, n <= 6)."""
    M, X, G = scoring
    rng = np.random.default_rng(11)
    for _ in range(12):
        m, n = rng.integers(1, 7, size=2)
        x = rng.integers(0, 4, size=m).astype(np.uint8)
        y = rng.integers(0, 4, size=n).astype(np.uint8)
        H = oracle.seqcmp(x, y, M, X, G)
        for i in range(1, m + 1):
            for j in range(1, n + 1):
                assert H[i - 1, j - 1] == max(_all_global_alignment_scores(x[:i], y[:j], M, X, G))


@pytest.mark.parametrize("kind", ["protein", "bytes"])
def test_nw_brute_force_any_byte_residues(kind):
    """alphabet = 0 inputs (ASCII letters, bytes >= 0x80): the oracle still equals the maximum
    over all alignments -- only equality of codes enters s(x_i, y_j)."""
    M, X, G = 2, -1, -1
    for t in range(8):
        x, y = workloads.seqcmp_inputs(int(3 + t % 4), int(6 - t % 3), kind=kind, seed_x=40 + t, seed_y=80 + t)
        if t % 2:   # force some matches
            y[: min(len(x), len(y)) // 2] = x[: min(len(x), len(y)) // 2]
        H = oracle.seqcmp(x, y, M, X, G)
        for i in range(1, len(x) + 1):
            for j in range(1, len(y) + 1):
                assert H[i - 1, j - 1] == max(_all_global_alignment_scores(x[:i], y[:j], M, X, G))


def test_nw_invariant_under_residue_relabelling():
    """A bijection of the byte alphabet leaves the grid unchanged (s depends on x_i == y_j only);
    0x80..0xff codes behave like any other (no sign-extension artefacts)."""
    x, y = workloads.seqcmp_inputs(200, 230, kind="bytes")
    perm = np.random.default_rng(5).permutation(256).astype(np.uint8)
    for local in (False, True):
        H = oracle.seqcmp(x, y, 2, -1, -1, local=local)
        assert np.array_equal(H, oracle.seqcmp(perm[x], perm[y], 2, -1, -1, local=local))
    px, py = workloads.seqcmp_inputs(150, kind="protein")
    assert set(np.unique(px)) <= set(workloads.PROTEIN) and len(np.unique(px)) == 20
    codes = {c: i for i, c in enumerate(workloads.PROTEIN)}
    assert np.array_equal(oracle.seqcmp(px, py, 1, -1, -1),
                          oracle.seqcmp(np.array([codes[c] for c in px], np.uint8),
                                        np.array([codes[c] for c in py], np.uint8), 1, -1, -1))


def test_sw_local_brute_force():
    """Smith-Waterman H[i][j] == max(0, best alignment of a suffix of x[:i] with a suffix of y[:j])."""
    M, X, G = 2, -1, -1
    rng = np.random.default_rng(12)
    for _ in range(6):
        m, n = rng.integers(1, 6, size=2)
        x = rng.integers(0, 4, size=m).astype(np.uint8)
        y = rng.integers(0, 4, size=n).astype(np.uint8)
        H = oracle.seqcmp(x, y, M, X, G, local=True)
        for i in range(1, m + 1):
            for j in range(1, n + 1):
                best = 0
                for a in range(0, i):
                    for b in range(0, j):
                        best = max(best, max(_all_global_alignment_scores(x[a:i], y[b:j], M, X, G)))
                assert H[i - 1, j - 1] == best


def test_nw_closed_form_identical_sequences():
    # x == y: best is min(i,j) matches plus |i-j| gaps (for M >= 0 >= G, X <= M)
    x, y = workloads.seqcmp_inputs(300, kind="identical")
    H = oracle.seqcmp(x, y, 1, -1, -1)
    i = np.arange(1, 301)[:, None]
    j = np.arange(1, 301)[None, :]
    assert np.array_equal(H, np.minimum(i, j) * 1 + np.abs(i - j) * -1)


@pytest.mark.parametrize("scoring,expect", [((1, -1, -1), lambda i, j: -np.maximum(i, j)),
                                            ((1, -1, -2), lambda i, j: np.minimum(i, j) * -1 + np.abs(i - j) * -2)])
def test_nw_closed_form_disjoint_alphabets(scoring, expect):
    # no match possible: min(i,j) mismatches + |i-j| gaps whenever X >= 2G
    x, y = workloads.seqcmp_inputs(257, 301, kind="disjoint")
    H = oracle.seqcmp(x, y, *scoring)
    i = np.arange(1, 258)[:, None]
    j = np.arange(1, 302)[None, :]
    assert np.array_equal(H, expect(i, j))


def test_nw_transpose_and_reversal_symmetry():
    x, y = workloads.seqcmp_inputs(97, 131)
    H = oracle.seqcmp(x, y, 1, -1, -1)
    Ht = oracle.seqcmp(y, x, 1, -1, -1)
    assert np.array_equal(H, Ht.T)
    Hr = oracle.seqcmp(x[::-1].copy(), y[::-1].copy(), 1, -1, -1)
    assert Hr[-1, -1] == H[-1, -1]


def test_nw_row_prefix_is_exact_prefix():
    x, y = workloads.seqcmp_inputs(200)
    full = oracle.seqcmp(x, y)
    part = oracle.seqcmp(x, y, m_compute=37)
    assert np.array_equal(full[:37], part[:37])
    assert not part[37:].any()


# ---------------------------------------------------------------- anti-diagonal order
def _antidiag_profile(m, n):
    return [sum(1 for i in range(m) for j in range(n) if i + j == t) for t in range(m + n - 1)]


def test_fig1_diagonal_profile():
    g = _read_golden("fig1_profile.txt")
    prof = _antidiag_profile(int(g["rows"]), int(g["cols"]))
    assert prof == [int(v) for v in g["profile"]]
    mx = max(prof)
    assert [t for t, v in enumerate(prof) if v == mx] == [int(v) for v in g["max_iterations"]]


def _nw_antidiagonal(x, y, M, X, G):
    """Test-only evaluator: whole anti-diagonals at once (numpy), no code shared with the oracle."""
    m, n = len(x), len(y)
    A = np.zeros((m + 1, n + 1), dtype=np.int64)
    A[0, :] = np.arange(n + 1) * G
    A[:, 0] = np.arange(m + 1) * G
    for t in range(2, m + n + 1):
        i = np.arange(max(1, t - n), min(m, t - 1) + 1)
        j = t - i
        s = np.where(x[i - 1] == y[j - 1], M, X)
        A[i, j] = np.maximum(np.maximum(A[i - 1, j - 1] + s, A[i - 1, j] + G), A[i, j - 1] + G)
    return A[1:, 1:]


def test_nw_rowmajor_equals_antidiagonal_order():
    x, y = workloads.seqcmp_inputs(123, 77)
    assert np.array_equal(oracle.seqcmp(x, y, 1, -1, -1), _nw_antidiagonal(x, y, 1, -1, -1))


# ---------------------------------------------------------------- synthetic
def test_synthetic_int_closed_forms():
    m, n = 173, 211
    u, v, top, left = workloads.synthetic_inputs(m, n, 2)
    i0, i1, f = oracle.synthetic(u, v, top, left, tsize=3)
    i = np.arange(1, m + 1)[:, None]
    j = np.arange(1, n + 1)[None, :]
    assert np.array_equal(i0, (i - 1) + (j - 1))
    assert np.array_equal(i1, i * j)


@pytest.mark.parametrize("b", [0.5, 0.625, 0.75, 0.875])
@pytest.mark.parametrize("tsize", [0, 7, 1000])
def test_synthetic_constant_field_fixed_point(b, tsize):
    """u = 1, v = b, boundary floats = b  =>  every cell is exactly b.

    (b+b)+b = 3b is exact for these b; 3b * fl(1/3) = b(1 + 2^-24 * 0.5) rounds to b for
    b in [0.5,1); c = (1*b)*2^-12 exactly, and fma(b, 1-2^-12, b*2^-12) = b exactly."""
    m, n, d = 40, 33, 2
    u = np.ones(m, np.float32)
    v = np.full(n, b, np.float32)
    top = np.full((d, n + 1), b, np.float32)
    left = np.full((d, m + 1), b, np.float32)
    i0, i1, f = oracle.synthetic(u, v, top, left, tsize=tsize)
    assert np.all(f == np.float32(b))


@pytest.mark.parametrize("tsize", [1, 10, 100])
def test_synthetic_iteration_closed_form(tsize):
    """x_T = uv + A^T (x_0 - uv) in exact arithmetic (A = 1 - 2^-12, c = uv 2^-12).

    Each fma rounds once (<= 2^-24 relative) and errors are damped by A < 1, so the fp32
    result lies within (T+2) 2^-24 |x| of the closed form.  A wrong A, c scale or trip count
    (off by one: 2^-12 A^T |x_0 - uv|) breaks this bound."""
    m, n, d = 24, 29, 1
    u, v, top, left = workloads.synthetic_inputs(m, n, d, seed_u=21, seed_v=22, seed_b=23)
    i0, i1, f = oracle.synthetic(u, v, top, left, tsize=tsize)
    F = np.zeros((m + 1, n + 1), np.float32)
    F[0, :] = top[0]
    F[1:, 0] = left[0, 1:]
    F[1:, 1:] = f[0]
    A = 1.0 - 2.0 ** -12
    for i in range(1, m + 1):
        for j in range(1, n + 1):
            x0 = np.float32(np.float32(F[i - 1, j] + F[i - 1, j - 1]) + F[i, j - 1]) * np.float32(1 / 3)
            uv = float(np.float32(u[i - 1] * v[j - 1]))
            exact = uv + A ** tsize * (float(x0) - uv)
            err = abs(float(F[i, j]) - exact)
            bound = (tsize + 2) * 2.0 ** -24 * max(abs(exact), 1.0)
            assert err <= bound


def test_synthetic_values_in_range_and_distinct():
    m = 96
    u, v, top, left = workloads.synthetic_inputs(m, m, 3)
    i0, i1, f = oracle.synthetic(u, v, top, left, tsize=11)
    assert f.min() >= 0.25 and f.max() < 1.0
    deep = f[:, 32:, 32:]
    assert len(np.unique(deep)) > 0.9 * deep.size


def test_synthetic_row_prefix_is_exact_prefix():
    u, v, top, left = workloads.synthetic_inputs(50, 60, 2)
    a = oracle.synthetic(u, v, top, left, 5)
    b = oracle.synthetic(u, v, top, left, 5, m_compute=17)
    assert np.array_equal(a[0][:17], b[0][:17]) and np.array_equal(a[2][:, :17], b[2][:, :17])


# ---------------------------------------------------------------- nash
def test_lowbias32_matches_published_inverse():
    """lowbias32 (C. Wellons, hash-prospector) has the published inverse
    x ^= x>>16; x *= 0x43021123; x ^= x>>15 ^ x>>30; x *= 0x1d69e2a5; x ^= x>>16."""
    assert pow(0x846CA68B, -1, 1 << 32) == 0x43021123
    assert pow(0x7FEB352D, -1, 1 << 32) == 0x1D69E2A5

    def inv(x):
        x ^= x >> 16
        x = (x * 0x43021123) & 0xFFFFFFFF
        x ^= (x >> 15) ^ (x >> 30)
        x = (x * 0x1D69E2A5) & 0xFFFFFFFF
        x ^= x >> 16
        return x

    rng = np.random.default_rng(5)
    for v in list(rng.integers(0, 1 << 32, size=300)) + [0, 1, 0xFFFFFFFF, 0x80000000]:
        v = int(v)
        assert inv(oracle.lowbias32(v)) == v
    assert oracle.lowbias32(0) == 0


def test_nash_solver_textbook_games():
    g = _read_golden("nash_textbook_games.txt")
    assert len(g["game"]) >= 3
    for rec in g["game"]:
        name = rec[0]
        a = rec.index("A"), rec.index("B"), rec.index("expected")
        A = np.array([int(t) for t in rec[a[0] + 1:a[1]]]).reshape(2, 2)
        B = np.array([int(t) for t in rec[a[1] + 1:a[2]]]).reshape(2, 2)
        exp = tuple(int(t) for t in rec[a[2] + 1:])
        assert oracle.nash_solve(A, B) == exp, name


def test_nash_solver_all_ties_every_profile_is_equilibrium():
    n = 5
    Z = np.zeros((n, n), np.int32)
    assert oracle.nash_solve(Z, Z) == (n * n, 0, 0, 0)


def test_nash_solver_vs_deviation_enumeration():
    rng = np.random.default_rng(9)
    for _ in range(200):
        n = int(rng.integers(1, 7))
        A = rng.integers(0, 4, size=(n, n))
        B = rng.integers(0, 4, size=(n, n))
        ne = [(a, b) for a, b in itertools.product(range(n), range(n))
              if not any(A[a2, b] > A[a, b] for a2 in range(n))
              and not any(B[a, b2] > B[a, b] for b2 in range(n))]
        first = ne[0][0] * n + ne[0][1] if ne else -1
        exp = (len(ne), first, int(A.flat[first]) if ne else -1, int(B.flat[first]) if ne else -1)
        assert oracle.nash_solve(A, B) == exp


def test_nash_grid_expected_equilibrium_count():
    """For iid uniform{0..255} payoffs, E[#pure NE] = n^2 q^2 with
    q = P(entry >= the n-1 others) = sum_k (1/256) ((k+1)/256)^(n-1).  The hash-derived
    payoffs must reproduce this (within 5 sigma) and the first-NE fields must be consistent."""
    n = 16
    m = 72
    r, c, top, left = workloads.nash_inputs(m, m)
    out = oracle.nash(r, c, top, left, nstrat=n)
    q = sum((1 / 256) * ((k + 1) / 256) ** (n - 1) for k in range(256))
    expect = n * n * q * q
    p0 = out[0].astype(np.float64)
    sigma = p0.std() / math.sqrt(p0.size)
    assert abs(p0.mean() - expect) < 5 * sigma + 1e-3
    none = out[0] == 0
    assert np.all(out[1][none] == -1) and np.all(out[2][none] == -1) and np.all(out[3][none] == -1)
    some = ~none
    assert np.all((out[1][some] >= 0) & (out[1][some] < n * n))
    assert np.all((out[2][some] >= 0) & (out[2][some] <= 255))


def test_nash_cell_matches_grid_and_w_enters_key():
    m = 6
    r, c, top, left = workloads.nash_inputs(m, m)
    out = oracle.nash(r, c, top, left, nstrat=8)
    N = out[:, 2, 3]
    W = out[:, 3, 2]
    NW = out[:, 2, 2]
    assert oracle.nash_cell(8, N, NW, W, int(r[3]), int(c[3])) == tuple(int(v) for v in out[:, 3, 3])
    # W, N, NW, r, c all enter the key: perturbing any of them changes some cell output
    base = tuple(int(v) for v in out[:, 3, 3])
    for which in range(5):
        changed = False
        for bit in range(8):
            args = [N.copy(), NW.copy(), W.copy(), int(r[3]), int(c[3])]
            if which < 3:
                args[which][bit % 4] ^= 1 << bit
            else:
                args[which] ^= 1 << bit
            changed |= oracle.nash_cell(8, *args) != base
        assert changed, which


def test_oracle_rejects_bad_arguments():
    with pytest.raises(ValueError):
        oracle.nash(np.zeros(2, np.uint32), np.zeros(2, np.uint32), np.zeros((4, 3), np.int32),
                    np.zeros((4, 3), np.int32), nstrat=65)
