"""CPU check of the generation-8 NW ramp-up (wf_nw8.cu, Warp constructor).

Lane l of a warp starts on row 1 - l.  Instead of predicating its state updates until it reaches
row 1, the kernel extends the row-0 boundary H[0][j] = j g (P:150-157 with DESIGN.md R2) to
virtual rows r <= 0 by V(r, j) = j g + r c, c = max(1, g, max(match, mismatch) - g).  These
tests pin the two facts the kernel relies on, independently of the kernel and of the oracle:
V is a fixed point of the recurrence for every score a virtual cell may draw, and a grid
computed through any number of virtual rows equals the grid computed from the true boundary.
"""
from __future__ import annotations

import numpy as np
import pytest


def c_of(match, mismatch, gap):
    return max(1, gap, max(match, mismatch) - gap)


@pytest.mark.parametrize("gap", list(range(-64, 65, 4)) + [64])
def test_virtual_rows_are_a_fixed_point(gap):
    """max(V(r-1,j)+g, V(r,j-1)+g, V(r-1,j-1)+s) == V(r,j) for s in {match, mismatch}, over the
    ABI range [-64, 64] of every scoring parameter."""
    sc = np.arange(-64, 65)
    M, X = np.meshgrid(sc, sc, indexing="ij")
    c = np.maximum(np.maximum(1, gap), np.maximum(M, X) - gap)
    for r in (-31, -5, 0):
        for j in (1, 7, 40000):
            V = lambda rr, jj: jj * gap + rr * c  # noqa: E731
            for s in (M, X):
                h = np.maximum(np.maximum(V(r - 1, j) + gap, V(r, j - 1) + gap), V(r - 1, j - 1) + s)
                assert np.array_equal(h, V(r, j))


def _grid(x, y, M, X, g, virt, rng):
    m, n = len(x), len(y)
    c = c_of(M, X, g)
    H = np.zeros((m + virt + 1, n + 1), dtype=np.int64)   # row index r + virt
    H[0, :] = np.arange(n + 1) * g - virt * c
    for r in range(-virt + 1, m + 1):
        i = r + virt
        H[i, 0] = r * g if r >= 0 else r * c
        for j in range(1, n + 1):
            s = (M if x[r - 1] == y[j - 1] else X) if r >= 1 else int(rng.choice((M, X)))
            H[i, j] = max(H[i - 1, j] + g, H[i, j - 1] + g, H[i - 1, j - 1] + s)
    return H[virt + 1:, 1:]


@pytest.mark.parametrize("seed", range(40))
def test_grid_through_virtual_rows_equals_the_boundary_grid(seed):
    rng = np.random.default_rng(seed)
    M, X, g = (int(v) for v in rng.integers(-64, 65, size=3))
    x = rng.integers(0, 4, size=int(rng.integers(1, 10)))
    y = rng.integers(0, 4, size=int(rng.integers(1, 9)))
    ref = _grid(x, y, M, X, g, 0, rng)
    for virt in (1, 5, 31):
        assert np.array_equal(_grid(x, y, M, X, g, virt, rng), ref)
