"""Per-row 64-bit hashes of output planes -- test infrastructure ("full-grid
parity for C5 uses per-row hashes ... precomputed by the same oracle binary").

The hash holds none of the method's arithmetic.  For row r of a grid with planes p = 0..P-1
(each row n 32-bit words, ints or fp32 bit patterns):

    h[r] = sum_p sum_j  word_p[r][j] * C[p][j]   (mod 2**64)

with C a fixed table of odd 64-bit constants drawn from PCG64(0x5EED).  Any change of one
word changes h (odd multipliers are invertible mod 2**64).  The same function hashes the
oracle's planes (tools/make_c5_golden.py) and the GPU planes (tests), so a row matches iff
its hash matches, up to a 2**-64 collision chance per differing row.
"""
from __future__ import annotations

import numpy as np

_SEED = 0x5EED


def constants(nplanes: int, n: int) -> np.ndarray:
    rng = np.random.Generator(np.random.PCG64(_SEED))
    c = rng.integers(0, 1 << 63, size=(nplanes, n), dtype=np.int64).astype(np.uint64)
    return (c << np.uint64(1)) | np.uint64(1)


def row_hashes(planes, chunk: int = 512) -> np.ndarray:
    """planes: sequence of (m, n) arrays with 4-byte elements (numpy, or anything with
    ``__getitem__`` row slicing returning numpy-convertible blocks).  Returns uint64[m]."""
    m, n = planes[0].shape
    C = constants(len(planes), n)
    h = np.zeros(m, dtype=np.uint64)
    with np.errstate(over="ignore"):
        for r0 in range(0, m, chunk):
            r1 = min(m, r0 + chunk)
            acc = np.zeros(r1 - r0, dtype=np.uint64)
            for p, pl in enumerate(planes):
                blk = np.ascontiguousarray(np.asarray(pl[r0:r1])).view(np.uint32).astype(np.uint64)
                acc += (blk * C[p][None, :]).sum(axis=1, dtype=np.uint64)
            h[r0:r1] = acc
    return h
