"""Seeded synthetic input generators and the BASELINE.json configs.

This module is shared by the oracle-side tests, the GPU parity tests and bench.py.
It holds NONE of the method's arithmetic: it only draws inputs (input
recipe; SURVEY.md §8(d) "Synthetic inputs").  Generators are numpy
``Generator(PCG64(seed))`` draws, deterministic per seed.
"""
from __future__ import annotations

from dataclasses import dataclass, field

import numpy as np

# Default seeds.
SEED_X, SEED_Y = 1, 2          # sequence comparison
SEED_U, SEED_V, SEED_SYN_B = 3, 4, 5   # synthetic
SEED_R, SEED_C, SEED_NASH_B = 6, 7, 8  # nash


def _rng(seed: int) -> np.random.Generator:
    return np.random.Generator(np.random.PCG64(seed))


def unit_half_open_f32(rng: np.random.Generator, shape) -> np.ndarray:
    """fp32 uniform on [0.5, 1): (2^23 + k) * 2^-24, k uniform in [0, 2^23) -- exact, never 1.0."""
    k = rng.integers(0, 1 << 23, size=shape, dtype=np.int64)
    return ((k + (1 << 23)).astype(np.float64) * 2.0 ** -24).astype(np.float32)


PROTEIN = b"ACDEFGHIKLMNPQRSTVWY"   # the 20 standard amino-acid one-letter codes


def seqcmp_inputs(m: int, n: int | None = None, kind: str = "random", seed_x: int = SEED_X,
                  seed_y: int = SEED_Y, alphabet: int = 4, mutation: float = 0.10):
    """DNA-like residue codes in {0..alphabet-1} (uint8).

    kind: 'random' (x, y independent uniform), 'identical' (y = x), 'disjoint'
    (x over {0,1}, y over {2,3}), 'mutated' (y = x with `mutation` of positions redrawn),
    'protein' (ASCII amino-acid letters, PROTEIN), 'dna_ascii' (b"ACGT"), 'bytes' (any byte
    value 0..255, including 0x80..0xff) -- the wf_params.alphabet = 0 inputs.
    """
    n = m if n is None else n
    rx, ry = _rng(seed_x), _rng(seed_y)
    if kind == "random":
        x = rx.integers(0, alphabet, size=m, dtype=np.uint8)
        y = ry.integers(0, alphabet, size=n, dtype=np.uint8)
    elif kind == "identical":
        x = rx.integers(0, alphabet, size=max(m, n), dtype=np.uint8)
        x, y = x[:m].copy(), x[:n].copy()
    elif kind == "disjoint":
        x = rx.integers(0, 2, size=m, dtype=np.uint8)
        y = (ry.integers(0, 2, size=n, dtype=np.uint8) + 2).astype(np.uint8)
    elif kind in ("protein", "dna_ascii"):
        letters = np.frombuffer(PROTEIN if kind == "protein" else b"ACGT", dtype=np.uint8)
        x = letters[rx.integers(0, len(letters), size=m)]
        y = letters[ry.integers(0, len(letters), size=n)]
    elif kind == "bytes":
        x = rx.integers(0, 256, size=m, dtype=np.uint8)
        y = ry.integers(0, 256, size=n, dtype=np.uint8)
    elif kind == "mutated":
        base = rx.integers(0, alphabet, size=max(m, n), dtype=np.uint8)
        x = base[:m].copy()
        y = base[:n].copy()
        mask = ry.random(n) < mutation
        y[mask] = ry.integers(0, alphabet, size=int(mask.sum()), dtype=np.uint8)
    else:
        raise ValueError(kind)
    return x, y


def synthetic_inputs(m: int, n: int | None, dsize: int, seed_u: int = SEED_U, seed_v: int = SEED_V,
                     seed_b: int = SEED_SYN_B):
    """u (m), v (n) in [0.5,1); boundary floats top (dsize, n+1), left (dsize, m+1) in [0.5,1).

    left[:, 0] is set equal to top[:, 0] (the shared corner (0,0))."""
    n = m if n is None else n
    u = unit_half_open_f32(_rng(seed_u), m)
    v = unit_half_open_f32(_rng(seed_v), n)
    rb = _rng(seed_b)
    top = unit_half_open_f32(rb, (dsize, n + 1))
    left = unit_half_open_f32(rb, (dsize, m + 1))
    left[:, 0] = top[:, 0]
    return u, v, top, left


def nash_inputs(m: int, n: int | None = None, seed_r: int = SEED_R, seed_c: int = SEED_C,
                seed_b: int = SEED_NASH_B):
    """r (m), c (n) uint32; boundary planes top (4, n+1), left (4, m+1) int32 in [0, 255]."""
    n = m if n is None else n
    r = _rng(seed_r).integers(0, 1 << 32, size=m, dtype=np.uint64).astype(np.uint32)
    c = _rng(seed_c).integers(0, 1 << 32, size=n, dtype=np.uint64).astype(np.uint32)
    rb = _rng(seed_b)
    top = rb.integers(0, 256, size=(4, n + 1), dtype=np.int32)
    left = rb.integers(0, 256, size=(4, m + 1), dtype=np.int32)
    left[:, 0] = top[:, 0]
    return r, c, top, left


@dataclass(frozen=True)
class Config:
    """One BASELINE.json config."""
    name: str
    fn: str            # 'seqcmp' | 'synthetic' | 'nash'
    dim: int
    tsize: int = 0
    dsize: int = 0
    gpus: tuple = (1,)
    note: str = ""
    extra: dict = field(default_factory=dict)

    @property
    def cells(self) -> int:
        return self.dim * self.dim

    def bytes_per_cell(self) -> int:
        """Algorithmic output bytes per cell (each output cell written once)."""
        if self.fn == "seqcmp":
            return 4
        if self.fn == "synthetic":
            return 8 + 4 * self.dsize
        return 16


NASH_N = 16  # strategies per player for the Nash stand-in (reading R8)

CONFIGS = {
    "C1": Config("C1", "seqcmp", 512, note="sequence comparison (Needleman-Wunsch) dim=512, 1 GPU"),
    "C2": Config("C2", "synthetic", 2048, tsize=100, dsize=1,
                 note="synthetic wavefront dim=2048 tsize=100 dsize=1 float, 1 GPU"),
    "C3": Config("C3", "nash", 4096, tsize=NASH_N, dsize=4, gpus=(1, 2),
                 note="Nash equilibrium wavefront dim=4096, 1/2 GPUs"),
    "C4": Config("C4", "seqcmp", 32768, gpus=(1, 2, 4, 8),
                 note="sequence comparison dim=32768, 1/2/4/8 GPUs"),
    "C5a": Config("C5a", "synthetic", 16384, tsize=10, dsize=1, gpus=(1, 2, 4, 8)),
    "C5b": Config("C5b", "synthetic", 16384, tsize=10, dsize=5, gpus=(1, 2, 4, 8)),
    "C5c": Config("C5c", "synthetic", 16384, tsize=1000, dsize=1, gpus=(1, 2, 4, 8)),
    "C5d": Config("C5d", "synthetic", 16384, tsize=1000, dsize=5, gpus=(1, 2, 4, 8)),
}
