"""Plain sequential CPU oracle for the wavefront sweep -- TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s ``cpu_baseline`` leg /
``--impl reference`` arm may import this package.  The product path
(``paper_conf_ppopp_mohantyc14_b200``) never imports it, and it never imports the
product path: the two share no code.

The arithmetic lives in ``oracle.c`` (single thread, row-major, ``-O2
-ffp-contract=off``); this module only compiles it with gcc and marshals numpy
arrays.  Citations per function are in ``oracle.h``/``oracle.c``.

Parity status per function:
  seqcmp     pinned: textbook worked examples (tests/golden), brute-force enumeration of all
             alignments (m, n <= 6), closed forms (identical / disjoint sequences).
  synthetic  pinned: closed forms i0=(i-1)+(j-1), i1=i*j; constant-field fixed point;
             per-cell closed form of the FMA iteration (x_T = uv + A^T (x_0 - uv)).
  nash       solver pinned on textbook 2x2 games and a brute-force deviation check;
             expected-count closed form for random games.  The hash-derived payoffs are
             this build's definition (reading R8): "parity unpinned" beyond those pins.
"""
from __future__ import annotations

import ctypes
import os
import subprocess
import threading

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "oracle.c")
_HDR = os.path.join(_HERE, "oracle.h")
_LIB = os.path.join(_HERE, "liboracle.so")
_CFLAGS = ["-O2", "-std=c11", "-ffp-contract=off", "-fno-fast-math", "-fPIC", "-shared"]
_lock = threading.Lock()
_lib = None


def build(force: bool = False) -> str:
    """Compile liboracle.so with gcc (plain C, no FMA contraction)."""
    stale = (not os.path.exists(_LIB)) or any(
        os.path.getmtime(p) > os.path.getmtime(_LIB) for p in (_SRC, _HDR))
    if force or stale:
        tmp = _LIB + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", *_CFLAGS, "-o", tmp, _SRC, "-lm"])
        os.replace(tmp, _LIB)
    return _LIB


def lib() -> ctypes.CDLL:
    global _lib
    with _lock:
        if _lib is None:
            build()
            L = ctypes.CDLL(_LIB)
            P = ctypes.c_void_p
            i32 = ctypes.c_int32
            L.oracle_seqcmp.argtypes = [ctypes.c_int] * 3 + [P, P, i32, i32, i32, ctypes.c_int, P]
            L.oracle_synthetic.argtypes = [ctypes.c_int] * 5 + [P] * 7
            L.oracle_nash.argtypes = [ctypes.c_int] * 4 + [P] * 5
            L.oracle_lowbias32.argtypes = [ctypes.c_uint32]
            L.oracle_lowbias32.restype = ctypes.c_uint32
            L.oracle_nash_solve.argtypes = [ctypes.c_int, P, P, P]
            L.oracle_nash_cell.argtypes = [ctypes.c_int, P, P, P, ctypes.c_uint32, ctypes.c_uint32, P]
            for f in (L.oracle_seqcmp, L.oracle_synthetic, L.oracle_nash, L.oracle_nash_solve,
                      L.oracle_nash_cell):
                f.restype = ctypes.c_int
            _lib = L
    return _lib


def _ptr(a: np.ndarray | None):
    if a is None:
        return None
    assert a.flags.c_contiguous
    return a.ctypes.data


def _check(rc: int, what: str) -> None:
    if rc != 0:
        raise ValueError(f"oracle_{what}: invalid arguments")


def seqcmp(x: np.ndarray, y: np.ndarray, match: int = 1, mismatch: int = -1, gap: int = -1,
           local: bool = False, m_compute: int | None = None, out: np.ndarray | None = None) -> np.ndarray:
    """H[1..m][1..n] of Needleman-Wunsch (local=False) or Smith-Waterman (local=True)."""
    x = np.ascontiguousarray(x, dtype=np.uint8)
    y = np.ascontiguousarray(y, dtype=np.uint8)
    m, n = len(x), len(y)
    H = out if out is not None else np.zeros((m, n), dtype=np.int32)
    assert H.shape == (m, n) and H.dtype == np.int32
    rc = lib().oracle_seqcmp(m, n, m_compute or 0, _ptr(x), _ptr(y), match, mismatch, gap,
                             1 if local else 0, _ptr(H))
    _check(rc, "seqcmp")
    return H


def synthetic(u: np.ndarray, v: np.ndarray, top: np.ndarray, left: np.ndarray, tsize: int,
              m_compute: int | None = None):
    """(i0, i1, f) planes of the synthetic application; f has shape (dsize, m, n)."""
    u = np.ascontiguousarray(u, dtype=np.float32)
    v = np.ascontiguousarray(v, dtype=np.float32)
    top = np.ascontiguousarray(top, dtype=np.float32)
    left = np.ascontiguousarray(left, dtype=np.float32)
    m, n = len(u), len(v)
    dsize = top.shape[0]
    assert top.shape == (dsize, n + 1) and left.shape == (dsize, m + 1)
    i0 = np.zeros((m, n), dtype=np.int32)
    i1 = np.zeros((m, n), dtype=np.int32)
    f = np.zeros((dsize, m, n), dtype=np.float32)
    rc = lib().oracle_synthetic(m, n, m_compute or 0, tsize, dsize, _ptr(u), _ptr(v), _ptr(top),
                                _ptr(left), _ptr(i0), _ptr(i1), _ptr(f))
    _check(rc, "synthetic")
    return i0, i1, f


def nash(r: np.ndarray, c: np.ndarray, top: np.ndarray, left: np.ndarray, nstrat: int = 16,
         m_compute: int | None = None) -> np.ndarray:
    """Planes p0..p3 (shape (4, m, n)) of the Nash stand-in."""
    r = np.ascontiguousarray(r, dtype=np.uint32)
    c = np.ascontiguousarray(c, dtype=np.uint32)
    top = np.ascontiguousarray(top, dtype=np.int32)
    left = np.ascontiguousarray(left, dtype=np.int32)
    m, n = len(r), len(c)
    assert top.shape == (4, n + 1) and left.shape == (4, m + 1)
    out = np.zeros((4, m, n), dtype=np.int32)
    rc = lib().oracle_nash(m, n, m_compute or 0, nstrat, _ptr(r), _ptr(c), _ptr(top), _ptr(left),
                           _ptr(out))
    _check(rc, "nash")
    return out


def lowbias32(x: int) -> int:
    return int(lib().oracle_lowbias32(int(x) & 0xFFFFFFFF))


def nash_solve(A: np.ndarray, B: np.ndarray) -> tuple[int, int, int, int]:
    A = np.ascontiguousarray(A, dtype=np.int32)
    B = np.ascontiguousarray(B, dtype=np.int32)
    n = A.shape[0]
    assert A.shape == (n, n) and B.shape == (n, n)
    out = np.zeros(4, dtype=np.int32)
    _check(lib().oracle_nash_solve(n, _ptr(A), _ptr(B), _ptr(out)), "nash_solve")
    return tuple(int(v) for v in out)


def nash_cell(nstrat: int, N, NW, W, r: int, c: int) -> tuple[int, int, int, int]:
    a = [np.ascontiguousarray(np.asarray(v, dtype=np.int64).astype(np.int32)) for v in (N, NW, W)]
    out = np.zeros(4, dtype=np.int32)
    _check(lib().oracle_nash_cell(nstrat, _ptr(a[0]), _ptr(a[1]), _ptr(a[2]), r & 0xFFFFFFFF,
                                  c & 0xFFFFFFFF, _ptr(out)), "nash_cell")
    return tuple(int(v) for v in out)
