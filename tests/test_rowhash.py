"""The per-row hash used for the C5 full-grid parity (tests/_rowhash.py) and its golden files.

CPU-only: the hash must notice any single changed word (in any plane, any column), must not
depend on the chunking, and the committed golden files must have one hash per C5 row."""
import os

import numpy as np

import workloads
from _rowhash import constants, row_hashes

GOLDEN = os.path.join(os.path.dirname(__file__), "golden")


def test_hash_detects_any_single_word_change():
    rng = np.random.default_rng(0)
    planes = [rng.integers(-2**31, 2**31, size=(37, 53), dtype=np.int64).astype(np.int32) for _ in range(3)]
    planes.append(rng.random((37, 53), dtype=np.float32))
    h0 = row_hashes(planes)
    for p, (i, j) in [(0, (0, 0)), (1, (36, 52)), (2, (17, 3)), (3, (5, 40))]:
        mod = [q.copy() for q in planes]
        mod[p].view(np.uint32)[i, j] ^= np.uint32(1 << (i % 32))
        h1 = row_hashes(mod)
        assert h1[i] != h0[i] and np.array_equal(np.delete(h1, i), np.delete(h0, i))


def test_hash_independent_of_chunking_and_swaps():
    rng = np.random.default_rng(1)
    planes = [rng.integers(0, 1000, size=(70, 20), dtype=np.int32) for _ in range(2)]
    assert np.array_equal(row_hashes(planes, chunk=7), row_hashes(planes, chunk=512))
    # swapping two words of a row, or the two planes, changes the hash (position-weighted)
    sw = [q.copy() for q in planes]
    sw[0][3, [1, 2]] = sw[0][3, [2, 1]]
    if planes[0][3, 1] != planes[0][3, 2]:
        assert row_hashes(sw)[3] != row_hashes(planes)[3]
    assert not np.array_equal(row_hashes(planes[::-1]), row_hashes(planes))
    assert np.all(constants(2, 20) & np.uint64(1) == 1)


def test_c5_golden_files_cover_every_row():
    for name in ("C5a", "C5b", "C5c", "C5d"):
        h = np.load(os.path.join(GOLDEN, f"c5_rowhash_{name}.npy"))
        assert h.dtype == np.uint64 and h.shape == (workloads.CONFIGS[name].dim,)
        assert len(np.unique(h)) == h.size   # rows of a wavefront grid are all distinct
