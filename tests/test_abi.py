"""C-ABI boundary tests that need no GPU: the library loads, exports every symbol that
include/wf.h declares, and validates parameters (WF_EINVAL with a message naming the field).
"""
from __future__ import annotations

import ctypes
import os
import re

import pytest

from paper_conf_ppopp_mohantyc14_b200 import _abi
from paper_conf_ppopp_mohantyc14_b200.wf import make_params, query

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _declared_symbols():
    src = open(os.path.join(ROOT, "include", "wf.h")).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(wf_[a-z_]+)\s*\(", src)))


def test_library_exports_every_declared_symbol():
    lib = _abi.lib()
    declared = _declared_symbols()
    assert set(declared) == set(_abi.EXPORTS)
    for name in declared:
        assert hasattr(lib, name), name
    assert lib.wf_abi_version() == 1
    assert b"sm_100a" in lib.wf_build_info()


def test_struct_sizes_match_header_layout():
    # offsets follow the C declaration order with natural alignment
    assert ctypes.sizeof(_abi.WfParams) == 16 * 4 + 8 + 6 * 4
    assert ctypes.sizeof(_abi.WfDist) == 16
    assert _abi.WfParams.watchdog_cycles.offset == 64


def _err(fn, dim, **kw):
    with pytest.raises(_abi.WfError) as ei:
        query(fn, dim, **kw)
    return ei.value


@pytest.mark.parametrize("kw,field", [
    (dict(fn="seqcmp", dim=0), "dim"),
    (dict(fn="seqcmp", dim=70000), "dim"),
    (dict(fn="seqcmp", dim=100, cols=-3), "cols"),
    (dict(fn="seqcmp", dim=100, tsize=5), "tsize"),
    (dict(fn="seqcmp", dim=100, dsize=1), "dsize"),
    (dict(fn="seqcmp", dim=100, match=100, mismatch=-1, gap=-1), "match"),
    (dict(fn="seqcmp", dim=100, gap=-65, match=1, mismatch=-1), "gap"),
    (dict(fn="synthetic", dim=100, dsize=9), "dsize"),
    (dict(fn="synthetic", dim=100, dsize=1, tsize=-1), "tsize"),
    (dict(fn="seqcmp", dim=100, lane_cols=3), "lane_cols"),
    (dict(fn="seqcmp", dim=100, warps=9), "warps"),
    (dict(fn="seqcmp", dim=100, skew=5), "skew"),
    (dict(fn="seqcmp", dim=100, ngpus=9), "ngpus"),
    (dict(fn=7, dim=100), "fn"),
])
def test_query_rejects_bad_params_naming_the_field(kw, field):
    fn = kw.pop("fn")
    dim = kw.pop("dim")
    e = _err(fn, dim, **kw)
    assert e.status == _abi.WF_EINVAL
    assert field in str(e)


def test_nccl_transport_is_accepted_and_edge_calls_validate():
    """transport = NCCL is the host-staged fallback (include/wf.h wf_edge_*):
    the planner accepts it, and the edge calls reject NULL arguments without a GPU."""
    lay = query("seqcmp", 1024, ngpus=2, transport="nccl")
    assert lay.col_begin == 0 and lay.col_end > 0
    L = _abi.lib()
    n = ctypes.c_size_t()
    assert L.wf_edge_bytes(None, ctypes.byref(n)) == _abi.WF_EINVAL
    assert L.wf_edge_export(None, None, None) == _abi.WF_EINVAL
    assert L.wf_edge_import(None, None, None) == _abi.WF_EINVAL
    e = _err("seqcmp", 1024, ngpus=2, transport=7)
    assert e.status == _abi.WF_EINVAL and "transport" in str(e)


def test_strip_axis():
    """wf_params.strip = rows per hand-off block: generation 8 compiles 8 / 16 / 32 for its main
    tilings (default 16, reported by wf_query); other strips, and any strip on a generation with a
    fixed block, are refused by name."""
    assert query("seqcmp", 1000).strip == 16
    for s in (8, 16, 32):
        assert query("seqcmp", 1000, lane_cols=2, warps=4, strip=s).strip == s
        assert query("seqcmp", 1000, lane_cols=4, warps=2, strip=s, ngpus=2).strip == s
    assert query("seqcmp", 1000, lane_cols=1, warps=4).strip == 16
    for kw in (dict(strip=24), dict(strip=8, lane_cols=1, warps=4), dict(strip=16, kernel=4),
               dict(strip=16, skew=2, lane_cols=4, warps=1)):
        e = _err("seqcmp", 1000, **kw)
        assert e.status == _abi.WF_EUNSUPPORTED and "strip" in str(e)
    assert query("synthetic", 100, tsize=10, dsize=1).strip == 0
    assert _err("synthetic", 100, tsize=10, dsize=1, strip=16).status == _abi.WF_EUNSUPPORTED
    assert _err("seqcmp", 1000, strip=-1).status == _abi.WF_EINVAL


def test_reserved_fields_must_be_zero():
    p = make_params("seqcmp", 64)
    p.reserved[1] = 1
    lay = _abi.WfLayout()
    st = _abi.lib().wf_query(ctypes.byref(p), 0, ctypes.byref(lay))
    assert st == _abi.WF_EINVAL and b"reserved" in _abi.lib().wf_last_error(None)


def test_local_alignment_layout_and_bad_flag():
    # Smith-Waterman (local = 1) is built: same single int32 plane as global alignment
    lay = query("seqcmp", 64, local=1)
    assert lay.nplanes == 1 and lay.plane_is_float == [False]
    assert _err("seqcmp", 64, local=2).status == _abi.WF_EINVAL


def test_layout_single_slab():
    lay = query("seqcmp", 1000, lane_cols=4, warps=2, skew=1)
    assert (lay.nplanes, lay.col_begin, lay.col_end) == (1, 0, 1000)
    assert lay.band_cols == 256 and lay.nbands == 4
    assert lay.min_pitch == 1000 and lay.bytes_out == 1000 * 1000 * 4
    lay = query("synthetic", 33, tsize=3, dsize=5)
    assert lay.nplanes == 7 and lay.nbound == 5
    assert lay.plane_is_float == [False, False, True, True, True, True, True]
    assert lay.min_pitch == 36


@pytest.mark.parametrize("dim,G", [(32768, 8), (1000, 3), (4096, 2), (777, 2)])
def test_layout_slabs_partition_columns(dim, G):
    lays = [query("seqcmp", dim, ngpus=G, rank=g) for g in range(G)]
    assert lays[0].col_begin == 0 and lays[-1].col_end == dim
    for a, b in zip(lays, lays[1:]):
        assert a.col_end == b.col_begin
        # every slab but the last is a whole number of bands
        assert a.width % a.band_cols == 0
    assert sum(l.width for l in lays) == dim


def test_nash_layout_one_column_per_warp():
    lay = query("nash", 4096, tsize=16, dsize=4)
    assert lay.nplanes == 4 and lay.nbound == 4 and lay.plane_is_float == [False] * 4
    # default band width follows the autotune winner for C3 (profiles/autotune_C3.json)
    assert (lay.lane_cols, lay.warps, lay.skew) == (1, 2, 1)
    assert lay.band_cols == 2 and lay.nbands == 2048
    lays = [query("nash", 4096, tsize=16, dsize=4, ngpus=2, rank=g) for g in range(2)]
    assert lays[0].col_end == lays[1].col_begin == 2048


@pytest.mark.parametrize("kw,field", [(dict(tsize=0, dsize=4), "tsize"), (dict(tsize=65, dsize=4), "tsize"),
                                      (dict(tsize=16, dsize=3), "dsize")])
def test_nash_rejects_bad_params(kw, field):
    e = _err("nash", 100, **kw)
    assert e.status == _abi.WF_EINVAL and field in str(e)


def test_nash_rejects_multi_column_lanes():
    e = _err("nash", 100, tsize=16, dsize=4, lane_cols=2)
    assert e.status == _abi.WF_EUNSUPPORTED


def test_slab_count_too_large_is_rejected():
    e = _err("seqcmp", 300, ngpus=4, rank=0, lane_cols=4, warps=2)
    assert e.status == _abi.WF_EINVAL and "empty" in str(e)


def test_null_context_calls_are_rejected():
    L = _abi.lib()
    assert L.wf_destroy(None) == _abi.WF_OK
    assert L.wf_sync(None) == _abi.WF_EINVAL
    assert L.wf_run(None, None, None) == _abi.WF_EINVAL
    assert L.wf_last_error(None)  # never NULL


def test_create_without_dist_rejects_multi_slab():
    p = make_params("seqcmp", 128, ngpus=2)
    ctx = ctypes.c_void_p()
    st = _abi.lib().wf_create(ctypes.byref(p), None, ctypes.byref(ctx))
    assert st == _abi.WF_EINVAL and not ctx.value


def test_halo_overlap_validation():
    """NEXT-4 halo (include/wf.h wf_params.halo): whole bands of the generation-8 NW sweep,
    multi-slab only; slab g > 0 computes halo more columns but outputs the same ones."""
    base = query("seqcmp", 4096, rank=1, ngpus=2)
    lay = query("seqcmp", 4096, rank=1, ngpus=2, halo=base.band_cols)
    assert (lay.col_begin, lay.col_end) == (base.col_begin, base.col_end)
    assert lay.nbands == base.nbands + 1
    assert query("seqcmp", 4096, rank=0, ngpus=2, halo=base.band_cols).nbands == base.nbands
    for kw, st in ((dict(halo=100), _abi.WF_EINVAL), (dict(halo=-256), _abi.WF_EINVAL),
                   (dict(halo=256, ngpus=1), _abi.WF_EINVAL), (dict(halo=256, local=1), _abi.WF_EUNSUPPORTED),
                   (dict(halo=256, kernel=4), _abi.WF_EUNSUPPORTED), (dict(halo=256 * 8), _abi.WF_EINVAL)):
        kw.setdefault("ngpus", 2)
        e = _err("seqcmp", 4096, **kw)
        assert e.status == st and "halo" in str(e), (kw, e)
    e = _err("synthetic", 4096, tsize=10, dsize=1, ngpus=2, halo=32)
    assert e.status == _abi.WF_EUNSUPPORTED
