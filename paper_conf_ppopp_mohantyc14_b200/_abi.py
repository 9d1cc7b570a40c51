"""ctypes mirror of include/wf.h (argument marshalling only; no computation here).

Loading fails loudly if libwf.so is missing: there is no CPU or eager fallback.
"""
from __future__ import annotations

import ctypes
import os

HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(HERE, "libwf.so")

WF_MAX_PLANES = 10
WF_IPC_HANDLE_BYTES = 64

WF_OK, WF_EINVAL, WF_ENOMEM, WF_ECUDA, WF_ECOMM, WF_ETIMEOUT, WF_EUNSUPPORTED, WF_ESTATE = range(8)
STATUS_NAMES = {0: "WF_OK", 1: "WF_EINVAL", 2: "WF_ENOMEM", 3: "WF_ECUDA", 4: "WF_ECOMM", 5: "WF_ETIMEOUT",
                6: "WF_EUNSUPPORTED", 7: "WF_ESTATE"}
WF_FN_SYNTHETIC, WF_FN_NASH, WF_FN_SEQCMP = 0, 1, 2
FN_IDS = {"synthetic": WF_FN_SYNTHETIC, "nash": WF_FN_NASH, "seqcmp": WF_FN_SEQCMP}
WF_TRANSPORT_P2P, WF_TRANSPORT_NCCL = 0, 1

# every symbol include/wf.h declares (checked by tests/test_abi.py)
EXPORTS = ("wf_query", "wf_create", "wf_run", "wf_sync", "wf_destroy", "wf_last_error", "wf_link_local",
           "wf_ipc_handle", "wf_connect", "wf_last_run_ms", "wf_abi_version", "wf_build_info", "wf_debug_trace",
           "wf_local_best", "wf_edge_bytes", "wf_edge_export", "wf_edge_import")


class WfParams(ctypes.Structure):
    _fields_ = [("dim", ctypes.c_int32), ("cols", ctypes.c_int32), ("fn", ctypes.c_int32),
                ("tsize", ctypes.c_int32), ("dsize", ctypes.c_int32), ("lane_cols", ctypes.c_int32),
                ("warps", ctypes.c_int32), ("skew", ctypes.c_int32), ("strip", ctypes.c_int32),
                ("ngpus", ctypes.c_int32), ("match", ctypes.c_int32), ("mismatch", ctypes.c_int32),
                ("gap", ctypes.c_int32), ("local", ctypes.c_int32), ("transport", ctypes.c_uint32),
                ("max_ctas", ctypes.c_uint32), ("watchdog_cycles", ctypes.c_uint64),
                ("alphabet", ctypes.c_int32), ("kernel", ctypes.c_int32), ("halo", ctypes.c_int32),
                ("reserved", ctypes.c_int32 * 3)]


class WfDist(ctypes.Structure):
    _fields_ = [("rank", ctypes.c_int32), ("world", ctypes.c_int32), ("device", ctypes.c_int32),
                ("device_share", ctypes.c_int32)]


class WfLayout(ctypes.Structure):
    _fields_ = [("nplanes", ctypes.c_int32), ("plane_bytes", ctypes.c_int32 * WF_MAX_PLANES),
                ("plane_is_float", ctypes.c_int32 * WF_MAX_PLANES), ("nbound", ctypes.c_int32),
                ("col_begin", ctypes.c_int32), ("col_end", ctypes.c_int32), ("min_pitch", ctypes.c_int64),
                ("bytes_out", ctypes.c_int64), ("lane_cols", ctypes.c_int32), ("warps", ctypes.c_int32),
                ("skew", ctypes.c_int32), ("band_cols", ctypes.c_int32), ("nbands", ctypes.c_int32),
                ("strip", ctypes.c_int32), ("reserved", ctypes.c_int32 * 4)]


class WfIo(ctypes.Structure):
    _fields_ = [("row_in", ctypes.c_void_p), ("col_in", ctypes.c_void_p),
                ("top", ctypes.c_void_p * WF_MAX_PLANES), ("left", ctypes.c_void_p * WF_MAX_PLANES),
                ("out", ctypes.c_void_p * WF_MAX_PLANES), ("out_pitch", ctypes.c_int64)]


class WfError(RuntimeError):
    def __init__(self, status: int, msg: str):
        super().__init__(f"{STATUS_NAMES.get(status, status)}: {msg}")
        self.status = status


_lib = None


def lib() -> ctypes.CDLL:
    """Load libwf.so (built by paper_conf_ppopp_mohantyc14_b200.build).  No fallback."""
    global _lib
    if _lib is None:
        if not os.path.exists(LIB_PATH):
            raise ImportError(f"libwf.so not built ({LIB_PATH}); run `python -m paper_conf_ppopp_mohantyc14_b200.build`"
                              " -- there is no CPU fallback")
        L = ctypes.CDLL(LIB_PATH)
        P = ctypes.c_void_p
        L.wf_query.argtypes = [ctypes.POINTER(WfParams), ctypes.c_int32, ctypes.POINTER(WfLayout)]
        L.wf_create.argtypes = [ctypes.POINTER(WfParams), ctypes.POINTER(WfDist), ctypes.POINTER(P)]
        L.wf_run.argtypes = [P, ctypes.POINTER(WfIo), P]
        L.wf_sync.argtypes = [P]
        L.wf_destroy.argtypes = [P]
        L.wf_last_error.argtypes = [P]
        L.wf_last_error.restype = ctypes.c_char_p
        L.wf_link_local.argtypes = [P, P]
        L.wf_ipc_handle.argtypes = [P, P]
        L.wf_connect.argtypes = [P, P, P]
        L.wf_last_run_ms.argtypes = [P, ctypes.POINTER(ctypes.c_float)]
        i32p = ctypes.POINTER(ctypes.c_int32)
        L.wf_local_best.argtypes = [P, i32p, i32p, i32p]
        L.wf_debug_trace.argtypes = [P, P, ctypes.c_size_t, ctypes.POINTER(ctypes.c_int32)]
        L.wf_debug_trace.restype = ctypes.c_int
        L.wf_abi_version.argtypes = []
        L.wf_abi_version.restype = ctypes.c_int32
        L.wf_build_info.argtypes = []
        L.wf_build_info.restype = ctypes.c_char_p
        L.wf_edge_bytes.argtypes = [P, ctypes.POINTER(ctypes.c_size_t)]
        L.wf_edge_export.argtypes = [P, P, P]
        L.wf_edge_import.argtypes = [P, P, P]
        for name in ("wf_query", "wf_create", "wf_run", "wf_sync", "wf_destroy", "wf_link_local",
                     "wf_ipc_handle", "wf_connect", "wf_last_run_ms", "wf_local_best", "wf_edge_bytes",
                     "wf_edge_export", "wf_edge_import"):
            getattr(L, name).restype = ctypes.c_int
        _lib = L
    return _lib


def check(status: int, ctx=None) -> None:
    if status != WF_OK:
        msg = lib().wf_last_error(ctx).decode(errors="replace")
        raise WfError(status, msg)
