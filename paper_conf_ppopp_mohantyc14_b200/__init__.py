"""B200-native (sm_100a) wavefront sweep -- the hot path of Mohanty & Cole, PMAM'14
(dblp conf/ppopp/MohantyC14): a[i][j] = f(a[i-1][j], a[i][j-1], a[i-1][j-1]).

The compute path is libwf.so (hand-written CUDA for sm_100a behind the C ABI in
include/wf.h).  This package only marshals arguments; importing the binding when the
library is missing raises -- there is no CPU fallback.
"""
from ._abi import WfError, lib  # noqa: F401

__all__ = ["WfError", "lib", "Wavefront", "LocalSlabs", "query", "make_params"]


def __getattr__(name):
    if name in ("Wavefront", "LocalSlabs", "query", "make_params", "to_device"):
        from . import wf
        return getattr(wf, name)
    raise AttributeError(name)
