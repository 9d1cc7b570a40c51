"""C-ABI state rules that need a device (include/wf.h): slab linking is validated (same problem
and tuning, adjacent columns, before the first run), a device error of a completed run is
reported by the next wf_run, and a context connects only before its first run.
(wf_link_local, epoch pairing, wf_run error word)."""
from __future__ import annotations

import numpy as np
import pytest

torch = pytest.importorskip("torch")
if not torch.cuda.is_available():
    pytest.skip("needs a CUDA device", allow_module_level=True)

import workloads  # noqa: E402
from paper_conf_ppopp_mohantyc14_b200 import _abi  # noqa: E402
from paper_conf_ppopp_mohantyc14_b200.wf import Wavefront  # noqa: E402

from _gpu_helpers import dev_inputs  # noqa: E402

pytestmark = pytest.mark.gpu


def _slab(rank, G=2, dim=300, **kw):
    return Wavefront("seqcmp", dim, rank=rank, device=torch.cuda.current_device(), ngpus=G, device_share=G, **kw)


def test_link_rejects_a_different_tuning():
    a, b = _slab(0, lane_cols=2, warps=4), _slab(1, lane_cols=4, warps=2)
    try:
        with pytest.raises(_abi.WfError) as ei:
            a.link(b)
        assert ei.value.status == _abi.WF_EINVAL
    finally:
        a.close()
        b.close()


def test_link_rejects_a_different_strip():
    a, b = _slab(0, strip=8), _slab(1, strip=32)
    try:
        with pytest.raises(_abi.WfError) as ei:
            a.link(b)
        assert ei.value.status == _abi.WF_EINVAL
    finally:
        a.close()
        b.close()


def test_link_rejects_non_adjacent_slabs():
    a, c = _slab(0, G=3, dim=1000), _slab(2, G=3, dim=1000)
    try:
        with pytest.raises(_abi.WfError) as ei:
            a.link(c)
        assert ei.value.status == _abi.WF_EINVAL
    finally:
        a.close()
        c.close()


def test_link_after_a_run_is_a_state_error():
    dim = 300
    x, y = workloads.seqcmp_inputs(dim)
    dev = torch.device("cuda", torch.cuda.current_device())
    a, b = _slab(0, dim=dim), _slab(1, dim=dim, watchdog_cycles=20_000_000)
    row_in, col_in, _, _ = dev_inputs("seqcmp", (x, y), dev)
    b.run(row_in, col_in)   # slab 1 alone: its west ring is never written -> a quick watchdog
    try:
        with pytest.raises(_abi.WfError) as ei:
            a.link(b)
        assert ei.value.status == _abi.WF_ESTATE
    finally:
        try:
            b.sync()
        except _abi.WfError:
            pass
        a.close()
        b.close()


def test_next_run_reports_the_previous_runs_timeout_once():
    dim = 256
    x, y = workloads.seqcmp_inputs(dim)
    dev = torch.device("cuda", torch.cuda.current_device())
    w = Wavefront("seqcmp", dim, rank=1, device=torch.cuda.current_device(), ngpus=2, watchdog_cycles=20_000_000)
    try:
        row_in, col_in, _, _ = dev_inputs("seqcmp", (x, y), dev)
        w.run(row_in, col_in)
        torch.cuda.synchronize()
        with pytest.raises(_abi.WfError) as ei:   # the completed run's watchdog error, without wf_sync
            w.run(row_in, col_in)
        assert ei.value.status == _abi.WF_ETIMEOUT
        w.run(row_in, col_in)                     # reported once; the next run is enqueued
        with pytest.raises(_abi.WfError) as ei:
            w.sync()
        assert ei.value.status == _abi.WF_ETIMEOUT
    finally:
        w.close()


def test_connect_after_a_run_is_a_state_error():
    dim = 128
    x, y = workloads.seqcmp_inputs(dim)
    dev = torch.device("cuda", torch.cuda.current_device())
    w = Wavefront("seqcmp", dim)
    try:
        row_in, col_in, _, _ = dev_inputs("seqcmp", (x, y), dev)
        w.run(row_in, col_in)
        w.sync()
        with pytest.raises(_abi.WfError) as ei:
            w.connect(None, None)
        assert ei.value.status == _abi.WF_ESTATE
    finally:
        w.close()
