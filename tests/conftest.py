import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
# virtual-slab tests run up to 4 slab streams per device; keep every stream on its own hardware
# queue (paper_conf_ppopp_mohantyc14_b200.wf.LocalSlabs)
os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)

# The race / liveness runs (tools/xbuild_jitter.sh) run the GPU tests against the
# jitter build of the library; the product path always loads its in-tree libwf.so.
if os.environ.get("WF_TEST_LIB"):
    from paper_conf_ppopp_mohantyc14_b200 import _abi
    _abi.LIB_PATH = os.path.abspath(os.environ["WF_TEST_LIB"])


def pytest_configure(config):
    config.addinivalue_line("markers", "gpu: needs a CUDA device (B200, sm_100a)")
    config.addinivalue_line("markers", "slow: long-running (large configs)")
