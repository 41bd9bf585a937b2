import os
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)
# hardware queues for concurrent tenant streams; must precede CUDA init
os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")


def pytest_configure(config):
    config.addinivalue_line("markers", "gpu: needs a CUDA device (B200, sm_100a)")
    config.addinivalue_line("markers", "slow: longer CPU test")


@pytest.fixture(scope="session")
def oracle_lib():
    from oracle import tenants
    tenants.build()
    return tenants


@pytest.fixture(scope="session")
def occ():
    """cuda_occupancy.h evaluated on CPU for an sm_100 device (library pin)."""
    import ctypes
    import subprocess
    src = os.path.join(ROOT, "tests", "shims", "occ_shim.cpp")
    out = os.path.join(ROOT, "tests", "shims", "libocc_shim.so")
    if not os.path.exists(out) or os.path.getmtime(out) < os.path.getmtime(src):
        subprocess.check_call(["g++", "-O1", "-fPIC", "-shared", "-I/usr/local/cuda/include",
                               src, "-o", out])
    lib = ctypes.CDLL(out)
    return lib.occ_blocks_per_sm
