import os
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)

# culi_eval_text reads small host texts with the host reader unless told otherwise (CULI_F_DEVICE_READ);
# the tests' *_text calls are there to exercise the device reader (§8(f)2), so they force it everywhere
# (tests/test_gpu_reader.py::test_small_host_text_uses_host_reader covers the size-based default).
os.environ.setdefault("CULI_DEVICE_READ", "1")


def pytest_configure(config):
    config.addinivalue_line("markers", "gpu: needs a CUDA device (B200, sm_100a)")
    config.addinivalue_line("markers", "slow: long-running test")


@pytest.fixture(scope="session")
def oracle_mod():
    import oracle
    oracle.build()
    return oracle
