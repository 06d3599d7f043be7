import os
import sys

import pytest

# Virtual-rank tests of the device-driven exchange (test_dist.py) run G ranks on G CUDA streams
# of one process whose kernels wait on each other: every stream needs its own hardware queue
# (the default of 8 connections would let a waiting kernel block a peer's stream behind it).
os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)


def pytest_configure(config):
    config.addinivalue_line("markers", "gpu: needs a CUDA device (B200); run with -m gpu")
    config.addinivalue_line("markers", "slow: long-running (full-size configs)")


@pytest.fixture(scope="session")
def golden_dir():
    return os.path.join(os.path.dirname(os.path.abspath(__file__)), "golden")
