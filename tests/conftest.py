import os
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)


def pytest_configure(config):
    config.addinivalue_line("markers", "gpu: needs a B200 (runs through the CUDA C-ABI library)")
    config.addinivalue_line("markers", "slow: long CPU test")
    # libjp.so is a build artefact (git-ignored): build it once if this checkout
    # has none yet (nvcc cross-compiles sm_100a without a GPU); never rebuilt here
    so = os.path.join(ROOT, "paper_conf_icpp_hanzlw13_b200", "libjp.so")
    if not os.path.exists(so) and not os.environ.get("JP_LIB"):
        import subprocess
        subprocess.check_call(["make", "-s", "-j", str(os.cpu_count() or 4), "-C",
                               os.path.join(ROOT, "paper_conf_icpp_hanzlw13_b200", "csrc")])


@pytest.fixture(scope="session")
def golden_dir():
    return os.path.join(ROOT, "tests", "golden")
