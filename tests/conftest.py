import json
import os
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)

GOLDEN = os.path.join(ROOT, "tests", "golden")


def pytest_configure(config):
    config.addinivalue_line("markers", "gpu: needs a CUDA B200 (sm_100a) device")
    config.addinivalue_line("markers", "slow: long-running CPU test")


def golden(name):
    with open(os.path.join(GOLDEN, name)) as f:
        return json.load(f)


@pytest.fixture(scope="session", autouse=True)
def ensure_built():
    """Build libaol.so / liboracle.so / the C example if a checkout arrives without them (they are
    git-ignored build products)."""
    pkg = os.path.join(ROOT, "paper_conf_ipps_guortgbs11_b200", "libaol.so")
    if not (os.path.exists(pkg) and os.path.exists(os.path.join(ROOT, "oracle", "liboracle.so"))):
        import __graft_entry__

        __graft_entry__.build()
    yield


@pytest.fixture(scope="session")
def orc():
    import oracle

    oracle.lib()
    return oracle
