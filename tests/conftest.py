import os
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)


def pytest_configure(config):
    config.addinivalue_line("markers", "gpu: needs a B200 (run via gpurun)")
    config.addinivalue_line("markers", "slow: full-size configs (minutes)")


def pytest_collection_modifyitems(config, items):
    # keep the CPU tier fast unless explicitly asked for full-size oracle runs
    if os.environ.get("MCM_FULL", "0") == "1":
        return
    skip = pytest.mark.skip(reason="full-size oracle run; set MCM_FULL=1")
    for it in items:
        if "slow" in it.keywords and "gpu" not in it.keywords:
            it.add_marker(skip)
