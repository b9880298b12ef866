import os
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)


def pytest_configure(config):
    config.addinivalue_line("markers", "gpu: needs a CUDA device (B200); run via gpurun")
    config.addinivalue_line("markers", "slow: long-running CPU test")


@pytest.fixture(scope="session")
def orc():
    import oracle
    oracle.build_oracle()
    return oracle


@pytest.hookimpl(hookwrapper=True)
def pytest_pyfunc_call(pyfuncitem):
    """Engine 4 (sparse ligand) legitimately refuses shapes whose atom-grid plane ring does not fit in shared
    memory (DOCK_E_UNSUPPORTED): such parametrisations are skipped, not failed."""
    outcome = yield
    exc = outcome.excinfo
    params = getattr(getattr(pyfuncitem, "callspec", None), "params", {})
    if exc and params.get("engine") == 4 and type(exc[1]).__name__ == "DockError" and \
            getattr(exc[1], "status", 0) == -2 and "ineligible" in str(exc[1]):
        outcome.force_exception(pytest.skip.Exception(f"sparse engine ineligible: {exc[1]}", _use_item_location=True))
