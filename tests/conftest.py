"""pytest configuration: the ``gpu`` marker and shared builds.

``-m "not gpu"`` runs here (no GPU): oracle pins, generator, host logic, C-ABI symbol
checks, gloo multi-process tests. ``-m gpu`` runs on a B200 (parity through the C-ABI).
"""
import os
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)
GOLDEN = os.path.join(ROOT, "tests", "golden")


def pytest_configure(config):
    config.addinivalue_line("markers", "gpu: needs a CUDA device (B200, sm_100a)")
    config.addinivalue_line("markers", "slow: long-running CPU test")


@pytest.fixture(scope="session", autouse=True)
def _built():
    import lmgen
    import oracle
    lmgen.build()
    oracle.build()
    yield


def read_golden_paths(name="paths_4cube.txt"):
    """Parse a golden path fixture: [(name, p1, p2, [(coord, len), ...]), ...]."""
    out = []
    with open(os.path.join(GOLDEN, name)) as fh:
        for line in fh:
            line = line.strip()
            if not line or line.startswith("#"):
                continue
            nm, pts, pairs = (x.strip() for x in line.split("|"))
            v = [float(t) for t in pts.split()]
            pr = [(int(a), float(b)) for a, b in (t.split(":") for t in pairs.split())] if pairs else []
            out.append((nm, v[:3], v[3:], pr))
    return out
