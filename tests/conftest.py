import os
import subprocess
import sys

import numpy as np
import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)


def pytest_configure(config):
    config.addinivalue_line("markers", "gpu: needs a CUDA GPU (B200)")
    config.addinivalue_line("markers", "slow: long-running (full-size parity)")


def pytest_sessionstart(session):
    # Build every in-tree native artefact once (no-op when up to date).
    subprocess.run(["make", "-s", "-C", ROOT, "all"], check=True)


def load_golden(path):
    """Parse a tests/golden fixture: `table <name> <cols...>` blocks of int rows and
    `expect <query>` blocks of result rows (group codes..., sum, count)."""
    tables, expect = {}, {}
    cur = None
    with open(path) as f:
        for line in f:
            line = line.split("#", 1)[0].strip()
            if not line:
                continue
            tok = line.split()
            if tok[0] == "table":
                cur = ("table", tok[1], tok[2:])
                tables[tok[1]] = {c: [] for c in tok[2:]}
            elif tok[0] == "expect":
                cur = ("expect", tok[1])
                expect[tok[1]] = []
            elif cur[0] == "table":
                vals = [int(v) for v in tok]
                assert len(vals) == len(cur[2]), line
                for c, v in zip(cur[2], vals):
                    tables[cur[1]][c].append(v)
            else:
                expect[cur[1]].append(tuple(int(v) for v in tok))
    db = {t: {c: np.asarray(v, dtype=np.int32) for c, v in cols.items()}
          for t, cols in tables.items()}
    return db, expect


@pytest.fixture(scope="session")
def handcrafted():
    return load_golden(os.path.join(ROOT, "tests", "golden", "handcrafted_ssb.txt"))
