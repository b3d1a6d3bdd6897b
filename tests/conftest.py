import os
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)
GOLDEN = os.path.join(ROOT, "tests", "golden")


def pytest_configure(config):
    config.addinivalue_line("markers", "gpu: needs a B200 (run via gpurun)")
    config.addinivalue_line("markers", "slow: long-running")


def read_golden(name):
    """Parse a golden fixture: '# section' lines start a section; other '#' lines
    are commentary/citations.  Returns {section: [[numbers...], ...]}."""
    sections, cur = {}, None
    with open(os.path.join(GOLDEN, name)) as f:
        for line in f:
            s = line.strip()
            if not s:
                continue
            if s.startswith("#"):
                word = s[1:].strip()
                if word and " " not in word:
                    cur = word
                    sections[cur] = []
                continue
            sections.setdefault(cur, []).append([float(t) for t in s.split()])
    return sections


@pytest.fixture
def golden():
    return read_golden
