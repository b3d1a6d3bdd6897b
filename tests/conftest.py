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
    # the library's on-disk cubin cache (SKL_CACHE_DIR), in a directory fresh for
    # this session: the many short-lived contexts of the tests compile each
    # (skeleton, types, options) program once instead of once per context; a
    # test that sets its own directory (test_abi's cache test) still can
    if "SKL_CACHE_DIR" not in os.environ:
        import tempfile
        os.environ["SKL_CACHE_DIR"] = tempfile.mkdtemp(prefix="skl_test_cache_")


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
