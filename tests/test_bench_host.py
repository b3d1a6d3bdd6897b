"""Host logic of bench.py (no GPU): the statistics, the exit-status rule, the
roofline helpers, the Mandelbrot row dealing, and the reference arm's JSON line
(the CPU oracle on a bounded sample)."""
import json
import os
import subprocess
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import bench  # noqa: E402


def test_stats_median_min_mean():
    st = bench.stats([3.0, 1.0, 2.0, 10.0])
    assert st == {"median": 2.5, "mean": 4.0, "min": 1.0, "n": 4}


def test_all_checks_ok():
    assert bench.all_checks_ok({"a": {"check": "ok"}, "b": {"ms": 1.0}})
    assert not bench.all_checks_ok({"a": {"check": "ok"}, "b": {"check": "FAIL"}})
    assert not bench.all_checks_ok({"error": "skeleton section exceeded 600 s"})


def test_row_order_is_a_permutation_dealt_round_robin():
    for G in (1, 2, 3, 8):
        o = bench.row_order(3072, G)
        assert sorted(o.tolist()) == list(range(3072))
        if G > 1:
            # the block of device g holds rows g, g + G, g + 2G, ..., the ones
            # nearest the image's middle first
            lo, hi = bench.S_block(3072, G, 1)
            assert sorted(o[lo:hi].tolist()) == np.arange(1, 3072, G)[: hi - lo].tolist()
            d = np.abs(o[lo:hi] - 3071 / 2.0)
            assert np.all(np.diff(d) >= 0)


def test_roofline_helpers():
    P = {"hbm_gbs": 6000.0, "sm_max_mhz": 2000.0, "source": "test"}
    r = bench.roof_hbm(6e9, 1.0, P, ngpu=2)     # 6 GB in 1 ms = 6000 GB/s on 2 GPUs
    assert r["achieved"] == 6000.0 and r["peak"] == 12000.0 and r["frac"] == 0.5
    a = bench.roof_alu(148 * 128 * 2e9 * 1e-3, 1.0, P, 148)   # exactly the peak for 1 ms
    assert abs(a["frac"] - 1.0) < 1e-12
    n = bench.roof_nvlink(8 * 450e6, 1.0, 8)                   # 450 MB into each of 8 GPUs in 1 ms
    assert n["achieved"] == 450.0 and n["frac"] == 0.5 and n["bound"] == "nvlink"


def test_reference_arm_line():
    out = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--impl", "reference", "--steps", "1",
                          "--warmup", "3"], capture_output=True, text=True, timeout=600, cwd=ROOT)
    assert out.returncode == 0, out.stderr[-2000:]
    line = json.loads(out.stdout.strip().splitlines()[-1])
    assert line["impl"] == "reference" and line["unit"] == "elements/s" and line["value"] > 0
    assert line["cpu_baseline"]["kind"] == "oracle" and line["cpu_baseline"]["cores"] == 1
    assert line["e2e"]["h2d_bytes_per_step"] == 0
