"""bench.py end to end in its multi-device modes on ONE GPU (the driver runs
N > 1 under torchrun, one process per GPU; nothing else exercises the bench's
own code in that mode before it): two ranks sharing the GPU over the IPC
transport, and one process with two logical devices; a short run of the dot
product and redistribution lines must exit 0 with every parity check ok."""
import json
import os
import subprocess
import sys

import pytest

from gpu_util import require_gpu

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
pytestmark = pytest.mark.gpu


def _run(cmd, env):
    out = subprocess.run(cmd, capture_output=True, text=True, timeout=900, cwd=ROOT, env={**os.environ, **env})
    assert out.returncode == 0, out.stderr[-3000:]
    line = json.loads(out.stdout.strip().splitlines()[-1])
    assert line["n_gpus"] == 2
    for k, v in line["skeletons"].items():
        if isinstance(v, dict) and "check" in v:
            assert v["check"] == "ok", k
    return line


def test_bench_two_ranks_on_one_gpu():
    require_gpu()
    _run([sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node", "2",
          "--master-addr", "127.0.0.1", "--master-port", "29541", "bench.py", "--gpus", "2",
          "--skeletons", "dot,redist", "--steps", "3", "--warmup", "3"],
         {"SKL_BENCH_SHARE_GPU": "1"})


def test_bench_two_logical_devices():
    require_gpu()
    _run([sys.executable, "bench.py", "--gpus", "2", "--skeletons", "dot,redist", "--steps", "3", "--warmup", "3"],
         {"SKL_BENCH_LOGICAL": "1"})
