"""Host-side cost of skeleton calls: wall-clock time to ENQUEUE a call (no
synchronisation; the GPU is kept busy by a long spin kernel so the host never
waits for it) on 1 and 4 logical devices of one GPU, next to the GPU time of
the same call.  Shows whether iterated stencils on several GPUs are
host-launch-bound.  HOST_G="1,4" HOST_N=200"""
import os
import sys
import time

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from paper_conf_pact_steuwerg13_b200 import apps as A  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import inputs as I  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import skl as S  # noqa: E402

N = int(os.environ.get("HOST_N", "200"))
for G in (int(g) for g in os.environ.get("HOST_G", "1,4").split(",")):
    c = S.Context(G, devices=[0] * G)
    streams = [torch.cuda.Stream() for _ in range(G)]
    for g, st in enumerate(streams):
        c.set_stream(g, st.cuda_stream)
    c.set_option("block_threads", 128)
    gau = S.MapOverlap(c, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
    c.set_option("block_threads", 256)
    a = S.Matrix.from_numpy(c, I.image_f32(I.SEED_GAUSS, 2048, 2048))
    b = S.Matrix(c, S.F32, 2048, 2048)
    neg = S.Map(c, A.NEG, S.F32, S.F32)
    v = S.Vector.from_numpy(c, np.ones(1 << 16, np.float32))
    vo = neg(v)
    addf = S.Reduce(c, A.ADD, S.F32)
    cases = {
        "MapOverlap 2048^2 (ping-pong)": lambda i: gau(a, out=b) if i % 2 == 0 else gau(b, out=a),
        "Map 2^16": lambda i: neg(v, out=vo),
        "Reduce 2^16": lambda i: addf(v),
    }
    for name, fn in cases.items():
        for i in range(10):
            fn(i)
        torch.cuda.synchronize()
        # keep the GPU busy far longer than the enqueue loop takes
        for st in streams:
            with torch.cuda.stream(st):
                torch.cuda._sleep(int(2e9))
        t0 = time.perf_counter()
        for i in range(N):
            fn(i)
        t1 = time.perf_counter()
        torch.cuda.synchronize()
        # GPU time per call (events on the first stream around N calls, no spin)
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(streams[0])
        for i in range(N):
            fn(i)
        e1.record(streams[0])
        torch.cuda.synchronize()
        print(f"G={G} {name:32s} host enqueue {(t1 - t0) / N * 1e6:8.1f} us/call   "
              f"stream-0 time {e0.elapsed_time(e1) / N * 1e3:8.1f} us/call", flush=True)
    c.finalize()
