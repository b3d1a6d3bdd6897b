"""Iterated Gaussian 8192^2 (10 iterations, ping-pong) on G logical devices of
one GPU, replayed as one CUDA graph: event time per step, to separate the
multi-device overhead (barriers, halo push, partial waves) from the stencil.
ITER_G="1,2,4" ITER_PUSH=1 ITER_ROWS=8192 ITER_ONCE=1 (one replay each, for ncu
launch lists)"""
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from paper_conf_pact_steuwerg13_b200 import apps as A  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import inputs as I  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import skl as S  # noqa: E402

R = int(os.environ.get("ITER_ROWS", "8192"))
C = 8192
img = I.image_f32(I.SEED_GAUSS, R, C)
once = os.environ.get("ITER_ONCE") == "1"
for G in (int(g) for g in os.environ.get("ITER_G", "1,2,4").split(",")):
    c = S.Context(G, devices=[0] * G)
    streams = [torch.cuda.Stream() for _ in range(G)]
    for g, st in enumerate(streams):
        c.set_stream(g, st.cuda_stream)
    c.set_option("halo_push", int(os.environ.get("ITER_PUSH", "1")))
    c.set_option("block_threads", 128)
    gau = S.MapOverlap(c, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
    a = S.Matrix.from_numpy(c, img)
    b = S.Matrix(c, S.F32, R, C)
    t = S.Matrix(c, S.F32, R, C)

    def run10():
        gau(a, out=b)
        for k in range(9):
            gau(b, out=t) if k % 2 == 0 else gau(t, out=b)

    run10()
    g = c.capture(run10)
    torch.cuda.synchronize()
    if once:
        g.launch()
        torch.cuda.synchronize()
        print(f"G={G}: ran once", flush=True)
    else:
        ts = []
        for _ in range(12):
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(streams[0])
            g.launch()
            e1.record(streams[0])
            torch.cuda.synchronize()
            ts.append(e0.elapsed_time(e1))
        print(f"G={G} push={os.environ.get('ITER_PUSH', '1')} rows={R}: "
              f"{np.median(ts[2:]):.4f} ms per 10 iterations",
              flush=True)
    g.destroy()
    c.finalize()
