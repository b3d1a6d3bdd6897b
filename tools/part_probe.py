"""One GPU's part of the 8192^2 stencils at G = 1, 2, 4, 8 (8192/G rows x 8192),
per launch configuration: how a smaller grid (fewer waves) changes the best
tiles-per-block / rows-per-thread choice.  Event-timed, L2 flushed, median of 20.
PART_CFGS="name:key=v,key=v;..."  name in gauss, sobel_tuned, ident_u8"""
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from paper_conf_pact_steuwerg13_b200 import apps as A  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import inputs as I  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import skl as S  # noqa: E402


def timeit(fn, flush, reps=20):
    for _ in range(3):
        fn()
    torch.cuda.synchronize()
    torch.cuda._sleep(int(reps * 4e5))
    ts = []
    for _ in range(reps):
        flush.zero_()
        flush.sum()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        fn()
        b.record()
        ts.append((a, b))
    torch.cuda.synchronize()
    return float(np.median([a.elapsed_time(b) for a, b in ts]))


flush = torch.empty(64 << 20, dtype=torch.float32, device="cuda")
C = 8192
for cfg in os.environ.get("PART_CFGS", "gauss:mo_kt=2;gauss:mo_kt=1").split(";"):
    name, opts = cfg.split(":") if ":" in cfg else (cfg, "")
    o = dict(kv.split("=") for kv in opts.split(",") if kv)
    line = []
    for G in (1, 2, 4, 8):
        R = 8192 // G
        c = S.Context(1)
        st = torch.cuda.Stream()
        torch.cuda.set_stream(st)
        c.set_stream(0, st.cuda_stream)
        if name == "gauss":
            c.set_option("block_threads", 128)
        for k, v in o.items():
            c.set_option(k, int(v))
        if name == "gauss":
            mo = S.MapOverlap(c, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
            img = I.image_f32(I.SEED_GAUSS, R, C)
        else:
            mo = S.MapOverlap(c, A.SOBEL_TUNED if name == "sobel_tuned" else A.IDENT2D_U8, S.U8, S.U8, 1,
                              S.NEUTRAL, 0)
            img = I.image_u8(I.SEED_SOBEL, R, C)
        m = S.Matrix.from_numpy(c, img)
        out = mo(m)
        ms = timeit(lambda: mo(m, out=out), flush)
        line.append(f"G={G} {ms * 1e3:7.1f} us (x{G}: {ms * 1e3 * G:7.1f})")
        c.finalize()
    print(f"{cfg:40s} " + "  ".join(line), flush=True)
