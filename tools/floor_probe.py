"""Event-timing floor on one GPU: an L2 flush, then event -> X -> event, median
of 50, for X = nothing, a 1-element Map (one tiny kernel), and the 8192^2
identity u8 stencil (skl_mo2d_t).  Separates the launch / event overhead from
a kernel's own duration (ncu gpu__time_duration)."""
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from paper_conf_pact_steuwerg13_b200 import apps as A  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import inputs as I  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import skl as S  # noqa: E402


def timeit(fn, flush, reps=50):
    for _ in range(3):
        fn()
    torch.cuda.synchronize()
    torch.cuda._sleep(int(reps * 4e5))
    ts = []
    for _ in range(reps):
        flush.zero_()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        fn()
        b.record()
        ts.append((a, b))
    torch.cuda.synchronize()
    v = [a.elapsed_time(b) * 1e3 for a, b in ts]
    return float(np.median(v)), float(np.min(v))


c = S.Context(1)
s = torch.cuda.Stream()
torch.cuda.set_stream(s)
c.set_stream(0, s.cuda_stream)
flush = torch.empty(64 << 20, dtype=torch.float32, device="cuda")
tiny = S.Vector.from_numpy(c, np.ones(1, np.float32))
neg = S.Map(c, A.NEG, S.F32, S.F32)
to = neg(tiny)
img = S.Matrix.from_numpy(c, I.image_u8(I.SEED_SOBEL, 8192, 8192))
mo = S.MapOverlap(c, A.IDENT2D_U8, S.U8, S.U8, 1, S.NEUTRAL, 0)
out = mo(img)
z = torch.zeros(1, device="cuda")
for name, fn in (("nothing", lambda: None), ("torch tiny kernel", lambda: z.add_(1.0)),
                 ("skl 1-element Map", lambda: neg(tiny, out=to)), ("identity u8 8192^2", lambda: mo(img, out=out))):
    med, mn = timeit(fn, flush)
    print(f"{name:22s} median {med:7.2f} us  min {mn:7.2f} us", flush=True)
c.finalize()
