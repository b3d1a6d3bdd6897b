"""Minimal driver for ncu captures: runs one skeleton workload at its BASELINE
size a few times (no oracle, no timing).  Usage under gpurun, e.g.

  ncu --set full --clock-control none --import-source on -k regex:skl_scan -s 1 -c 1 \
      -o gpurun_out/prof_scan python tools/prof_driver.py scan_i32
"""
import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

from paper_conf_pact_steuwerg13_b200 import apps as A  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import inputs as I  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import skl as S  # noqa: E402


def main(which: str, reps: int = 3):
    ctx = S.Context(1)
    ctx.set_option("xfer_chunks", 1)   # one launch per call: the captured kernel is the bench step's
    if which == "mandel":
        # the bench's configuration
        ctx.set_option("block_threads", 1024)
        ctx.set_option("map_unroll", 1)
        ctx.set_option("map_interleave", 1)
        m = S.Map(ctx, A.mandelbrot_blocktest(1000, 12), S.F32X2, S.U32)
        x = S.Matrix(ctx, S.F32X2, 3072, 4096).copy_in(I.mandel_grid(3072, 4096))
        o = m(x)
        for _ in range(reps):
            m(x, out=o)
    elif which in ("scan_i32", "scan_f32"):
        n = 1 << 30
        dt = S.I32 if which == "scan_i32" else S.F32
        sc = S.Scan(ctx, A.ADD_I32 if dt == S.I32 else A.ADD, dt)
        v = S.Vector(ctx, dt, n).set_distribution(S.BLOCK)
        v.fill(1)
        o = sc(v)
        for _ in range(reps):
            sc(v, out=o)
    elif which in ("sobel", "gauss"):
        if which == "sobel":
            mo = S.MapOverlap(ctx, A.SOBEL, S.U8, S.U8, 1, S.NEUTRAL, 0)
            x = S.Matrix.from_numpy(ctx, I.image_u8(5, 8192, 8192))
        else:
            ctx.set_option("block_threads", 128)   # bench.py's Gaussian configuration
            mo = S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
            ctx.set_option("block_threads", 256)
            x = S.Matrix.from_numpy(ctx, I.image_f32(6, 8192, 8192))
        o = mo(x)
        for _ in range(reps):
            mo(x, out=o)
    elif which in ("dot", "dot28"):
        n = 1 << 20 if which == "dot" else 1 << 28
        a = S.Vector(ctx, S.F32, n).set_distribution(S.BLOCK).fill(1.0)
        b = S.Vector(ctx, S.F32, n).set_distribution(S.BLOCK).fill(2.0)
        mult, sm = S.Zip(ctx, A.MULT, S.F32, S.F32, S.F32), S.Reduce(ctx, A.SUM, S.F32)
        s = sm(mult(a, b))
        for _ in range(reps):
            sm(mult(a, b), out=s)   # fused Zip -> Reduce (one kernel)
    elif which in ("allpairs_dot", "allpairs_manhattan"):
        d = 4096 if which == "allpairs_dot" else 128
        ap = S.Allpairs(ctx, A.MULT if which == "allpairs_dot" else A.ABSDIFF, S.F32, S.F32, reduce=A.ADD)
        a = S.Matrix.from_numpy(ctx, I.uniform_f32(81, 4096 * d).reshape(4096, d)).set_distribution(S.BLOCK)
        b = S.Matrix.from_numpy(ctx, I.uniform_f32(82, 4096 * d).reshape(4096, d)).set_distribution(S.COPY)
        c = ap(a, b)
        for _ in range(reps):
            ap(a, b, out=c)
    elif which == "lmosem":
        N, nev = 150, 10_000_000
        evd = ctx.struct_type("Event", A.EVENT_DECL, A.EVENT_SIZE, 4)
        ctx.set_option("map_unroll", 1)
        lm = S.Map(ctx, A.lmosem_map(N), evd, S.VOID, extra=[S.F32 | S.PTR, S.F32 | S.PTR])
        ev = S.Vector(ctx, evd, nev).set_distribution(S.BLOCK)
        from paper_conf_pact_steuwerg13_b200.lmosem import ListModeOSEM
        events = I.lmosem_events(7, nev, N)
        ev.copy_in(np.ascontiguousarray(events[ListModeOSEM.path_order(events, N)]))   # bench.py's order
        f = S.Vector(ctx, S.F32, N ** 3).set_distribution(S.COPY).fill(1.0)
        c = S.Vector(ctx, S.F32, N ** 3).set_distribution(S.COPY).fill(0.0)
        for _ in range(reps):
            lm(ev, f, (c, S.WRITE))
    ctx.sync()
    ctx.finalize()


if __name__ == "__main__":
    main(sys.argv[1], int(sys.argv[2]) if len(sys.argv) > 2 else 3)
