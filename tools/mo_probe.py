"""MapOverlap probe on one GPU: 8192^2 identity u8 / Sobel (paper form and the
tuned user function apps.SOBEL_TUNED) / identity f32 / Gaussian, timed with CUDA events (L2
flushed), each checked against the oracle on row bands.

  python tools/mo_probe.py [names] [--once]      names: ident_u8,sobel,sobel_tuned,ident_f32,gauss,
                                                 file:<path> (a u8 user function checked as Sobel)
  MO_OPTS="key=value,..."  library options (skl_set_option) for every context
  MO_PER_EVENT=k           k launches between one event pair (time per launch = total / k)
  MO_NOFLUSH=1             no L2 flush before the timed launches

--once runs each kernel a single time (for ncu -k regex:skl_mo launch lists).
"""
import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import oracle as O  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import apps as A  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import inputs as I  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import skl as S  # noqa: E402

R = C = 8192


def opts():
    out = {}
    for kv in filter(None, os.environ.get("MO_OPTS", "").split(",")):
        k, v = kv.split("=")
        out[k] = int(v)
    return out


def timeit(fn, flush, reps=20, warm=3, flush_on=True):
    for _ in range(warm):
        fn()
    torch.cuda.synchronize()
    torch.cuda._sleep(int(reps * 4e5))
    ts = []
    for _ in range(reps):
        if flush_on:
            flush.zero_()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        fn()
        b.record()
        ts.append((a, b))
    torch.cuda.synchronize()
    return float(np.median([a.elapsed_time(b) for a, b in ts]))


def main():
    names = [a for a in sys.argv[1:] if not a.startswith("--")] or ["ident_u8", "sobel", "sobel_tuned", "ident_f32",
                                                                   "gauss"]
    once = "--once" in sys.argv
    flush = torch.empty(64 << 20, dtype=torch.float32, device="cuda")
    img8 = I.image_u8(I.SEED_SOBEL, R, C)
    img32 = I.image_f32(I.SEED_GAUSS, R, C)
    for name in names:
        c = S.Context(1)
        s = torch.cuda.Stream()
        torch.cuda.set_stream(s)
        c.set_stream(0, s.cuda_stream)
        o = opts()
        if (name in ("gauss", "ident_f32") or name.startswith("gfile:")) and "block_threads" not in o:
            o["block_threads"] = 128
        for k, v in o.items():
            c.set_option(k, v)
        if name == "ident_u8":
            mo, img, st, d, b = S.MapOverlap(c, A.IDENT2D_U8, S.U8, S.U8, 1, S.NEUTRAL, 0), img8, O.OS_IDENT, 1, O.OB_NEUTRAL
        elif name == "sobel":
            mo, img, st, d, b = S.MapOverlap(c, A.SOBEL, S.U8, S.U8, 1, S.NEUTRAL, 0), img8, O.OS_SOBEL, 1, O.OB_NEUTRAL
        elif name == "sobel_tuned":
            mo, img, st, d, b = (S.MapOverlap(c, A.SOBEL_TUNED, S.U8, S.U8, 1, S.NEUTRAL, 0), img8, O.OS_SOBEL, 1,
                                 O.OB_NEUTRAL)
        elif name.startswith("file:"):   # a Sobel-semantics u8 user function from a file
            mo, img, st, d, b = (S.MapOverlap(c, open(name[5:]).read(), S.U8, S.U8, 1, S.NEUTRAL, 0), img8,
                                 O.OS_SOBEL, 1, O.OB_NEUTRAL)
        elif name.startswith("gfile:"):   # an f32 user function from a file checked as the Gaussian
            mo, img, st, d, b = (S.MapOverlap(c, open(name[6:]).read(), S.F32, S.F32, 2, S.NEAREST, 0.0), img32,
                                 O.OS_GAUSS5, 2, O.OB_NEAREST)
        elif name == "ident_f32":
            mo, img, st, d, b = (S.MapOverlap(c, A.IDENT2D, S.F32, S.F32, 1, S.NEAREST, 0.0), img32, O.OS_IDENT, 1,
                                 O.OB_NEAREST)
        else:
            mo, img, st, d, b = (S.MapOverlap(c, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0), img32, O.OS_GAUSS5, 2,
                                 O.OB_NEAREST)
        mi = S.Matrix.from_numpy(c, img)
        out = mo(mi)
        if once:
            torch.cuda.synchronize()
            mo(mi, out=out)
            torch.cuda.synchronize()
            print(f"{name}: ran once", flush=True)
        else:
            per = int(os.environ.get("MO_PER_EVENT", "1"))   # launches between one event pair

            def many():
                for _ in range(per):
                    mo(mi, out=out)
            ms = timeit(many, flush, flush_on=os.environ.get("MO_NOFLUSH") != "1") / per
            full = out.to_numpy()
            ok = True
            if name.startswith(("file:", "gfile:")):   # whole image
                ok = bool(np.array_equal(full, O.mapoverlap2d(st, img, d, b, 0)))
            for r0 in (0, 4000, R - 64):
                lo, hi = max(0, r0 - 8), min(R, r0 + 72)
                ref = O.mapoverlap2d(st, img[lo:hi], d, b, 0)
                ok &= bool(np.array_equal(full[r0:r0 + 64], ref[r0 - lo:r0 - lo + 64]))
            byt = (2 if img.dtype == np.uint8 else 8) * R * C
            print(f"{name:10s} {o}: {ms * 1e3:7.1f} us  {byt / (ms / 1e3) / 1e9:6.0f} GB/s  "
                  f"({byt / (ms / 1e3) / 1e9 / 6548.2:.3f} of HBM)  bitexact={ok}", flush=True)
        c.finalize()


if __name__ == "__main__":
    main()
