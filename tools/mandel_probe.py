"""Mandelbrot headline probe on one GPU: the per-pixel blocktest user function
in several launch configurations, each timed (CUDA events, L2 flushed, median
of 20) and checked bit for bit against the oracle on the whole 4096x3072 image.
(The two-pixel packed fp32x2 variant measured with it in round 2 -
profiles/sweeps/sweep_r02_mandel_pairs.log - is in the history of
paper_conf_pact_steuwerg13_b200/apps.py, commit "Mandelbrot user function for
two neighbouring pixels".)

  MANDEL_CFGS="kind,block,unroll,interleave,B[,THxTW];..."   kind: single (blocktest
  user function, B iterations per block) or plain (the A22 loop); THxTW: pixels stored in
  TH x TW warp tiles (application-level layout, restored on download)
  MANDEL_ILJ=j     elements per lane of the interleaved Map kernel (map_il_elems)
  MANDEL_EVERY=k   only rows 0, k, 2k, ... (one GPU's share of the image at k GPUs
                   with the bench's round-robin row dealing)
  MANDEL_ORDER=center  those rows ordered nearest-the-middle first
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

ROWS, COLS, MAX = 3072, 4096, 1000


def timeit(fn, flush, reps=20, warm=3):
    for _ in range(warm):
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
    return float(np.median([a.elapsed_time(b) for a, b in ts]))


def main():
    flush = torch.empty(64 << 20, dtype=torch.float32, device="cuda")
    global ROWS
    every = int(os.environ.get("MANDEL_EVERY", "1"))
    rows = np.arange(0, ROWS, every)
    if os.environ.get("MANDEL_ORDER") == "center":
        # the rows nearest the image's middle (the costliest) first
        rows = rows[np.argsort(np.abs(rows - (ROWS - 1) / 2.0), kind="stable")]
    grid = np.ascontiguousarray(I.mandel_grid(ROWS, COLS)[rows])
    ROWS = grid.shape[0]
    ref, tot = O.mandelbrot(grid, MAX)
    cfgs = os.environ.get("MANDEL_CFGS", "single,1024,1,1,12;single,512,1,1,12")
    for cfg in cfgs.split(";"):
        kind, bt, un, il, B = cfg.split(",")[:5]
        tile = cfg.split(",")[5] if len(cfg.split(",")) > 5 else ""
        perm = np.arange(ROWS * COLS)
        if tile:
            th, tw = (int(v) for v in tile.split("x"))
            perm = perm.reshape(ROWS // th, th, COLS // tw, tw).transpose(0, 2, 1, 3).reshape(-1)
        c = S.Context(1)
        st = torch.cuda.Stream()
        torch.cuda.set_stream(st)
        c.set_stream(0, st.cuda_stream)
        c.set_option("block_threads", int(bt))
        c.set_option("map_unroll", int(un))
        c.set_option("map_interleave", int(il))
        if os.environ.get("MANDEL_ILJ"):
            c.set_option("map_il_elems", int(os.environ["MANDEL_ILJ"]))
        src = A.mandelbrot(MAX) if kind == "plain" else A.mandelbrot_blocktest(MAX, int(B))
        m = S.Map(c, src, S.F32X2, S.U32)
        x = S.Matrix(c, S.F32X2, ROWS, COLS).copy_in(np.ascontiguousarray(grid.reshape(-1, 2)[perm]))
        o = S.Matrix(c, S.U32, ROWS, COLS)
        m(x, out=o)
        ms = timeit(lambda: m(x, out=o), flush)
        got = np.empty(ROWS * COLS, np.uint32)
        got[perm] = o.to_numpy(np.uint32).reshape(-1)
        got = got.reshape(ROWS, COLS)
        ok = bool(np.array_equal(got, ref))
        print(f"mandel {cfg}: {ms:.4f} ms  {8 * tot / (ms / 1e3) / 1e12:.2f} TFLOP/s (8 ops/iter)  bitexact={ok}",
              flush=True)
        c.finalize()


if __name__ == "__main__":
    main()
