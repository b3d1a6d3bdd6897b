"""Parameter sweeps on one GPU (work-group size / unroll knobs, user-function
variants).  Prints one line per configuration: device ms per call (CUDA events,
L2 flushed), plus a parity flag against the oracle where cheap.

  python tools/sweep.py mandel|lmosem|scan|mo|mows
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

FLUSH = None


def ctx_with(opts):
    global FLUSH
    c = S.Context(1)
    s = torch.cuda.Stream()
    torch.cuda.set_stream(s)
    c.set_stream(0, s.cuda_stream)
    for k, v in opts.items():
        c.set_option(k, v)
    if FLUSH is None:
        FLUSH = torch.empty(64 << 20, dtype=torch.float32, device="cuda")
    return c


def timeit(fn, reps=10, warm=3):
    for _ in range(warm):
        fn()
    torch.cuda.synchronize()
    torch.cuda._sleep(int(reps * 4e5))   # host-ahead pre-roll (as bench.py)
    ts = []
    for _ in range(reps):
        FLUSH.zero_()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        fn()
        b.record()
        ts.append((a, b))
    torch.cuda.synchronize()
    return float(np.median([a.elapsed_time(b) for a, b in ts]))


def dot20():
    """fused dot product at 2^20 (BASELINE config 0) in a CUDA graph, cold and warm,
    DOT_CFGS="block,..." """
    n = 1 << 20
    a, b = I.uniform_f32(1, n), I.uniform_f32(2, n)
    for bt in (int(x) for x in os.environ.get("DOT_CFGS", "256").split(",")):
        c = ctx_with({"block_threads": bt})
        va = S.Vector.from_numpy(c, a).set_distribution(S.BLOCK)
        vb = S.Vector.from_numpy(c, b).set_distribution(S.BLOCK)
        mult, sm = S.Zip(c, A.MULT, S.F32, S.F32, S.F32), S.Reduce(c, A.SUM, S.F32)
        s = sm(mult(va, vb))
        g = c.capture(lambda: sm(mult(va, vb), out=s))
        cold = timeit(g.launch, reps=30)
        ts = []
        torch.cuda.synchronize()
        torch.cuda._sleep(int(30 * 4e5))
        for _ in range(30):
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record()
            g.launch()
            e1.record()
            ts.append((e0, e1))
        torch.cuda.synchronize()
        warm = float(np.median([x.elapsed_time(y) for x, y in ts]))
        ref = O.reduce_(O.OP_ADD_F32, O.zip_(O.OZ_MULT_F32, a, b))
        ok = abs(float(s.scalar()) - ref) <= 1e-5 * abs(ref)
        print(f"dot20 block={bt}: cold {cold * 1e3:.2f} us  warm {warm * 1e3:.2f} us  ok={ok}", flush=True)
        g.destroy()
        # floor of this measurement: a graph with one tiny kernel (fill of 4 floats)
        tiny = S.Vector(c, S.F32, 4).set_distribution(S.BLOCK).fill(0.0)
        g0 = c.capture(lambda: tiny.fill(1.0))
        ts = []
        torch.cuda.synchronize()
        torch.cuda._sleep(int(30 * 4e5))
        for _ in range(30):
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record()
            g0.launch()
            e1.record()
            ts.append((e0, e1))
        torch.cuda.synchronize()
        print(f"   one-kernel graph floor: {float(np.median([x.elapsed_time(y) for x, y in ts])) * 1e3:.2f} us", flush=True)
        # and a plain torch kernel between the same events
        t = torch.zeros(4, device="cuda")
        ts = []
        torch.cuda.synchronize()
        torch.cuda._sleep(int(30 * 4e5))
        for _ in range(30):
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record()
            t.add_(1.0)
            e1.record()
            ts.append((e0, e1))
        torch.cuda.synchronize()
        print(f"   one torch kernel: {float(np.median([x.elapsed_time(y) for x, y in ts])) * 1e3:.2f} us", flush=True)
        c.finalize()


def allpairs():
    """AP_CFGS="tile[:bk],...": 4096^3 dot and 4096x4096x128 Manhattan, zip-reduce form"""
    for cfg in os.environ.get("AP_CFGS", "0").split(","):
        tile, bk = (int(v) for v in (cfg.split(":") + ["0"])[:2])
        c = ctx_with({"ap_tile": tile, "ap_bk": bk})
        for name, z, dd in (("dot", A.MULT, 4096), ("manhattan", A.ABSDIFF, 128)):
            a = I.uniform_f32(81, 4096 * dd).reshape(4096, dd)
            b = I.uniform_f32(82, 4096 * dd).reshape(4096, dd)
            ap = S.Allpairs(c, z, S.F32, S.F32, reduce=A.ADD)
            ma, mb = S.Matrix.from_numpy(c, a), S.Matrix.from_numpy(c, b)
            o = ap(ma, mb)
            ms = timeit(lambda: ap(ma, mb, out=o), reps=5)
            cg = o.to_numpy()
            fn = O.AP_DOT if z == A.MULT else O.AP_MANHATTAN
            ok = np.array_equal(cg[:16, :40], O.allpairs(fn, a[:16], b[:40]))
            tf = 2.0 * 4096 * 4096 * dd / (ms / 1e3) / 1e12
            print(f"allpairs {name:9s} tile={tile} bk={bk}: {ms:.4f} ms  {tf:.2f} TFLOP/s  bitexact={ok}", flush=True)
        c.finalize()


def mandel():
    """MANDEL_CFGS="fn,block,unroll,interleave;..." (fn: plain | unroll4)"""
    grid = I.mandel_grid(3072, 4096)
    ref = None
    cfgs = [t.split(",") for t in os.environ.get("MANDEL_CFGS", "unroll4,512,2,0").split(";")]
    for name, bt, un, il in cfgs:
        bt, un, il = int(bt), int(un), int(il)
        if name == "plain":
            src = A.mandelbrot(1000)
        elif name.startswith("btest"):
            src = A.mandelbrot_blocktest(1000, int(name[5:] or 8))
        else:
            src = A.mandelbrot_unrolled(1000, int(name[6:] or 4))
        c = ctx_with({"block_threads": bt, "map_unroll": un, "map_interleave": il})
        m = S.Map(c, src, S.F32X2, S.U32)
        x = S.Matrix(c, S.F32X2, 3072, 4096).copy_in(grid)
        o = m(x)
        ms = timeit(lambda: m(x, out=o))
        out = o.to_numpy()
        if ref is None:
            ref, tot = O.mandelbrot(grid, 1000)
        ok = np.array_equal(out, ref)
        print(f"mandel {name:8s} block={bt:4d} unroll={un} interleave={il}: {ms:.4f} ms  "
              f"{8 * tot / (ms / 1e3) / 1e12:.2f} TFLOP/s  bitexact={ok}", flush=True)
        c.finalize()


def lmosem():
    N, nev = 150, 10_000_000
    events = I.lmosem_events(7, nev, N)
    for bt in (128, 256):
        for un in (1, 4):
            c = ctx_with({"block_threads": bt, "map_unroll": un})
            evd = c.struct_type("Event", A.EVENT_DECL, A.EVENT_SIZE, 4)
            lm = S.Map(c, A.lmosem_map(N), evd, S.VOID, extra=[S.F32 | S.PTR, S.F32 | S.PTR])
            ev = S.Vector(c, evd, nev).set_distribution(S.BLOCK)
            ev.copy_in(events)
            f = S.Vector(c, S.F32, N ** 3).set_distribution(S.COPY).fill(1.0)
            cc = S.Vector(c, S.F32, N ** 3).set_distribution(S.COPY).fill(0.0)
            ms = timeit(lambda: lm(ev, f, (cc, S.WRITE)), reps=5, warm=1)
            print(f"lmosem block={bt} unroll={un}: {ms:.3f} ms  {nev / (ms / 1e3) / 1e9:.3f} Gevents/s", flush=True)
            c.finalize()


def scan():
    """configurations from SCAN_CFGS="variant,block,chunks,minb;..." (default: the shipped one)"""
    n = 1 << 30
    cfgs = [tuple(int(x) for x in t.split(",")) for t in os.environ.get("SCAN_CFGS", "3,256,8,4").split(";")]
    for var, bt, ch, mb in cfgs:
        pers, fs, ns = 1, 16, 1
        if True:
            if True:
                c = ctx_with({"block_threads": bt, "scan_chunks": ch, "scan_variant": var, "scan_minb": mb})
                sc = S.Scan(c, A.ADD_I32, S.I32)
                v = S.Vector(c, S.I32, n).set_distribution(S.BLOCK).fill(1)
                o = sc(v)
                ms = timeit(lambda: sc(v, out=o), reps=5)
                p, f, cnt = o.local_part(0)

                class View:
                    __cuda_array_interface__ = {"shape": (cnt,), "typestr": "<i4", "data": (p, False),
                                                "version": 3, "strides": None}
                c.sync()
                got = torch.as_tensor(View(), device="cuda")
                idx = torch.tensor([0, 1, 8191, 8192, 123456789, n // 2, n - 2, n - 1], device="cuda")
                ok = bool(torch.equal(got[idx].long(), idx + 1))   # scan of ones = 1..n
                print(f"scan i32 variant={var} block={bt} chunks={ch} minb={mb}: {ms:.3f} ms  "
                      f"{8 * n / (ms / 1e3) / 1e9:.0f} GB/s ok={ok}", flush=True)
                c.finalize()


def copy():
    """Map identity over 2^30 int32 (read 4 B + write 4 B per element): the
    skeleton's streaming ceiling, for comparison with Scan and the measured copy."""
    n = 1 << 30
    for bt in (256, 512):
        for un in (1, 2, 4, 8):
            c = ctx_with({"block_threads": bt, "map_unroll": un})
            m = S.Map(c, "int id(int x){ return x; }", S.I32, S.I32)
            v = S.Vector(c, S.I32, n).set_distribution(S.BLOCK).fill(1)
            o = m(v)
            ms = timeit(lambda: m(v, out=o), reps=5)
            print(f"map-copy i32 block={bt} unroll={un}: {ms:.3f} ms  {8 * n / (ms / 1e3) / 1e9:.0f} GB/s", flush=True)
            c.finalize()


def mo():
    img8 = I.image_u8(5, 8192, 8192)
    imgf = I.image_f32(6, 8192, 8192)
    # MO_CFGS="block,rh,cw_u8,cw_f32;..." (0 = the library's automatic choice)
    cfgs = [tuple(int(x) for x in t.split(",")) for t in os.environ.get("MO_CFGS", "256,0,0,0").split(";")]
    for cfg in cfgs:
        bt, rh, cw8, cw32 = cfg[:4]
        c = ctx_with({"block_threads": bt, "mo_minb": cfg[4] if len(cfg) > 4 else 0,
                      "mo_persist": cfg[5] if len(cfg) > 5 else 0})
        for name, src, t, d, bnd, img in (("ident_u8", A.IDENT2D_U8, S.U8, 1, S.NEUTRAL, img8),
                                          ("sobel", A.SOBEL, S.U8, 1, S.NEUTRAL, img8),
                                          ("ident_f32", A.IDENT2D, S.F32, 2, S.NEAREST, imgf),
                                          ("gauss", A.gaussian5(), S.F32, 2, S.NEAREST, imgf)):
            c.set_option("mo_rh", rh)
            c.set_option("mo_cw", cw8 if t == S.U8 else cw32)
            m = S.MapOverlap(c, src, t, t, d, bnd, 0)
            x = S.Matrix.from_numpy(c, img)
            o = m(x)
            ms = timeit(lambda: m(x, out=o))
            bpp = 2 * img.itemsize
            ok = ""
            if name in ("sobel", "gauss"):
                sub = img[3990:4074]
                ref = (O.mapoverlap2d(O.OS_SOBEL, sub, 1, O.OB_NEUTRAL, 0) if name == "sobel"
                       else O.mapoverlap2d(O.OS_GAUSS5, sub, 2, O.OB_NEAREST, 0.0))[10:74]
                ok = f" bitexact={np.array_equal(o.to_numpy()[4000:4064], ref)}"
            print(f"mo {name:9s} block={bt} rh={rh} cw={cw8 if t == S.U8 else cw32} minb={cfg[4] if len(cfg) > 4 else 0} persist={cfg[5] if len(cfg) > 5 else 0}: {ms:.4f} ms  "
                  f"{bpp * img.size / (ms / 1e3) / 1e9:.0f} GB/s{ok}", flush=True)
            x.destroy()
            o.destroy()
        c.finalize()


def mows():
    """TMA / warp-specialised MapOverlap (mo_ws) against the one-tile-per-block
    kernel.  MOWS_CFGS="block,rh,cw,ws,stages,wsminb;..." (0 = automatic).  The
    full output image is compared with the plain kernel's (bit-exact)."""
    img8 = I.image_u8(5, 8192, 8192)
    imgf = I.image_f32(6, 8192, 8192)
    cfgs = [tuple(int(x) for x in t.split(",")) for t in
            os.environ.get("MOWS_CFGS", "256,0,0,0,4,0").split(";")]
    work = [w for w in (("ident_u8", A.IDENT2D_U8, S.U8, 1, S.NEUTRAL, img8),
                        ("sobel", A.SOBEL, S.U8, 1, S.NEUTRAL, img8),
                        ("ident_f32", A.IDENT2D, S.F32, 2, S.NEAREST, imgf),
                        ("gauss", A.gaussian5(), S.F32, 2, S.NEAREST, imgf))
            if w[0] in os.environ.get("MOWS_WORK", "ident_u8,sobel,ident_f32,gauss").split(",")]
    refs = {}
    c0 = ctx_with({"block_threads": 256 if True else 0})
    for name, src, t, d, bnd, img in work:
        if name == "gauss":
            c0.set_option("block_threads", 128)
        m = S.MapOverlap(c0, src, t, t, d, bnd, 0)
        c0.set_option("block_threads", 256)
        x = S.Matrix.from_numpy(c0, img)
        o = m(x)
        ms = timeit(lambda: m(x, out=o))
        refs[name] = o.to_numpy()
        print(f"mows {name:9s} plain (bench config): {ms:.4f} ms", flush=True)
        x.destroy()
        o.destroy()
    c0.finalize()
    for cfg in cfgs:
        bt, rh, cw, ws, st, wm = cfg
        c = ctx_with({"block_threads": bt, "mo_ws": ws, "mo_ws_stages": st, "mo_ws_minb": wm,
                      "mo_rh": rh, "mo_cw": cw})
        for name, src, t, d, bnd, img in work:
            m = S.MapOverlap(c, src, t, t, d, bnd, 0)
            x = S.Matrix.from_numpy(c, img)
            o = m(x)
            n0 = c.counter("tma_launches")
            ms = timeit(lambda: m(x, out=o))
            tma = c.counter("tma_launches") > n0
            ok = np.array_equal(o.to_numpy(), refs[name])
            bpp = 2 * img.itemsize
            print(f"mows {name:9s} block={bt} rh={rh} cw={cw} ws={ws} stages={st} wsminb={wm} tma={tma}: "
                  f"{ms:.4f} ms  {bpp * img.size / (ms / 1e3) / 1e9:.0f} GB/s same={ok}", flush=True)
            x.destroy()
            o.destroy()
        c.finalize()


def e2e():
    """headline end to end (pinned host -> copy_in -> Mandelbrot Map -> copy_out)
    against the PCIe floor, for E2E_CHUNKS="4,8,16,32" transfer chunks"""
    R, Cc = 3072, 4096
    ctx_with({}).finalize()   # creates the L2 flush buffer
    grid = I.mandel_grid(R, Cc)
    pin_in = torch.empty(grid.nbytes, dtype=torch.uint8, pin_memory=True)
    pin_in.numpy()[:] = grid.view(np.uint8).ravel()
    pin_out = torch.empty(R * Cc * 4, dtype=torch.uint8, pin_memory=True)
    dev_in = torch.empty(grid.nbytes, dtype=torch.uint8, device="cuda")
    dev_out = torch.empty(R * Cc * 4, dtype=torch.uint8, device="cuda")
    h2d = timeit(lambda: dev_in.copy_(pin_in, non_blocking=True))
    d2h = timeit(lambda: pin_out.copy_(dev_out, non_blocking=True))
    print(f"PCIe pinned H2D {grid.nbytes / 1e6:.0f} MB: {h2d:.3f} ms ({grid.nbytes / h2d / 1e6:.1f} GB/s); "
          f"D2H {R * Cc * 4 / 1e6:.0f} MB: {d2h:.3f} ms ({R * Cc * 4 / d2h / 1e6:.1f} GB/s)", flush=True)
    for cfg in os.environ.get("E2E_CHUNKS", "4,8,16,32").split(","):
        ch, taper = (int(v) for v in (cfg.split(":") + ["1"])[:2])   # "chunks[:taper]"
        c = ctx_with({"xfer_chunks": ch, "xfer_taper": taper, "block_threads": 128, "map_unroll": 1,
                      "map_interleave": 1, "map_il_elems": 1})
        # E2E_FN=cheap: a trivial function of the same types (the pipeline without compute)
        src = ("uint cheap(float2 c){ return (uint)c.x; }" if os.environ.get("E2E_FN") == "cheap"
               else A.mandelbrot_blocktest(1000, 12))
        m = S.Map(c, src, S.F32X2, S.U32)
        e_in = S.Matrix(c, S.F32X2, R, Cc).set_distribution(S.BLOCK)
        e_out = S.Matrix(c, S.U32, R, Cc)

        def step():
            e_in.copy_in_ptr(pin_in.data_ptr(), grid.nbytes)
            m(e_in, out=e_out)
            e_out.copy_out_part(0, pin_out.numpy())

        ms = timeit(step, reps=10)
        dev = timeit(lambda: m(e_in, out=e_out), reps=10)
        print(f"e2e chunks={ch} taper={taper}: {ms:.3f} ms (kernel alone {dev:.3f} ms)", flush=True)
        c.finalize()


if __name__ == "__main__":
    for w in sys.argv[1:]:
        globals()[w]()
