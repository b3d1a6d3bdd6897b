"""Chunked host<->device transfers (implicit upload/download):
an upload of >= 4 MB goes to the device in chunks on a copy stream; a Map/Zip
consumes the chunks as they arrive (one launch per chunk) and its output chunks
stream back to the host while later chunks compute.  Every other consumer waits
for all chunks.  Results must be those of the unchunked path (bit-exact)."""
import numpy as np
import pytest

import oracle as O
from gpu_util import rel_l2, require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu

N = (3 << 20) + 5      # 12 MB of fp32: chunked (>= 4 MB), ragged last chunk


@pytest.fixture(scope="module", params=[1, 2])
def ctx(request):
    require_gpu()
    G = request.param
    c = S.Context(G, devices=[0] * G)
    yield c
    c.finalize()


def _launches(ctx, fn):
    l0 = ctx.counter("launches")
    r = fn()
    return r, ctx.counter("launches") - l0


def test_pipelined_map_roundtrip(ctx):
    x = I.uniform_f32(51, N) - np.float32(0.5)
    sq = S.Map(ctx, A.SQP1, S.F32, S.F32)
    v = S.Vector(ctx, S.F32, N).set_distribution(S.BLOCK)
    out = S.Vector(ctx, S.F32, N)
    sq(S.Vector.from_numpy(ctx, x), out=out)      # compile
    v.copy_in(x)
    _, k = _launches(ctx, lambda: sq(v, out=out))
    assert k > ctx.ndev                            # one launch per chunk
    assert np.array_equal(out.to_numpy(), O.map_(O.OM_SQP1_F32, x))
    # per-device download of a chunked output (each device's part streams out)
    want = O.map_(O.OM_SQP1_F32, x)
    for g in range(ctx.ndev):
        v.copy_in(x)
        sq(v, out=out)
        buf = np.empty(N, np.float32)
        first, n = out.copy_out_part(g, buf)
        assert n > 0 and np.array_equal(buf[:n], want[first:first + n])


def test_other_consumers_wait_for_all_chunks(ctx):
    x = I.uniform_f32(52, N)
    v = S.Vector(ctx, S.F32, N).set_distribution(S.BLOCK)
    v.copy_in(x)
    s = float(S.Reduce(ctx, A.SUM, S.F32)(v).scalar())
    ref = O.reduce_(O.OP_ADD_F32, x)
    assert abs(s - ref) <= 1e-5 * abs(ref)
    v.copy_in(x)
    sc = S.Scan(ctx, A.ADD, S.F32)(v).to_numpy()
    assert rel_l2(sc, O.scan(O.OP_ADD_F32, x)) <= 1e-5
    v.copy_in(x)
    v.set_distribution(S.COPY)                     # redistribution after a chunked upload
    assert np.array_equal(v.to_numpy(), x)


def test_in_place_zip_and_chained(ctx):
    x, y = I.uniform_f32(53, N), I.uniform_f32(54, N)
    add = S.Zip(ctx, A.ADD, S.F32, S.F32, S.F32)
    neg = S.Map(ctx, A.NEG, S.F32, S.F32)
    vx = S.Vector(ctx, S.F32, N).set_distribution(S.BLOCK)
    vy = S.Vector(ctx, S.F32, N).set_distribution(S.BLOCK)
    vx.copy_in(x)
    vy.copy_in(y)
    add(vx, vy, out=vx)                            # in place, both inputs chunked
    neg(vx, out=vx)                                # consumes the Zip's output chunks
    assert np.array_equal(vx.to_numpy(), -O.zip_(O.OZ_ADD_F32, x, y))


def test_matrix_stencil_after_chunked_upload(ctx):
    img = I.image_f32(I.SEED_GAUSS, 1100, 1024)    # 4.5 MB
    m = S.Matrix(ctx, S.F32, 1100, 1024).set_distribution(S.OVERLAP, 2)
    m.copy_in(img)
    gau = S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
    assert np.array_equal(gau(m).to_numpy(), O.mapoverlap2d(O.OS_GAUSS5, img, 2, O.OB_NEAREST, 0.0))


def test_repeated_uploads_and_destroy_while_pending(ctx):
    x = I.uniform_f32(55, N)
    v = S.Vector(ctx, S.F32, N).set_distribution(S.BLOCK)
    for _ in range(3):
        v.copy_in(x)                               # never consumed
    v.destroy()
    w = S.Vector(ctx, S.F32, N).set_distribution(S.BLOCK)
    w.copy_in(x)
    assert np.array_equal(w.to_numpy(), x)


def test_unchunked_option(ctx):
    ctx.set_option("xfer_chunks", 1)
    try:
        x = I.uniform_f32(56, N)
        sq = S.Map(ctx, A.SQP1, S.F32, S.F32)
        v = S.Vector(ctx, S.F32, N).set_distribution(S.BLOCK)
        out = S.Vector(ctx, S.F32, N)
        sq(S.Vector.from_numpy(ctx, x), out=out)
        v.copy_in(x)
        _, k = _launches(ctx, lambda: sq(v, out=out))
        assert k == ctx.ndev
        assert np.array_equal(out.to_numpy(), O.map_(O.OM_SQP1_F32, x))
    finally:
        ctx.set_option("xfer_chunks", 8)
