"""skl_set_allocator: with torch's caching allocator every
device buffer of the library comes from torch (PyTorch as device-memory
plumbing); results are unchanged and the memory returns to torch at finalize."""
import numpy as np
import pytest

import oracle as O
from gpu_util import rel_l2, require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu


@pytest.mark.parametrize("G", [1, 2])
def test_torch_allocator_end_to_end(G):
    require_gpu()
    import torch
    torch.cuda.synchronize()
    base = torch.cuda.memory_allocated(0)
    ctx = S.Context(G, devices=[0] * G)
    try:
        ctx.use_torch_allocator()
        n = (1 << 20) + 7
        a, b = I.uniform_f32(I.SEED_DOT_A, n), I.uniform_f32(I.SEED_DOT_B, n)
        mult, add = S.Zip(ctx, A.MULT, S.F32, S.F32, S.F32), S.Reduce(ctx, A.SUM, S.F32)
        va, vb = S.Vector.from_numpy(ctx, a), S.Vector.from_numpy(ctx, b)
        got = float(add(mult(va, vb)).scalar())
        ref = O.reduce_(O.OP_ADD_F32, O.zip_(O.OZ_MULT_F32, a, b))
        assert abs(got - ref) <= 1e-5 * abs(ref)
        assert torch.cuda.memory_allocated(0) >= base + 2 * 4 * n   # the inputs live in torch's pool
        xi = I.uniform_int(3, 100003, -1000, 1000)
        sc = S.Scan(ctx, A.ADD_I32, S.I32)
        assert np.array_equal(sc(S.Vector.from_numpy(ctx, xi)).to_numpy(), O.scan(O.OP_ADD_I32, xi))
        img = I.image_f32(I.SEED_GAUSS, 130, 97)
        gau = S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
        assert np.array_equal(gau(S.Matrix.from_numpy(ctx, img)).to_numpy(),
                              O.mapoverlap2d(O.OS_GAUSS5, img, 2, O.OB_NEAREST, 0.0))
        x = I.uniform_f32(5, 4097)
        v = S.Vector.from_numpy(ctx, x).set_distribution(S.COPY)
        v.set_distribution(S.BLOCK)
        assert rel_l2(v.to_numpy(), x) == 0
    finally:
        ctx.finalize()
    torch.cuda.synchronize()
    assert torch.cuda.memory_allocated(0) == base


def test_allocator_only_before_containers():
    require_gpu()
    ctx = S.Context(1)
    try:
        keep = S.Vector(ctx, S.F32, 10).fill(1.0)   # noqa: F841 - a live container
        with pytest.raises(S.SklError) as e:
            ctx.use_torch_allocator()
        assert e.value.name == "INVALID_ARG"
    finally:
        ctx.finalize()
