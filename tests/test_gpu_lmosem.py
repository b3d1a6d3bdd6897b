"""Iterative list-mode OSEM over several subsets (reading
A29) on 1 and 3 devices: f goes block -> copy and c copy(+) -> block at every
subset.  Checked against the oracle's one-subset function applied subset by
subset (each next subset starts from the oracle's image rounded to fp32, the
precision the GPU keeps f in): relative L2 <= 1e-4 (north_star)."""
import numpy as np
import pytest

import oracle as O
from gpu_util import rel_l2, require_gpu
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S
from paper_conf_pact_steuwerg13_b200.lmosem import ListModeOSEM


def test_subset_bounds_cover_once():
    for nev, nsub in ((10, 3), (7, 7), (1000003, 10), (5, 1)):
        b = ListModeOSEM.subset_bounds(nev, nsub)
        assert b[0][0] == 0 and b[-1][1] == nev
        assert all(b[i][1] == b[i + 1][0] for i in range(nsub - 1))
        sizes = [hi - lo for lo, hi in b]
        assert max(sizes) - min(sizes) <= 1


def _oracle_osem(events, N, f0, nsub, passes):
    f = f0.astype(np.float32)
    for _ in range(passes):
        for lo, hi in ListModeOSEM.subset_bounds(events.shape[0], nsub):
            _, fn, _, _ = O.lmosem(events[lo:hi], N, f)
            f = fn.astype(np.float32)
    return f


@pytest.mark.gpu
@pytest.mark.parametrize("G", [1, 3])
@pytest.mark.parametrize("nsub,passes", [(3, 1), (2, 2)])
def test_osem_subsets_match_oracle(G, nsub, passes):
    require_gpu()
    N, nev = 16, 9001
    ctx = S.Context(G, devices=[0] * G)
    try:
        events = I.lmosem_events(I.SEED_LMOSEM, nev, N)
        f0 = (1.0 + 0.5 * I.uniform_f32(9, N ** 3)).astype(np.float32)
        osem = ListModeOSEM(ctx, N)
        osem.load_events(events, nsub)
        osem.set_image(f0)
        p2p0 = ctx.counter("p2p_bytes")
        osem.iterate(passes)
        got = osem.image()
        want = _oracle_osem(events, N, f0, nsub, passes)
        assert rel_l2(got, want) <= 1e-4
        if G > 1:   # the image and the correction moved between devices every subset
            assert ctx.counter("p2p_bytes") - p2p0 >= nsub * passes * (G - 1) * N ** 3 * 4
        osem.destroy()
    finally:
        ctx.finalize()
