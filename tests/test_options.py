"""Host logic of skl_set_option (include/skl.h): every key the header documents
is accepted with a valid value, out-of-range values and unknown keys fail with
SKL_ERR_INVALID_ARG.  Runs on an offline context (no GPU)."""
import os
import re

import pytest

from paper_conf_pact_steuwerg13_b200 import skl as S

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
VALID = {"ap_tile": 2, "scan_chunks": 8, "mo_ws_stages": 3, "ap_bk": 32, "block_threads": 128,
         "scan_variant": 6, "combine_peer": 2, "combine_unroll": 4, "mo_kt": 3}


def documented_keys():
    h = open(os.path.join(ROOT, "include", "skl.h")).read()
    i, j = h.find("/* Options:"), h.find("skl_status skl_set_option")
    return sorted(set(re.findall(r'"([a-z_0-9]+)"', h[i:j])))


@pytest.fixture(scope="module")
def ctx():
    c = S.Context.offline()
    yield c
    c.finalize()


def test_header_documents_the_new_keys():
    keys = documented_keys()
    for k in ("mo_ws", "mo_ws_stages", "ap_hybrid", "ap_bk", "combine_peer", "combine_unroll"):
        assert k in keys, k


@pytest.mark.parametrize("key", documented_keys())
def test_documented_key_accepted(ctx, key):
    ctx.set_option(key, VALID.get(key, 1))


@pytest.mark.parametrize("key,value", [("combine_peer", 3), ("combine_unroll", 9), ("mo_ws_stages", 1),
                                       ("mo_ws_stages", 9), ("mo_ws_minb", 33), ("ap_bk", 8), ("ap_tile", 3),
                                       ("no_such_key", 1)])
def test_invalid_value_rejected(ctx, key, value):
    with pytest.raises(S.SklError) as e:
        ctx.set_option(key, value)
    assert e.value.name == "INVALID_ARG"
