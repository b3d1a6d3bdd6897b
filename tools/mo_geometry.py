"""Print the register-block geometry the library chose for a MapOverlap (the
SKL_RH / SKL_CW / SKL_MO_KT / SKL_MO_HEAVY defines of its compiled program)."""
import os
import re
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from paper_conf_pact_steuwerg13_b200 import apps as A  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import skl as S  # noqa: E402

ctx = S.Context(1)
for name in ("IDENT2D_U8", "SOBEL", "SOBEL_TUNED"):
    mo = S.MapOverlap(ctx, getattr(A, name), S.U8, S.U8, 1, S.NEUTRAL, 0)
    src = mo.source()
    geo = {k: re.findall(r"#define %s (\S+)" % k, src) for k in ("SKL_RH", "SKL_CW", "SKL_MO_KT", "SKL_MO_HEAVY")}
    print(name, geo, flush=True)
ctx.finalize()
