"""Build tuning variants of libmpcgs.so (extra -D defines) under variants/.

usage: python tools/build_variants.py NAME=DEF1,DEF2 NAME2=... ; bench with
MPCGS_LIB=variants/libmpcgs_NAME.so python bench.py ...
"""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
from paper_conf_ipps_davistzw17_b200 import _build  # noqa: E402

os.makedirs(os.path.join(ROOT, "variants"), exist_ok=True)
for spec in sys.argv[1:]:
    name, _, defs = spec.partition("=")
    out = os.path.join(ROOT, "variants", f"libmpcgs_{name}.so")
    _build.build(force=True, out=out, defines=[d for d in defs.split(",") if d])
    print("built", out, flush=True)
