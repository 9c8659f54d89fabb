"""One query per process, for bisecting sanitizer reports (tools/sanitize.py
runs them all).  python tools/san_exp.py MODE AGG [CHUNK [PASS [STAGES]]]"""
import os
import sys

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import oracle  # noqa: E402
from datagen import configs as C  # noqa: E402
from datagen import polygons as PG  # noqa: E402
from paper_journals_pvldb_zacharatoudasf17_b200 import rj  # noqa: E402

mode, agg = sys.argv[1], sys.argv[2]
chunk = int(sys.argv[3]) if len(sys.argv) > 3 else 0
variant = int(sys.argv[4]) if len(sys.argv) > 4 else -1
stages = int(sys.argv[5]) if len(sys.argv) > 5 else 0
polys = C.polygon_set("c1b")
flat = PG.flatten(polys)
pts = C.c1_points(20000)
x, y = pts["x"], pts["y"]
col = (np.arange(len(x)) % 7).astype(np.int32)
R = rj.RasterJoin(C.C1_BOX)
if chunk:
    R.set_option(rj.OPT_CHUNK, chunk)
R.set_option(rj.OPT_PASS, variant)
if stages:
    R.set_option(rj.OPT_STAGES, stages)
R.load_points(x, y, [col])
R.load_polygons(flat)
cnt, _ = R.query(W=1024, H=1024, mode=mode, agg=agg, agg_column=0 if agg != "count" else -1)
P = oracle.Polys(flat, C.C1_BOX)
ocnt = oracle.query(P, x, y, W=1024, H=1024, mode="bounded" if mode == "bounded" else "accurate")[0]
print("ok" if np.array_equal(cnt, ocnt) else "MISMATCH", mode, agg, chunk)
