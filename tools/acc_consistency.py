"""Full-size accurate-mode self-consistency (no oracle needed): at 1e9 points
the exact variants -- accurate raster join through the label kernel, the
pixel-tile kernel, and the index join (PIP for every point) -- must give the
same counts (all equal the exact GROUP BY).  Reports every polygon
where two variants disagree, for a query path's configuration matrix.
    python tools/acc_consistency.py [--config C3] [--points N]"""
import argparse
import json
import os
import sys

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import bench  # noqa: E402
from datagen import configs as C  # noqa: E402
from paper_journals_pvldb_zacharatoudasf17_b200 import rj  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--config", default="C3")
ap.add_argument("--points", type=int, default=1_000_000_000)
ap.add_argument("--prefix", type=int, default=0, help="also compare on the first N points with the oracle")
args = ap.parse_args()
box, polys_name, recipe, q, desc = bench.workload(args.config)
x, y, cols = bench.gen_points(recipe, args.points, 0, pinned=True)
flat = C.array_polys(polys_name)
R = rj.RasterJoin(box)
R.load_points(x, y, cols)
R.load_polygons(flat)
res = {}
for name, opts, kw in [("index", {}, dict(mode="index")),
                       ("acc_label", {rj.OPT_PASS: 0}, dict(mode="accurate")),
                       ("acc_tile", {rj.OPT_PASS: 1}, dict(mode="accurate")),
                       ("acc_count", {}, dict(mode="accurate", agg="count")),
                       ("acc_label_nograph", {rj.OPT_PASS: 0, rj.OPT_GRAPHS: 0}, dict(mode="accurate")),
                       ("acc_label_nofused", {rj.OPT_PASS: 0, rj.OPT_FUSED_POLY: 0}, dict(mode="accurate"))]:
    for k, v in opts.items():
        R.set_option(k, v)
    qq = dict(q, **kw)
    outs = []
    for rep in range(3):
        cnt, val = R.query(**qq)
        st = R.stats()
        outs.append((cnt.copy(), st["n_boundary"]))
    for k in opts:
        R.set_option(k, -1 if k == rj.OPT_PASS else 1)
    res[name] = outs
    print(name, [int(c.sum()) for c, _ in outs], [nb for _, nb in outs], flush=True)
ref = res["index"][0][0]
for name, outs in res.items():
    for rep, (cnt, nb) in enumerate(outs):
        d = np.nonzero(cnt != ref)[0]
        if len(d):
            print("DIFF", name, rep, "polygons", len(d), "first", d[:8].tolist(),
                  "delta", (cnt[d[:8]].astype(np.int64) - ref[d[:8]].astype(np.int64)).tolist(), flush=True)
print("done")
