"""Localise a full-size accurate vs index-join disagreement: bisect the canvas
with query windows (Z20: windows partition the points) until single pixels,
then show each pixel's points, the oracle's exact counts for them, and
whether the oracle (O9) and the kernels' boundary pieces flag the pixel.
    python tools/acc_bisect.py [--config C3] [--points N]"""
import argparse
import os
import sys

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import bench  # noqa: E402
import oracle  # noqa: E402
from datagen import configs as C  # noqa: E402
from paper_journals_pvldb_zacharatoudasf17_b200 import rj  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--config", default="C3")
ap.add_argument("--points", type=int, default=1_000_000_000)
args = ap.parse_args()
box, polys_name, recipe, q, desc = bench.workload(args.config)
x, y, cols = bench.gen_points(recipe, args.points, 0, pinned=True)
flat = C.array_polys(polys_name)
R = rj.RasterJoin(box)
R.set_option(rj.OPT_GRAPHS, 0)
R.load_points(x, y, cols)
R.load_polygons(flat)
W, H = q["W"], q["H"]


def diff(view):
    a, _ = R.query(W=W, H=H, mode="accurate", view=view)
    b, _ = R.query(W=W, H=H, mode="index", view=view)
    return a, b


stack = [(0, 0, W, H)]
bad = []
while stack:
    v = stack.pop()
    a, b = diff(v)
    if np.array_equal(a, b):
        continue
    c0, r0, c1, r1 = v
    if c1 - c0 == 1 and r1 - r0 == 1:
        bad.append((v, a, b))
        continue
    if c1 - c0 >= r1 - r0:
        m = (c0 + c1) // 2
        stack += [(c0, r0, m, r1), (m, r0, c1, r1)]
    else:
        m = (r0 + r1) // 2
        stack += [(c0, r0, c1, m), (c0, m, c1, r1)]
print("bad pixels", len(bad))
P = oracle.Polys(flat, box)
omask = oracle.boundary_mask(P, W, H)
qx = np.array([oracle.quantize(float(t), box[0], box[2]) for t in x[:0]])
for v, a, b in bad[:10]:
    c0, r0 = v[0], v[1]
    d = np.nonzero(a != b)[0]
    print("pixel", (c0, r0), "accurate", {int(k): int(a[k]) for k in d}, "index", {int(k): int(b[k]) for k in d})
    # points of this pixel (vectorised O1/O2 on the float32 inputs)
    fx = np.floor((x.astype(np.float64) - box[0]) / (box[2] - box[0]) * 2.0 ** 30).astype(np.int64)
    fy = np.floor((y.astype(np.float64) - box[1]) / (box[3] - box[1]) * 2.0 ** 30).astype(np.int64)
    sel = np.nonzero(((fx * W) >> 30 == c0) & ((fy * H) >> 30 == r0))[0]
    print("  points", len(sel), "first", sel[:5].tolist(), "x,y", list(zip(x[sel[:3]].tolist(), y[sel[:3]].tolist())))
    oc, _, _ = oracle.query(P, x[sel], y[sel], W=W, H=H, mode="accurate")
    ob, _, _ = oracle.query(P, x[sel], y[sel], W=W, H=H, mode="bounded")
    nz = np.nonzero(oc)[0]
    print("  oracle exact", {int(k): int(oc[k]) for k in nz}, "oracle bounded", {int(k): int(ob[k]) for k in np.nonzero(ob)[0]})
    print("  oracle O9 boundary:", bool((omask[r0, c0 >> 5] >> (c0 & 31)) & 1))
    bnd, cov = R.boundary_pieces(W=W, H=H, view=(max(0, c0 - 2), max(0, r0 - 2), min(W, c0 + 3), min(H, r0 + 3)))
    print("  kernel boundary piece:", bool((bnd[r0, c0 >> 5] >> (c0 & 31)) & 1), "covered:", bool((cov[r0, c0 >> 5] >> (c0 & 31)) & 1))
    # neighbourhood of the oracle mask
    for rr in range(r0 - 2, r0 + 3):
        print("   ", "".join("#" if (omask[rr, cc >> 5] >> (cc & 31)) & 1 else "." for cc in range(c0 - 4, c0 + 5)),
              "".join("#" if (bnd[rr, cc >> 5] >> (cc & 31)) & 1 else "." for cc in range(c0 - 4, c0 + 5)))
