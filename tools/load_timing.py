"""Load-time costs (S1 quantise + Morton sort, S6 edge grid), not part of the
query metric: rj_load_polygons per polygon set and rj_load_points per point
count, wall clock around the synchronous C-ABI calls (best of 3).
    python tools/load_timing.py [--points N]"""
import argparse
import json
import os
import sys
import time

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from datagen import configs as C  # noqa: E402
from datagen import polygons as PG  # noqa: E402
from paper_journals_pvldb_zacharatoudasf17_b200 import rj  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--points", type=int, default=200_000_000)
args = ap.parse_args()
out = {}
for name, box, flat in (("c1b", C.C1_BOX, PG.flatten(C.polygon_set("c1b"))),
                        ("neighborhoods", C.NYC_BOX, C.array_polys("neighborhoods")),
                        ("tracts", C.NYC_BOX, C.array_polys("tracts")),
                        ("counties", C.US_BOX, C.array_polys("counties"))):
    R = rj.RasterJoin(box)
    best = 1e9
    for _ in range(3):
        t0 = time.perf_counter()
        R.load_polygons(flat)
        best = min(best, time.perf_counter() - t0)
    out[name] = {"polygons": int(len(flat[0]) - 1), "vertices": int(len(flat[2])), "load_polygons_ms": best * 1e3}
    R.close()
import bench  # noqa: E402
import torch  # noqa: E402
x, y, cols = bench.gen_points("taxi_t", args.points, 0, pinned=True)
R = rj.RasterJoin(C.NYC_BOX)
R.set_option(rj.OPT_KEEP_LOAD_SCRATCH, 1)
ts = []
for _ in range(3):
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    R.load_points(x, y, cols)
    ts.append(time.perf_counter() - t0)
dx, dy, dc = torch.from_numpy(x).cuda(), torch.from_numpy(y).cuda(), [torch.from_numpy(c).cuda() for c in cols]
td = []
for _ in range(3):
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    R.load_points(dx, dy, dc)
    td.append(time.perf_counter() - t0)
out["load_points"] = {"points": args.points, "host_pinned_ms": min(ts) * 1e3, "device_resident_ms": min(td) * 1e3,
                      "host_pinned_Gpts_s": args.points / min(ts) / 1e9,
                      "device_resident_Gpts_s": args.points / min(td) / 1e9}
print(json.dumps(out))
