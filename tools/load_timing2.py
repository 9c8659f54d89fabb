"""Where the load-then-query time goes (C2, 1e9 points, pinned host columns):
wall time of rj_load_points and of the first rj_query, repeated."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import bench
from datagen import configs as C
from paper_journals_pvldb_zacharatoudasf17_b200 import rj

box, polys, recipe, q, _ = bench.workload("C2")
n = int(float(sys.argv[1])) if len(sys.argv) > 1 else 1_000_000_000
x, y, cols = bench.gen_points(recipe, n, 0, pinned=True)
R = rj.RasterJoin(box)
R.load_polygons(C.array_polys(polys))
desc = rj.make_desc(**q)
cnt = np.zeros(R.n_poly, np.uint64); val = np.zeros(R.n_poly, np.float64)
for it in range(int(os.environ.get("ITERS", "4"))):
    torch.cuda.synchronize()
    t0 = time.perf_counter(); R.load_points(x, y, cols); t1 = time.perf_counter()
    rj.rj_query(R.ctx, desc, cnt, val); t2 = time.perf_counter()
    rj.rj_query(R.ctx, desc, cnt, val); t3 = time.perf_counter()
    print(f"load {1e3*(t1-t0):.1f} ms  first query {1e3*(t2-t1):.1f} ms  second query {1e3*(t3-t2):.1f} ms", flush=True)
