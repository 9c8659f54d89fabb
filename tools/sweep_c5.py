"""C5 (BASELINE.json configs[4]): canvas-resolution / epsilon-bound sweep on
1e9 taxi-shaped points x 260 neighbourhoods, COUNT, no filter -- the
accuracy-vs-time experiment of PAPER.md Fig. 12 on B200.

For W = H in 1024 .. 32768 (epsilon = w * sqrt(2) / W on the 57.92 km
domain, reading Z3) it reports
  - bounded and accurate query latency (device, graph-replayed, mean of K),
  - the bounded result's per-polygon % error against the accurate (exact)
    count: median / p95 / max (as Fig. 12b),
  - the worst-case interval of P:797-810 (must contain the exact count for
    every polygon, O10) and the expected interval's estimate error
    (Z22),
  - the accurate count's invariance across W (it is exact at every W).

    python tools/sweep_c5.py [--points 1e9] [--steps 10] > profiles/...jsonl
"""
from __future__ import annotations

import argparse
import json
import math
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import bench  # noqa: E402
from datagen import configs as C  # noqa: E402
from paper_journals_pvldb_zacharatoudasf17_b200 import rj  # noqa: E402


def timed(R, desc, stream, steps):
    n = R.n_poly
    d_cnt = torch.zeros(n, dtype=torch.int64, device="cuda")
    d_sum = torch.zeros(n, dtype=torch.float64, device="cuda")

    def step():
        with torch.cuda.stream(stream):
            rj.rj_query_device(R.ctx, desc, d_cnt, d_sum)
        stream.synchronize()

    for _ in range(3):
        step()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    torch.cuda.synchronize()
    e0.record(stream)
    for _ in range(steps):
        step()
    e1.record(stream)
    torch.cuda.synchronize()
    return e0.elapsed_time(e1) / steps, d_cnt.cpu().numpy().astype(np.int64)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--points", type=float, default=1e9)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--sizes", default="1024,2048,4096,8192,16384,32768")
    args = ap.parse_args()
    n = int(args.points)
    box = C.NYC_BOX
    x, y, cols = bench.gen_points("taxi", n, 0)
    stream = torch.cuda.Stream()
    R = rj.RasterJoin(box, device=0, stream=stream.cuda_stream)
    R.load_polygons(C.array_polys("neighborhoods"))
    R.load_points(x, y, cols)
    del x, y, cols
    exact = None
    w_dom = box[2] - box[0]
    for W in [int(v) for v in args.sizes.split(",")]:
        ms_b, cb = timed(R, rj.make_desc(W=W, H=W, mode="bounded"), stream, args.steps)
        ms_a, ca = timed(R, rj.make_desc(W=W, H=W, mode="accurate"), stream, args.steps)
        if exact is None:
            exact = ca
        cnt, _, ep, em, xp, xm = R.query_interval_ex(W=W, H=W)
        cnt = cnt.astype(np.int64)
        assert np.array_equal(cnt, cb)
        ok = exact > 0
        err = np.abs(cb[ok] - exact[ok]) / exact[ok] * 100.0
        est = cnt - xp + xm
        est_err = np.abs(est[ok] - exact[ok]) / exact[ok] * 100.0
        holds = bool(np.all((exact >= cnt - ep.astype(np.int64)) & (exact <= cnt + em.astype(np.int64))))
        width = (ep + em).astype(np.float64)[ok] / exact[ok] * 100.0
        line = {
            "W": W, "epsilon_m": w_dom * math.sqrt(2.0) / W, "points": n, "polygons": int(R.n_poly),
            "bounded_ms": ms_b, "accurate_ms": ms_a,
            "bounded_points_per_s": n / (ms_b / 1e3), "accurate_points_per_s": n / (ms_a / 1e3),
            "accurate_equals_exact_at_every_W": bool(np.array_equal(ca, exact)),
            "tiling_sum_ok": bool(cb.sum() == exact.sum()),
            "pct_error": {"median": float(np.median(err)), "p95": float(np.percentile(err, 95)),
                          "max": float(err.max())},
            "worst_case_interval_holds": holds,
            "worst_case_width_pct": {"median": float(np.median(width)), "max": float(width.max())},
            "expected_estimate_pct_error": {"median": float(np.median(est_err)),
                                            "p95": float(np.percentile(est_err, 95)),
                                            "max": float(est_err.max())},
        }
        print(json.dumps(line), flush=True)
    R.close()


if __name__ == "__main__":
    main()
