"""Full-size oracle parity:
every BASELINE.json configuration at its full point count, through the exact
launch configuration bench.py times (library defaults, the bench's context
stream, rj_query_device + rj_finalize_device, the same seeded points from
bench.gen_points), compared element by element with the CPU oracle run on
the same host arrays: COUNT bit-exact, SUM/AVG within 1e-9 relative (reading
Z23; integer SUM bit-exact).  The exact result is the plain GROUP BY over
exact point-in-polygon; bounded mode is the pixel-centre rule
(P:550-562).

    python tools/fullsize_parity.py [--only C2,C3,...] [--out FILE]
Writes one JSON line per case (points, oracle seconds and threads, GPU ms,
pass/fail) to --out (default gpurun_out/fullsize_parity.jsonl).
"""
from __future__ import annotations

import argparse
import json
import os
import sys
import time

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import bench  # noqa: E402
import oracle  # noqa: E402
from datagen import configs as C  # noqa: E402

# name, bench config, points, i0, query overrides
CASES = [
    ("C2", "C2", 1_000_000_000, 0, {}),
    ("C3-accurate", "C3", 1_000_000_000, 0, {}),
    ("C3-bounded", "C3", 1_000_000_000, 0, {"mode": "bounded"}),
    ("C4-rank-shard", "C4", 250_000_000, 750_000_000, {}),
    ("C5-1024-bounded", "C5", 1_000_000_000, 0, {"W": 1024, "H": 1024}),
    ("C5-1024-accurate", "C5", 1_000_000_000, 0, {"W": 1024, "H": 1024, "mode": "accurate"}),
    ("C5-32768-bounded", "C5", 1_000_000_000, 0, {}),
    ("C5-32768-accurate", "C5", 1_000_000_000, 0, {"mode": "accurate"}),
]


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--only", default="")
    ap.add_argument("--out", default=os.path.join(ROOT, "gpurun_out", "fullsize_parity.jsonl"))
    args = ap.parse_args()
    import torch

    from paper_journals_pvldb_zacharatoudasf17_b200 import rj

    only = set(args.only.split(",")) if args.only else None
    os.makedirs(os.path.dirname(args.out), exist_ok=True)
    cache = {}
    for name, cfg, n, i0, over in CASES:
        if only and name not in only:
            continue
        box, polys_name, recipe, q, desc = bench.workload(cfg)
        q = dict(q, **over)
        key = (recipe, n, i0)
        if key not in cache:
            cache.clear()
            cache[key] = bench.gen_points(recipe, n, i0, pinned=True)
        x, y, cols = cache[key]
        flat = C.array_polys(polys_name)
        stream = torch.cuda.Stream()
        R = rj.RasterJoin(box, stream=stream.cuda_stream)
        R.load_points(x, y, cols)
        R.load_polygons(flat)
        desc_q = rj.make_desc(**q)
        W, H = rj.rj_resolve_canvas(R.ctx, desc_q)
        npl = R.n_poly
        d_cnt = torch.zeros(npl, dtype=torch.int64, device="cuda")
        d_sum = torch.zeros(npl, dtype=torch.float64, device="cuda")
        d_val = torch.zeros(npl, dtype=torch.float64, device="cuda")
        for _ in range(3):                                  # graph capture + replay, as bench.py
            with torch.cuda.stream(stream):
                rj.rj_query_device(R.ctx, desc_q, d_cnt, d_sum)
                rj.rj_finalize_device(R.ctx, desc_q.agg, d_cnt, d_sum, d_val)
            stream.synchronize()
        R.set_option(rj.OPT_TIMING, 1)
        with torch.cuda.stream(stream):
            rj.rj_query_device(R.ctx, desc_q, d_cnt, d_sum)
            rj.rj_finalize_device(R.ctx, desc_q.agg, d_cnt, d_sum, d_val)
        stream.synchronize()
        st = R.stats()
        g_cnt = d_cnt.cpu().numpy().astype(np.uint64)
        g_val = d_val.cpu().numpy()
        R.close()
        P = oracle.Polys(flat, box)
        preds = [(c_, op, v) for c_, op, v in q.get("preds", [])]
        agg_col = q.get("agg_column", -1)
        t0 = time.perf_counter()
        o_cnt, o_sum, kept = oracle.query(P, x, y, cols=cols, preds=preds, agg_col=agg_col, W=W, H=H,
                                          mode=q["mode"])
        o_s = time.perf_counter() - t0
        count_ok = bool(np.array_equal(g_cnt, o_cnt))
        rel = 0.0
        if q["agg"] == "sum":
            o_val = o_sum
        elif q["agg"] == "avg":
            o_val = oracle.avg(o_cnt, o_sum)
        else:
            o_val = o_cnt.astype(np.float64)
        both_nan = np.isnan(g_val) & np.isnan(o_val)
        den = np.where(o_val == 0, 1.0, np.abs(o_val))
        err = np.where(both_nan, 0.0, np.abs(g_val - o_val) / den)
        rel = float(np.nanmax(err)) if len(err) else 0.0
        exact_int = q["agg"] == "count" or (q["agg"] == "sum" and cols[0].dtype == np.int32 and agg_col == 0)
        val_ok = bool(np.array_equal(g_val, o_val)) if exact_int else rel <= 1e-9
        rec = {"case": name, "workload": desc, "points": n, "first_point": i0, "canvas": [W, H], "mode": q["mode"],
               "agg": q["agg"], "polygons": npl, "n_filtered_gpu": st["n_filtered"], "n_filtered_oracle": kept,
               "n_boundary": st["n_boundary"], "count_bitexact": count_ok, "value_max_rel_err": rel,
               "value_exact_required": exact_int, "pass": count_ok and val_ok and st["n_filtered"] == kept,
               "gpu_query_ms": st["ms_total"], "oracle_s": o_s, "oracle_threads": len(os.sched_getaffinity(0)),
               "launch": "bench.py configuration: library defaults, rj_query_device + rj_finalize_device on the "
                         "bench stream, graph replay"}
        print(json.dumps(rec), flush=True)
        with open(args.out, "a") as f:
            f.write(json.dumps(rec) + "\n")


if __name__ == "__main__":
    main()
