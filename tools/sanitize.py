"""Drive every librj kernel variant once on small C1/C1b inputs, for
compute-sanitizer (memcheck / racecheck / synccheck / initcheck; SURVEY.md
4.5 and 7 step 4).  Each query is also checked against the CPU oracle so a
run under a sanitizer proves the same launches are still correct.

    compute-sanitizer --tool racecheck python tools/sanitize.py [--quick]

Variants: tile (COUNT; in-lane and warp-merged runs) and label (SUM/AVG) point-pass kernels, bounded and
accurate, index join, the exact chooser, windows, a fine canvas, streamed
queries (host and device columns, ragged batches), worst-case and expected
intervals, MIN/MAX and multi-aggregate, graph replay, the debug kernels and
a two-rank sharded query (rj_query_device + rj_finalize_device).
"""
from __future__ import annotations

import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import oracle  # noqa: E402
from datagen import configs as C  # noqa: E402
from datagen import polygons as PG  # noqa: E402
from paper_journals_pvldb_zacharatoudasf17_b200 import rj  # noqa: E402


def device_paths(R, S, P, x, y, cols, chk):
    """Device-resident inputs: a streamed query over torch device columns and
    the multi-GPU path's calls (device partials + finalize)."""
    import torch
    dx, dy = torch.from_numpy(x).cuda(), torch.from_numpy(y).cuda()
    dc = [torch.from_numpy(c).cuda() for c in cols]
    cnt, _ = S.query_stream(dx, dy, dc, W=1024, H=1024, mode="accurate", agg="avg", agg_column=1)
    chk(cnt, oracle.query(P, x, y, W=1024, H=1024, mode="accurate")[0], "stream-dev")
    # device partials + finalize (the multi-GPU path's calls)
    d_cnt = torch.zeros(P.n, dtype=torch.int64, device="cuda")
    d_sum = torch.zeros(P.n, dtype=torch.float64, device="cuda")
    d_val = torch.zeros(P.n, dtype=torch.float64, device="cuda")
    q = rj.make_desc(agg="avg", agg_column=1, W=1024, H=1024, mode="accurate")
    rj.rj_query_device(R.ctx, q, d_cnt, d_sum)
    torch.cuda.synchronize()
    rj.rj_finalize_device(R.ctx, "avg", d_cnt, d_sum, d_val)
    torch.cuda.synchronize()
    chk(d_cnt.cpu().numpy().astype(np.uint64), oracle.query(P, x, y, W=1024, H=1024, mode="accurate")[0], "device")


def main():
    quick = "--quick" in sys.argv
    n = 20_000 if quick else 60_000
    polys = C.polygon_set("c1b")
    flat = PG.flatten(polys)
    pts = C.c1_points(n)
    ax, ay = PG.c1b_points(polys)
    x = np.concatenate([pts["x"], ax])
    y = np.concatenate([pts["y"], ay])
    rng = np.random.default_rng(3)
    ti = rng.integers(-50, 50, len(x)).astype(np.int32)
    tf = rng.normal(5, 3, len(x)).astype(np.float32)
    cols = [ti, tf]
    P = oracle.Polys(flat, C.C1_BOX)
    R = rj.RasterJoin(C.C1_BOX)
    R.set_option(rj.OPT_CHUNK, 4096)             # many work items, heavy-cell split
    R.load_points(x, y, cols)
    R.load_polygons(flat)
    ok = 0

    def chk(cnt, ocnt, tag):
        nonlocal ok
        assert np.array_equal(cnt, ocnt), tag
        ok += 1

    for W in (1024, 333, 8192):
        for mode in ("bounded", "accurate", "index", "exact"):
            om = "bounded" if mode == "bounded" else "accurate"
            for variant in (-1, 0, 1):
                R.set_option(rj.OPT_PASS, variant)
                # COUNT: in-lane runs (default) and warp-merged runs (variant 1)
                R.set_option(rj.OPT_LANE_RUNS, 2 if variant == 1 else 0)
                for agg, col in (("count", -1), ("sum", 0), ("avg", 1)):
                    preds = [(0, ">=", -30)]
                    cnt, _ = R.query(W=W, H=W, mode=mode, agg=agg, agg_column=col, preds=preds)
                    ocnt, _, _ = oracle.query(P, x, y, cols=cols, preds=preds, W=W, H=W, mode=om)
                    chk(cnt, ocnt, (W, mode, variant, agg))
    R.set_option(rj.OPT_PASS, -1)
    R.set_option(rj.OPT_LANE_RUNS, 0)
    for _ in range(3):                            # graph capture + replay
        cnt, _ = R.query(W=1024, H=1024, mode="accurate")
    chk(cnt, oracle.query(P, x, y, W=1024, H=1024, mode="accurate")[0], "graph")
    view = (100, 50, 700, 900)
    cnt, _ = R.query(W=1024, H=1024, mode="accurate", view=view)
    chk(cnt, oracle.query(P, x, y, W=1024, H=1024, mode="accurate", view=view)[0], "view")
    cnt, _, ep, em = R.query_interval(W=512, H=512)
    chk(cnt, oracle.query(P, x, y, W=512, H=512)[0], "interval")
    R.query_interval_ex(W=512, H=512)
    cnt, vals = R.query_multi([("min", 1), ("max", 0), ("avg", 1), ("count", 0)], W=1024, H=1024, mode="accurate")
    chk(cnt, oracle.query(P, x, y, W=1024, H=1024, mode="accurate")[0], "multi")
    R.query(W=1024, H=1024, mode="bounded", agg="min", agg_column=1)
    R.spans(W=300, H=300)
    R.boundary_mask(W=300, H=300)
    R.membership(W=300, H=300, mode="accurate")
    R.point_canvas(W=256, H=256)
    # streamed queries: host, ragged batches, device columns
    S = rj.RasterJoin(C.C1_BOX)
    S.load_polygons(flat)
    S.set_option(rj.OPT_STREAM_BATCH, 4097)
    for mode in ("bounded", "accurate", "index"):
        om = "bounded" if mode == "bounded" else "accurate"
        cnt, _ = S.query_stream(x, y, cols, W=777, H=777, mode=mode, agg="sum", agg_column=0)
        chk(cnt, oracle.query(P, x, y, W=777, H=777, mode=om)[0], ("stream", mode))
    device_paths(R, S, P, x, y, cols, chk)
    R.close()
    S.close()
    import gc
    import torch
    gc.collect()
    torch.cuda.synchronize()
    torch.cuda.empty_cache()                      # memcheck --leak-check: only librj's frees count
    print(f"sanitize driver: {ok} checked queries bit-exact")


if __name__ == "__main__":
    main()
