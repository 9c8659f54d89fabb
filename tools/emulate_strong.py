"""Strong-scaling projection on ONE GPU: run every rank's
share of a P-way sharded query one after the other on cuda:0 and take the
slowest rank, for index-range shards (spatially random points, whole-canvas
polygon pass per rank) and for x-strip shards (dist.strip_splitters'
quantile rule + per-rank pixel window).  projected efficiency =
T(1 GPU) / (P x max_r T_r); a second figure adds the one all-reduce of the
packed partials as measured on one GPU (world size 1, a lower bound of the
NVSwitch latency; allreduce_standin_ms).  Not a bench line: evidence for the
shard design until a multi-GPU box is available.

    python tools/emulate_strong.py [--config C3] [--points 1e9] [--ranks 2,4,8]
"""
from __future__ import annotations

import argparse
import json
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import bench  # noqa: E402
from datagen import configs as C  # noqa: E402
from paper_journals_pvldb_zacharatoudasf17_b200 import dist as rjdist  # noqa: E402
from paper_journals_pvldb_zacharatoudasf17_b200 import rj  # noqa: E402


def time_query(R, desc, stream, steps, graph_step=False):
    """ms per step of the bench's step (query + finalise + D2H of the
    results + stream sync); graph_step: the step captured once as one CUDA
    graph (every kernel and copy still runs every step)."""
    n = R.n_poly
    d_cnt = torch.zeros(n, dtype=torch.int64, device="cuda")
    d_sum = torch.zeros(n, dtype=torch.float64, device="cuda")
    d_val = torch.zeros(n, dtype=torch.float64, device="cuda")
    h_cnt = torch.zeros(n, dtype=torch.int64, pin_memory=True)
    h_val = torch.zeros(n, dtype=torch.float64, pin_memory=True)

    def body():
        rj.rj_query_device(R.ctx, desc, d_cnt, d_sum)
        rj.rj_finalize_device(R.ctx, desc.agg, d_cnt, d_sum, d_val)
        h_cnt.copy_(d_cnt, non_blocking=True)
        h_val.copy_(d_val, non_blocking=True)

    def step():
        with torch.cuda.stream(stream):
            body()
        stream.synchronize()

    for _ in range(3):
        step()
    if graph_step:
        g = torch.cuda.CUDAGraph()
        with torch.cuda.graph(g, stream=stream, capture_error_mode="relaxed"):
            body()

        def step():                                  # noqa: F811
            with torch.cuda.stream(stream):          # replay on the timed stream
                g.replay()
            stream.synchronize()
        step()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    torch.cuda.synchronize()
    e0.record(stream)
    for _ in range(steps):
        step()
    e1.record(stream)
    torch.cuda.synchronize()
    st = R.stats()
    return e0.elapsed_time(e1) / steps, h_cnt.numpy().copy(), st


def allreduce_standin_ms(n_poly, stream, iters=200):
    """The one collective of a sharded query, measured the only way one GPU
    allows: a world-size-1 NCCL all-reduce of the packed partials (2 n_poly
    binary64, rj_pack_partials' layout) on the query stream.  A lower bound
    of the 8-rank latency over NVSwitch (NCCL still launches its kernel)."""
    import torch.distributed as dist
    os.environ.setdefault("MASTER_ADDR", "127.0.0.1")
    os.environ.setdefault("MASTER_PORT", str(29500 + os.getpid() % 1000))
    if not dist.is_initialized():
        dist.init_process_group("nccl", rank=0, world_size=1, device_id=torch.device("cuda", 0))
    buf = torch.zeros(2 * n_poly, dtype=torch.float64, device="cuda")
    with torch.cuda.stream(stream):
        for _ in range(10):
            dist.all_reduce(buf)
    stream.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    with torch.cuda.stream(stream):
        e0.record(stream)
        for _ in range(iters):
            dist.all_reduce(buf)
        e1.record(stream)
    stream.synchronize()
    return e0.elapsed_time(e1) / iters


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--config", default="C3")
    ap.add_argument("--points", type=float, default=1e9)
    ap.add_argument("--ranks", default="2,4,8")
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--only-rank", type=int, default=-1, help="profile: run only this rank's spatial shard")
    ap.add_argument("--poly-weight", type=float, default=0.0, help="strip cost weight of the domain width")
    ap.add_argument("--spatial-only", action="store_true")
    ap.add_argument("--graph-step", action="store_true", help="capture each rank's whole step as one CUDA graph")
    ap.add_argument("--skip-t1", action="store_true", help="profiling: skip the one-GPU query (T1 = NaN)")
    args = ap.parse_args()
    n = int(args.points)
    box, polys_name, recipe, q, desc_s = bench.workload(args.config)
    x, y, cols = bench.gen_points(recipe, n, 0)
    stream = torch.cuda.Stream()
    R = rj.RasterJoin(box, device=0, stream=stream.cuda_stream)
    R.set_option(rj.OPT_TIMING, 1)
    R.load_polygons(C.array_polys(polys_name))
    R.load_points(x, y, cols)
    desc = rj.make_desc(**q)
    W, H = rj.rj_resolve_canvas(R.ctx, desc)
    if args.skip_t1:
        t1, c1, st1 = float("nan"), np.zeros(R.n_poly, np.int64), {"ms_polygon": float("nan")}
    else:
        t1, c1, st1 = time_query(R, desc, stream, args.steps, args.graph_step)
    ar_ms = allreduce_standin_ms(R.n_poly, stream)
    out = {"config": desc_s, "points": n, "canvas": [W, H], "t1_ms": t1,
           "t1_polygon_ms": st1["ms_polygon"], "allreduce_1gpu_ms": ar_ms, "ranks": {}}
    sample = torch.from_numpy(x[np.linspace(0, n - 1, 1 << 20).astype(np.int64)].astype(np.float64))
    for P in [int(v) for v in args.ranks.split(",")]:
        sp = rjdist.splitters_from_sample(sample, P, box, args.poly_weight)
        dest = np.empty(n, dtype=np.uint8)
        for a in range(0, n, 1 << 26):              # chunked: int64 ranks for 1e9 points would be 8 GB
            dest[a:a + (1 << 26)] = rjdist.strip_of(torch.from_numpy(x[a:a + (1 << 26)]), sp).numpy()
        res = {}
        for kind in (("spatial",) if args.only_rank >= 0 or args.spatial_only else ("range", "spatial")):
            per, tot = [], np.zeros_like(c1)
            for r in (range(P) if args.only_rank < 0 else [args.only_rank]):
                if kind == "range":
                    lo, hi = rjdist.shard_range(n, r, P)
                    sel = slice(lo, hi)
                    d = desc
                else:
                    sel = dest == r
                    d = rj.make_desc(**q, view=rjdist.strip_window(box, sp, r, P, desc))
                R.load_points(np.ascontiguousarray(x[sel]), np.ascontiguousarray(y[sel]),
                              [np.ascontiguousarray(c[sel]) for c in cols])
                ms, cnt, st = time_query(R, d, stream, args.steps, args.graph_step)
                tot += cnt
                per.append({"ms": ms, "points": int(R.n_input), "polygon_ms": st["ms_polygon"],
                            "point_pass_ms": st["ms_point_pass"]})
            worst = max(p["ms"] for p in per)
            res[kind] = {"max_rank_ms": worst, "projected_efficiency": t1 / (P * worst),
                         "projected_efficiency_with_allreduce": t1 / (P * (worst + ar_ms)),
                         "sum_equals_1gpu": bool(np.array_equal(tot, c1)) if args.only_rank < 0 else None,
                         "per_rank": per}
        out["ranks"][P] = res
        print(json.dumps({"P": P, **{k: {kk: vv for kk, vv in v.items() if kk != "per_rank"}
                                       for k, v in res.items()}}), flush=True)
    R.close()
    print(json.dumps(out), flush=True)


if __name__ == "__main__":
    main()
