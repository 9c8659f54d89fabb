"""Check that a caller-side CUDA-graph capture of the bench step (query +
finalise + D2H) replays the whole query: results after a replay must equal
the eager results, for COUNT and SUM, with and without timing events."""
import sys

import numpy as np
import torch

sys.path.insert(0, ".")
import bench  # noqa: E402
from datagen import configs as C  # noqa: E402
from paper_journals_pvldb_zacharatoudasf17_b200 import rj  # noqa: E402

box, polys_name, recipe, q, desc_s = bench.workload("C4")
x, y, cols = bench.gen_points(recipe, 5_000_000, 0)
for agg in ("count", "sum"):
    for timing in (0, 1):
        stream = torch.cuda.Stream()
        R = rj.RasterJoin(box, device=0, stream=stream.cuda_stream)
        R.set_option(rj.OPT_TIMING, timing)
        R.load_polygons(C.array_polys(polys_name))
        R.load_points(x, y, cols)
        desc = rj.make_desc(**dict(q, agg=agg))
        n = R.n_poly
        d_cnt = torch.zeros(n, dtype=torch.int64, device="cuda")
        d_sum = torch.zeros(n, dtype=torch.float64, device="cuda")
        d_val = torch.zeros(n, dtype=torch.float64, device="cuda")
        h_cnt = torch.zeros(n, dtype=torch.int64, pin_memory=True)

        def body():
            rj.rj_query_device(R.ctx, desc, d_cnt, d_sum)
            rj.rj_finalize_device(R.ctx, desc.agg, d_cnt, d_sum, d_val)
            h_cnt.copy_(d_cnt, non_blocking=True)

        for _ in range(3):
            with torch.cuda.stream(stream):
                body()
            stream.synchronize()
        ref = h_cnt.clone()
        g = torch.cuda.CUDAGraph()
        with torch.cuda.graph(g, stream=stream, capture_error_mode="relaxed"):
            body()
        h_cnt.fill_(-1)
        d_cnt.fill_(-1)
        torch.cuda.synchronize()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(stream)
        with torch.cuda.stream(stream):
            g.replay()
        e1.record(stream)
        torch.cuda.synchronize()
        print(agg, "timing", timing, "replay ms", round(e0.elapsed_time(e1), 4), "equal", torch.equal(h_cnt, ref),
              flush=True)
        R.close()
