import numpy as np, torch, sys
sys.path.insert(0, ".")
from datagen import configs as C
from datagen import polygons as PG
from paper_journals_pvldb_zacharatoudasf17_b200 import rj
polys = C.polygon_set("c1"); flat = PG.flatten(polys)
pts = C.c1_points(100000)
stream = torch.cuda.Stream()
R = rj.RasterJoin(C.C1_BOX, stream=stream.cuda_stream)
R.load_points(pts["x"], pts["y"]); R.load_polygons(flat)
desc = rj.make_desc(W=1024, H=1024)
n = R.n_poly
d_cnt = torch.zeros(n, dtype=torch.int64, device="cuda"); d_sum = torch.zeros(n, dtype=torch.float64, device="cuda")
for _ in range(3):
    with torch.cuda.stream(stream):
        rj.rj_query_device(R.ctx, desc, d_cnt, d_sum)
    stream.synchronize()
ref = d_cnt.cpu().clone()
g = torch.cuda.CUDAGraph()
with torch.cuda.graph(g, stream=stream, capture_error_mode="relaxed"):
    print("capturing:", torch.cuda.is_current_stream_capturing(), "cur", torch.cuda.current_stream().cuda_stream, "ctx", rj.rj_get_stream(R.ctx))
    rj.rj_query_device(R.ctx, desc, d_cnt, d_sum)
print("launches in capture", R.stats()["launches"])
d_cnt.fill_(-1); torch.cuda.synchronize()
g.replay(); torch.cuda.synchronize()
print("after replay equal:", torch.equal(d_cnt.cpu(), ref), d_cnt[:5].tolist(), ref[:5].tolist())

# the bench / emulate_strong step: timing events on, finalise, D2H copies
R.set_option(rj.OPT_TIMING, 1)
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
g2 = torch.cuda.CUDAGraph()
with torch.cuda.graph(g2, stream=stream, capture_error_mode="relaxed"):
    body()
print("launches in capture 2", R.stats()["launches"])
h_cnt.fill_(-1); d_cnt.fill_(-1); torch.cuda.synchronize()
e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
e0.record(stream); g2.replay(); e1.record(stream); torch.cuda.synchronize()
print("replay 2 ms", e0.elapsed_time(e1), "equal:", torch.equal(h_cnt, ref), R.stats()["ms_point_pass"])
