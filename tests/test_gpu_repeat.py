"""Repeated and interleaved queries on one context (GPU).

A repeated query key (canvas, level, mode, window, loaded data) reuses the
polygon pass's buffer sizes of the previous query and skips its two
device->host size reads; polygons whose footprint misses the query window
are culled from the polygon pass.  Neither may change a result: every query
of an interleaved sequence -- including after reloading points or polygons,
which must invalidate the sizes -- is compared with the oracle."""
import numpy as np
import pytest

import oracle
from datagen import configs as C
from datagen import polygons as PG

pytestmark = pytest.mark.gpu

rjmod = pytest.importorskip("paper_journals_pvldb_zacharatoudasf17_b200.rj")


@pytest.fixture(scope="module", autouse=True)
def _gpu():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("needs a CUDA device")


QUERIES = [
    dict(W=1024, H=1024, mode="bounded"),
    dict(W=1024, H=1024, mode="accurate"),
    dict(W=512, H=512, mode="bounded", view=(100, 50, 300, 400)),
    dict(W=512, H=512, mode="accurate", view=(0, 0, 256, 512)),
    dict(W=777, H=555, mode="bounded"),
]


def _oracle(P, x, y, cols, q):
    return oracle.query(P, x, y, cols=cols, agg_col=0, W=q["W"], H=q["H"], mode=q["mode"],
                        view=q.get("view"))


def test_interleaved_and_reloaded():
    polys = C.polygon_set("c1b")
    flat = PG.flatten(polys)
    pts = C.c1_points(200_000)
    ax, ay = PG.c1b_points(polys)
    x = np.concatenate([pts["x"], ax])
    y = np.concatenate([pts["y"], ay])
    fav = (np.arange(len(x)) % 5).astype(np.int32)
    R = rjmod.RasterJoin(C.C1_BOX)
    R.load_points(x, y, [fav])
    R.load_polygons(flat)
    P = oracle.Polys(flat, C.C1_BOX)
    want = [_oracle(P, x, y, [fav], q) for q in QUERIES]
    for rep in range(3):
        for q, (oc, os_, _) in zip(QUERIES, want):
            cnt, val = R.query(agg="sum", agg_column=0, **q)
            assert np.array_equal(cnt, oc), (rep, q)
            assert np.array_equal(val, os_), (rep, q)
    # new points: the cached sizes (pieces depend on the non-empty point cells) must not be reused
    k = len(x) // 3
    R.load_points(x[:k], y[:k], [fav[:k]])
    for q in QUERIES[:3] + QUERIES[:3]:
        oc, os_, _ = _oracle(P, x[:k], y[:k], [fav[:k]], q)
        cnt, val = R.query(agg="sum", agg_column=0, **q)
        assert np.array_equal(cnt, oc) and np.array_equal(val, os_), q
    # new polygons
    flat2 = C.array_polys("c1")
    R.load_polygons(flat2)
    P2 = oracle.Polys(flat2, C.C1_BOX)
    for q in QUERIES + QUERIES:
        oc, os_, _ = _oracle(P2, x[:k], y[:k], [fav[:k]], q)
        cnt, val = R.query(agg="sum", agg_column=0, **q)
        assert np.array_equal(cnt, oc) and np.array_equal(val, os_), q
    R.close()


def test_window_culls_polygons_exactly():
    """Windows that cut through, touch and miss polygons (C1: P0 occupies
    columns 100..199 at 1024^2): the culled polygon pass equals the oracle."""
    flat = C.array_polys("c1")
    pts = C.c1_points(100_000)
    R = rjmod.RasterJoin(C.C1_BOX)
    R.load_points(pts["x"], pts["y"])
    R.load_polygons(flat)
    P = oracle.Polys(flat, C.C1_BOX)
    for view in [(0, 0, 100, 1024), (0, 0, 101, 1024), (199, 0, 200, 1024), (200, 0, 201, 1024),
                 (600, 600, 1024, 1024), (500, 90, 520, 110), (0, 0, 1024, 100), (0, 0, 1024, 101)]:
        for mode in ("bounded", "accurate"):
            oc, _, _ = oracle.query(P, pts["x"], pts["y"], W=1024, H=1024, mode=mode, view=view)
            cnt, _ = R.query(W=1024, H=1024, mode=mode, view=view)
            assert np.array_equal(cnt, oc), (view, mode)
    R.close()


def test_graph_replay_matches_eager():
    """RJ_OPT_GRAPHS: the 2nd identical call is captured, later ones replay
    the graph.  Results, launch counts and the timing events must match the
    eager path; a changed filter constant or output buffer is a new key."""
    import torch
    flat = C.array_polys("neighborhoods")
    pts = C.taxi(400_000, fare=True)
    R = rjmod.RasterJoin(C.NYC_BOX)
    R.load_points(pts["x"], pts["y"], [pts["t"], pts["fare"]])
    R.load_polygons(flat)
    R.set_option(rjmod.OPT_TIMING, 1)
    n = R.n_poly
    outs = {}
    for graphs in (0, 1):
        R.set_option(rjmod.OPT_GRAPHS, graphs)
        for mode in ("bounded", "accurate"):
            for t_lo in (C.T_2012[0], C.T_2012[0] + 86400 * 30):
                q = rjmod.make_desc(agg="avg", agg_column=1, preds=[(0, ">=", t_lo)], W=2048, H=2048, mode=mode)
                d_cnt = torch.zeros(n, dtype=torch.int64, device="cuda")
                d_sum = torch.zeros(n, dtype=torch.float64, device="cuda")
                res = []
                for rep in range(4):
                    d_cnt.fill_(-1)
                    d_sum.fill_(-1.0)
                    torch.cuda.synchronize()            # the context has its own stream
                    rjmod.rj_query_device(R.ctx, q, d_cnt, d_sum)
                    torch.cuda.synchronize()
                    st = R.stats()
                    assert st["ms_point_pass"] > 0 and st["ms_polygon"] > 0
                    res.append((d_cnt.cpu().numpy().copy(), d_sum.cpu().numpy().copy(), st["launches"]))
                for r in res[1:]:                       # fp64 sums: atomic order may differ
                    assert np.array_equal(r[0], res[0][0]) and np.allclose(r[1], res[0][1], rtol=1e-12, atol=0)
                    assert r[2] == res[0][2]
                cnt, val = R.query(agg="avg", agg_column=1, preds=[(0, ">=", t_lo)], W=2048, H=2048, mode=mode)
                cnt2, val2 = R.query(agg="avg", agg_column=1, preds=[(0, ">=", t_lo)], W=2048, H=2048, mode=mode)
                cnt3, val3 = R.query(agg="avg", agg_column=1, preds=[(0, ">=", t_lo)], W=2048, H=2048, mode=mode)
                assert np.array_equal(cnt, cnt3) and np.allclose(val, val3, rtol=1e-12, atol=0, equal_nan=True)
                assert np.array_equal(cnt.astype(np.int64), res[0][0])
                outs[(graphs, mode, t_lo)] = (res[0][0], res[0][1])
    for k, v in outs.items():
        if k[0] == 1:
            e = outs[(0,) + k[1:]]
            assert np.array_equal(v[0], e[0]) and np.allclose(v[1], e[1], rtol=1e-12, atol=0), k
    R.close()


@pytest.mark.parametrize("agg", ["count", "sum"])
def test_caller_graph_capture(agg):
    """A caller may capture a whole query step (rj_query_device +
    rj_finalize_device + the D2H copies) into its own CUDA graph on the
    context's stream: the library then runs inside that capture (no
    internal graph), and every replay recomputes the result -- checked by
    poisoning the outputs before each replay."""
    import torch
    flat = PG.flatten(C.polygon_set("c1b"))
    pts = C.c1_points(300_000)
    fav = (np.arange(len(pts["x"])) % 9).astype(np.int32)
    stream = torch.cuda.Stream()
    R = rjmod.RasterJoin(C.C1_BOX, stream=stream.cuda_stream)
    R.set_option(rjmod.OPT_TIMING, 1)
    R.load_points(pts["x"], pts["y"], [fav])
    R.load_polygons(flat)
    P = oracle.Polys(flat, C.C1_BOX)
    desc = rjmod.make_desc(agg=agg, agg_column=0 if agg == "sum" else -1, W=777, H=555, mode="accurate")
    n = R.n_poly
    d_cnt = torch.zeros(n, dtype=torch.int64, device="cuda")
    d_sum = torch.zeros(n, dtype=torch.float64, device="cuda")
    d_val = torch.zeros(n, dtype=torch.float64, device="cuda")
    h_cnt = torch.zeros(n, dtype=torch.int64, pin_memory=True)

    def body():
        rjmod.rj_query_device(R.ctx, desc, d_cnt, d_sum)
        rjmod.rj_finalize_device(R.ctx, desc.agg, d_cnt, d_sum, d_val)
        h_cnt.copy_(d_cnt, non_blocking=True)

    for _ in range(3):                                   # internal graph captured and replayed
        with torch.cuda.stream(stream):
            body()
        stream.synchronize()
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g, stream=stream, capture_error_mode="relaxed"):
        body()
    ocnt, osum, _ = oracle.query(P, pts["x"], pts["y"], cols=[fav], agg_col=0, W=777, H=555, mode="accurate")
    for _ in range(2):
        h_cnt.fill_(-1)
        d_cnt.fill_(-1)
        d_val.fill_(-1.0)
        torch.cuda.synchronize()
        with torch.cuda.stream(stream):
            g.replay()
        stream.synchronize()
        assert np.array_equal(h_cnt.numpy().astype(np.uint64), ocnt)
        if agg == "sum":
            assert np.array_equal(d_val.cpu().numpy(), osum)
    assert R.stats()["ms_point_pass"] > 0
    R.close()
