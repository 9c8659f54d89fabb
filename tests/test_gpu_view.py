"""GPU parity of viewport windows and canvases beyond 32768^2 (SURVEY.md 8(f)
NEXT-2: multi-canvas rendering P:625-633, LOD zoom P:640-650; readings Z20,
Z21) against oracle O12.

Bar: COUNT and membership bit-exact, integer SUM exact, float SUM/AVG and
MIN/MAX as the other parity tests; windows tiling the canvas add up to the
whole canvas exactly."""
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


def rel_close(g, o, tol=1e-9):
    g = np.asarray(g, np.float64)
    o = np.asarray(o, np.float64)
    ok = (np.isnan(g) & np.isnan(o)) | (np.abs(g - o) <= tol * np.abs(o)) | ((o == 0) & (g == 0))
    return bool(np.all(ok)), np.nonzero(~ok)[0]


@pytest.fixture(scope="module")
def c1():
    polys = C.polygon_set("c1b")
    flat = PG.flatten(polys)
    pts = C.c1_points(150_000)
    ax, ay = PG.c1b_points(polys)
    x = np.concatenate([pts["x"], ax])
    y = np.concatenate([pts["y"], ay])
    rng = np.random.default_rng(71)
    ti = rng.integers(-50, 50, len(x)).astype(np.int32)
    tf = rng.normal(5, 3, len(x)).astype(np.float32)
    R = rjmod.RasterJoin(C.C1_BOX)
    R.load_points(x, y, [ti, tf])
    R.load_polygons(flat)
    return R, oracle.Polys(flat, C.C1_BOX), x, y, [ti, tf]


VIEWS = [(0, 0, 1024, 1024), (123, 201, 650, 977), (0, 0, 1, 1), (1023, 0, 1024, 1024), (500, 500, 501, 900),
         (96, 96, 313, 129)]


@pytest.mark.parametrize("mode", ["bounded", "accurate", "index"])
@pytest.mark.parametrize("view", VIEWS)
def test_view_count_bitexact(c1, mode, view):
    R, P, x, y, cols = c1
    cnt, _ = R.query(W=1024, H=1024, mode=mode, view=view)
    ocnt, _, kept = oracle.query(P, x, y, W=1024, H=1024, mode="bounded" if mode == "bounded" else "accurate",
                                 view=view)
    assert np.array_equal(cnt, ocnt), (mode, view)


@pytest.mark.parametrize("mode", ["bounded", "accurate"])
@pytest.mark.parametrize("variant", [0, 1])
def test_view_sum_both_kernels(c1, mode, variant):
    R, P, x, y, cols = c1
    R.set_option(rjmod.OPT_PASS, variant)
    try:
        for view in [(123, 201, 650, 977), (0, 0, 1, 1), (699, 0, 700, 1100), (500, 500, 501, 900), (96, 96, 313, 129)]:
            cnt, val = R.query(W=700, H=1100, mode=mode, agg="sum", agg_column=0, view=view,
                               preds=[(1, ">", 2.0)])
            ocnt, osum, _ = oracle.query(P, x, y, cols=cols, agg_col=0, preds=[(1, ">", 2.0)], W=700, H=1100,
                                         mode=mode, view=view)
            assert np.array_equal(cnt, ocnt), view
            assert np.array_equal(val, osum), view          # integer attribute: exact
    finally:
        R.set_option(rjmod.OPT_PASS, -1)


@pytest.mark.parametrize("mode", ["bounded", "accurate"])
def test_view_tiles_add_up(c1, mode):
    # multi-canvas: every point-polygon pair counted exactly once
    R, P, x, y, cols = c1
    full_c, full_s = R.query(W=1024, H=1024, mode=mode, agg="sum", agg_column=0)
    cs, rs = (0, 100, 101, 640, 1024), (0, 333, 1000, 1024)
    tc = np.zeros_like(full_c)
    ts = np.zeros_like(full_s)
    for i in range(len(cs) - 1):
        for j in range(len(rs) - 1):
            c, s = R.query(W=1024, H=1024, mode=mode, agg="sum", agg_column=0,
                           view=(cs[i], rs[j], cs[i + 1], rs[j + 1]))
            tc += c
            ts += s
    assert np.array_equal(tc, full_c) and np.array_equal(ts, full_s)


def test_view_membership_and_spans(c1):
    R, P, x, y, cols = c1
    view = (123, 201, 650, 977)
    for mode in ("bounded", "accurate"):
        g = R.membership(W=1024, H=1024, mode=mode, view=view)
        o = oracle.membership(P, x, y, W=1024, H=1024, mode=mode, view=view)
        assert np.array_equal(g, o), mode
    sp = R.spans(W=1024, H=1024, view=view)
    assert len(sp) and sp[:, 1].min() >= 201 and sp[:, 1].max() < 977
    assert sp[:, 2].min() >= 123 and sp[:, 3].max() <= 650
    full = R.spans(W=1024, H=1024)
    # clipping the whole canvas's spans gives the window's pixel set
    k = (full[:, 1] >= 201) & (full[:, 1] < 977)
    lo = np.maximum(full[k, 2], 123)
    hi = np.minimum(full[k, 3], 650)
    keep = lo < hi
    want = sorted(zip(full[k, 0][keep], full[k, 1][keep], lo[keep], hi[keep]))
    assert sorted(map(tuple, sp.tolist())) == [tuple(map(int, t)) for t in want]


def test_view_label_canvas_paths(c1):
    # streamed query, MIN/MAX and multi-aggregate run on a window-sized label canvas
    R, P, x, y, cols = c1
    view = (123, 201, 650, 977)
    for mode in ("bounded", "accurate", "index"):
        om = "bounded" if mode == "bounded" else "accurate"
        ocnt, osum, _ = oracle.query(P, x, y, cols=cols, agg_col=0, W=1024, H=1024, mode=om, view=view)
        cnt, val = R.query_stream(x, y, cols, W=1024, H=1024, mode=mode, agg="sum", agg_column=0, view=view)
        assert np.array_equal(cnt, ocnt) and np.array_equal(val, osum), mode
        mn, mx = oracle.query_minmax(P, x, y, cols, 1, W=1024, H=1024, mode=om, view=view)
        cnt, vals = R.query_multi([("min", 1), ("max", 1), ("avg", 1)], W=1024, H=1024, mode=mode, view=view)
        assert np.array_equal(cnt, ocnt), mode
        assert np.array_equal(vals[0][cnt > 0], mn[cnt > 0]) and np.array_equal(vals[1][cnt > 0], mx[cnt > 0])
        _, ofs, _ = oracle.query(P, x, y, cols=cols, agg_col=1, W=1024, H=1024, mode=om, view=view)
        ok, bad = rel_close(vals[2], oracle.avg(ocnt, ofs))
        assert ok, (mode, bad)


def test_view_lod_closed_form(c1):
    # LOD zoom: W = 8192 on [0,1024)^2, window columns [0, 1200)
    # end at x = 150: the pixel-aligned square P0 = [100,200)^2 counts the
    # points of [100,150) x [100,200), in both modes
    R, P, x, y, cols = c1
    want = int(np.sum((x >= 100) & (x < 150) & (y >= 100) & (y < 200)))
    for mode in ("bounded", "accurate"):
        cnt, _ = R.query(W=8192, H=8192, mode=mode, view=(0, 0, 1200, 8192))
        assert cnt[0] == want and cnt[9] == 0, mode
    Wf, Hf, v = rjmod.lod_view(C.C1_BOX, (100, 100, 150, 200), 1000)
    cnt, _ = R.query(W=Wf, H=Hf, mode="accurate", view=v)
    assert cnt[0] == want


@pytest.mark.parametrize("W", [40000, 81912, 131072])
@pytest.mark.parametrize("mode", ["bounded", "accurate"])
def test_high_resolution_parity(c1, W, mode):
    # reading Z21: one canvas up to 2^17 a side (eps = 1 m on NYC is 81912)
    R, P, x, y, cols = c1
    cnt, val = R.query(W=W, H=W, mode=mode, agg="sum", agg_column=0)
    ocnt, osum, _ = oracle.query(P, x, y, cols=cols, agg_col=0, W=W, H=W, mode=mode)
    assert np.array_equal(cnt, ocnt)
    assert np.array_equal(val, osum)
    cnt, _ = R.query(W=W, H=W, mode=mode)
    assert np.array_equal(cnt, ocnt)
    # a zoomed window of the fine canvas
    view = (W // 10, W // 10, W // 10 + 5000, W // 10 + 7000)
    cnt, _ = R.query(W=W, H=W, mode=mode, view=view)
    ocnt, _, _ = oracle.query(P, x, y, W=W, H=W, mode=mode, view=view)
    assert np.array_equal(cnt, ocnt)


@pytest.mark.parametrize("W,H,view", [(64, 70000, None), (131072, 131072, (60000, 0, 60512, 131072))])
def test_label_canvas_taller_than_grid_y(c1, W, H, view):
    """Label-canvas paths (MIN/MAX, multi-aggregate, streamed) on windows
    more than 65535 rows high: the label canvas init strides rows over
    gridDim.y (a launch with gridDim.y = height failed)."""
    R, P, x, y, cols = c1
    for mode in ("bounded", "accurate"):
        ocnt, osum, _ = oracle.query(P, x, y, cols=cols, agg_col=0, W=W, H=H, mode=mode, view=view)
        mn, mx = oracle.query_minmax(P, x, y, cols, 1, W=W, H=H, mode=mode, view=view)
        cnt, v = R.query(W=W, H=H, mode=mode, agg="min", agg_column=1, view=view)
        assert np.array_equal(cnt, ocnt), mode
        assert np.array_equal(v[cnt > 0], mn[cnt > 0])
        cnt, vals = R.query_multi([("max", 1), ("sum", 0)], W=W, H=H, mode=mode, view=view)
        assert np.array_equal(cnt, ocnt) and np.array_equal(vals[0][cnt > 0], mx[cnt > 0])
        assert np.array_equal(vals[1], osum)
        cnt, val = R.query_stream(x, y, cols, W=W, H=H, mode=mode, agg="sum", agg_column=0, view=view)
        assert np.array_equal(cnt, ocnt) and np.array_equal(val, osum), mode
        assert ocnt.sum() > 0


def test_view_errors(c1):
    R, P, x, y, cols = c1
    for view in ((0, 0, 1025, 10), (5, 0, 5, 10), (-1, 0, 3, 3), (0, 7, 3, 3)):
        with pytest.raises(rjmod.RJError) as e:
            R.query(W=1024, H=1024, view=view)
        assert e.value.status == -1, view
    with pytest.raises(rjmod.RJError) as e:
        R.query_interval(W=1024, H=1024, view=(0, 0, 10, 10))
    assert e.value.status == -1


def test_view_taxi_prefix_window():
    """C2-shaped prefix: a Manhattan-sized window of an eps = 1 m canvas."""
    flat = C.array_polys("neighborhoods")
    pts = C.taxi(1_000_000)
    R = rjmod.RasterJoin(C.NYC_BOX)
    R.load_points(pts["x"], pts["y"], [pts["t"]])
    R.load_polygons(flat)
    P = oracle.Polys(flat, C.NYC_BOX)
    W = 81912
    view = (30000, 30000, 46000, 50000)
    preds = [(0, ">=", C.T_2012[0]), (0, "<", C.T_2012[1])]
    for mode in ("bounded", "accurate"):
        cnt, _ = R.query(W=W, H=W, mode=mode, preds=preds, view=view)
        ocnt, _, kept = oracle.query(P, pts["x"], pts["y"], cols=[pts["t"]], preds=preds, W=W, H=W, mode=mode,
                                     view=view)
        assert np.array_equal(cnt, ocnt), mode
        assert int(cnt.sum()) == kept          # exact tiling inside the window
