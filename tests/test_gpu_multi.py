"""GPU parity of MIN/MAX and multi-aggregate queries (
PAPER.md P:754-766 distributive aggregates, P:1278-1283 several aggregates
per pass) against oracle O11 (or_query_minmax, IEEE totalOrder, reading
Z16) and O5-O8.

Bar: MIN/MAX are values of the input column -> identical (NaN iff the
oracle's NaN, same sign bit, -0 vs +0 distinguished); COUNT bit-exact;
integer SUM exact; float SUM/AVG within 1e-9 relative."""
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


def same_values(g, o):
    g = np.asarray(g, np.float64)
    o = np.asarray(o, np.float64)
    ok = (np.isnan(g) & np.isnan(o) & (np.signbit(g) == np.signbit(o))) | \
         ((g == o) & (np.signbit(g) == np.signbit(o)))
    return bool(np.all(ok)), np.nonzero(~ok)[0]


def rel_close(g, o, tol=1e-9):
    g = np.asarray(g, np.float64)
    o = np.asarray(o, np.float64)
    ok = (np.isnan(g) & np.isnan(o)) | (np.abs(g - o) <= tol * np.abs(o)) | ((o == 0) & (g == 0))
    return bool(np.all(ok)), np.nonzero(~ok)[0]


@pytest.fixture(scope="module")
def c1():
    polys = C.polygon_set("c1b")
    flat = PG.flatten(polys)
    pts = C.c1_points(200_000)
    ax, ay = PG.c1b_points(polys)
    x = np.concatenate([pts["x"], ax])
    y = np.concatenate([pts["y"], ay])
    rng = np.random.default_rng(51)
    ti = rng.integers(-2**31, 2**31 - 1, len(x), dtype=np.int64).astype(np.int32)
    ti[:2] = [-2**31, 2**31 - 1]
    tf = rng.normal(0, 100, len(x)).astype(np.float32)
    tf[::101] = np.nan
    tf[::103] = -0.0
    tf[::107] = 0.0
    tf[::211] = -np.inf
    neg_nan = np.frombuffer(np.uint32(0xFFC00000).tobytes(), np.float32)[0]
    tf[5::997] = neg_nan
    tc = rng.integers(-50, 50, len(x)).astype(np.int32)
    cols = [ti, tf, tc]
    R = rjmod.RasterJoin(C.C1_BOX)
    R.load_points(x, y, cols)
    R.load_polygons(flat)
    return R, oracle.Polys(flat, C.C1_BOX), x, y, cols


@pytest.mark.parametrize("mode", ["bounded", "accurate", "index"])
@pytest.mark.parametrize("col", [0, 1])
def test_min_max_single(c1, mode, col):
    R, P, x, y, cols = c1
    om = "bounded" if mode == "bounded" else "accurate"
    preds = [(2, ">=", -30)]
    mn, mx = oracle.query_minmax(P, x, y, cols, col, preds=preds, W=1024, H=1024, mode=om)
    ocnt, _, _ = oracle.query(P, x, y, cols=cols, preds=preds, W=1024, H=1024, mode=om)
    for agg, exp in (("min", mn), ("max", mx)):
        cnt, val = R.query(W=1024, H=1024, mode=mode, agg=agg, agg_column=col, preds=preds)
        assert np.array_equal(cnt, ocnt), agg
        ok, bad = same_values(val, exp)
        assert ok, (agg, bad, val[bad[:5]], exp[bad[:5]])


@pytest.mark.parametrize("mode", ["bounded", "accurate"])
def test_multi_aggregates(c1, mode):
    R, P, x, y, cols = c1
    preds = [(2, "<", 40)]
    aggs = [("count", 0), ("sum", 2), ("avg", 1), ("min", 1), ("max", 0), ("min", 0)]
    for chunk in (aggs[:4], aggs[2:]):
        cnt, vals = R.query_multi(chunk, W=777, H=555, mode=mode, preds=preds)
        ocnt, _, _ = oracle.query(P, x, y, cols=cols, preds=preds, W=777, H=555, mode=mode)
        assert np.array_equal(cnt, ocnt)
        for k, (agg, col) in enumerate(chunk):
            if agg == "count":
                assert np.array_equal(vals[k], ocnt.astype(np.float64))
            elif agg in ("sum", "avg"):
                c_, s_, _ = oracle.query(P, x, y, cols=cols, preds=preds, agg_col=col, W=777, H=555, mode=mode)
                exp = s_ if agg == "sum" else oracle.avg(c_, s_)
                if agg == "sum" and col == 2:
                    assert np.array_equal(vals[k], exp)
                ok, bad = rel_close(vals[k], exp)
                assert ok, (agg, col, bad)
            else:
                mn, mx = oracle.query_minmax(P, x, y, cols, col, preds=preds, W=777, H=555, mode=mode)
                ok, bad = same_values(vals[k], mn if agg == "min" else mx)
                assert ok, (agg, col, bad)


def test_stream_min_max(c1):
    R, P, x, y, cols = c1
    R.set_option(rjmod.OPT_STREAM_BATCH, 50_000)
    mn, mx = oracle.query_minmax(P, x, y, cols, 1, W=512, H=512, mode="accurate")
    for agg, exp in (("min", mn), ("max", mx)):
        _, val = R.query_stream(x, y, cols, W=512, H=512, mode="accurate", agg=agg, agg_column=1)
        ok, bad = same_values(val, exp)
        assert ok, (agg, bad)


def test_tracts_fare_multi():
    """C3 shape on a 1M-point prefix: AVG/MIN/MAX(fare) + COUNT in one pass."""
    flat = C.array_polys("tracts")
    pts = C.taxi(1_000_000, fare=True)
    cols = [pts["t"], pts["fare"]]
    R = rjmod.RasterJoin(C.NYC_BOX)
    R.load_points(pts["x"], pts["y"], cols)
    R.load_polygons(flat)
    P = oracle.Polys(flat, C.NYC_BOX)
    cnt, vals = R.query_multi([("avg", 1), ("min", 1), ("max", 1), ("count", 0)], W=8192, H=8192, mode="accurate")
    oc, osum, _ = oracle.query(P, pts["x"], pts["y"], cols=cols, agg_col=1, W=8192, H=8192, mode="accurate")
    mn, mx = oracle.query_minmax(P, pts["x"], pts["y"], cols, 1, W=8192, H=8192, mode="accurate")
    assert np.array_equal(cnt, oc)
    ok, bad = rel_close(vals[0], oracle.avg(oc, osum))
    assert ok, bad
    assert same_values(vals[1], mn)[0] and same_values(vals[2], mx)[0]
    assert np.array_equal(vals[3], oc.astype(np.float64))


def test_multi_errors(c1):
    R = c1[0]
    with pytest.raises(rjmod.RJError):
        R.query_multi([], W=64)
    with pytest.raises(rjmod.RJError):
        R.query_multi([("min", 0)] * 5, W=64)
    with pytest.raises(rjmod.RJError):
        R.query_multi([("max", 9)], W=64)
    import torch
    d = torch.zeros(R.n_poly, dtype=torch.int64, device="cuda")
    with pytest.raises(rjmod.RJError):
        rjmod.rj_query_device(R.ctx, rjmod.make_desc(agg="min", agg_column=0, W=64), d, d)
