"""GPU parity of the streamed one-shot query (rj_query_stream, SURVEY.md 8(f)
NEXT-2: points not loaded, read once in batches with copy/compute overlap;
PAPER.md P:786-790).  Same bar as the loaded path: COUNT bit-exact,
integer SUM exact, float SUM/AVG within 1e-9 relative, against the oracle on
the same seeded points -- over batch boundaries (ragged last batch), host
pageable / pinned / device inputs, overlapping polygons (MULTI pixels), both
coordinate dtypes and every mode."""
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
    polys = C.polygon_set("c1b")                       # overlapping polygons, holes
    flat = PG.flatten(polys)
    pts = C.c1_points(200_000)
    ax, ay = PG.c1b_points(polys)                      # points on vertices / edges / centres
    x = np.concatenate([pts["x"], ax, [np.nan, -5.0, 1024.0, 3.0]])
    y = np.concatenate([pts["y"], ay, [1.0, 2.0, 3.0, 1e9]])
    rng = np.random.default_rng(21)
    ti = rng.integers(-50, 50, len(x)).astype(np.int32)
    tf = rng.normal(5, 3, len(x)).astype(np.float32)
    R = rjmod.RasterJoin(C.C1_BOX)
    R.load_polygons(flat)
    return R, oracle.Polys(flat, C.C1_BOX), x, y, [ti, tf]


CASES = [
    dict(agg="count", preds=[]),
    dict(agg="sum", agg_column=0, preds=[(1, "<", 6.0)]),
    dict(agg="avg", agg_column=1, preds=[(0, ">=", -20), (0, "<", 30)]),
]


def check(cnt, val, ocnt, osum, cs):
    assert np.array_equal(cnt, ocnt), cs
    if cs["agg"] == "sum":
        assert np.array_equal(val, osum), cs                  # integer attribute: exact
    elif cs["agg"] == "avg":
        ok, bad = rel_close(val, oracle.avg(ocnt, osum))
        assert ok, (cs, bad)


@pytest.mark.parametrize("mode", ["bounded", "accurate", "index", "exact"])
@pytest.mark.parametrize("batch", [1 << 24, 4097])
def test_stream_c1_modes(c1, mode, batch):
    R, P, x, y, cols = c1
    R.set_option(rjmod.OPT_STREAM_BATCH, batch)
    for W in (1024, 777):
        for cs in CASES:
            cnt, val = R.query_stream(x, y, cols, W=W, H=W, mode=mode, **cs)
            om = "bounded" if mode == "bounded" else "accurate"
            ocnt, osum, kept = oracle.query(P, x, y, cols=cols, preds=cs["preds"],
                                            agg_col=cs.get("agg_column", -1), W=W, H=W, mode=om)
            check(cnt, val, ocnt, osum, cs)
            st = R.stats()
            assert st["n_filtered"] == kept


def test_stream_pinned_and_device_inputs(c1):
    import torch
    R, P, x, y, cols = c1
    R.set_option(rjmod.OPT_STREAM_BATCH, 65536)
    ocnt, osum, _ = oracle.query(P, x, y, cols=cols, preds=[(1, "<", 6.0)], agg_col=0, W=2048, H=2048,
                                 mode="accurate")
    xt, yt = torch.from_numpy(x.astype(np.float32)), torch.from_numpy(y.astype(np.float32))
    ct = [torch.from_numpy(c) for c in cols]
    o32 = oracle.query(P, xt.numpy(), yt.numpy(), cols=cols, preds=[(1, "<", 6.0)], agg_col=0, W=2048,
                       H=2048, mode="accurate")
    variants = {
        "pinned": ([xt.pin_memory(), yt.pin_memory()], [c.pin_memory() for c in ct], o32),
        "device": ([xt.cuda(), yt.cuda()], [c.cuda() for c in ct], o32),
        "mixed": ([xt.cuda(), yt.pin_memory()], [ct[0], ct[1].cuda()], o32),
        "f64 host": ([x, y], cols, (ocnt, osum, None)),
    }
    for name, (xy, cc, (oc, os_, _)) in variants.items():
        cnt, val = R.query_stream(xy[0], xy[1], cc, W=2048, H=2048, mode="accurate", agg="sum", agg_column=0,
                                  preds=[(1, "<", 6.0)])
        assert np.array_equal(cnt, oc), name
        assert np.array_equal(val, os_), name


def test_stream_equals_loaded_path_taxi():
    """C2 shape on a 2M-point prefix: the streamed and the loaded paths agree
    with each other and with the oracle, bounded and accurate."""
    flat = C.array_polys("neighborhoods")
    pts = C.taxi(2_000_000)
    preds = [(0, ">=", C.T_2012[0]), (0, "<", C.T_2012[1])]
    R = rjmod.RasterJoin(C.NYC_BOX)
    R.load_points(pts["x"], pts["y"], [pts["t"]])
    R.load_polygons(flat)
    R.set_option(rjmod.OPT_STREAM_BATCH, 300_000)
    P = oracle.Polys(flat, C.NYC_BOX)
    for mode in ("bounded", "accurate"):
        c_load, _ = R.query(W=8192, H=8192, preds=preds, mode=mode)
        c_str, _ = R.query_stream(pts["x"], pts["y"], [pts["t"]], W=8192, H=8192, preds=preds, mode=mode)
        ocnt, _, _ = oracle.query(P, pts["x"], pts["y"], cols=[pts["t"]], preds=preds, W=8192, H=8192, mode=mode)
        assert np.array_equal(c_str, ocnt), mode
        assert np.array_equal(c_load, c_str), mode


def test_stream_tracts_avg_accurate():
    flat = C.array_polys("tracts")
    pts = C.taxi(1_000_000, fare=True)
    R = rjmod.RasterJoin(C.NYC_BOX)
    R.load_polygons(flat)
    P = oracle.Polys(flat, C.NYC_BOX)
    cnt, val = R.query_stream(pts["x"], pts["y"], [pts["t"], pts["fare"]], W=8192, H=8192, mode="accurate",
                              agg="avg", agg_column=1)
    ocnt, osum, _ = oracle.query(P, pts["x"], pts["y"], cols=[pts["t"], pts["fare"]], agg_col=1, W=8192,
                                 H=8192, mode="accurate")
    assert np.array_equal(cnt, ocnt)
    ok, bad = rel_close(val, oracle.avg(ocnt, osum))
    assert ok, bad


def test_stream_empty_and_errors(c1):
    R, P, x, y, cols = c1
    cnt, val = R.query_stream(np.zeros(0), np.zeros(0), W=64, agg="count")
    assert cnt.sum() == 0
    with pytest.raises(rjmod.RJError):
        R.query_stream(x, y, cols, W=64, agg="sum", agg_column=5)      # column out of range
    with pytest.raises(rjmod.RJError):
        R.set_option(rjmod.OPT_STREAM_BATCH, 10)
    R2 = rjmod.RasterJoin(C.C1_BOX)
    with pytest.raises(rjmod.RJError):
        R2.n_poly = 1
        R2.query_stream(x, y, W=64)                                    # no polygons loaded
