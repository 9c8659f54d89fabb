"""GPU parity of the index-join variant (RJ_INDEX_JOIN: grid-indexed PIP for
every filtered point, Proc. IndexJoin) and of the exact
chooser (RJ_EXACT).  Both are exact, so the oracle
reference is its accurate mode (the plain even-odd PIP definition, O4):
COUNT and membership bit-exact, SUM/AVG within 1e-9 relative."""
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


def ctx(box, flat, x, y, cols=()):
    R = rjmod.RasterJoin(box)
    R.load_points(x, y, cols)
    R.load_polygons(flat)
    return R


def rel_close(g, o, tol=1e-9):
    g = np.asarray(g, np.float64)
    o = np.asarray(o, np.float64)
    ok = (np.isnan(g) & np.isnan(o)) | (np.abs(g - o) <= tol * np.abs(o)) | ((o == 0) & (g == 0))
    return bool(np.all(ok)), np.nonzero(~ok)[0]


@pytest.fixture(scope="module")
def c1():
    polys = C.polygon_set("c1b")
    flat = PG.flatten(polys)
    pts = C.c1_points()
    ax, ay = PG.c1b_points(polys)
    x = np.concatenate([pts["x"], ax])
    y = np.concatenate([pts["y"], ay])
    rng = np.random.default_rng(12)
    ti = rng.integers(-50, 50, len(x)).astype(np.int32)
    tf = rng.normal(5, 3, len(x)).astype(np.float32)
    return flat, x, y, [ti, tf]


@pytest.mark.parametrize("variant", [-1, 0, 1])
@pytest.mark.parametrize("W", [64, 1024, 3001])
def test_index_join_c1(c1, variant, W):
    """Every point through the edge grid: identical to the exact oracle at
    every canvas size (the canvas only shapes the point tiles)."""
    flat, x, y, cols = c1
    R = ctx(C.C1_BOX, flat, x, y, cols)
    R.set_option(rjmod.OPT_PASS, variant)
    P = oracle.Polys(flat, C.C1_BOX)
    for cs in (dict(agg="count", preds=[]),
               dict(agg="sum", agg_column=0, preds=[(1, "<", 6.0)]),
               dict(agg="avg", agg_column=1, preds=[(0, ">=", -20)])):
        cnt, val = R.query(W=W, H=W, mode="index", **cs)
        ocnt, osum, kept = oracle.query(P, x, y, cols=cols, preds=cs["preds"], agg_col=cs.get("agg_column", -1),
                                        W=W, H=W, mode="accurate")
        assert np.array_equal(cnt, ocnt), cs
        st = R.stats()
        assert st["mode"] == 2 and st["n_boundary"] == st["n_filtered"] == kept
        assert st["n_pieces"] == 0 and st["n_crossings"] == 0          # no polygon pass
        if cs["agg"] == "sum":
            assert np.array_equal(val, osum)                              # integer attribute: exact
        elif cs["agg"] == "avg":
            ok, bad = rel_close(val, oracle.avg(ocnt, osum))
            assert ok, bad
    R.close()


def test_index_join_membership(c1):
    flat, x, y, cols = c1
    R = ctx(C.C1_BOX, flat, x, y, cols)
    P = oracle.Polys(flat, C.C1_BOX)
    g = R.membership(W=512, H=512, mode="index")
    o = oracle.membership(P, x, y, W=512, H=512, mode="accurate")
    assert np.array_equal(g, o)


def test_index_join_tracts_avg():
    """C3 shape (tracts, AVG(fare)) on a 1M-point prefix."""
    flat = C.array_polys("tracts")
    pts = C.taxi(1_000_000, fare=True)
    R = ctx(C.NYC_BOX, flat, pts["x"], pts["y"], [pts["t"], pts["fare"]])
    P = oracle.Polys(flat, C.NYC_BOX)
    cnt, val = R.query(W=8192, H=8192, mode="index", agg="avg", agg_column=1)
    ocnt, osum, _ = oracle.query(P, pts["x"], pts["y"], cols=[pts["t"], pts["fare"]], agg_col=1,
                                 W=8192, H=8192, mode="accurate")
    assert np.array_equal(cnt, ocnt)
    ok, bad = rel_close(val, oracle.avg(ocnt, osum))
    assert ok, bad


def test_index_join_empty_and_tiny():
    flat = PG.flatten(C.polygon_set("c1"))
    P = oracle.Polys(flat, C.C1_BOX)
    for n in (0, 1, 9, 257):
        pts = C.c1_points(n) if n else {"x": np.zeros(0), "y": np.zeros(0)}
        R = ctx(C.C1_BOX, flat, pts["x"], pts["y"])
        cnt, _ = R.query(W=1024, mode="index", agg="count")
        ocnt, _, _ = oracle.query(P, pts["x"], pts["y"], W=1024, H=1024, mode="accurate")
        assert np.array_equal(cnt, ocnt), n
        R.close()


def test_exact_chooser(c1):
    """RJ_EXACT resolves to one of the exact variants and returns the exact
    result; a handful of points picks the index join (the polygon pass would
    dominate), 16M points on the coarse C1b polygons pick the raster join."""
    flat, x, y, cols = c1
    P = oracle.Polys(flat, C.C1_BOX)
    R = ctx(C.C1_BOX, flat, x[:1000], y[:1000])
    cnt, _ = R.query(W=2048, H=2048, mode="exact")
    ocnt, _, _ = oracle.query(P, x[:1000], y[:1000], W=2048, H=2048, mode="accurate")
    assert np.array_equal(cnt, ocnt)
    assert R.stats()["mode"] == 2
    R.close()
    pts = C.c1_points(16_000_000)
    R = ctx(C.C1_BOX, flat, pts["x"], pts["y"])
    cnt, _ = R.query(W=1024, H=1024, mode="exact")
    st = R.stats()
    assert st["mode"] == 1 and 0.0 < st["est_boundary_frac"] < 0.5
    ocnt, _, _ = oracle.query(P, pts["x"], pts["y"], W=1024, H=1024, mode="accurate")
    assert np.array_equal(cnt, ocnt)
