"""GPU parity of the bounded-mode result intervals (rj_query_interval,
SURVEY.md 8(f) NEXT-1, reading Z13 / oracle O10) and of
the point canvas Fpt (S2, Proc. DrawPoints P:519-527).

Bar: the per-pixel count canvas and eps+/eps- are integers -> bit-exact
against the oracle (or_pixel_counts, or_error_interval); the paper's
"100 % confidence" invariant accurate in [bounded - eps+, bounded + eps-]
must hold on every polygon."""
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


@pytest.fixture(scope="module")
def c1():
    polys = C.polygon_set("c1b")
    flat = PG.flatten(polys)
    pts = C.c1_points(300_000)
    ax, ay = PG.c1b_points(polys)
    x = np.concatenate([pts["x"], ax])
    y = np.concatenate([pts["y"], ay])
    rng = np.random.default_rng(31)
    ti = rng.integers(-50, 50, len(x)).astype(np.int32)
    R = rjmod.RasterJoin(C.C1_BOX)
    R.load_points(x, y, [ti])
    R.load_polygons(flat)
    return R, oracle.Polys(flat, C.C1_BOX), x, y, [ti]


@pytest.mark.parametrize("W,H", [(16, 16), (200, 200), (1024, 1024), (777, 555)])
def test_point_canvas_bitexact(c1, W, H):
    R, P, x, y, cols = c1
    preds = [(0, ">=", -10)]
    g = R.point_canvas(W=W, H=H, preds=preds)
    o = oracle.pixel_counts(x, y, C.C1_BOX, cols=cols, preds=preds, W=W, H=H)
    assert np.array_equal(g, o)


@pytest.mark.parametrize("W,H", [(16, 16), (64, 64), (200, 200), (777, 555)])
@pytest.mark.parametrize("chunk", [None, 1000])
def test_interval_bitexact_and_holds(c1, W, H, chunk):
    R, P, x, y, cols = c1
    if chunk:
        R.set_option(rjmod.OPT_CHUNK, chunk)          # heavy cells split over work items
    preds = [(0, "<", 25)]
    cnt, val, ep, em = R.query_interval(W=W, H=H, preds=preds, agg="sum", agg_column=0)
    if chunk:
        R.set_option(rjmod.OPT_CHUNK, 65536)
    ob, osum, _ = oracle.query(P, x, y, cols=cols, preds=preds, agg_col=0, W=W, H=H, mode="bounded")
    oa, _, _ = oracle.query(P, x, y, cols=cols, preds=preds, W=W, H=H, mode="accurate")
    counts = oracle.pixel_counts(x, y, C.C1_BOX, cols=cols, preds=preds, W=W, H=H)
    oep, oem = oracle.error_interval(P, W, H, counts)
    assert np.array_equal(cnt, ob)
    assert np.array_equal(val, osum)
    assert np.array_equal(ep, oep)
    assert np.array_equal(em, oem)
    b, a = cnt.astype(np.int64), oa.astype(np.int64)
    assert np.all(a >= b - ep.astype(np.int64)) and np.all(a <= b + em.astype(np.int64))


def test_interval_taxi_neighbourhoods():
    """C2/C5 shape on a 1M-point prefix at 512^2 (the oracle's O10 is
    O(n_poly x W x H)); invariant at 4096^2."""
    flat = C.array_polys("neighborhoods")
    pts = C.taxi(1_000_000)
    R = rjmod.RasterJoin(C.NYC_BOX)
    R.load_points(pts["x"], pts["y"], [pts["t"]])
    R.load_polygons(flat)
    P = oracle.Polys(flat, C.NYC_BOX)
    cnt, _, ep, em = R.query_interval(W=512, H=512)
    counts = oracle.pixel_counts(pts["x"], pts["y"], C.NYC_BOX, W=512, H=512)
    oep, oem = oracle.error_interval(P, 512, 512, counts)
    assert np.array_equal(ep, oep) and np.array_equal(em, oem)
    for W in (512, 4096):
        cnt, _, ep, em = R.query_interval(W=W, H=W)
        acc, _ = R.query(W=W, H=W, mode="accurate")
        b, a = cnt.astype(np.int64), acc.astype(np.int64)
        assert np.all(a >= b - ep.astype(np.int64)) and np.all(a <= b + em.astype(np.int64)), W
    # finer canvas -> tighter intervals
    _, _, ep1, em1 = R.query_interval(W=1024, H=1024)
    _, _, ep2, em2 = R.query_interval(W=8192, H=8192)
    assert (ep2 + em2).sum() < (ep1 + em1).sum()


def test_interval_rejects_other_modes(c1):
    R = c1[0]
    with pytest.raises(rjmod.RJError):
        R.query_interval(W=64, mode="accurate")


def _close(g, o, scale):
    """binary64 sums of f * Fpt by two different area computations (Green
    edge integrals vs ring clipping): within 1e-9 of the worst-case mass."""
    return np.all(np.abs(g - o) <= 1e-9 * (scale + 1.0))


@pytest.mark.parametrize("W,H", [(16, 16), (64, 64), (200, 200), (777, 555), (1024, 1024)])
def test_expected_interval_parity(c1, W, H):
    # P:811-827, reading Z22 / oracle O13
    R, P, x, y, cols = c1
    preds = [(0, "<", 25)]
    cnt, _, ep, em, xp, xm = R.query_interval_ex(W=W, H=H, preds=preds)
    counts = oracle.pixel_counts(x, y, C.C1_BOX, cols=cols, preds=preds, W=W, H=H)
    oep, oem = oracle.error_interval(P, W, H, counts)
    oxp, oxm = oracle.expected_interval(P, W, H, counts)
    assert np.array_equal(ep, oep) and np.array_equal(em, oem)
    assert _close(xp, oxp, oep.astype(np.float64)), (xp, oxp)
    assert _close(xm, oxm, oem.astype(np.float64)), (xm, oxm)
    assert np.all(xp <= ep + 1e-9) and np.all(xm <= em + 1e-9)
    # the plain call gives the same worst case
    c2, _, ep2, em2 = R.query_interval(W=W, H=H, preds=preds)
    assert np.array_equal(c2, cnt) and np.array_equal(ep2, ep) and np.array_equal(em2, em)


def test_expected_interval_taxi_neighbourhoods():
    """Tiling with shared vertices, 1M taxi-shaped points, 256^2 (parity)
    and the estimate's quality at 2048^2 against the accurate count."""
    flat = C.array_polys("neighborhoods")
    pts = C.taxi(1_000_000)
    R = rjmod.RasterJoin(C.NYC_BOX)
    R.load_points(pts["x"], pts["y"])
    R.load_polygons(flat)
    P = oracle.Polys(flat, C.NYC_BOX)
    _, _, ep, em, xp, xm = R.query_interval_ex(W=256, H=256)
    counts = oracle.pixel_counts(pts["x"], pts["y"], C.NYC_BOX, W=256, H=256)
    oxp, oxm = oracle.expected_interval(P, 256, 256, counts)
    assert _close(xp, oxp, ep.astype(np.float64)) and _close(xm, oxm, em.astype(np.float64))
    cnt, _, ep, em, xp, xm = R.query_interval_ex(W=2048, H=2048)
    acc, _ = R.query(W=2048, H=2048, mode="accurate")
    b, a = cnt.astype(np.float64), acc.astype(np.float64)
    est = b - xp + xm
    assert np.abs(a - est).sum() < 0.5 * np.abs(a - b).sum()
