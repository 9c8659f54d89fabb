"""Parity at BASELINE.json's full sizes, in the launch configuration bench.py
times (library defaults).  The oracle cannot aggregate 1e9 points per test,
so full-size runs are checked through properties that hold at any size --
exact tilings partition the filtered points (lemma L6), shards add up to the
whole (distributivity), the filtered / out-of-domain counts equal
independent numpy counts -- plus oracle parity on prefixes of the same data
in the same launch configuration."""
import numpy as np
import pytest

import oracle
from datagen import configs as C

pytestmark = [pytest.mark.gpu, pytest.mark.slow]

rjmod = pytest.importorskip("paper_journals_pvldb_zacharatoudasf17_b200.rj")


@pytest.fixture(scope="module", autouse=True)
def _gpu():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("needs a CUDA device")


def ctx(box, flat, x, y, cols):
    R = rjmod.RasterJoin(box)
    n_ood = R.load_points(x, y, cols)
    R.load_polygons(flat)
    return R, n_ood


@pytest.fixture(scope="module")
def c2_full():
    n = 1_000_000_000
    return C.taxi(n), C.array_polys("neighborhoods")


def test_c2_full_tiling_filter_and_domain(c2_full):
    pts, flat = c2_full
    preds = [(0, ">=", C.T_2012[0]), (0, "<", C.T_2012[1])]
    R, n_ood = ctx(C.NYC_BOX, flat, pts["x"], pts["y"], [pts["t"]])
    ood = int(np.count_nonzero((pts["x"] >= np.float32(57920.0)) | (pts["y"] >= np.float32(57920.0))))
    assert n_ood == ood
    cnt, _ = R.query(W=8192, H=8192, mode="bounded", preds=preds)
    st = R.stats()
    inside = (pts["x"] < np.float32(57920.0)) & (pts["y"] < np.float32(57920.0))
    t = pts["t"]
    want = int(np.count_nonzero(inside & (t >= C.T_2012[0]) & (t < C.T_2012[1])))
    assert st["n_filtered"] == want
    assert int(cnt.sum()) == want                      # exact tiling: each point in one polygon
    # accurate mode on the same resident data partitions the points too
    cnt_a, _ = R.query(W=8192, H=8192, mode="accurate", preds=preds)
    assert int(cnt_a.sum()) == want
    R.close()


def test_c2_full_shards_add_up(c2_full):
    pts, flat = c2_full
    preds = [(0, ">=", C.T_2012[0]), (0, "<", C.T_2012[1])]
    n = len(pts["x"])
    R, _ = ctx(C.NYC_BOX, flat, pts["x"], pts["y"], [pts["t"]])
    whole, _ = R.query(W=8192, H=8192, mode="bounded", preds=preds)
    R.close()
    acc = np.zeros_like(whole)
    for lo, hi in ((0, n // 3), (n // 3, n)):
        S, _ = ctx(C.NYC_BOX, flat, pts["x"][lo:hi], pts["y"][lo:hi], [pts["t"][lo:hi]])
        c, _ = S.query(W=8192, H=8192, mode="bounded", preds=preds)
        acc += c
        S.close()
    assert np.array_equal(acc, whole)


@pytest.mark.parametrize("mode", ["bounded", "accurate"])
def test_c2_prefix_parity_full_launch(c2_full, mode):
    """A 4e6-point prefix through the full-size launch path vs the oracle."""
    pts, flat = c2_full
    n = 4_000_000
    preds = [(0, ">=", C.T_2012[0]), (0, "<", C.T_2012[1])]
    x, y, t = pts["x"][:n], pts["y"][:n], pts["t"][:n]
    R, _ = ctx(C.NYC_BOX, flat, x, y, [t])
    cnt, _ = R.query(W=8192, H=8192, mode=mode, preds=preds)
    P = oracle.Polys(flat, C.NYC_BOX)
    ocnt, _, _ = oracle.query(P, x, y, cols=[t], preds=preds, W=8192, H=8192, mode=mode)
    assert np.array_equal(cnt, ocnt)
    R.close()


def test_c3_full_accurate_avg():
    n = 1_000_000_000
    pts = C.taxi(n, fare=True)
    flat = C.array_polys("tracts")
    R, n_ood = ctx(C.NYC_BOX, flat, pts["x"], pts["y"], [pts["t"], pts["fare"]])
    cnt, avg = R.query(W=8192, H=8192, mode="accurate", agg="avg", agg_column=1)
    st = R.stats()
    assert int(cnt.sum()) == st["n_points"] == n - n_ood
    assert st["n_boundary"] > 0
    ok = np.isfinite(avg) | (cnt == 0)
    assert ok.all() and np.all(avg[cnt > 0] >= 2.5)      # fares are >= 2.5 by construction
    R.close()
    # prefix parity vs the oracle (AVG to 1e-9)
    m = 2_000_000
    cols = [pts["t"][:m], pts["fare"][:m]]
    R, _ = ctx(C.NYC_BOX, flat, pts["x"][:m], pts["y"][:m], cols)
    cnt, avg = R.query(W=8192, H=8192, mode="accurate", agg="avg", agg_column=1)
    P = oracle.Polys(flat, C.NYC_BOX)
    ocnt, osum, _ = oracle.query(P, pts["x"][:m], pts["y"][:m], cols=cols, agg_col=1, W=8192, H=8192,
                                 mode="accurate")
    assert np.array_equal(cnt, ocnt)
    oavg = oracle.avg(ocnt, osum)
    both = np.isnan(avg) & np.isnan(oavg)
    assert np.all(both | (np.abs(avg - oavg) <= 1e-9 * np.abs(oavg)))
    R.close()


def test_c4_shard_sum_exact():
    """One rank's shard of C4 (2e9 points over 8 GPUs = 2.5e8): SUM(fav) is
    exact (integer attribute), tiling holds, prefix matches the oracle."""
    n = 250_000_000
    pts = C.twitter(n)
    flat = C.array_polys("counties")
    R, n_ood = ctx(C.US_BOX, flat, pts["x"], pts["y"], [pts["fav"]])
    cnt, s = R.query(epsilon=1000.0, mode="bounded", agg="sum", agg_column=0)
    assert int(cnt.sum()) == n - n_ood
    inside = (pts["x"] < np.float32(4.6e6)) & (pts["y"] < np.float32(2.9e6))
    assert float(s.sum()) == float(pts["fav"][inside].astype(np.int64).sum())
    R.close()
    m = 2_000_000
    R, _ = ctx(C.US_BOX, flat, pts["x"][:m], pts["y"][:m], [pts["fav"][:m]])
    cnt, s = R.query(epsilon=1000.0, mode="bounded", agg="sum", agg_column=0)
    P = oracle.Polys(flat, C.US_BOX)
    ocnt, osum, _ = oracle.query(P, pts["x"][:m], pts["y"][:m], cols=[pts["fav"][:m]], agg_col=0, W=6506,
                                 H=4102, mode="bounded")
    assert np.array_equal(cnt, ocnt) and np.array_equal(s, osum)
    R.close()


@pytest.mark.parametrize("W", [1024, 32768])
def test_c5_resolution_extremes_tiling(W):
    n = 1_000_000_000
    pts = C.taxi(n)
    flat = C.array_polys("neighborhoods")
    R, n_ood = ctx(C.NYC_BOX, flat, pts["x"], pts["y"], [])
    for mode in ("bounded", "accurate"):
        cnt, _ = R.query(W=W, H=W, mode=mode)
        assert int(cnt.sum()) == n - n_ood, mode
    R.close()
