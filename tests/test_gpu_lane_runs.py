"""GPU parity of the COUNT tile kernel's two window variants (pass.cu):
runs of equal pixels merged inside each lane only (process_lane_runs, the
default) and merged across the lanes of a warp (process, RJ_OPT_LANE_RUNS
= 2), against the CPU oracle and each other.

Bar (BASELINE.json north_star): per-polygon COUNT
bit-exact in both modes.  Cases: canvases from one pixel to 32768^2 (cells
of odd sizes), small work items that split heavy cells (ragged tails),
pixel-border adversarial points (C1b), hot pixels (one pixel holding a
whole work item, i.e. 32 lanes reducing into one word), filters.
"""
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
    pts = C.c1_points()
    ax, ay = PG.c1b_points(polys)
    x = np.concatenate([pts["x"], ax])
    y = np.concatenate([pts["y"], ay])
    t = (np.arange(len(x)) % 100 - 50).astype(np.int32)
    return flat, x, y, [t]


def ctx(box, flat, x, y, cols, runs, chunk=None):
    R = rjmod.RasterJoin(box)
    R.set_option(rjmod.OPT_LANE_RUNS, runs)
    if chunk:
        R.set_option(rjmod.OPT_CHUNK, chunk)
    R.load_points(x, y, cols)
    R.load_polygons(flat)
    return R


@pytest.mark.parametrize("W,H", [(1, 1), (5, 7), (64, 64), (333, 517), (1024, 1024), (4096, 4096),
                                 (32768, 32768)])
@pytest.mark.parametrize("mode", ["bounded", "accurate"])
@pytest.mark.parametrize("runs,chunk", [(1, None), (1, 256), (2, 256)])
def test_count_bitexact(c1, W, H, mode, runs, chunk):
    flat, x, y, cols = c1
    R = ctx(C.C1_BOX, flat, x, y, cols, runs, chunk)
    P = oracle.Polys(flat, C.C1_BOX)
    cnt, _ = R.query(W=W, H=H, mode=mode)
    ocnt, _, kept = oracle.query(P, x, y, W=W, H=H, mode=mode)
    assert np.array_equal(cnt, ocnt)
    assert R.stats()["n_filtered"] == kept


@pytest.mark.parametrize("preds", [[(0, ">=", -10), (0, "<", 25)], [(0, "==", 7)], [(0, "<", -60)]])
def test_filters(c1, preds):
    flat, x, y, cols = c1
    R = ctx(C.C1_BOX, flat, x, y, cols, 1, 512)
    P = oracle.Polys(flat, C.C1_BOX)
    for mode in ("bounded", "accurate"):
        cnt, _ = R.query(W=2048, H=2048, mode=mode, preds=preds)
        ocnt, _, kept = oracle.query(P, x, y, cols, W=2048, H=2048, mode=mode, preds=preds)
        assert np.array_equal(cnt, ocnt)
        assert R.stats()["n_filtered"] == kept


def test_both_variants_agree_taxi():
    """1.5M taxi-shaped points, 260 neighbourhoods, three canvases, both
    modes: identical counts from both window variants."""
    pts = C.taxi(1_500_000)
    flat = C.array_polys("neighborhoods")
    R = rjmod.RasterJoin(C.NYC_BOX)
    R.load_points(pts["x"], pts["y"], [pts["t"]])
    R.load_polygons(flat)
    preds = [(0, ">=", C.T_2012[0]), (0, "<", C.T_2012[1])]
    for W in (1024, 8192, 32768):
        for mode in ("bounded", "accurate"):
            R.set_option(rjmod.OPT_LANE_RUNS, 1)
            a, _ = R.query(W=W, H=W, mode=mode, preds=preds)
            R.set_option(rjmod.OPT_LANE_RUNS, 2)
            b, _ = R.query(W=W, H=W, mode=mode, preds=preds)
            assert np.array_equal(a, b), (W, mode)
    R.close()


def test_hot_pixel():
    """65535 points on one pixel in one work item: every lane of every
    window reduces into the same tile word; the neighbour pixel (another
    polygon) stays empty."""
    sq = lambda x0, y0, x1, y1: [np.array([(x0, y0), (x1, y0), (x1, y1), (x0, y1)], dtype=np.float64)]
    flat = PG.flatten([sq(10.0, 10.0, 30.0, 30.0), sq(11.0, 10.0, 12.0, 30.0), sq(200.0, 200.0, 230.0, 230.0)])
    x = np.concatenate([np.full(65535, 10.5), np.full(7, 210.5)])
    y = np.concatenate([np.full(65535, 20.5), np.full(7, 210.5)])
    for runs in (1, 2):
        R = ctx(C.C1_BOX, flat, x, y, [], runs, 65535)
        for mode in ("bounded", "accurate"):
            cnt, _ = R.query(W=1024, H=1024, mode=mode)
            assert cnt.tolist() == [65535, 0, 7], (runs, mode)
        with pytest.raises(Exception):
            R.set_option(rjmod.OPT_LANE_RUNS, 3)
        R.close()
