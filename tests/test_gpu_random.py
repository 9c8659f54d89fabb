"""Randomised GPU-vs-oracle parity (seeded): random domains, random
non-convex / self-intersecting rings with holes, vertices on a coarse grid,
on half-units and at random positions, points placed on vertices, on edge
midpoints, on the grid and uniformly; random canvases (non power of two,
1..3000 a side), windows, filters, aggregates and modes.  COUNT bit-exact,
SUM of an integer column bit-exact, SUM of a float column within 1e-9."""
import numpy as np
import pytest

import oracle

pytestmark = pytest.mark.gpu

rjmod = pytest.importorskip("paper_journals_pvldb_zacharatoudasf17_b200.rj")


@pytest.fixture(scope="module", autouse=True)
def _gpu():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("needs a CUDA device")


def _ring(rng, cx, cy, r, k, snap, shuffle=False):
    ang = np.sort(rng.uniform(0, 2 * np.pi, k))
    if shuffle:
        rng.shuffle(ang)                                   # self-intersecting
    rad = r * rng.uniform(0.3, 1.0, k)
    pts = np.stack([cx + rad * np.cos(ang), cy + rad * np.sin(ang)], 1)
    if snap:
        pts = np.round(pts / snap) * snap
    return pts


def _case(seed):
    rng = np.random.default_rng(seed)
    w, h = rng.uniform(50, 5000), rng.uniform(50, 5000)
    x0, y0 = rng.uniform(-1e4, 1e4), rng.uniform(-1e4, 1e4)
    box = (x0, y0, x0 + w, y0 + h)
    snap = [None, w / 64, w / 128, 0.5][rng.integers(4)]
    polys = []
    for _ in range(rng.integers(3, 10)):
        cx, cy = x0 + rng.uniform(0.1, 0.9) * w, y0 + rng.uniform(0.1, 0.9) * h
        r = min(w, h) * rng.uniform(0.05, 0.4)
        outer = _ring(rng, cx, cy, r, rng.integers(3, 40), snap, shuffle=rng.random() < 0.15)
        rings = [outer]
        if rng.random() < 0.3:
            rings.append(_ring(rng, cx, cy, r * 0.25, rng.integers(3, 10), snap))
        for q in rings:
            q[:, 0] = np.clip(q[:, 0], x0, x0 + w)
            q[:, 1] = np.clip(q[:, 1], y0, y0 + h)
        polys.append(rings)
    rings = [q for p in polys for q in p]
    n_ring = [len(p) for p in polys]
    pro = np.concatenate([[0], np.cumsum(n_ring)]).astype(np.uint32)
    rvo = np.concatenate([[0], np.cumsum([len(q) for q in rings])]).astype(np.uint32)
    vx = np.concatenate([q[:, 0] for q in rings]).astype(np.float64)
    vy = np.concatenate([q[:, 1] for q in rings]).astype(np.float64)
    flat = (pro, rvo, vx, vy)
    n = int(rng.integers(1, 40000))
    x = rng.uniform(x0, x0 + w, n)
    y = rng.uniform(y0, y0 + h, n)
    k = min(n, len(vx))                                     # points on vertices and edge midpoints
    x[:k] = vx[:k]
    y[:k] = vy[:k]
    m = min(n - k, len(vx) - 1)
    if m > 0:
        x[k:k + m] = 0.5 * (vx[:m] + vx[1:m + 1])
        y[k:k + m] = 0.5 * (vy[:m] + vy[1:m + 1])
    if snap:
        g = slice(k + max(m, 0), min(n, k + max(m, 0) + 2000))
        x[g] = np.round(x[g] / snap) * snap
        y[g] = np.round(y[g] / snap) * snap
    ti = rng.integers(-100, 100, n).astype(np.int32)
    tf = rng.normal(3.0, 2.0, n).astype(np.float32)
    W, H = int(rng.integers(1, 3000)), int(rng.integers(1, 3000))
    view = None
    if rng.random() < 0.3:
        c0, r0 = int(rng.integers(0, W)), int(rng.integers(0, H))
        view = (c0, r0, int(rng.integers(c0 + 1, W + 1)), int(rng.integers(r0 + 1, H + 1)))
    preds = [] if rng.random() < 0.4 else [(0, [">=", "<", "<=", ">"][rng.integers(4)], float(rng.integers(-80, 80)))]
    f64 = rng.random() < 0.5
    if not f64:
        x, y = x.astype(np.float32), y.astype(np.float32)
    return box, flat, x, y, [ti, tf], W, H, view, preds


@pytest.mark.parametrize("seed", range(24))
def test_random_parity(seed):
    box, flat, x, y, cols, W, H, view, preds = _case(seed)
    P = oracle.Polys(flat, box)
    R = rjmod.RasterJoin(box)
    R.load_points(x, y, cols)
    R.load_polygons(flat)
    for mode in ("bounded", "accurate", "index"):
        if mode == "index" and view is not None:
            continue
        oc, oi, _ = oracle.query(P, x, y, cols=cols, preds=preds, agg_col=0, W=W, H=H,
                                 mode="accurate" if mode == "index" else mode, view=view)
        _, of, _ = oracle.query(P, x, y, cols=cols, preds=preds, agg_col=1, W=W, H=H,
                                mode="accurate" if mode == "index" else mode, view=view)
        cnt, si = R.query(W=W, H=H, mode=mode, agg="sum", agg_column=0, preds=preds, view=view)
        assert np.array_equal(cnt, oc), (seed, mode)
        assert np.array_equal(si, oi), (seed, mode)
        _, sf = R.query(W=W, H=H, mode=mode, agg="sum", agg_column=1, preds=preds, view=view)
        # reading Z23: 1e-9 relative to the sum of |values| (condition-number
        # normalised; equals 1e-9 relative for same-sign data, and stays
        # meaningful when mixed signs cancel) -- the oracle's SUM of |col|
        _, oabs, _ = oracle.query(P, x, y, cols=[cols[0], np.abs(cols[1])], preds=preds, agg_col=1, W=W, H=H,
                                  mode="accurate" if mode == "index" else mode, view=view)
        assert np.all(np.abs(sf - of) <= 1e-9 * oabs), (seed, mode, sf, of, oabs)
    R.close()
