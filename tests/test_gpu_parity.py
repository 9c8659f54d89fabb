"""GPU parity: the CUDA path (through the C ABI) against the CPU oracle,
element by element on the same seeded inputs.

Bar (BASELINE.json north_star): COUNT, pixel spans,
boundary mask and point membership bit-exact; SUM/AVG within 1e-9 relative
(exact for integer attributes).  Sizes span many tiles / work items and a
ragged tail; the edge cases cover empty and degenerate inputs.
"""
import math

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


def gpu_ctx(box, polys_flat, x, y, cols=(), chunk=None):
    R = rjmod.RasterJoin(box)
    if chunk:
        R.set_option(rjmod.OPT_CHUNK, chunk)
    R.load_points(x, y, cols)
    R.load_polygons(polys_flat)
    return R


def rel_close(g, o, tol=1e-9):
    g = np.asarray(g, np.float64)
    o = np.asarray(o, np.float64)
    both_nan = np.isnan(g) & np.isnan(o)
    ok = both_nan | (np.abs(g - o) <= tol * np.abs(o)) | ((o == 0) & (g == 0))
    return bool(np.all(ok)), np.nonzero(~ok)[0]


# ------------------------------------------------------------------------ C1
@pytest.fixture(scope="module")
def c1():
    polys = C.polygon_set("c1b")
    flat = PG.flatten(polys)
    pts = C.c1_points()
    ax, ay = PG.c1b_points(polys)
    x = np.concatenate([pts["x"], ax])
    y = np.concatenate([pts["y"], ay])
    rng = np.random.default_rng(11)
    ti = rng.integers(-50, 50, len(x)).astype(np.int32)
    tf = rng.normal(5, 3, len(x)).astype(np.float32)
    tf[::97] = np.nan
    return flat, x, y, [ti, tf]


@pytest.mark.parametrize("mode", ["bounded", "accurate"])
@pytest.mark.parametrize("chunk", [None, 256])
def test_c1_count_bitexact(c1, mode, chunk):
    flat, x, y, cols = c1
    R = gpu_ctx(C.C1_BOX, flat, x, y, cols, chunk=chunk)
    P = oracle.Polys(flat, C.C1_BOX)
    cnt, val = R.query(W=1024, H=1024, mode=mode)
    ocnt, _, kept = oracle.query(P, x, y, W=1024, H=1024, mode=mode)
    assert np.array_equal(cnt, ocnt), (cnt, ocnt)
    assert np.array_equal(val, ocnt.astype(np.float64))
    st = R.stats()
    assert st["n_filtered"] == kept == len(x)
    if mode == "accurate":
        assert st["n_boundary"] > 0


@pytest.mark.parametrize("W,H", [(1, 1), (5, 7), (64, 64), (333, 517), (1000, 700), (4096, 4096), (32768, 32768)])
@pytest.mark.parametrize("mode", ["bounded", "accurate"])
def test_c1_resolutions(c1, W, H, mode):
    flat, x, y, cols = c1
    R = gpu_ctx(C.C1_BOX, flat, x, y, cols)
    P = oracle.Polys(flat, C.C1_BOX)
    cnt, _ = R.query(W=W, H=H, mode=mode)
    ocnt, _, _ = oracle.query(P, x, y, W=W, H=H, mode=mode)
    assert np.array_equal(cnt, ocnt)


def _merge_touching(sp):
    """(row, lo, hi) spans sorted by (row, lo) -> maximal runs.  Even-odd
    pairing of sorted thresholds can emit two spans that touch ([a,b), [b,c)
    for a self-intersecting ring); the pixel set is what is unique."""
    out = []
    for r, lo, hi in sp.tolist():
        if out and out[-1][0] == r and out[-1][2] == lo:
            out[-1][2] = hi
        else:
            out.append([r, lo, hi])
    return np.asarray(out, dtype=np.int64).reshape(-1, 3)


@pytest.mark.parametrize("W,H", [(1024, 1024), (333, 517), (64, 48)])
def test_pixel_spans_bitexact(c1, W, H):
    flat, x, y, cols = c1
    R = gpu_ctx(C.C1_BOX, flat, x, y, cols)
    P = oracle.Polys(flat, C.C1_BOX)
    sp = R.spans(W=W, H=H)
    for pid in range(P.n):
        g = _merge_touching(sp[sp[:, 0] == pid][:, 1:].astype(np.int64))
        o = oracle.pixel_spans(P, pid, W, H).astype(np.int64)
        assert np.array_equal(g, o), pid


@pytest.mark.parametrize("W,H", [(1024, 1024), (200, 300), (4096, 4096)])
def test_boundary_mask_bitexact(c1, W, H):
    flat, x, y, cols = c1
    R = gpu_ctx(C.C1_BOX, flat, x, y, cols)
    P = oracle.Polys(flat, C.C1_BOX)
    g = R.boundary_mask(W=W, H=H)
    o = oracle.boundary_mask(P, W, H)
    assert np.array_equal(g, o)


def _unpack_bits(bits, W):
    """uint32[H, ceil(W/32)] -> bool[H, W] (bit i % 32 of word i / 32)."""
    b = np.unpackbits(bits.view(np.uint8), axis=1, bitorder="little")
    return b[:, :W].astype(bool)


@pytest.fixture(scope="module")
def c1_dense():
    """C1b polygons with 2M uniform points, so every point cell of the
    canvases below holds points and the kernels' tiles cover every pixel."""
    polys = C.polygon_set("c1b")
    flat = PG.flatten(polys)
    rng = np.random.default_rng(20171117)
    x = rng.uniform(0, 1024, 2_000_000)
    y = rng.uniform(0, 1024, 2_000_000)
    return flat, x, y, [(np.arange(len(x)) % 5).astype(np.int32)]


@pytest.mark.parametrize("W,H", [(1024, 1024), (200, 300), (4096, 4096), (777, 1500)])
@pytest.mark.parametrize("agg,variant", [("count", -1), ("sum", 0), ("sum", 1)])
def test_boundary_pieces_bitexact(c1_dense, W, H, agg, variant):
    """S5 as the hot path uses it: the boundary pixels the accurate kernels
    paint into their tiles from k_bnd_pieces (pixel-tile kernel for COUNT and
    RJ_OPT_PASS=1, label kernel for SUM) equal O9's supercover mask
     on every pixel the tiles cover -- over-marking
    would be invisible in counts (lemma L4) and only cost time."""
    flat, x, y, cols = c1_dense
    R = gpu_ctx(C.C1_BOX, flat, x, y, cols)
    R.set_option(rjmod.OPT_PASS, variant)
    P = oracle.Polys(flat, C.C1_BOX)
    kw = dict(W=W, H=H, agg=agg, agg_column=0 if agg == "sum" else -1)
    bnd, cov = R.boundary_pieces(**kw)
    bnd, cov = _unpack_bits(bnd, W), _unpack_bits(cov, W)
    o = _unpack_bits(oracle.boundary_mask(P, W, H), W)
    assert np.array_equal(bnd, o & cov)
    # every point's pixel is covered, and with 2M uniform points every pixel is
    q = lambda v, n: (np.floor(v * (1 << 20)).astype(np.int64) * n) >> 30
    assert cov[q(y, H), q(x, W)].all()
    assert cov.all()
    assert o.sum() > 0
    # a window: pieces are clipped to it
    view = (W // 5, H // 7, W - W // 3, H - H // 9)
    bnd, cov = R.boundary_pieces(view=view, **kw)
    bnd, cov = _unpack_bits(bnd, W), _unpack_bits(cov, W)
    win = np.zeros((H, W), dtype=bool)
    win[view[1]:view[3], view[0]:view[2]] = True
    assert np.array_equal(cov, win)
    assert np.array_equal(bnd, o & win)
    R.close()


@pytest.mark.parametrize("mode", ["bounded", "accurate"])
@pytest.mark.parametrize("variant", [0, 1])
@pytest.mark.parametrize("W,H", [(1024, 1024), (333, 517)])
def test_fused_membership_fingerprint(c1, mode, variant, W, H):
    """Point membership through the fused kernels themselves (the label and
    the pixel-tile kernel, RJ_OPT_PASS 0 / 1), not the separate diagnostic
    kernel: two columns of uniformly random full-range int32 attributes are
    summed per polygon.  Every partial sum is an integer below 2^53
    (< 1.1e5 points x 2^31), so fp64 SUM is exact on both sides and must be
    bit-identical; a polygon whose GPU point set differs from the oracle's
    in any point changes the sum of a random column except with probability
    ~2^-32 per column (P:681-726 exact join, P:550-554 bounded)."""
    flat, x, y, _ = c1
    rng = np.random.default_rng(1729 + W)
    fa = rng.integers(-2**31, 2**31, len(x), dtype=np.int64).astype(np.int32)
    fb = rng.integers(-2**31, 2**31, len(x), dtype=np.int64).astype(np.int32)
    R = gpu_ctx(C.C1_BOX, flat, x, y, [fa, fb])
    R.set_option(rjmod.OPT_PASS, variant)
    P = oracle.Polys(flat, C.C1_BOX)
    for col in (0, 1):
        cnt, val = R.query(W=W, H=H, mode=mode, agg="sum", agg_column=col)
        ocnt, osum, _ = oracle.query(P, x, y, cols=[fa, fb], agg_col=col, W=W, H=H, mode=mode)
        assert np.array_equal(cnt, ocnt), col
        assert np.array_equal(val, osum), col
        assert np.all(np.abs(osum) < 2.0 ** 53)
    R.close()


@pytest.mark.parametrize("mode", ["bounded", "accurate"])
@pytest.mark.parametrize("W", [1024, 97])
def test_point_membership_bitexact(c1, mode, W):
    flat, x, y, cols = c1
    R = gpu_ctx(C.C1_BOX, flat, x, y, cols)
    P = oracle.Polys(flat, C.C1_BOX)
    preds = [(0, ">=", -20.5), (1, "<", 7.25)]
    g = R.membership(W=W, H=W, mode=mode, preds=preds)
    o = oracle.membership(P, x, y, cols=cols, preds=preds, W=W, H=W, mode=mode)
    assert np.array_equal(g, o)


@pytest.mark.parametrize("mode,variant", [("bounded", 0), ("bounded", 1), ("accurate", 0), ("accurate", 1),
                                          ("bounded", -1), ("accurate", -1)])
def test_sum_avg_filters(c1, mode, variant):
    """Both point-pass kernels (label: default for bounded SUM/AVG; tile:
    RJ_OPT_PASS = 1) against the oracle."""
    flat, x, y, cols = c1
    R = gpu_ctx(C.C1_BOX, flat, x, y, cols)
    R.set_option(rjmod.OPT_PASS, variant)
    P = oracle.Polys(flat, C.C1_BOX)
    cases = [
        dict(agg="sum", agg_column=0, preds=[]),                                   # integer SUM: exact
        dict(agg="sum", agg_column=1, preds=[(0, ">", -10.5)]),
        dict(agg="avg", agg_column=1, preds=[(1, ">=", 2.0), (1, "<=", 8.0)]),
        dict(agg="avg", agg_column=0, preds=[(0, "==", 7.0)]),
        dict(agg="count", preds=[(0, "==", 7.5)]),                                 # never
        dict(agg="count", preds=[(0, "<", 1e12), (1, ">", -1e30)]),
        dict(agg="avg", agg_column=0, preds=[(0, ">=", 10), (0, "<", 10)]),       # empty range: NaN
    ]
    for cs in cases:
        cnt, val = R.query(W=1024, H=1024, mode=mode, **cs)
        pc = [(c_, op, v) for c_, op, v in cs["preds"]]
        ocnt, osum, _ = oracle.query(P, x, y, cols=cols, preds=pc, agg_col=cs.get("agg_column", -1),
                                     W=1024, H=1024, mode=mode)
        assert np.array_equal(cnt, ocnt), cs
        if cs["agg"] == "sum":
            if cs["agg_column"] == 0:
                assert np.array_equal(val, osum), cs
            ok, bad = rel_close(val, osum)
            assert ok, (cs, bad)
        elif cs["agg"] == "avg":
            ok, bad = rel_close(val, oracle.avg(ocnt, osum))
            assert ok, (cs, bad)


@pytest.mark.parametrize("mode", ["bounded", "accurate"])
def test_label_widths_many_polygons(mode):
    """Polygon ids beyond 16 bits through the label kernel (SUM/AVG): a grid
    of 257^2 = 66049 squares (non-dyadic side), and its first 1000 squares;
    SUM of an integer attribute is bit-exact in both."""
    m = 257
    s = 1024.0 / m
    ii, jj = np.meshgrid(np.arange(m), np.arange(m), indexing="xy")
    x0, y0 = (ii.ravel() * s), (jj.ravel() * s)
    x1, y1 = np.minimum(1024.0, x0 + s), np.minimum(1024.0, y0 + s)
    n = m * m
    vx = np.stack([x0, x1, x1, x0], 1).ravel()
    vy = np.stack([y0, y0, y1, y1], 1).ravel()
    pts = C.c1_points(20000)
    rng = np.random.default_rng(5)
    fav = rng.integers(0, 9, 20000).astype(np.int32)
    for k in (1000, n):
        flat = (np.arange(k + 1, dtype=np.uint32), np.arange(k + 1, dtype=np.uint32) * 4, vx[:4 * k], vy[:4 * k])
        R = gpu_ctx(C.C1_BOX, flat, pts["x"], pts["y"], [fav])
        P = oracle.Polys(flat, C.C1_BOX)
        cnt, val = R.query(W=700, H=700, mode=mode, agg="sum", agg_column=0)
        ocnt, osum, _ = oracle.query(P, pts["x"], pts["y"], cols=[fav], agg_col=0, W=700, H=700, mode=mode)
        assert np.array_equal(cnt, ocnt), k
        assert np.array_equal(val, osum), k
        R.close()


# ------------------------------------------------------------- edge cases
def test_empty_and_degenerate_point_sets():
    flat = PG.flatten(C.polygon_set("c1"))
    P = oracle.Polys(flat, C.C1_BOX)
    for n in (0, 1, 7, 8, 9, 255, 257):
        pts = C.c1_points(n) if n else {"x": np.zeros(0), "y": np.zeros(0)}
        R = gpu_ctx(C.C1_BOX, flat, pts["x"], pts["y"])
        for mode in ("bounded", "accurate"):
            cnt, val = R.query(W=1024, mode=mode, agg="count")
            ocnt, _, _ = oracle.query(P, pts["x"], pts["y"], W=1024, H=1024, mode=mode)
            assert np.array_equal(cnt, ocnt), n
        R.close()
    # all points out of domain (and on x = X1 exactly, NaN)
    x = np.array([-1.0, 1024.0, 5.0, np.nan, 2000.0])
    y = np.array([5.0, 5.0, 1024.0, 5.0, -3.0])
    R = rjmod.RasterJoin(C.C1_BOX)
    assert R.load_points(x, y) == 5
    R.load_polygons(flat)
    cnt, val = R.query(W=64, mode="accurate", agg="count")
    assert cnt.sum() == 0 and R.stats()["n_points"] == 0


def test_float32_coords_and_device_pointers():
    import torch
    flat = PG.flatten(C.polygon_set("c1"))
    P = oracle.Polys(flat, C.C1_BOX)
    pts = C.c1_points(50000)
    x32, y32 = pts["x"].astype(np.float32), pts["y"].astype(np.float32)
    R = rjmod.RasterJoin(C.C1_BOX)
    R.load_points(torch.from_numpy(x32).cuda(), torch.from_numpy(y32).cuda())
    R.load_polygons(flat)
    cnt, _ = R.query(W=777, H=555, mode="accurate")
    ocnt, _, _ = oracle.query(P, x32, y32, W=777, H=555, mode="accurate")
    assert np.array_equal(cnt, ocnt)


def test_errors():
    flat = PG.flatten(C.polygon_set("c1"))
    R = rjmod.RasterJoin(C.C1_BOX)
    with pytest.raises(rjmod.RJError) as e:
        R.n_poly = 10
        R.query(W=64)
    assert e.value.status == -1                       # query before load
    pts = C.c1_points(100)
    R.load_points(pts["x"], pts["y"], [np.zeros(100, np.int32)])
    R.load_polygons(flat)
    for kw in (dict(agg="sum", agg_column=3), dict(preds=[(5, "<", 1)]), dict(preds=[(0, "<", 1)] * 6)):
        with pytest.raises((rjmod.RJError, ValueError)):
            R.query(W=64, **kw)
    with pytest.raises(rjmod.RJError) as e:
        R.query(W=131073)                             # reading Z21: cap 2^17
    assert e.value.status == -3
    bad = PG.flatten([[np.array([(0, 0), (2000, 0), (0, 5)], float)]])
    with pytest.raises(rjmod.RJError) as e:
        R.load_polygons(bad)
    assert e.value.status == -2
    tri2 = (np.array([0, 1], np.uint32), np.array([0, 2], np.uint32), np.zeros(2), np.zeros(2))
    with pytest.raises(rjmod.RJError) as e:
        R.load_polygons(tri2)
    assert e.value.status == -1


# ------------------------------------------------------ realistic workloads
@pytest.mark.parametrize("W", [8192, 4096, 1500])
def test_taxi_neighborhoods_bounded_time_filter(W):
    """C2 shape on a 2M-point prefix: COUNT, calendar-2012 filter, bounded."""
    flat = C.array_polys("neighborhoods")
    pts = C.taxi(2_000_000)
    R = gpu_ctx(C.NYC_BOX, flat, pts["x"], pts["y"], [pts["t"]])
    P = oracle.Polys(flat, C.NYC_BOX)
    preds = [(0, ">=", C.T_2012[0]), (0, "<", C.T_2012[1])]
    cnt, _ = R.query(W=W, H=W, mode="bounded", preds=preds)
    ocnt, _, kept = oracle.query(P, pts["x"], pts["y"], cols=[pts["t"]], preds=preds, W=W, H=W, mode="bounded")
    assert np.array_equal(cnt, ocnt)
    assert int(cnt.sum()) == kept == R.stats()["n_filtered"]          # exact tiling


def test_tracts_accurate_avg_fare():
    """C3 shape on a 1M-point prefix: AVG(fare), accurate, 8192^2."""
    flat = C.array_polys("tracts")
    pts = C.taxi(1_000_000, fare=True)
    R = gpu_ctx(C.NYC_BOX, flat, pts["x"], pts["y"], [pts["t"], pts["fare"]])
    P = oracle.Polys(flat, C.NYC_BOX)
    cnt, val = R.query(W=8192, H=8192, mode="accurate", agg="avg", agg_column=1)
    ocnt, osum, kept = oracle.query(P, pts["x"], pts["y"], cols=[pts["t"], pts["fare"]], agg_col=1,
                                    W=8192, H=8192, mode="accurate")
    assert np.array_equal(cnt, ocnt)
    ok, bad = rel_close(val, oracle.avg(ocnt, osum))
    assert ok, bad
    st = R.stats()
    assert st["n_boundary"] > 0 and int(cnt.sum()) == kept


def test_counties_sum_fav_epsilon():
    """C4 shape on a 1M-point prefix: SUM(fav) + COUNT, bounded, eps = 1 km."""
    flat = C.array_polys("counties")
    pts = C.twitter(1_000_000)
    R = gpu_ctx(C.US_BOX, flat, pts["x"], pts["y"], [pts["fav"]])
    P = oracle.Polys(flat, C.US_BOX)
    cnt, val = R.query(epsilon=1000.0, mode="bounded", agg="sum", agg_column=0)
    assert R.stats()["W"] == 6506 and R.stats()["H"] == 4102
    ocnt, osum, _ = oracle.query(P, pts["x"], pts["y"], cols=[pts["fav"]], agg_col=0, W=6506, H=4102,
                                 mode="bounded")
    assert np.array_equal(cnt, ocnt)
    assert np.array_equal(val, osum)            # integer attribute: bit-exact


def test_sharding_sums_to_unsharded():
    """Point shards add up (distributive aggregates)."""
    flat = C.array_polys("neighborhoods")
    pts = C.taxi(600_000, fare=True)
    whole = gpu_ctx(C.NYC_BOX, flat, pts["x"], pts["y"], [pts["fare"]])
    c_all, s_all = whole.query(W=4096, mode="accurate", agg="sum", agg_column=0)
    acc_c = np.zeros_like(c_all)
    acc_s = np.zeros_like(s_all)
    for lo, hi in ((0, 200_000), (200_000, 450_000), (450_000, 600_000)):
        R = gpu_ctx(C.NYC_BOX, flat, pts["x"][lo:hi], pts["y"][lo:hi], [pts["fare"][lo:hi]])
        c, s = R.query(W=4096, mode="accurate", agg="sum", agg_column=0)
        acc_c += c
        acc_s += s
    assert np.array_equal(acc_c, c_all)
    ok, _ = rel_close(acc_s, s_all)
    assert ok


# ---------------------------------------------- nearly axis-parallel edges
def _sliver_set():
    """C1 polygons plus a quad whose right edge is nearly vertical (dx = 3
    lattice units over 800 world units) and whose top edge is nearly
    horizontal: within a pixel row the right edge's x-extent lies strictly
    between two consecutive lattice values inside one pixel's extent.  Round
    2's full-size C3 parity run found tract edges of this kind whose
    boundary pixels the supercover skipped (O9)."""
    u = 2.0 ** -20
    quad = [np.array([(200.0, 100.0), (300.0 + u, 100.0), (300.0 + 4 * u, 900.0 + u), (200.0, 900.0 + 4 * u)], float)]
    tall = [np.array([(600.0, 50.0), (600.0 + 2 * u, 50.0), (600.0 + 3 * u, 1000.0), (599.0, 1000.0)], float)]
    return C.polygon_set("c1") + [quad, tall]


@pytest.mark.parametrize("W,H", [(1024, 1024), (333, 517), (4096, 4096), (8192, 8192)])
def test_nearly_axis_parallel_edges(W, H):
    polys = _sliver_set()
    flat = PG.flatten(polys)
    rng = np.random.default_rng(W + H)
    n = 400_000
    x = rng.uniform(0, 1024, n)
    y = rng.uniform(0, 1024, n)
    # a third of the points hug the nearly vertical edges (inside and outside)
    k = n // 3
    x[:k // 2] = 300.0 + rng.uniform(-0.6, 0.6, k // 2)
    x[k // 2:k] = 600.0 + rng.uniform(-0.6, 0.6, k - k // 2)
    fav = rng.integers(-1000, 1000, n).astype(np.int32)
    R = gpu_ctx(C.C1_BOX, flat, x, y, [fav])
    P = oracle.Polys(flat, C.C1_BOX)
    o = oracle.boundary_mask(P, W, H)
    assert np.array_equal(R.boundary_mask(W=W, H=H), o)
    bnd, cov = R.boundary_pieces(W=W, H=H)
    ob = _unpack_bits(o, W)
    assert np.array_equal(_unpack_bits(bnd, W), ob & _unpack_bits(cov, W))
    for mode in ("bounded", "accurate"):
        for variant in (0, 1):
            R.set_option(rjmod.OPT_PASS, variant)
            cnt, val = R.query(W=W, H=H, mode=mode, agg="sum", agg_column=0)
            ocnt, osum, _ = oracle.query(P, x, y, cols=[fav], agg_col=0, W=W, H=H, mode=mode)
            assert np.array_equal(cnt, ocnt), (mode, variant)
            assert np.array_equal(val, osum), (mode, variant)
    cnt, _ = R.query_stream(x, y, [fav], W=W, H=H, mode="accurate")
    assert np.array_equal(cnt, oracle.query(P, x, y, W=W, H=H, mode="accurate")[0])
    if W <= 1024:
        c_, v_, ep, em = R.query_interval(W=W, H=H)
        counts = oracle.pixel_counts(x, y, C.C1_BOX, W=W, H=H)
        oep, oem = oracle.error_interval(P, W, H, counts)
        assert np.array_equal(ep, oep) and np.array_equal(em, oem)
    R.close()
