"""Pins for the CPU oracle (-m "not gpu").

The oracle (oracle/rj_oracle.c) is checked against what the paper and the
mathematics fix, never against itself: closed forms (half-open rectangle
range counts, pixel-aligned polygons), special cases that reduce to a
textbook test (convex polygon = intersection of half-planes), symmetry,
invariants (an exact tiling partitions the points, the worst-case interval of
PAPER.md P:797-810 holds, bounded converges to accurate) and
brute force on tiny inputs.  Each pin is chosen so that a plausible mistake
(a dropped term, a wrong sign or index, a transposed operand, a closed
instead of half-open bound, reciprocal-multiply quantisation) fails it.
"""
import math

import numpy as np
import pytest

import datagen
import oracle
from datagen import configs as C
from datagen import polygons as PG

TWO30 = 1 << 30
C1 = C.C1_BOX


def rect_count(x, y, a, b, c, d):
    return int(np.sum((x >= a) & (x < b) & (y >= c) & (y < d)))


# ------------------------------------------------------------------- O1 / O2
def test_quantize_dyadic_closed_form():
    # domain [0,1024): (x/1024)*2^30 = x*2^20 exactly for <=20 fractional bits
    rng = np.random.default_rng(1)
    ks = rng.integers(0, 1024 << 20, size=2000)
    for k in ks:
        assert oracle.quantize(k / float(1 << 20), 0.0, 1024.0) == k
    assert oracle.quantize(1024.0, 0.0, 1024.0) == TWO30          # X1 -> exactly 2^30
    assert oracle.quantize(0.0, 0.0, 1024.0) == 0
    assert oracle.quantize(-1e-9, 0.0, 1024.0) == -1               # floor, not truncation
    assert oracle.quantize(float("nan"), 0.0, 1.0) == np.iinfo(np.int64).min


def test_quantize_division_not_reciprocal():
    # X1 must map to exactly 2^30 for every domain (a reciprocal multiply fails
    # this on ~14 % of random domains, SURVEY.md 7 hard part 1)
    rng = np.random.default_rng(2)
    for _ in range(20000):
        x0 = rng.uniform(-1e7, 1e7)
        x1 = x0 + 10 ** rng.uniform(-3, 7)
        assert oracle.quantize(x1, x0, x1) == TWO30
        assert oracle.quantize(x0, x0, x1) == 0


def test_quantize_monotone():
    rng = np.random.default_rng(3)
    v = np.sort(rng.uniform(0, 57920, 5000))
    q = [oracle.quantize(t, 0.0, 57920.0) for t in v]
    assert all(a <= b for a, b in zip(q, q[1:]))


def test_pixel_centre_closed_form_pow2():
    L = oracle.lib()
    for i in range(0, 1024, 7):
        assert L.or_centre(i, 1024) == i * (1 << 20) + (1 << 19)
        assert L.or_pixel(i * (1 << 20), 1024) == i
        assert L.or_pixel(i * (1 << 20) - 1, 1024) == i - 1


@pytest.mark.parametrize("W", [1, 2, 3, 5, 7, 11, 13, 1000, 1024, 4102, 6506, 8191, 32768, 81912, 131072])
def test_pixel_extent_and_centre(W):
    # qlo(i) is the first lattice point of pixel i; the centre lies in the pixel
    L = oracle.lib()
    idx = sorted(set([0, 1, W // 2, W - 2, W - 1]) & set(range(W)))
    for i in idx:
        lo, hi, c = L.or_qlo(i, W), L.or_qhi(i, W), L.or_centre(i, W)
        assert L.or_pixel(lo, W) == i and L.or_pixel(hi, W) == i
        assert lo == 0 or L.or_pixel(lo - 1, W) == i - 1
        assert lo <= c <= hi
        # centre = floor of the exact midpoint of the real interval [i, i+1) * 2^30/W
        assert c == math.floor((2 * i + 1) * (1 << 29) / W) or c == ((2 * i + 1) * (1 << 29)) // W
    assert L.or_qhi(W - 1, W) == TWO30 - 1


def test_resolve_epsilon():
    # NYC-like width 57,920 m: eps 80/40/20/10 m -> 1024/2048/4096/8192
    # (the paper: eps = 20 m ~ "approximately 4k x 4k")
    for eps, W in ((80, 1024), (40, 2048), (20, 4096), (10, 8192)):
        assert oracle.resolve(57920.0, 57920.0, eps) == (W, W)
    assert oracle.resolve(4.6e6, 2.9e6, 1000.0) == (6506, 4102)   # C4, eps = 1 km
    # reading Z21: canvases up to 2^17 a side (eps = 1 m on NYC: ceil(57920 sqrt 2) = 81912)
    assert oracle.resolve(57920.0, 57920.0, 1.0) == (81912, 81912)
    assert oracle.resolve(131072.0 / math.sqrt(2.0), 1.0, 1.0)[0] in (131072,)  # the cap itself
    assert oracle.resolve(57920.0, 57920.0, 0.5) is None            # 163824 > 131072
    assert oracle.resolve(1.0, 1.0, 0.0) is None
    assert oracle.resolve(1.0, 1.0, float("nan")) is None


# ----------------------------------------------------------------------- O3
def _lattice_polys(rings_list, box=(0.0, 0.0, 1024.0, 1024.0)):
    return oracle.Polys(PG.flatten(rings_list), box)


def test_rectangle_half_open_ties():
    # axis-aligned rectangle [a,b) x [c,d) in lattice units: inside iff a<=px<b, c<=py<d
    rng = np.random.default_rng(4)
    for _ in range(40):
        a, b = sorted(rng.integers(0, 1000, 2)) ; b += 2
        c, d = sorted(rng.integers(0, 1000, 2)) ; d += 2
        S = 1.0 / (1 << 20)   # lattice unit in world units on [0,1024)
        poly = [[np.array([(a, c), (b, c), (b, d), (a, d)], dtype=np.float64) * S]]
        if rng.integers(2):    # orientation must not matter
            poly = [[poly[0][0][::-1].copy()]]
        P = _lattice_polys(poly)
        for px in (a - 1, a, a + 1, b - 1, b, b + 1):
            for py in (c - 1, c, c + 1, d - 1, d, d + 1):
                assert P.pnpoly(0, px, py) == (a <= px < b and c <= py < d)


def test_unit_squares_partition():
    # 4 unit squares tiling [0,2)^2 (world units): every lattice point on a
    # shared edge or vertex lands in exactly one square
    sq = lambda x, y: [np.array([(x, y), (x + 1, y), (x + 1, y + 1), (x, y + 1)], dtype=np.float64)]
    P = _lattice_polys([sq(0, 0), sq(1, 0), sq(0, 1), sq(1, 1)])
    U = 1 << 20
    for px in (0, 1, U - 1, U, U + 1, 2 * U - 1):
        for py in (0, 1, U - 1, U, U + 1, 2 * U - 1):
            owners = [k for k in range(4) if P.pnpoly(k, px, py)]
            assert len(owners) == 1
            assert owners[0] == (px >= U) + 2 * (py >= U)
    assert not any(P.pnpoly(k, 2 * U, 5) for k in range(4))


def _on_edge(ring, px, py):
    for (xa, ya), (xb, yb) in zip(ring, np.roll(ring, -1, axis=0)):
        if (xb - xa) * (py - ya) - (yb - ya) * (px - xa) == 0 and min(xa, xb) <= px <= max(xa, xb) \
                and min(ya, yb) <= py <= max(ya, yb):
            return True
    return False


def _hull(pts):
    """Andrew's monotone chain, strictly convex, CCW."""
    P = sorted(set(map(tuple, pts)))
    if len(P) < 3:
        return np.array(P)
    cross = lambda o, a, b: (a[0] - o[0]) * (b[1] - o[1]) - (a[1] - o[1]) * (b[0] - o[0])
    lo, hi = [], []
    for p in P:
        while len(lo) >= 2 and cross(lo[-2], lo[-1], p) <= 0:
            lo.pop()
        lo.append(p)
    for p in reversed(P):
        while len(hi) >= 2 and cross(hi[-2], hi[-1], p) <= 0:
            hi.pop()
        hi.append(p)
    return np.array(lo[:-1] + hi[:-1], dtype=np.float64)


def test_convex_equals_halfplanes():
    # textbook special case: for a CCW convex polygon, a point off the boundary
    # is inside iff it is strictly left of every edge
    rng = np.random.default_rng(5)
    for trial in range(60):
        k = rng.integers(3, 12)
        ang = np.sort(rng.uniform(0, 2 * np.pi, k))
        R = rng.uniform(50, 400)
        cx, cy = rng.uniform(R, 1024 - R, 2)
        raw = np.stack([np.round(cx + R * np.cos(ang)), np.round(cy + R * np.sin(ang))], 1)
        ring = _hull(raw)         # strictly convex CCW ring (rounding can break convexity)
        if len(ring) < 3:
            continue
        P = _lattice_polys([[ring]])
        U = 1 << 20
        lat = (ring * U).astype(np.int64)
        pts = rng.integers(int((cx - R - 5) * U), int((cx + R + 5) * U), size=(400, 2))
        for px, py in pts:
            if _on_edge(lat, px, py):
                continue
            cr = [(xb - xa) * (py - ya) - (yb - ya) * (px - xa)
                  for (xa, ya), (xb, yb) in zip(lat, np.roll(lat, -1, axis=0))]
            assert P.pnpoly(0, px, py) == all(c > 0 for c in cr)


def test_symmetry_mirror_and_rotate():
    # even-odd membership off the boundary is invariant under mirroring and a
    # 90-degree rotation of polygon and point together (catches a ray-direction
    # or inequality-direction mistake that the tie pins might not)
    rng = np.random.default_rng(6)
    polys = C.polygon_set("c1b")
    U = 1 << 20
    for pid, poly in enumerate(polys):
        mir = [[np.stack([1024.0 - r[:, 0], r[:, 1]], 1) for r in poly]]
        rot = [[np.stack([1024.0 - r[:, 1], r[:, 0]], 1) for r in poly]]
        P0, PM, PR = _lattice_polys([poly]), _lattice_polys(mir), _lattice_polys(rot)
        lat = [np.round(r * U).astype(np.int64) for r in poly]
        pts = rng.integers(1, 1024 * U - 1, size=(300, 2))
        for px, py in pts:
            if any(_on_edge(r, px, py) for r in lat):
                continue
            v = P0.pnpoly(0, px, py)
            assert PM.pnpoly(0, 1024 * U - px, py) == v
            assert PR.pnpoly(0, 1024 * U - py, px) == v


# -------------------------------------------------------------- C1 closed forms
@pytest.fixture(scope="module")
def c1():
    polys = oracle.Polys(C.array_polys("c1"), C1)
    pts = C.c1_points()
    ax, ay = PG.c1b_points(C.polygon_set("c1b"))
    x = np.concatenate([pts["x"], ax])
    y = np.concatenate([pts["y"], ay])
    return polys, x, y


def test_c1_closed_forms(c1):
    polys, x, y = c1
    cb, _, kb = oracle.query(polys, x, y, W=1024, H=1024, mode="bounded")
    ca, _, ka = oracle.query(polys, x, y, W=1024, H=1024, mode="accurate")
    assert kb == ka == len(x)
    r = lambda *a: rect_count(x, y, *a)
    # P0 square on pixel borders: both modes
    assert cb[0] == ca[0] == r(100, 200, 100, 200)
    # P1 vertices on pixel centres: bounded uses centres, accurate the points
    assert cb[1] == r(300, 400, 100, 200)
    assert ca[1] == r(300.5, 400.5, 100.5, 200.5)
    # P4 L-shape
    L = r(100, 300, 400, 450) + r(100, 150, 450, 600)
    assert cb[4] == ca[4] == L
    # P6 annulus (hole)
    assert cb[6] == ca[6] == r(700, 950, 400, 650) - r(775, 875, 475, 575)
    # P7 comb
    comb = r(100, 400, 700, 750) + r(150, 200, 750, 950) + r(250, 300, 750, 950) + r(350, 400, 750, 950)
    assert cb[7] == ca[7] == comb
    # P8 square overlapping the hexagon (multi-count is allowed)
    assert cb[8] == ca[8] == r(820, 1000, 150, 330)
    # P9 shares x=200 with P0: x = 200 exactly counts in P9, not P0
    assert cb[9] == ca[9] == r(200, 300, 100, 200)
    assert np.sum((x == 200) & (y >= 100) & (y < 200)) > 0


def test_c1_convex_polys_halfplane(c1):
    # P2 triangle and P3 hexagon (convex, CCW): accurate count = points strictly
    # left of all edges, plus boundary points, which are decided by the tie rule;
    # compare on off-boundary points only, with numpy cross products
    polys, x, y = c1
    U = 1 << 20
    qx = np.floor(x * U).astype(np.int64)
    qy = np.floor(y * U).astype(np.int64)
    bits = oracle.membership(polys, x, y, W=1024, H=1024, mode="accurate")
    for pid in (2, 3):
        ring = np.round(C.polygon_set("c1")[pid][0] * U).astype(np.int64)
        ins = np.ones(len(x), dtype=bool)
        zero = np.zeros(len(x), dtype=bool)
        for (xa, ya), (xb, yb) in zip(ring, np.roll(ring, -1, axis=0)):
            cr = (xb - xa) * (qy - ya) - (yb - ya) * (qx - xa)
            ins &= cr > 0
            zero |= cr == 0
        got = (bits >> np.uint64(pid)) & np.uint64(1)
        assert np.array_equal(got[~zero].astype(bool), ins[~zero])


# ---------------------------------------------------------- O2/O3 pixel spans
# or_pixel_spans is the expected value of the GPU span test (S3): its pins are
# closed forms in exact integer arithmetic on the REAL pixel centres
# cx(i) = (2i+1)*512/W world units on the C1 domain [0,1024) (P:561-562
# pixel-centre rule), not the oracle's floored lattice centres: for a
# rectilinear polygon with integer or half-integer vertices, floor(c*2^20) >= k
# iff c*2^20 >= k for an integer lattice value k, so the two agree exactly.

# rectilinear C1 polygons as signed half-open rectangles (x0, x1, y0, y1, sign)
_RECTS = {
    0: [(100, 200, 100, 200, 1)],
    1: [(300.5, 400.5, 100.5, 200.5, 1)],
    4: [(100, 300, 400, 450, 1), (100, 150, 450, 600, 1)],                    # L-shape
    6: [(700, 950, 400, 650, 1), (775, 875, 475, 575, -1)],                   # annulus
    7: [(100, 400, 700, 750, 1)] + [(a, a + 50, 750, 950, 1) for a in (150, 250, 350)],   # comb
    8: [(820, 1000, 150, 330, 1)],
    9: [(200, 300, 100, 200, 1)],
}


def _centre_in(v0, v1, k, n):
    """v0 <= (2k+1)*512/n < v1 for integer arrays k (2*v integer): exact."""
    t = (2 * k + 1) * 1024
    return (int(round(2 * v0)) * n <= t) & (t < int(round(2 * v1)) * n)


def _runs(row_mask):
    out = []
    for r in range(row_mask.shape[0]):
        m = np.concatenate([[0], row_mask[r].astype(np.int8), [0]])
        d = np.diff(m)
        for lo, hi in zip(np.nonzero(d == 1)[0], np.nonzero(d == -1)[0]):
            out.append((r, lo, hi))
    return np.asarray(out, dtype=np.int64).reshape(-1, 3)


@pytest.mark.parametrize("W,H", [(1024, 1024), (333, 517), (64, 48), (1500, 97)])
def test_pixel_spans_rectilinear_closed_form(W, H):
    polys = oracle.Polys(PG.flatten(C.polygon_set("c1")), C1)
    cols, rows = np.arange(W, dtype=np.int64), np.arange(H, dtype=np.int64)
    for pid, rects in _RECTS.items():
        m = np.zeros((H, W), dtype=np.int64)
        for x0, x1, y0, y1, sg in rects:
            m += sg * np.outer(_centre_in(y0, y1, rows, H), _centre_in(x0, x1, cols, W)).astype(np.int64)
        assert m.min() >= 0 and m.max() <= 1
        got = oracle.pixel_spans(polys, pid, W, H).astype(np.int64)
        assert np.array_equal(got, _runs(m)), (pid, W, H)
    # the hand-readable case: P0 at 1024^2 is rows 100..199, each [100, 200);
    # P1's centres i + 0.5 lie in [300.5, 400.5) for i = 300..399
    sp0 = oracle.pixel_spans(polys, 0, 1024, 1024)
    assert sp0.tolist() == [[r, 100, 200] for r in range(100, 200)]
    sp1 = oracle.pixel_spans(polys, 1, 1024, 1024)
    assert sp1.tolist() == [[r, 300, 400] for r in range(100, 200)]
    # comb row 800 (y = 800.5): three teeth [150,200), [250,300), [350,400)
    sp7 = oracle.pixel_spans(polys, 7, 1024, 1024)
    assert sp7[sp7[:, 0] == 800][:, 1:].tolist() == [[150, 200], [250, 300], [350, 400]]
    # annulus row 500 crosses the hole: [700,775) and [875,950)
    sp6 = oracle.pixel_spans(polys, 6, 1024, 1024)
    assert sp6[sp6[:, 0] == 500][:, 1:].tolist() == [[700, 775], [875, 950]]


@pytest.mark.parametrize("W,H", [(1024, 1024), (333, 517), (777, 211)])
def test_pixel_spans_triangle_halfplanes(W, H):
    """P2 (convex triangle, CCW): a centre is inside iff it is strictly left of
    all three edges.  Exact integer orientation at the real centre
    ((2i+1)*512/W, (2r+1)*512/H), scaled by W*H; pixels whose centre lies
    within 2^-18 world units of an edge line are left out (the lattice floor
    moves a centre by < 2^-19; exact ties are the half-open rule's, pinned by
    test_rectangle_half_open_ties)."""
    polys = oracle.Polys(PG.flatten(C.polygon_set("c1")), C1)
    ring = np.asarray(C.polygon_set("c1")[2][0], dtype=np.int64)
    i = np.arange(W, dtype=np.int64)[None, :]
    r = np.arange(H, dtype=np.int64)[:, None]
    cxs = (2 * i + 1) * 512 * H           # centre x * W * H
    cys = (2 * r + 1) * 512 * W           # centre y * W * H
    ins = np.ones((H, W), dtype=bool)
    near = np.zeros((H, W), dtype=bool)
    for (xa, ya), (xb, yb) in zip(ring, np.roll(ring, -1, axis=0)):
        cr = (xb - xa) * (cys - ya * W * H) - (yb - ya) * (cxs - xa * W * H)
        ins &= cr > 0
        near |= np.abs(cr) <= math.hypot(xb - xa, yb - ya) * W * H * 2.0 ** -18
    got = np.zeros((H, W), dtype=bool)
    for row, lo, hi in oracle.pixel_spans(polys, 2, W, H).tolist():
        assert not got[row, lo:hi].any()               # spans are disjoint, sorted
        got[row, lo:hi] = True
    assert near.sum() < 0.02 * ins.sum() and ins.sum() > 0
    assert np.array_equal(got[~near], ins[~near]), (W, H)


# ------------------------------------------------------------------ filters/SUM
def test_filter_identity_and_sum_identities():
    polys = oracle.Polys(C.array_polys("c1"), C1)
    pts = C.c1_points(50000)
    x, y = pts["x"], pts["y"]
    rng = np.random.default_rng(7)
    ti = rng.integers(-1000, 1000, len(x)).astype(np.int32)
    tf = rng.normal(0, 10, len(x)).astype(np.float32)
    ones = np.ones(len(x), dtype=np.int32)
    preds = [(0, ">=", -250.5), (0, "<", 600.0), (1, ">", -3.25)]
    c, s, k = oracle.query(polys, x, y, cols=[ti, tf, ones], preds=preds, agg_col=2, mode="accurate")
    m = (ti >= -250.5) & (ti < 600) & (tf > np.float32(-3.25))
    c2, _, k2 = oracle.query(polys, x[m], y[m], mode="accurate")
    assert k == k2 == int(m.sum())
    assert np.array_equal(c, c2)                      # COUNT(filter) = COUNT(prefiltered)
    assert np.array_equal(s, c.astype(np.float64))    # attr == 1 => SUM == COUNT exactly
    # integer attribute over the P0 rectangle: exact closed form
    _, s0, _ = oracle.query(polys, x, y, cols=[ti], agg_col=0, mode="accurate")
    box = (x >= 100) & (x < 200) & (y >= 100) & (y < 200)
    assert s0[0] == float(ti[box].astype(np.int64).sum())
    # EQ on int32 with a non-integer constant never passes; NaN never passes
    c3, _, k3 = oracle.query(polys, x, y, cols=[ti], preds=[(0, "==", 0.5)])
    assert k3 == 0 and c3.sum() == 0
    tn = tf.copy(); tn[::2] = np.nan
    _, _, k4 = oracle.query(polys, x, y, cols=[tn], preds=[(0, "<=", 1e30)])
    assert k4 == len(x) // 2
    avg = oracle.avg(np.array([0, 4], np.uint64), np.array([0.0, 10.0]))
    assert math.isnan(avg[0]) and avg[1] == 2.5


# ------------------------------------------------------------------ invariants
@pytest.mark.parametrize("name,n,W", [("neighborhoods", 60000, 8192), ("tracts", 20000, 4096)])
def test_tiling_partition(name, n, W):
    # exact tiling of the domain: every kept point is in exactly one polygon, in
    # both modes (centre representatives are lattice points too)
    polys = oracle.Polys(C.array_polys(name), C.NYC_BOX)
    pts = C.taxi(n)
    for mode in ("bounded", "accurate"):
        bits_total = 0
        c, _, k = oracle.query(polys, pts["x"], pts["y"], W=W, H=W, mode=mode)
        assert int(c.sum()) == k
        assert k >= n - 5      # only float32 rounding onto x = 57920 may drop points
    # plus: no point double-counted (sum == kept and each point at least once)


def test_counties_partition():
    polys = oracle.Polys(C.array_polys("counties"), C.US_BOX)
    pts = C.twitter(20000)
    c, _, k = oracle.query(polys, pts["x"], pts["y"], W=6506, H=4102, mode="bounded")
    assert int(c.sum()) == k
    c, _, k = oracle.query(polys, pts["x"], pts["y"], mode="accurate")
    assert int(c.sum()) == k


@pytest.mark.parametrize("W", [16, 64, 200])
def test_error_interval_holds(W):
    # worst-case interval [A - e+, A + e-] of P:797-810 ("100 % confidence")
    polys = oracle.Polys(C.array_polys("c1b"), C1)
    pts = C.c1_points(30000)
    ax, ay = PG.c1b_points(C.polygon_set("c1b"))
    x = np.concatenate([pts["x"], ax]); y = np.concatenate([pts["y"], ay])
    cb, _, _ = oracle.query(polys, x, y, W=W, H=W, mode="bounded")
    ca, _, _ = oracle.query(polys, x, y, W=W, H=W, mode="accurate")
    cnt = oracle.pixel_counts(x, y, C1, W=W, H=W)
    ep, em = oracle.error_interval(polys, W, W, cnt)
    cb, ca = cb.astype(np.int64), ca.astype(np.int64)
    assert np.all(ca >= cb - ep.astype(np.int64)) and np.all(ca <= cb + em.astype(np.int64))
    assert np.any(ca != cb)          # non-trivial at this resolution


def _seg_dist(px, py, xa, ya, xb, yb):
    dx, dy = xb - xa, yb - ya
    L2 = dx * dx + dy * dy
    t = np.clip(((px - xa) * dx + (py - ya) * dy) / np.where(L2 > 0, L2, 1), 0, 1)
    return np.hypot(px - (xa + t * dx), py - (ya + t * dy))


def test_convergence_away_from_edges():
    # points farther than delta from every edge have bounded == accurate once the
    # pixel diagonal is below delta
    polys_l = C.polygon_set("c1")
    polys = oracle.Polys(C.array_polys("c1"), C1)
    pts = C.c1_points(20000)
    x, y = pts["x"], pts["y"]
    d = np.full(len(x), np.inf)
    for poly in polys_l:
        for r in poly:
            for (xa, ya), (xb, yb) in zip(r, np.roll(r, -1, axis=0)):
                d = np.minimum(d, _seg_dist(x, y, xa, ya, xb, yb))
    far = d > 1.5
    for W in (1024, 2048):        # diagonal sqrt(2) and sqrt(2)/2 < 1.5
        mb = oracle.membership(polys, x, y, W=W, H=W, mode="bounded")
        ma = oracle.membership(polys, x, y, W=W, H=W, mode="accurate")
        assert np.array_equal(mb[far], ma[far])
    mb = oracle.membership(polys, x, y, W=64, H=64, mode="bounded")
    ma = oracle.membership(polys, x, y, W=64, H=64, mode="accurate")
    assert not np.array_equal(mb[far], ma[far])   # and it is not trivially true


# --------------------------------------------------------------------- O9 mask
def test_boundary_mask_pixel_aligned_square():
    polys = oracle.Polys(PG.flatten([[np.array([(100, 100), (200, 100), (200, 200), (100, 200)], float)]]), C1)
    m = oracle.boundary_mask(polys, 1024, 1024)
    bits = np.unpackbits(m.view(np.uint8), bitorder="little").reshape(1024, -1)[:, :1024]
    want = np.zeros((1024, 1024), dtype=np.uint8)
    want[100:201, 100] = want[100:201, 200] = 1
    want[100, 100:201] = want[200, 100:201] = 1
    assert np.array_equal(bits, want)          # 400 pixels: a naive raster marks 99/199 too


def test_boundary_mask_diagonal():
    polys = oracle.Polys(PG.flatten([[np.array([(0.5, 0.5), (10.5, 10.5), (0.5, 10.5)], float)]]), C1)
    m = oracle.boundary_mask(polys, 1024, 1024)
    bits = np.unpackbits(m.view(np.uint8), bitorder="little").reshape(1024, -1)[:, :1024]
    diag = {(i, i) for i in range(11)}
    top = {(10, i) for i in range(11)}
    left = {(i, 0) for i in range(11)}
    got = {(r, c) for r, c in zip(*np.nonzero(bits))}
    assert got == diag | top | left


def _sliver_polys():
    """A quad whose right edge is nearly vertical (dx = 3 lattice units over
    800 world units, 2^-20 world units per lattice unit on the C1 domain) and
    whose top edge is nearly horizontal (dy = 3 units): in every pixel row /
    column its x- (y-) extent lies strictly between two consecutive lattice
    values inside ONE pixel's extent (the full-size C3 finding of round 2)."""
    u = 2.0 ** -20
    return [[np.array([(200.0, 100.0), (300.0 + u, 100.0), (300.0 + 4 * u, 900.0 + u), (200.0, 900.0 + 4 * u)], float)]]


def test_boundary_mask_nearly_axis_parallel_edges():
    """O9 on edges that never cross a lattice column (row) inside a pixel
    row (column): the closed pixel rectangles they pass through are the
    boundary pixels -- pixel column 300 on every row 100..900 (the right
    edge) and pixel row 900 on every column 200..300 (the top edge), closed
    form at 1024^2 where pixel i spans lattice [i 2^20, (i+1) 2^20 - 1]."""
    polys = oracle.Polys(PG.flatten(_sliver_polys()), C1)
    m = oracle.boundary_mask(polys, 1024, 1024)
    bits = np.unpackbits(m.view(np.uint8), bitorder="little").reshape(1024, -1)[:, :1024].astype(bool)
    assert bits[100:901, 300].all()                 # right edge: every row of its extent
    assert bits[900, 200:301].all()                 # top edge: every column
    assert bits[100:901, 200].all() and bits[100, 200:301].all()
    assert bits.sum() == 801 + 801 + 101 + 101 - 4


def test_boundary_mask_brute_force_tiny():
    # brute force over every lattice point of a tiny domain: a pixel is a
    # boundary pixel iff some lattice point of it lies on an edge, or its
    # lattice points do not all share the centre's membership -- check the
    # implication L4 (non-boundary => uniform membership) exhaustively
    rng = np.random.default_rng(8)
    S = 1 << 24                    # use only a 64 x 64 corner of the lattice, W = 2^30 / 2^24 ...
    W = 1 << 10                    # pixel = 2^20 lattice units; test region = 3x3 pixels at 2^18 sampling
    for trial in range(6):
        ring = rng.uniform(0.2, 2.8, size=(rng.integers(3, 7), 2))
        polys = oracle.Polys(PG.flatten([[ring]]), C1)
        m = oracle.boundary_mask(polys, W, W)
        for r in range(3):
            for i in range(3):
                isb = bool(m[r, i // 32] >> (i % 32) & 1)
                if isb:
                    continue
                L = oracle.lib()
                c = polys.pnpoly(0, L.or_centre(i, W), L.or_centre(r, W))
                xs = np.linspace(i << 20, ((i + 1) << 20) - 1, 17).astype(np.int64)
                ys = np.linspace(r << 20, ((r + 1) << 20) - 1, 17).astype(np.int64)
                for px in xs:
                    for py in ys:
                        assert polys.pnpoly(0, px, py) == c


# ---------------------------------------------------------------------- O11
def _minmax_brute(P, x, y, cols, agg_col, W, mode):
    """Per-polygon min / max from the (separately pinned) membership bits and
    numpy: the aggregation step of O11 checked by brute force."""
    bits = oracle.membership(P, x, y, cols=cols, W=W, H=W, mode=mode)
    v = cols[agg_col]
    mn = np.full(P.n, np.nan)
    mx = np.full(P.n, np.nan)
    for p in range(P.n):
        sel = ((bits >> np.uint64(p)) & np.uint64(1)).astype(bool)
        if sel.any():
            mn[p] = v[sel].min()
            mx[p] = v[sel].max()
    return mn, mx


@pytest.mark.parametrize("mode", ["bounded", "accurate"])
def test_minmax_brute_force(mode):
    polys = C.polygon_set("c1b")                  # overlaps + holes
    P = oracle.Polys(PG.flatten(polys), C1)
    pts = C.c1_points(20000)
    x, y = pts["x"], pts["y"]
    rng = np.random.default_rng(41)
    ti = rng.integers(-2**31, 2**31 - 1, len(x), dtype=np.int64).astype(np.int32)
    ti[:3] = [-2**31, 2**31 - 1, 0]
    tf = rng.normal(0, 1e6, len(x)).astype(np.float32)
    cols = [ti, tf]
    for col in (0, 1):
        mn, mx = oracle.query_minmax(P, x, y, cols, col, W=64, H=64, mode=mode)
        bmn, bmx = _minmax_brute(P, x, y, cols, col, 64, mode)
        assert np.array_equal(mn, bmn, equal_nan=True), col
        assert np.array_equal(mx, bmx, equal_nan=True), col
    # invariant with O7: min <= avg <= max on non-empty polygons
    cnt, s, _ = oracle.query(P, x, y, cols=cols, agg_col=1, W=64, H=64, mode=mode)
    a = oracle.avg(cnt, s)
    mn, mx = oracle.query_minmax(P, x, y, cols, 1, W=64, H=64, mode=mode)
    ne = cnt > 0
    assert np.all(mn[ne] <= a[ne] * (1 + 1e-12) + 1e-9) and np.all(a[ne] <= mx[ne] * (1 + 1e-12) + 1e-9)
    assert np.all(np.isnan(mn[~ne])) and np.all(np.isnan(mx[~ne]))


def test_minmax_total_order_special_values():
    # one unit square holding every point; IEEE 754 totalOrder on binary32
    sq = [[np.array([(0.0, 0.0), (4.0, 0.0), (4.0, 4.0), (0.0, 4.0)])]]
    far = [[np.array([(100.0, 100.0), (101.0, 100.0), (101.0, 101.0), (100.0, 101.0)])]]   # empty
    P = _lattice_polys(sq + far)
    neg_nan = np.frombuffer(np.uint32(0xFFC00000).tobytes(), np.float32)[0]
    cases = [
        ([0.0, -0.0], (-0.0, 0.0)),              # -0 < +0
        ([1.0, np.nan, -5.0], (-5.0, np.nan)),  # +NaN above everything
        ([neg_nan, 3.0], (neg_nan, 3.0)),       # -NaN below everything
        ([-np.inf, np.inf, 7.0], (-np.inf, np.inf)),
        ([2.5], (2.5, 2.5)),
    ]
    for vals, (emn, emx) in cases:
        k = len(vals)
        x = np.full(k, 1.5)
        y = np.full(k, 1.5)
        v = np.asarray(vals, np.float32)
        mn, mx = oracle.query_minmax(P, x, y, [v], 0, W=8, H=8, mode="accurate")
        for got, exp in ((mn[0], emn), (mx[0], emx)):
            if np.isnan(exp):
                assert np.isnan(got) and np.signbit(got) == np.signbit(exp), vals
            else:
                assert got == exp and np.signbit(got) == np.signbit(exp), vals
        assert np.isnan(mn[1]) and np.isnan(mx[1])          # polygon without points


# ---------------------------------------------------------------- O12 viewport
def _np_pixels(x, y, box, W, H):
    """O1 + O2 restated in numpy (binary64 division, then an exact shift):
    the pixel of every point, -1 for points off the domain."""
    qx = np.floor(((x.astype(np.float64) - box[0]) / (box[2] - box[0])) * 2.0 ** 30)
    qy = np.floor(((y.astype(np.float64) - box[1]) / (box[3] - box[1])) * 2.0 ** 30)
    ok = (qx >= 0) & (qx < 2 ** 30) & (qy >= 0) & (qy < 2 ** 30)
    ix = np.where(ok, (qx.astype(np.int64) * W) >> 30, -1)
    iy = np.where(ok, (qy.astype(np.int64) * H) >> 30, -1)
    return ix, iy


@pytest.mark.parametrize("mode", ["bounded", "accurate"])
def test_view_equals_point_subset(mode):
    # O12: a window query = the full query over the points whose pixel is in
    # the window (pixels recomputed independently in numpy)
    polys = C.polygon_set("c1")
    P = oracle.Polys(PG.flatten(polys), C1)
    pts = C.c1_points(60_000)
    x, y = pts["x"], pts["y"]
    a = (np.arange(len(x)) % 11).astype(np.int32)
    W, H = 700, 1100
    view = (123, 201, 650, 977)
    ix, iy = _np_pixels(x, y, C1, W, H)
    sel = (ix >= view[0]) & (ix < view[2]) & (iy >= view[1]) & (iy < view[3])
    cv, sv, kv = oracle.query(P, x, y, cols=[a], agg_col=0, W=W, H=H, mode=mode, view=view)
    cs, ss, ks = oracle.query(P, x[sel], y[sel], cols=[a[sel]], agg_col=0, W=W, H=H, mode=mode)
    assert kv == ks == int(sel.sum())
    assert np.array_equal(cv, cs) and np.array_equal(sv, ss)
    assert 0 < cv.sum() < oracle.query(P, x, y, W=W, H=H, mode=mode)[0].sum()


@pytest.mark.parametrize("mode", ["bounded", "accurate"])
def test_view_tiles_partition_the_canvas(mode):
    # multi-canvas rendering: windows tiling the canvas count
    # every point-polygon pair exactly once
    polys = C.polygon_set("c1b")
    P = oracle.Polys(PG.flatten(polys), C1)
    pts = C.c1_points(40_000)
    x, y = pts["x"], pts["y"]
    ax, ay = PG.c1b_points(polys)
    x, y = np.concatenate([x, ax]), np.concatenate([y, ay])
    a = (np.arange(len(x)) % 5).astype(np.int32)
    W, H = 1024, 1024
    full_c, full_s, full_k = oracle.query(P, x, y, cols=[a], agg_col=0, W=W, H=H, mode=mode)
    cs, xs = (0, 333, 334, 1024), (0, 512, 1000, 1024)
    tot_c = np.zeros_like(full_c)
    tot_s = np.zeros_like(full_s)
    tot_k = 0
    for i in range(3):
        for j in range(3):
            c, s, k = oracle.query(P, x, y, cols=[a], agg_col=0, W=W, H=H, mode=mode,
                                   view=(cs[i], xs[j], cs[i + 1], xs[j + 1]))
            tot_c += c
            tot_s += s
            tot_k += k
    assert tot_k == full_k
    assert np.array_equal(tot_c, full_c) and np.array_equal(tot_s, full_s)   # integer sums: exact


def test_view_lod_zoom_closed_form():
    # LOD: zooming into a window of a finer canvas.  At W = 8192
    # on [0,1024)^2 a pixel is 1/8 unit; the window of columns [0, 1200) ends
    # at x = 150, so the pixel-aligned square P0 = [100,200)^2 counts exactly
    # the points of [100,150) x [100,200), in both modes.
    polys = C.polygon_set("c1")
    P = oracle.Polys(PG.flatten(polys), C1)
    pts = C.c1_points(100_000)
    x, y = pts["x"], pts["y"]
    for mode in ("bounded", "accurate"):
        c, _, _ = oracle.query(P, x, y, W=8192, H=8192, mode=mode, view=(0, 0, 1200, 8192))
        assert c[0] == rect_count(x, y, 100, 150, 100, 200)
        assert c[9] == 0                                   # P9 = [200,300) x [100,200) is clipped
        c, _, _ = oracle.query(P, x, y, W=8192, H=8192, mode=mode, view=(768, 768, 1792, 1792))
        assert c[0] == rect_count(x, y, 100, 200, 100, 200)


def test_high_resolution_pixel_aligned():
    # reading Z21: at W = 131072 (2^17) on [0,1024)^2 pixels are 2^-7 units;
    # P1's vertices (x.5) are on pixel borders, so bounded = accurate =
    # #[300.5,400.5) x [100.5,200.5) (P1's accurate closed form)
    polys = C.polygon_set("c1")
    P = oracle.Polys(PG.flatten(polys), C1)
    pts = C.c1_points(100_000)
    x, y = pts["x"], pts["y"]
    for mode in ("bounded", "accurate"):
        c, _, _ = oracle.query(P, x, y, W=131072, H=131072, mode=mode)
        assert c[1] == rect_count(x, y, 300.5, 400.5, 100.5, 200.5)
        assert c[0] == rect_count(x, y, 100, 200, 100, 200)
