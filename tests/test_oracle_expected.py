"""Pins for oracle O13, the expected result interval (PAPER.md P:811-827,
reading Z22), -m "not gpu".

f_i(pixel) -- the fraction of the pixel's area inside polygon i -- is pinned
by closed forms (axis-aligned edges at quarter pixels, half-pixel
triangles, a hole), by area conservation against the shoelace formula, by
partition of unity over an exact tiling, and by lemma L4 (off the boundary
f is the centre's membership).  The sums E+ / E- are pinned by the
worst-case interval they must tighten and by the uniform-points estimate
they are meant to be.
"""
import numpy as np
import pytest

import oracle
from datagen import configs as C
from datagen import polygons as PG

C1 = C.C1_BOX


def _polys(rings_list, box=C1):
    return oracle.Polys(PG.flatten(rings_list), box)


def _sq(x0, y0, x1, y1, rev=False):
    r = np.array([(x0, y0), (x1, y0), (x1, y1), (x0, y1)], dtype=np.float64)
    return r[::-1].copy() if rev else r


@pytest.mark.parametrize("rev", [False, True])
def test_fraction_quarter_pixel_square(rev):
    # [100.25, 200.75)^2 at 1024^2 on [0,1024)^2: one world unit = one pixel
    P = _polys([[_sq(100.25, 100.25, 200.75, 200.75, rev)]])
    f = lambda i, r: oracle.area_fraction(P, 0, i, r, 1024, 1024)
    assert f(100, 150) == 0.75 and f(150, 100) == 0.75
    assert f(200, 150) == 0.75 and f(150, 200) == 0.75
    assert f(100, 100) == 0.5625 and f(200, 200) == 0.5625 and f(100, 200) == 0.5625
    assert f(150, 150) == 1.0
    assert f(99, 150) == 0.0 and f(201, 150) == 0.0 and f(150, 201) == 0.0


def test_fraction_half_pixel_triangles():
    P = _polys([[np.array([(10, 10), (12, 10), (10, 12)], dtype=np.float64)],
                [np.array([(0, 0), (1, 0), (0, 1)], dtype=np.float64)]])
    f = lambda p, i, r: oracle.area_fraction(P, p, i, r, 1024, 1024)
    assert f(0, 10, 10) == 1.0
    assert f(0, 11, 10) == 0.5 and f(0, 10, 11) == 0.5
    assert f(0, 11, 11) == 0.0
    assert f(1, 0, 0) == 0.5
    # a 2x coarser canvas: the 2x2-pixel triangle covers half of one pixel
    assert oracle.area_fraction(P, 0, 5, 5, 512, 512) == 0.5


@pytest.mark.parametrize("hole_rev", [False, True])
def test_fraction_hole_either_orientation(hole_rev):
    # annulus: outer [700,950)^2, hole [775.5, 875.5)^2; the hole's ring
    # orientation must not matter (even-odd, O3)
    P = _polys([[_sq(700, 700, 950, 950), _sq(775.5, 775.5, 875.5, 875.5, hole_rev)]])
    f = lambda i, r: oracle.area_fraction(P, 0, i, r, 1024, 1024)
    assert oracle.ring_sigma(P, 0, 0) == 1
    # a clockwise hole already has negative signed area: weight +1
    assert oracle.ring_sigma(P, 0, 1) == (1 if hole_rev else -1)
    assert f(775, 800) == 0.5 and f(875, 800) == 0.5
    assert f(775, 775) == 0.75
    assert f(800, 800) == 0.0 and f(720, 800) == 1.0


def _shoelace(r):
    x, y = r[:, 0], r[:, 1]
    return 0.5 * abs(np.dot(x, np.roll(y, -1)) - np.dot(np.roll(x, -1), y))


@pytest.mark.parametrize("W", [64, 100])
def test_fraction_conserves_area(W):
    # sum over the pixels of f x pixel area = the polygon's even-odd area
    # (outer ring minus holes; the C1 set has no self-intersections)
    polys = C.polygon_set("c1")
    P = oracle.Polys(PG.flatten(polys), C1)
    box_w = C1[2] - C1[0]
    for k, rings in enumerate(polys):
        want = _shoelace(rings[0]) - sum(_shoelace(h) for h in rings[1:])
        xs = np.concatenate([r[:, 0] for r in rings])
        ys = np.concatenate([r[:, 1] for r in rings])
        i0, i1 = int(xs.min() * W / box_w), min(W - 1, int(xs.max() * W / box_w))
        r0, r1 = int(ys.min() * W / box_w), min(W - 1, int(ys.max() * W / box_w))
        got = 0.0
        for r in range(r0, r1 + 1):
            for i in range(i0, i1 + 1):
                qx0, qx1 = oracle.lib().or_qlo(i, W), oracle.lib().or_qlo(i + 1, W)
                qy0, qy1 = oracle.lib().or_qlo(r, W), oracle.lib().or_qlo(r + 1, W)
                got += oracle.area_fraction(P, k, i, r, W, W) * (qx1 - qx0) * (qy1 - qy0)
        got *= (box_w / (1 << 30)) ** 2          # lattice units^2 -> world units^2
        assert abs(got - want) <= 1e-9 * want, (k, got, want)


def test_fraction_partition_of_unity_on_tiling():
    # an exact tiling of the domain: at every pixel the fractions add to 1
    flat = C.array_polys("tiles:24:4:7")
    P = oracle.Polys(flat, C.NYC_BOX)
    W = 24
    tot = np.zeros((W, W))
    for k in range(P.n):
        for r in range(W):
            for i in range(W):
                tot[r, i] += oracle.area_fraction(P, k, i, r, W, W)
    assert np.all(np.abs(tot - 1.0) <= 1e-9), np.abs(tot - 1.0).max()


def test_fraction_off_boundary_is_centre_membership():
    # lemma L4: a pixel outside polygon P's boundary set is wholly in or out
    P = oracle.Polys(C.array_polys("c1"), C1)
    W = 64
    for k in range(P.n):
        bits = oracle.boundary_mask(P, W, W, k, k + 1)
        for r in range(W):
            for i in range(W):
                if bits[r, i // 32] >> (i % 32) & 1:
                    continue
                cx, cy = oracle.lib().or_centre(i, W), oracle.lib().or_centre(r, W)
                assert oracle.area_fraction(P, k, i, r, W, W) == float(P.pnpoly(k, cx, cy))


@pytest.mark.parametrize("W", [16, 40])
def test_expected_interval_tightens_and_estimates(W):
    polys = oracle.Polys(C.array_polys("c1"), C1)
    pts = C.c1_points(400_000)
    x, y = pts["x"], pts["y"]
    cb, _, _ = oracle.query(polys, x, y, W=W, H=W, mode="bounded")
    ca, _, _ = oracle.query(polys, x, y, W=W, H=W, mode="accurate")
    cnt = oracle.pixel_counts(x, y, C1, W=W, H=W)
    ep, em = oracle.error_interval(polys, W, W, cnt)
    xp, xm = oracle.expected_interval(polys, W, W, cnt)
    assert np.all(xp >= 0) and np.all(xm >= 0)
    assert np.all(xp <= ep) and np.all(xm <= em)         # inside the worst case
    cb, ca = cb.astype(np.float64), ca.astype(np.float64)
    est = cb - xp + xm                                   # the uniform-points estimate
    # uniform points: the estimate is within a few standard deviations of the
    # exact count; the (wrong) literal reading f * Fpt for P+ is not
    sd = np.sqrt(ep + em + 1.0)
    assert np.all(np.abs(ca - est) <= 5 * sd), (ca, est, sd)
    assert np.abs(ca - est).sum() < 0.5 * np.abs(ca - cb).sum()
    lit = cb - (ep - xp) + xm                            # f instead of (1 - f) on P+
    assert np.abs(ca - lit).sum() > 2 * np.abs(ca - est).sum()
