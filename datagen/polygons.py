"""Seeded synthetic polygon sets (world coordinates, float64).

Shared input generator: holds none of Raster Join's arithmetic (no
quantisation, no pixel map, no point-in-polygon test).  A polygon is a list
of rings, a ring an (k, 2) float64 array of vertices without a repeated
closing vertex (the C-ABI convention, include/rj.h).

Sets:
  * c1_polygons()   -- the 10 hand-made C1 polygons (square on pixel borders,
    square on pixel centres, triangle, hexagon, L-shape, 10-point star,
    square annulus, comb, square overlapping the hexagon, square sharing the
    edge x=200 with P0) on the domain [0,1024)^2.
  * c1b_polygons()  -- adversarial extras: 0.3 px sliver, bow-tie, square on
    the domain edge x=1024, ring with collinear and repeated vertices.
  * tiling(...)     -- an exact tiling of a box: jittered quad lattice with
    wiggled shared edges (each shared edge generated once so both neighbours
    hold bit-identical vertices, no T-junctions), region-grown into n
    connected polygons whose boundaries are traced into rings (outer rings
    and holes).  Adapted from the paper's Voronoi+merge generator
     so that the union is exactly the box.
"""
from __future__ import annotations

import heapq
import math

import numpy as np


def _ring(pts):
    return np.asarray(pts, dtype=np.float64).reshape(-1, 2)


def c1_polygons():
    """C1 polygon set, SURVEY.md 8(d) 'C1 polygon set' table (ids = index)."""
    star = []
    for k in range(10):
        r = 120.0 if k % 2 == 0 else 50.0
        a = math.radians(90.0 + 36.0 * k)
        star.append((round(500.0 + r * math.cos(a)), round(500.0 + r * math.sin(a))))
    polys = [
        [_ring([(100, 100), (200, 100), (200, 200), (100, 200)])],                       # P0
        [_ring([(300.5, 100.5), (400.5, 100.5), (400.5, 200.5), (300.5, 200.5)])],       # P1
        [_ring([(500, 100), (700, 120), (560, 300)])],                                   # P2
        [_ring([(950, 200), (900, 287), (800, 287), (750, 200), (800, 113), (900, 113)])],  # P3
        [_ring([(100, 400), (300, 400), (300, 450), (150, 450), (150, 600), (100, 600)])],  # P4
        [_ring(star)],                                                                   # P5
        [_ring([(700, 400), (950, 400), (950, 650), (700, 650)]),                        # P6 outer
         _ring([(775, 475), (875, 475), (875, 575), (775, 575)])],                       # P6 hole
        [_ring([(100, 700), (400, 700), (400, 950), (350, 950), (350, 750), (300, 750),  # P7 comb
                (300, 950), (250, 950), (250, 750), (200, 750), (200, 950), (150, 950),
                (150, 750), (100, 750)])],
        [_ring([(820, 150), (1000, 150), (1000, 330), (820, 330)])],                     # P8
        [_ring([(200, 100), (300, 100), (300, 200), (200, 200)])],                       # P9
    ]
    return polys


def c1b_polygons():
    """Adversarial extra polygons (SURVEY.md 8(d) 'C1b')."""
    return [
        # slanted sliver 0.3 px wide: no pixel centre inside, but lattice points are
        [_ring([(600.0, 700.0), (600.3, 700.0), (680.3, 900.0), (680.0, 900.0)])],
        # bow-tie (self-intersecting; even-odd)
        [_ring([(450, 750), (550, 850), (550, 750), (450, 850)])],
        # square touching the domain edge x = 1024 (Q = 2^30)
        [_ring([(980, 900), (1024, 900), (1024, 1000), (980, 1000)])],
        # collinear and repeated consecutive vertices
        [_ring([(20, 20), (40, 20), (40, 20), (60, 20), (60, 60), (60, 60), (40, 60), (20, 60), (20, 40)])],
    ]


def c1b_points(polys, seed=20171102):
    """~2k adversarial points: vertices, edge midpoints, integer (pixel border)
    and half-integer (pixel centre) coordinates on [0,1024)^2."""
    rng = np.random.default_rng(seed)
    pts = []
    for poly in polys:
        for ring in poly:
            nxt = np.roll(ring, -1, axis=0)
            pts.append(ring)
            pts.append(0.5 * (ring + nxt))
    pts.append(rng.integers(0, 1024, size=(600, 2)).astype(np.float64))
    pts.append(rng.integers(0, 1024, size=(600, 2)).astype(np.float64) + 0.5)
    pts.append(np.stack([rng.integers(0, 1024, 300) + 0.5, rng.integers(0, 1024, 300).astype(np.float64)], 1))
    p = np.concatenate(pts, axis=0)
    p = p[(p[:, 0] >= 0) & (p[:, 0] < 1024) & (p[:, 1] >= 0) & (p[:, 1] < 1024)]
    return np.ascontiguousarray(p[:, 0]), np.ascontiguousarray(p[:, 1])


def flatten(polys):
    """polygons -> (poly_ring_off u32[n+1], ring_vert_off u32[nr+1], vx f64, vy f64)."""
    pro = [0]
    rvo = [0]
    xs, ys = [], []
    for poly in polys:
        for ring in poly:
            xs.append(ring[:, 0])
            ys.append(ring[:, 1])
            rvo.append(rvo[-1] + len(ring))
        pro.append(pro[-1] + len(poly))
    return (np.asarray(pro, dtype=np.uint32), np.asarray(rvo, dtype=np.uint32),
            np.ascontiguousarray(np.concatenate(xs)), np.ascontiguousarray(np.concatenate(ys)))


# --------------------------------------------------------------------- tiling
def _quantile_map(sample, lo, hi):
    """Monotone map u in [0,1] -> 0.5 u + 0.5 F^-1(u) (normalised), F the
    empirical marginal CDF of `sample` on [lo, hi); endpoints pinned."""
    s = np.sort((np.asarray(sample, dtype=np.float64) - lo) / (hi - lo))
    s = np.clip(s, 0.0, 1.0)
    q = np.linspace(0.0, 1.0, 1025)
    inv = np.quantile(s, q)
    inv[0], inv[-1] = 0.0, 1.0
    inv = np.maximum.accumulate(inv)

    def f(u):
        return 0.5 * u + 0.5 * np.interp(u, q, inv)
    return f


def tiling(n, s, box, seed, warp_sample=None, jitter=0.3, wiggle=0.1):
    """Exact tiling of `box` = (x0, y0, x1, y1) into ~n connected polygons.

    s: segments per shared lattice edge (power of two).  warp_sample: optional
    (xs, ys) point sample; the lattice is density-warped per axis so that
    polygons shrink where points are dense (tract-like sets).
    """
    x0, y0, x1, y1 = map(float, box)
    rng = np.random.default_rng(seed)
    w, h = x1 - x0, y1 - y0
    nq = 4 * n
    nx = max(2, int(round(math.sqrt(nq * w / h))))
    ny = max(2, int(round(nq / nx)))
    gu = np.linspace(0.0, 1.0, nx + 1)
    gv = np.linspace(0.0, 1.0, ny + 1)
    if warp_sample is not None:
        gu = _quantile_map(warp_sample[0], x0, x1)(gu)
        gv = _quantile_map(warp_sample[1], y0, y1)(gv)
        gu[0], gu[-1], gv[0], gv[-1] = 0.0, 1.0, 0.0, 1.0
    # lattice vertices (normalised), jittered by a fraction of the local spacing
    du = np.diff(gu)
    dv = np.diff(gv)
    U = np.repeat(gu[:, None], ny + 1, 1).copy()
    V = np.repeat(gv[None, :], nx + 1, 0).copy()
    for i in range(nx + 1):
        for j in range(ny + 1):
            if 0 < i < nx:
                U[i, j] += jitter * min(du[i - 1], du[i]) * rng.uniform(-1, 1)
            if 0 < j < ny:
                V[i, j] += jitter * min(dv[j - 1], dv[j]) * rng.uniform(-1, 1)
    X = x0 + U * w
    Y = y0 + V * h
    X[0, :], X[nx, :] = x0, x1          # borders exactly on the box
    Y[:, 0], Y[:, ny] = y0, y1

    levels = int(round(math.log2(s))) if s > 1 else 0
    # local scale per lattice vertex: smallest adjacent spacing in world units
    sx = np.minimum(np.r_[du[0], du] , np.r_[du, du[-1]]) * w
    sy = np.minimum(np.r_[dv[0], dv], np.r_[dv, dv[-1]]) * h
    local = {(i, j): float(min(sx[i], sy[j])) for i in range(nx + 1) for j in range(ny + 1)}
    edge_cache = {}

    def poly_edge(a, b):
        """Polyline (list of (x,y)) from lattice vertex a to b, generated once per
        undirected edge so both neighbours share identical vertices."""
        key = (a, b) if a < b else (b, a)
        if key not in edge_cache:
            p, q = key
            pa = np.array([X[p], Y[p]])
            pb = np.array([X[q], Y[q]])
            border = (p[0] == q[0] and p[0] in (0, nx)) or (p[1] == q[1] and p[1] in (0, ny))
            pts = [pa, pb]
            if not border:
                erng = np.random.default_rng([seed, 7, p[0], p[1], q[0], q[1]])
                # displacement bounded by the local cell size (not the edge
                # length) so that thin warped cells cannot fold over
                amp = wiggle * min(local[p], local[q])
                for _ in range(levels):
                    new = [pts[0]]
                    for u, v in zip(pts[:-1], pts[1:]):
                        d = v - u
                        nrm = np.array([-d[1], d[0]]) / max(np.hypot(d[0], d[1]), 1e-300)
                        m = 0.5 * (u + v) + nrm * amp * erng.uniform(-1, 1)
                        new += [m, v]
                    pts = new
                    amp *= 0.5
            edge_cache[key] = [tuple(map(float, t)) for t in pts]
        line = edge_cache[key]
        return line if key == (a, b) else line[::-1]

    # region growing: randomized multi-source Dijkstra over quad adjacency
    nqx, nqy = nx, ny
    owner = -np.ones((nqx, nqy), dtype=np.int64)
    seeds = rng.choice(nqx * nqy, size=min(n, nqx * nqy), replace=False)
    heap = []
    for rid, sq in enumerate(seeds):
        heapq.heappush(heap, (0.0, int(rid), int(sq // nqy), int(sq % nqy)))
    while heap:
        d, rid, i, j = heapq.heappop(heap)
        if owner[i, j] >= 0:
            continue
        owner[i, j] = rid
        for di, dj in ((1, 0), (-1, 0), (0, 1), (0, -1)):
            a, b = i + di, j + dj
            if 0 <= a < nqx and 0 <= b < nqy and owner[a, b] < 0:
                heapq.heappush(heap, (d + 1.0 + rng.uniform(0, 1.5), rid, a, b))
    nreg = int(owner.max()) + 1

    # boundary tracing: directed CCW quad edges whose other side is another region
    out_edges = [dict() for _ in range(nreg)]
    for i in range(nqx):
        for j in range(nqy):
            r = owner[i, j]
            v00, v10, v11, v01 = (i, j), (i + 1, j), (i + 1, j + 1), (i, j + 1)
            for (a, b), (ni, nj) in (((v00, v10), (i, j - 1)), ((v10, v11), (i + 1, j)),
                                     ((v11, v01), (i, j + 1)), ((v01, v00), (i - 1, j))):
                other = owner[ni, nj] if (0 <= ni < nqx and 0 <= nj < nqy) else -1
                if other != r:
                    out_edges[r].setdefault(a, []).append(b)
    polys = []
    for r in range(nreg):
        oe = out_edges[r]
        rings = []
        while oe:
            start = next(iter(oe))
            ring = []
            cur = start
            while True:
                nxts = oe[cur]
                nxt = nxts.pop()
                if not nxts:
                    del oe[cur]
                ring.extend(poly_edge(cur, nxt)[:-1])
                cur = nxt
                if cur == start and cur not in oe:
                    break
                if cur == start and cur in oe:
                    break
            rings.append(np.asarray(ring, dtype=np.float64))
        polys.append(rings)
    return polys
