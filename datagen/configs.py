"""Workload presets C1..C5 (BASELINE.json configs).

Each preset names its domain, polygon-set recipe, point recipe and query.
Seeds are 20171101 + config id.  Nothing here computes any part of the
method; the time-filter constants are calendar facts (seconds since
2009-01-01 UTC).
"""
from __future__ import annotations

import functools

import numpy as np

from . import polygons as P
from . import taxi_points, twitter_points, uniform_points

NYC_BOX = (0.0, 0.0, 57920.0, 57920.0)
US_BOX = (0.0, 0.0, 4600000.0, 2900000.0)
C1_BOX = (0.0, 0.0, 1024.0, 1024.0)

T_2012 = (94608000, 126230400)          # calendar 2012 [start, end)
T_JUNE_2012 = (107740800, 110332800)    # June 2012, the paper's Fig. 1 query

SEED = {k: 20171101 + k for k in range(1, 6)}


@functools.lru_cache(maxsize=None)
def polygon_set(name):
    """Named polygon sets -> list of polygons (list of rings)."""
    if name == "c1":
        return P.c1_polygons()
    if name == "c1b":
        return P.c1_polygons() + P.c1b_polygons()
    if name == "neighborhoods":          # ~260 neighbourhood-like polygons (C2, C5)
        return P.tiling(260, 16, NYC_BOX, seed=SEED[2])
    if name == "tracts":                 # ~2.2k census-tract-like, density-warped (C3)
        s = taxi_points(SEED[3] + 1000, 400000, t=False)
        return P.tiling(2200, 4, NYC_BOX, seed=SEED[3], warp_sample=(s["x"], s["y"]))
    if name == "counties":               # ~3.1k county-like on the US box (C4)
        return P.tiling(3100, 16, US_BOX, seed=SEED[4])
    if name.startswith("tiles:"):        # tiles:n:s:seed (tests)
        _, n, s, sd = name.split(":")
        return P.tiling(int(n), int(s), NYC_BOX, seed=int(sd))
    raise KeyError(name)


# Point generators per preset.  Each returns dict of numpy columns.
def c1_points(n=100_000, i0=0):
    x, y = uniform_points(SEED[1], n, C1_BOX, i0=i0)
    return {"x": x, "y": y}


def taxi(n, i0=0, fare=False, seed=None):
    return taxi_points(SEED[2] if seed is None else seed, n, i0=i0, t=True, fare=fare)


def twitter(n, i0=0, seed=None):
    return twitter_points(SEED[4] if seed is None else seed, n, i0=i0, fav=True)


CONFIGS = {
    "C1": dict(box=C1_BOX, polys="c1", n=100_000, W=1024, H=1024, agg="count", modes=("bounded", "accurate")),
    "C2": dict(box=NYC_BOX, polys="neighborhoods", n=1_000_000_000, W=8192, H=8192, agg="count",
               filter=("t", T_2012), modes=("bounded",)),
    "C3": dict(box=NYC_BOX, polys="tracts", n=1_000_000_000, W=8192, H=8192, agg="avg", agg_col="fare",
               modes=("accurate",)),
    "C4": dict(box=US_BOX, polys="counties", n=2_000_000_000, epsilon=1000.0, agg="sum", agg_col="fav",
               modes=("bounded",)),
    "C5": dict(box=NYC_BOX, polys="neighborhoods", n=1_000_000_000, W=None, agg="count",
               modes=("bounded", "accurate"), sweep=(1024, 2048, 4096, 8192, 16384, 32768)),
}


def array_polys(name):
    return P.flatten(polygon_set(name))


def np_f64(a):
    return np.ascontiguousarray(a, dtype=np.float64)
