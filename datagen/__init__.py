"""Seeded synthetic input generators shared by the oracle and the CUDA path.

This package draws inputs only (world-coordinate points, raw attribute
columns, polygon rings); it contains none of Raster Join's arithmetic.  The
point generators are C (gen_points.c, OpenMP, counter-based so the output is
a pure function of (seed, index) for any thread count); polygons are numpy
(polygons.py).  Workload presets live in configs.py.
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "libdatagen.so")
_lib = None


def build(force=False):
    src = os.path.join(_HERE, "gen_points.c")
    if force or not os.path.exists(_SO) or os.path.getmtime(_SO) < os.path.getmtime(src):
        subprocess.check_call(["gcc", "-O2", "-fopenmp", "-fPIC", "-shared", "-o", _SO, src, "-lm"])
    return _SO


def lib():
    global _lib
    if _lib is None:
        build()
        L = ctypes.CDLL(_SO)
        u64, vp, d = ctypes.c_uint64, ctypes.c_void_p, ctypes.c_double
        L.dg_u64.restype = u64
        L.dg_u64.argtypes = [u64, u64, u64]
        L.dg_uniform_points.restype = None
        L.dg_uniform_points.argtypes = [u64, u64, u64, d, d, d, d, vp, vp]
        L.dg_taxi_points.restype = None
        L.dg_taxi_points.argtypes = [u64, u64, u64, vp, vp, vp, vp]
        L.dg_twitter_points.restype = None
        L.dg_twitter_points.argtypes = [u64, u64, u64, vp, vp, vp]
        _lib = L
    return _lib


def _ptr(a):
    return None if a is None else a.ctypes.data


def uniform_points(seed, n, box, i0=0):
    x = np.empty(n, dtype=np.float64)
    y = np.empty(n, dtype=np.float64)
    lib().dg_uniform_points(seed, i0, n, *map(float, box), _ptr(x), _ptr(y))
    return x, y


def taxi_points(seed, n, i0=0, t=True, fare=False, out=None):
    """NYC-taxi-shaped points on [0,57920)^2: x, y f32 (+ t int32, fare f32)."""
    o = out or {}
    x = o.get("x", np.empty(n, dtype=np.float32))
    y = o.get("y", np.empty(n, dtype=np.float32))
    tt = o.get("t", np.empty(n, dtype=np.int32)) if t else None
    ff = o.get("fare", np.empty(n, dtype=np.float32)) if fare else None
    lib().dg_taxi_points(seed, i0, n, _ptr(x), _ptr(y), _ptr(tt), _ptr(ff))
    r = {"x": x, "y": y}
    if t:
        r["t"] = tt
    if fare:
        r["fare"] = ff
    return r


def twitter_points(seed, n, i0=0, fav=True, out=None):
    """Twitter-shaped points on [0,4.6e6)x[0,2.9e6): x, y f32 (+ fav int32)."""
    o = out or {}
    x = o.get("x", np.empty(n, dtype=np.float32))
    y = o.get("y", np.empty(n, dtype=np.float32))
    ff = o.get("fav", np.empty(n, dtype=np.int32)) if fav else None
    lib().dg_twitter_points(seed, i0, n, _ptr(x), _ptr(y), _ptr(ff))
    r = {"x": x, "y": y}
    if fav:
        r["fav"] = ff
    return r
