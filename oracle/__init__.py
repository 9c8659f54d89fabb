"""CPU oracle for Raster Join -- TEST INFRASTRUCTURE ONLY.

Only tests/, __graft_entry__.smoke() and bench.py (cpu_baseline and
--impl reference) may import this package.  The product package
(paper_journals_pvldb_zacharatoudasf17_b200) never imports it, and the two
share no code.  See rj_oracle.c for the definitions (SURVEY.md 8(c) O1-O10,
each citing PAPER.md) that this wraps.
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "liboracle.so")
_lib = None

OPS = {"<": 0, "<=": 1, ">": 2, ">=": 3, "==": 4}
DTYPES = {np.dtype(np.int32): 0, np.dtype(np.float32): 1, np.dtype(np.float64): 2}


def build(force=False):
    src = os.path.join(_HERE, "rj_oracle.c")
    if force or not os.path.exists(_SO) or os.path.getmtime(_SO) < os.path.getmtime(src):
        subprocess.check_call(["gcc", "-O2", "-fopenmp", "-ffp-contract=off", "-fPIC", "-shared",
                               "-o", _SO, src, "-lm"])
    return _SO


def lib():
    global _lib
    if _lib is None:
        build()
        L = ctypes.CDLL(_SO)
        i64, u64, i32, d, vp = ctypes.c_int64, ctypes.c_uint64, ctypes.c_int, ctypes.c_double, ctypes.c_void_p
        L.or_quantize.restype = i64
        L.or_quantize.argtypes = [d, d, d]
        for f in (L.or_pixel, L.or_centre, L.or_qlo, L.or_qhi):
            f.restype = i64
            f.argtypes = [i64, i64]
        L.or_resolve.restype = i32
        L.or_resolve.argtypes = [d, d, d, ctypes.POINTER(i32), ctypes.POINTER(i32)]
        L.or_polys_new.restype = vp
        L.or_polys_new.argtypes = [i64, vp, vp, vp, vp, d, d, d, d]
        L.or_polys_free.restype = None
        L.or_polys_free.argtypes = [vp]
        L.or_polys_vertex.restype = i64
        L.or_polys_vertex.argtypes = [vp, i64, i32]
        L.or_pnpoly.restype = i32
        L.or_pnpoly.argtypes = [vp, i64, i64, i64]
        L.or_query.restype = u64
        L.or_query.argtypes = [vp, u64, vp, vp, i32, d, d, d, d, i32, vp, vp, i32, i32, vp, vp, vp,
                               i32, i32, i32, i32, vp, vp, vp]
        L.or_query_minmax.restype = None
        L.or_query_minmax.argtypes = [vp, u64, vp, vp, i32, d, d, d, d, i32, vp, vp, i32, i32, vp, vp, vp,
                                      i32, i32, i32, vp, vp, vp]
        L.or_avg.restype = None
        L.or_avg.argtypes = [i64, vp, vp, vp]
        L.or_membership.restype = None
        L.or_membership.argtypes = [vp, u64, vp, vp, i32, d, d, d, d, i32, vp, vp, i32, vp, vp, vp,
                                    i32, i32, i32, vp, vp]
        L.or_pixel_spans.restype = i64
        L.or_pixel_spans.argtypes = [vp, i64, i32, i32, i64, vp]
        L.or_seg_rect.restype = i32
        L.or_seg_rect.argtypes = [i64] * 8
        L.or_boundary_mask.restype = None
        L.or_boundary_mask.argtypes = [vp, i64, i64, i32, i32, vp]
        L.or_pixel_counts.restype = None
        L.or_pixel_counts.argtypes = [u64, vp, vp, i32, d, d, d, d, i32, vp, vp, i32, vp, vp, vp,
                                      i32, i32, vp]
        L.or_error_interval.restype = None
        L.or_error_interval.argtypes = [vp, i32, i32, vp, vp, vp]
        L.or_ring_sigma.restype = i32
        L.or_ring_sigma.argtypes = [vp, i64, i64]
        L.or_area_fraction.restype = d
        L.or_area_fraction.argtypes = [vp, i64, i64, i64, i32, i32]
        L.or_expected_interval.restype = None
        L.or_expected_interval.argtypes = [vp, i32, i32, vp, vp, vp]
        _lib = L
    return _lib


def quantize(v, lo, hi):
    return lib().or_quantize(float(v), float(lo), float(hi))


def resolve(w, h, eps):
    W, H = ctypes.c_int(), ctypes.c_int()
    if lib().or_resolve(float(w), float(h), float(eps), ctypes.byref(W), ctypes.byref(H)) != 0:
        return None
    return W.value, H.value


class Polys:
    """Quantised polygon set held by the oracle (O1 applied by the oracle itself)."""

    def __init__(self, flat, box):
        pro, rvo, vx, vy = flat
        self._keep = (np.ascontiguousarray(pro, np.uint32), np.ascontiguousarray(rvo, np.uint32),
                      np.ascontiguousarray(vx, np.float64), np.ascontiguousarray(vy, np.float64))
        self.n = len(pro) - 1
        self.box = tuple(map(float, box))
        h = lib().or_polys_new(self.n, *(a.ctypes.data for a in self._keep), *self.box)
        if not h:
            raise ValueError("polygon vertex outside the closed domain [0, 2^30]")
        self.h = h

    def __del__(self):
        if getattr(self, "h", None):
            lib().or_polys_free(self.h)
            self.h = None

    def pnpoly(self, P, px, py):
        return bool(lib().or_pnpoly(self.h, P, int(px), int(py)))


class _Cols:
    def __init__(self, cols, preds):
        """cols: list of numpy arrays; preds: list of (col, op-string, value)."""
        self.cols = [np.ascontiguousarray(c) for c in cols]
        self.ptrs = (ctypes.c_void_p * max(1, len(self.cols)))(*[c.ctypes.data for c in self.cols])
        self.dt = np.asarray([DTYPES[c.dtype] for c in self.cols] or [0], dtype=np.int32)
        self.np = len(preds)
        self.pc = np.asarray([p[0] for p in preds] or [0], dtype=np.int32)
        self.po = np.asarray([OPS[p[1]] for p in preds] or [0], dtype=np.int32)
        self.pv = np.asarray([p[2] for p in preds] or [0.0], dtype=np.float64)

    def args(self):
        return (len(self.cols), ctypes.addressof(self.ptrs), self.dt.ctypes.data)

    def pargs(self):
        return (self.np, self.pc.ctypes.data, self.po.ctypes.data, self.pv.ctypes.data)


def _view(view):
    """O12 window (c0, r0, c1, r1) as an int32 array, or None (whole canvas)."""
    if view is None:
        return None, None
    v = np.ascontiguousarray(view, dtype=np.int32)
    assert v.shape == (4,)
    return v, v.ctypes.data


def _xy(x, y):
    x = np.ascontiguousarray(x)
    y = np.ascontiguousarray(y)
    assert x.dtype == y.dtype and x.dtype in (np.float32, np.float64)
    return x, y, int(x.dtype == np.float64)


def query(polys, x, y, cols=(), preds=(), agg_col=-1, W=1024, H=1024, mode="bounded", nthreads=0, view=None):
    """Returns (count u64[n_poly], sum f64[n_poly], n_filtered); view = O12 pixel window."""
    x, y, f64 = _xy(x, y)
    c = _Cols(cols, preds)
    v, vp = _view(view)
    cnt = np.zeros(polys.n, dtype=np.uint64)
    s = np.zeros(polys.n, dtype=np.float64)
    kept = lib().or_query(polys.h, len(x), x.ctypes.data, y.ctypes.data, f64, *polys.box, *c.args(),
                          int(agg_col), *c.pargs(), int(W), int(H), 0 if mode == "bounded" else 1,
                          int(nthreads), cnt.ctypes.data, s.ctypes.data, vp)
    return cnt, s, int(kept)


def query_minmax(polys, x, y, cols, agg_col, preds=(), W=1024, H=1024, mode="bounded", view=None):
    """O11: (min f64[n_poly], max f64[n_poly]) of column agg_col, NaN for empty polygons."""
    x, y, f64 = _xy(x, y)
    c = _Cols(cols, preds)
    v, vp = _view(view)
    mn = np.zeros(polys.n, dtype=np.float64)
    mx = np.zeros(polys.n, dtype=np.float64)
    lib().or_query_minmax(polys.h, len(x), x.ctypes.data, y.ctypes.data, f64, *polys.box, *c.args(),
                          int(agg_col), *c.pargs(), int(W), int(H), 0 if mode == "bounded" else 1,
                          mn.ctypes.data, mx.ctypes.data, vp)
    return mn, mx


def avg(cnt, s):
    cnt = np.ascontiguousarray(cnt, np.uint64)
    s = np.ascontiguousarray(s, np.float64)
    out = np.empty(len(cnt), dtype=np.float64)
    lib().or_avg(len(cnt), cnt.ctypes.data, s.ctypes.data, out.ctypes.data)
    return out


def membership(polys, x, y, cols=(), preds=(), W=1024, H=1024, mode="bounded", view=None):
    x, y, f64 = _xy(x, y)
    c = _Cols(cols, preds)
    v, vp = _view(view)
    bits = np.zeros(len(x), dtype=np.uint64)
    lib().or_membership(polys.h, len(x), x.ctypes.data, y.ctypes.data, f64, *polys.box, *c.args(),
                        *c.pargs(), int(W), int(H), 0 if mode == "bounded" else 1, bits.ctypes.data, vp)
    return bits


def pixel_spans(polys, P, W, H):
    cap = 1 << 16
    while True:
        out = np.zeros((cap, 3), dtype=np.int32)
        n = lib().or_pixel_spans(polys.h, P, int(W), int(H), cap, out.ctypes.data)
        if n <= cap:
            return out[:n]
        cap = int(n)


def seg_rect(*a):
    return bool(lib().or_seg_rect(*map(int, a)))


def boundary_mask(polys, W, H, p0=0, p1=None):
    wpr = (W + 31) // 32
    bits = np.zeros((H, wpr), dtype=np.uint32)
    lib().or_boundary_mask(polys.h, p0, polys.n if p1 is None else p1, int(W), int(H), bits.ctypes.data)
    return bits


def pixel_counts(x, y, box, cols=(), preds=(), W=1024, H=1024):
    x, y, f64 = _xy(x, y)
    c = _Cols(cols, preds)
    out = np.zeros((H, W), dtype=np.uint32)
    lib().or_pixel_counts(len(x), x.ctypes.data, y.ctypes.data, f64, *map(float, box), *c.args(), *c.pargs(),
                          int(W), int(H), out.ctypes.data)
    return out


def error_interval(polys, W, H, counts):
    counts = np.ascontiguousarray(counts, np.uint32)
    ep = np.zeros(polys.n, dtype=np.uint64)
    em = np.zeros(polys.n, dtype=np.uint64)
    lib().or_error_interval(polys.h, int(W), int(H), counts.ctypes.data, ep.ctypes.data, em.ctypes.data)
    return ep, em


def ring_sigma(polys, P, r):
    """O13: orientation(ring r) * (-1)^depth -- the ring's even-odd weight."""
    return int(lib().or_ring_sigma(polys.h, int(P), int(r)))


def area_fraction(polys, P, i, r, W, H):
    """O13: fraction of pixel (i, r)'s lattice rectangle inside polygon P."""
    return float(lib().or_area_fraction(polys.h, int(P), int(i), int(r), int(W), int(H)))


def expected_interval(polys, W, H, counts):
    """O13: (E+, E-) per polygon, binary64."""
    counts = np.ascontiguousarray(counts, np.uint32)
    ep = np.zeros(polys.n, dtype=np.float64)
    em = np.zeros(polys.n, dtype=np.float64)
    lib().or_expected_interval(polys.h, int(W), int(H), counts.ctypes.data, ep.ctypes.data, em.ctypes.data)
    return ep, em
