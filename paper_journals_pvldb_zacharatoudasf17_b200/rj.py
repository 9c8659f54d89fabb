"""Thin ctypes binding of librj (include/rj.h): argument marshalling only.

Every step of a query runs in librj's CUDA kernels; this module converts
numpy arrays / torch tensors to pointers and status codes to exceptions.
There is no fallback: if librj.so is missing or no sm_100 device is present
the calls raise.

    rj_create, rj_destroy, rj_load_points, rj_load_polygons, rj_query,
    rj_query_device, rj_pack_partials, rj_finalize_packed, rj_finalize_device,
    rj_query_stream, rj_query_interval, rj_query_interval_ex, rj_query_multi,
    rj_resolve_canvas(_domain), rj_resolve_window, rj_resolve_lod,
    rj_debug_pixel_spans, rj_debug_boundary_mask, rj_debug_boundary_pieces, rj_debug_pip_work,
    rj_debug_point_membership, rj_debug_point_canvas,
    rj_get_stats, rj_set_option  -- same names as the C ABI.

`RasterJoin` wraps a context with a Pythonic API.
"""
from __future__ import annotations

import ctypes
import os

import numpy as np

_PKG = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(_PKG, "librj.so")

RJ_OK = 0
STATUS = {0: "RJ_OK", -1: "RJ_ERR_INVALID_ARGUMENT", -2: "RJ_ERR_OUT_OF_DOMAIN", -3: "RJ_ERR_RESOLUTION",
          -4: "RJ_ERR_CAPACITY", -5: "RJ_ERR_OOM", -6: "RJ_ERR_CUDA"}
AGG = {"count": 0, "sum": 1, "avg": 2, "min": 3, "max": 4}
MODE = {"bounded": 0, "accurate": 1, "index": 2, "exact": 3}
OPS = {"<": 0, "<=": 1, ">": 2, ">=": 3, "==": 4}
DT_I32, DT_F32, DT_F64 = 0, 1, 2
OPT_TIMING, OPT_CHUNK, OPT_PASS, OPT_KEEP_LOAD_SCRATCH, OPT_TILE_SIDE, OPT_STAGES, OPT_STREAM_BATCH = 1, 2, 3, 4, 5, 6, 7
OPT_GRAPHS = 8
OPT_LANE_RUNS = 9
MAX_PRED = 5


class RJError(RuntimeError):
    def __init__(self, status, msg=""):
        self.status = status
        super().__init__(f"{STATUS.get(status, status)}: {msg}")


class rj_pred(ctypes.Structure):
    _fields_ = [("column", ctypes.c_int32), ("op", ctypes.c_int32), ("value", ctypes.c_double)]


class rj_query_desc(ctypes.Structure):
    _fields_ = [("agg", ctypes.c_int32), ("agg_column", ctypes.c_int32), ("n_pred", ctypes.c_int32),
                ("pred", rj_pred * MAX_PRED), ("canvas_w", ctypes.c_int32), ("canvas_h", ctypes.c_int32),
                ("epsilon", ctypes.c_double), ("mode", ctypes.c_int32), ("view", ctypes.c_int32 * 4)]


class rj_agg_spec(ctypes.Structure):
    _fields_ = [("agg", ctypes.c_int32), ("column", ctypes.c_int32)]


class rj_stats(ctypes.Structure):
    _fields_ = [("W", ctypes.c_int32), ("H", ctypes.c_int32), ("n_points", ctypes.c_uint64),
                ("n_filtered", ctypes.c_uint64), ("n_boundary", ctypes.c_uint64),
                ("n_crossings", ctypes.c_uint64), ("n_spans", ctypes.c_uint64), ("n_pieces", ctypes.c_uint64),
                ("n_items", ctypes.c_uint64), ("stream_bytes", ctypes.c_uint64), ("launches", ctypes.c_uint32),
                ("ms_polygon", ctypes.c_float), ("ms_point_pass", ctypes.c_float), ("ms_total", ctypes.c_float),
                ("pass_stages", ctypes.c_int32), ("pass_ctas_per_sm", ctypes.c_int32), ("level", ctypes.c_int32),
                ("mode", ctypes.c_int32), ("est_boundary_frac", ctypes.c_float)]

    def as_dict(self):
        return {k: getattr(self, k) for k, _ in self._fields_}


_lib = None


def lib():
    """Load librj.so (raises if it is missing: there is no fallback path)."""
    global _lib
    if _lib is None:
        if not os.path.exists(LIB_PATH):
            raise ImportError(f"librj.so not built at {LIB_PATH}; run __graft_entry__.build()")
        L = ctypes.CDLL(LIB_PATH)
        vp, i32, u32, u64, d = ctypes.c_void_p, ctypes.c_int32, ctypes.c_uint32, ctypes.c_uint64, ctypes.c_double
        qp = ctypes.POINTER(rj_query_desc)
        sig = {
            "rj_create": (i32, [ctypes.POINTER(vp), i32, vp, d, d, d, d]),
            "rj_destroy": (i32, [vp]),
            "rj_set_allocator": (i32, [vp, vp, vp, vp]),
            "rj_load_points": (i32, [vp, u64, vp, vp, i32, i32, vp, vp, ctypes.POINTER(u64)]),
            "rj_load_polygons": (i32, [vp, u32, vp, vp, vp, vp]),
            "rj_query": (i32, [vp, qp, vp, vp]),
            "rj_query_device": (i32, [vp, qp, vp, vp]),
            "rj_query_stream": (i32, [vp, qp, u64, vp, vp, i32, i32, vp, vp, vp, vp]),
            "rj_query_interval": (i32, [vp, qp, vp, vp, vp, vp]),
            "rj_query_interval_ex": (i32, [vp, qp, vp, vp, vp, vp, vp, vp]),
            "rj_query_multi": (i32, [vp, qp, i32, vp, vp, vp]),
            "rj_debug_point_canvas": (i32, [vp, qp, vp]),
            "rj_finalize_device": (i32, [vp, i32, u32, vp, vp, vp]),
            "rj_resolve_canvas": (i32, [vp, qp, ctypes.POINTER(i32), ctypes.POINTER(i32)]),
            "rj_resolve_canvas_domain": (i32, [d, d, d, d, qp, ctypes.POINTER(i32), ctypes.POINTER(i32)]),
            "rj_resolve_window": (i32, [d, d, d, d, qp, d, d, d, d, ctypes.POINTER(i32)]),
            "rj_resolve_lod": (i32, [d, d, d, d, d, d, d, d, i32, i32, ctypes.POINTER(i32), ctypes.POINTER(i32),
                                     ctypes.POINTER(i32)]),
            "rj_pack_partials": (i32, [vp, u32, vp, vp, vp]),
            "rj_finalize_packed": (i32, [vp, i32, u32, vp, vp, vp]),
            "rj_debug_pixel_spans": (i32, [vp, qp, u64, vp, ctypes.POINTER(u64)]),
            "rj_debug_boundary_mask": (i32, [vp, qp, vp]),
            "rj_debug_boundary_pieces": (i32, [vp, qp, vp, vp]),
            "rj_debug_pip_work": (i32, [vp, ctypes.POINTER(u64), ctypes.POINTER(u64)]),
            "rj_debug_point_membership": (i32, [vp, qp, vp]),
            "rj_get_stats": (i32, [vp, ctypes.POINTER(rj_stats)]),
            "rj_set_option": (i32, [vp, i32, ctypes.c_int64]),
            "rj_get_stream": (vp, [vp]),
            "rj_n_polygons": (u32, [vp]),
            "rj_n_points": (u64, [vp]),
            "rj_status_str": (ctypes.c_char_p, [i32]),
            "rj_last_error": (ctypes.c_char_p, [vp]),
            "rj_version": (ctypes.c_char_p, []),
        }
        for name, (res, args) in sig.items():
            f = getattr(L, name)
            f.restype = res
            f.argtypes = args
        _lib = L
    return _lib


EXPORTS = ["rj_create", "rj_destroy", "rj_set_allocator", "rj_load_points", "rj_load_polygons", "rj_query",
           "rj_query_device", "rj_query_stream", "rj_query_interval", "rj_query_interval_ex", "rj_query_multi", "rj_debug_point_canvas", "rj_finalize_device", "rj_resolve_canvas", "rj_resolve_canvas_domain",
           "rj_resolve_window", "rj_resolve_lod", "rj_pack_partials", "rj_finalize_packed",
           "rj_debug_pixel_spans", "rj_debug_boundary_mask", "rj_debug_boundary_pieces", "rj_debug_pip_work", "rj_debug_point_membership", "rj_get_stats",
           "rj_set_option", "rj_get_stream", "rj_n_polygons", "rj_n_points", "rj_status_str", "rj_last_error", "rj_version"]


def _check(status, ctx=None):
    if status != RJ_OK:
        msg = ""
        if ctx:
            m = lib().rj_last_error(ctx)
            msg = m.decode() if m else ""
        raise RJError(status, msg)


def _ptr(a):
    """Data pointer of a numpy array or torch tensor (host or device)."""
    if a is None:
        return None
    if hasattr(a, "data_ptr"):
        assert a.is_contiguous(), "tensors must be contiguous"
        return a.data_ptr()
    assert a.flags["C_CONTIGUOUS"], "arrays must be C-contiguous"
    return a.ctypes.data


def _dtype_code(a):
    name = str(a.dtype).replace("torch.", "")
    return {"float32": DT_F32, "float64": DT_F64, "int32": DT_I32}[name]


def make_desc(agg="count", agg_column=-1, preds=(), W=0, H=0, epsilon=0.0, mode="bounded", view=None):
    """view = (c0, r0, c1, r1): viewport pixel window of the W x H canvas (None = whole canvas)."""
    q = rj_query_desc()
    q.agg = AGG[agg] if isinstance(agg, str) else int(agg)
    q.agg_column = int(agg_column)
    if len(preds) > MAX_PRED:
        raise ValueError("at most 5 predicates")
    q.n_pred = len(preds)
    for k, (col, op, val) in enumerate(preds):
        q.pred[k].column = int(col)
        q.pred[k].op = OPS[op] if isinstance(op, str) else int(op)
        q.pred[k].value = float(val)
    q.canvas_w, q.canvas_h = int(W), int(H if H else W)
    q.epsilon = float(epsilon)
    q.mode = MODE[mode] if isinstance(mode, str) else int(mode)
    if view is not None:
        if len(view) != 4:
            raise ValueError("view = (c0, r0, c1, r1)")
        for k in range(4):
            q.view[k] = int(view[k])
    return q


def lod_view(box, viewport, W, H=None):
    """LOD zoom through rj_resolve_lod: the canvas resolution and
    pixel window that render the world rectangle viewport = (vx0, vy0, vx1,
    vy1) with about W x H pixels.  Returns (W_full, H_full, view)."""
    Wf, Hf, v = ctypes.c_int32(), ctypes.c_int32(), (ctypes.c_int32 * 4)()
    _check(lib().rj_resolve_lod(*map(float, box), *map(float, viewport), int(W), int(H or W), ctypes.byref(Wf),
                                ctypes.byref(Hf), v))
    return Wf.value, Hf.value, tuple(v)


def rj_resolve_window(box, desc, rect):
    """Pixel window (c0, r0, c1, r1) holding every point of the world
    rectangle rect = (wx0, wy0, wx1, wy1), half-open (+-inf allowed)."""
    v = (ctypes.c_int32 * 4)()
    _check(lib().rj_resolve_window(*map(float, box), ctypes.byref(desc), *map(float, rect), v))
    return tuple(v)


def rj_pack_partials(ctx, d_count, d_sum, d_packed):
    _check(lib().rj_pack_partials(ctx, len(d_count), _ptr(d_count), _ptr(d_sum), _ptr(d_packed)), ctx)


def rj_finalize_packed(ctx, agg, d_packed, d_count, d_value):
    a = AGG[agg] if isinstance(agg, str) else int(agg)
    _check(lib().rj_finalize_packed(ctx, a, len(d_count), _ptr(d_packed), _ptr(d_count), _ptr(d_value)), ctx)


# ---- C-ABI names ------------------------------------------------------------
def rj_create(device=0, stream=None, box=(0.0, 0.0, 1.0, 1.0)):
    h = ctypes.c_void_p()
    s = lib().rj_create(ctypes.byref(h), int(device), stream, *map(float, box))
    _check(s)
    return h


def rj_destroy(ctx):
    _check(lib().rj_destroy(ctx))


def rj_set_option(ctx, option, value):
    _check(lib().rj_set_option(ctx, int(option), int(value)), ctx)


def _order_after_producer(ctx, arrays):
    """Device tensors may still be in flight on torch's current stream: make
    the context's stream wait for it before librj reads them."""
    if not any(getattr(a, "is_cuda", False) for a in arrays):
        return
    import torch
    s = rj_get_stream(ctx)
    if s:
        torch.cuda.ExternalStream(s).wait_stream(torch.cuda.current_stream())
    else:
        torch.cuda.current_stream().synchronize()


def rj_load_points(ctx, x, y, cols=()):
    _order_after_producer(ctx, [x, y, *cols])
    n = len(x)
    ptrs = (ctypes.c_void_p * max(1, len(cols)))(*[_ptr(c) for c in cols])
    dts = (ctypes.c_int32 * max(1, len(cols)))(*[_dtype_code(c) for c in cols])
    ood = ctypes.c_uint64()
    _check(lib().rj_load_points(ctx, n, _ptr(x), _ptr(y), _dtype_code(x), len(cols), ptrs, dts,
                                ctypes.byref(ood)), ctx)
    return ood.value


def rj_load_polygons(ctx, flat):
    pro, rvo, vx, vy = (np.ascontiguousarray(flat[0], np.uint32), np.ascontiguousarray(flat[1], np.uint32),
                        np.ascontiguousarray(flat[2], np.float64), np.ascontiguousarray(flat[3], np.float64))
    _check(lib().rj_load_polygons(ctx, len(pro) - 1, _ptr(pro), _ptr(rvo), _ptr(vx), _ptr(vy)), ctx)


def rj_query(ctx, desc, count=None, value=None):
    _check(lib().rj_query(ctx, ctypes.byref(desc), _ptr(count), _ptr(value)), ctx)


def rj_query_stream(ctx, desc, x, y, cols=(), count=None, value=None):
    _order_after_producer(ctx, [x, y, *cols])
    n = len(x)
    ptrs = (ctypes.c_void_p * max(1, len(cols)))(*[_ptr(c) for c in cols])
    dts = (ctypes.c_int32 * max(1, len(cols)))(*[_dtype_code(c) for c in cols])
    _check(lib().rj_query_stream(ctx, ctypes.byref(desc), n, _ptr(x), _ptr(y), _dtype_code(x), len(cols), ptrs, dts,
                                 _ptr(count), _ptr(value)), ctx)


def rj_query_multi(ctx, desc, aggs, count=None, values=None):
    """aggs: [(agg, column)] with agg a name or code; values: float64[len(aggs), n_poly]."""
    specs = (rj_agg_spec * max(1, len(aggs)))(*[rj_agg_spec(AGG[a] if isinstance(a, str) else int(a), int(c))
                                                 for a, c in aggs])
    _check(lib().rj_query_multi(ctx, ctypes.byref(desc), len(aggs), ctypes.addressof(specs), _ptr(count),
                                _ptr(values)), ctx)


def rj_query_interval(ctx, desc, count=None, value=None, eps_plus=None, eps_minus=None):
    _check(lib().rj_query_interval(ctx, ctypes.byref(desc), _ptr(count), _ptr(value), _ptr(eps_plus),
                                   _ptr(eps_minus)), ctx)


def rj_query_interval_ex(ctx, desc, count=None, value=None, eps_plus=None, eps_minus=None, exp_plus=None,
                         exp_minus=None):
    _check(lib().rj_query_interval_ex(ctx, ctypes.byref(desc), _ptr(count), _ptr(value), _ptr(eps_plus),
                                      _ptr(eps_minus), _ptr(exp_plus), _ptr(exp_minus)), ctx)


def rj_debug_point_canvas(ctx, desc):
    W, H = rj_resolve_canvas(ctx, desc)
    out = np.zeros((H, W), dtype=np.uint32)
    _check(lib().rj_debug_point_canvas(ctx, ctypes.byref(desc), _ptr(out)), ctx)
    return out


def rj_query_device(ctx, desc, d_count, d_sum=None):
    _check(lib().rj_query_device(ctx, ctypes.byref(desc), _ptr(d_count), _ptr(d_sum)), ctx)


def rj_finalize_device(ctx, agg, d_count, d_sum, d_value):
    a = AGG[agg] if isinstance(agg, str) else int(agg)
    _check(lib().rj_finalize_device(ctx, a, len(d_count), _ptr(d_count), _ptr(d_sum), _ptr(d_value)), ctx)


def rj_resolve_canvas_domain(box, desc):
    W, H = ctypes.c_int32(), ctypes.c_int32()
    _check(lib().rj_resolve_canvas_domain(*map(float, box), ctypes.byref(desc), ctypes.byref(W), ctypes.byref(H)))
    return W.value, H.value


def rj_resolve_canvas(ctx, desc):
    W, H = ctypes.c_int32(), ctypes.c_int32()
    _check(lib().rj_resolve_canvas(ctx, ctypes.byref(desc), ctypes.byref(W), ctypes.byref(H)), ctx)
    return W.value, H.value


def rj_get_stream(ctx):
    """cudaStream_t (as an int) the context issues its work on."""
    return lib().rj_get_stream(ctx) or 0


def rj_get_stats(ctx):
    st = rj_stats()
    _check(lib().rj_get_stats(ctx, ctypes.byref(st)), ctx)
    return st.as_dict()


def rj_debug_pixel_spans(ctx, desc):
    n = ctypes.c_uint64()
    _check(lib().rj_debug_pixel_spans(ctx, ctypes.byref(desc), 0, None, ctypes.byref(n)), ctx)
    out = np.zeros((max(1, n.value), 4), dtype=np.uint32)
    _check(lib().rj_debug_pixel_spans(ctx, ctypes.byref(desc), n.value, _ptr(out), ctypes.byref(n)), ctx)
    return out[:n.value]


def rj_debug_boundary_mask(ctx, desc):
    W, H = rj_resolve_canvas(ctx, desc)
    bits = np.zeros((H, (W + 31) // 32), dtype=np.uint32)
    _check(lib().rj_debug_boundary_mask(ctx, ctypes.byref(desc), _ptr(bits)), ctx)
    return bits


def rj_debug_boundary_pieces(ctx, desc):
    """(bnd_bits, cover_bits), each uint32[H, ceil(W/32)]: the boundary pixels
    the accurate point-pass kernels painted into their tiles, and the pixels
    those tiles covered."""
    W, H = rj_resolve_canvas(ctx, desc)
    bnd = np.zeros((H, (W + 31) // 32), dtype=np.uint32)
    cov = np.zeros_like(bnd)
    _check(lib().rj_debug_boundary_pieces(ctx, ctypes.byref(desc), _ptr(bnd), _ptr(cov)), ctx)
    return bnd, cov


def rj_debug_pip_work(ctx):
    """(boundary points tested, edge-grid entries walked) of the last accurate query."""
    a, b = ctypes.c_uint64(), ctypes.c_uint64()
    _check(lib().rj_debug_pip_work(ctx, ctypes.byref(a), ctypes.byref(b)), ctx)
    return a.value, b.value


def rj_debug_point_membership(ctx, desc, n_input):
    bits = np.zeros(max(1, n_input), dtype=np.uint64)
    _check(lib().rj_debug_point_membership(ctx, ctypes.byref(desc), _ptr(bits)), ctx)
    return bits[:n_input]


# ---- Pythonic wrapper ----------------------------------------------------------
class RasterJoin:
    """One librj context on one CUDA device."""

    def __init__(self, box, device=0, stream=None):
        self.box = tuple(map(float, box))
        self.ctx = rj_create(device, stream, self.box)
        self.n_input = 0

    def close(self):
        if getattr(self, "ctx", None):
            rj_destroy(self.ctx)
            self.ctx = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def load_points(self, x, y, cols=()):
        self.n_input = len(x)
        return rj_load_points(self.ctx, x, y, cols)

    def load_polygons(self, flat):
        rj_load_polygons(self.ctx, flat)
        self.n_poly = int(lib().rj_n_polygons(self.ctx))

    def set_option(self, option, value):
        rj_set_option(self.ctx, option, value)

    def query(self, **kw):
        """Returns (count uint64[n_poly], value float64[n_poly])."""
        q = make_desc(**kw)
        cnt = np.zeros(self.n_poly, dtype=np.uint64)
        val = np.zeros(self.n_poly, dtype=np.float64)
        rj_query(self.ctx, q, cnt, val)
        return cnt, val

    def query_stream(self, x, y, cols=(), **kw):
        """Streamed one-shot query over points that are not loaded (host or
        device arrays, read once in batches).  Returns (count, value)."""
        q = make_desc(**kw)
        cnt = np.zeros(self.n_poly, dtype=np.uint64)
        val = np.zeros(self.n_poly, dtype=np.float64)
        rj_query_stream(self.ctx, q, x, y, cols, cnt, val)
        return cnt, val

    def query_multi(self, aggs, **kw):
        """Several aggregates in one pass: aggs = [("min", col), ("avg", col), ("count", 0), ...].
        Returns (count uint64[n_poly], values float64[len(aggs), n_poly])."""
        q = make_desc(**kw)
        cnt = np.zeros(self.n_poly, dtype=np.uint64)
        val = np.zeros((len(aggs), self.n_poly), dtype=np.float64)
        rj_query_multi(self.ctx, q, aggs, cnt, val)
        return cnt, val

    def query_interval(self, **kw):
        """Bounded query with worst-case intervals: (count, value, eps_plus, eps_minus)."""
        q = make_desc(**kw)
        out = [np.zeros(self.n_poly, dtype=t) for t in (np.uint64, np.float64, np.uint64, np.uint64)]
        rj_query_interval(self.ctx, q, *out)
        return tuple(out)

    def query_interval_ex(self, **kw):
        """Bounded query with worst-case and expected intervals:
        (count, value, eps_plus, eps_minus, exp_plus, exp_minus)."""
        q = make_desc(**kw)
        out = [np.zeros(self.n_poly, dtype=t)
               for t in (np.uint64, np.float64, np.uint64, np.uint64, np.float64, np.float64)]
        rj_query_interval_ex(self.ctx, q, *out)
        return tuple(out)

    def point_canvas(self, **kw):
        return rj_debug_point_canvas(self.ctx, make_desc(**kw))

    def stats(self):
        return rj_get_stats(self.ctx)

    def spans(self, **kw):
        return rj_debug_pixel_spans(self.ctx, make_desc(**kw))

    def boundary_mask(self, **kw):
        return rj_debug_boundary_mask(self.ctx, make_desc(**kw))

    def boundary_pieces(self, **kw):
        return rj_debug_boundary_pieces(self.ctx, make_desc(**kw))

    def membership(self, **kw):
        return rj_debug_point_membership(self.ctx, make_desc(**kw), self.n_input)
