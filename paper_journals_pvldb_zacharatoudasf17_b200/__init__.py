"""B200-native Raster Join (PVLDB 11(3), 2017): spatial aggregation of points
over arbitrary polygons via a point draw + polygon rasterisation, hand-written
CUDA for sm_100a behind the C ABI in include/rj.h.

The package holds only the hot path: csrc/ (CUDA kernels + C ABI, built into
librj.so) and the ctypes binding (rj.py).  It never imports oracle/.
"""
from .rj import (RasterJoin, RJError, lib, make_desc, rj_create, rj_debug_boundary_mask,  # noqa: F401
                 rj_debug_pixel_spans, rj_debug_point_membership, rj_destroy, rj_finalize_device,
                 rj_get_stats, rj_load_points, rj_load_polygons, rj_query, rj_query_device,
                 rj_resolve_canvas, rj_resolve_canvas_domain, rj_set_option)

__all__ = ["RasterJoin", "RJError", "lib", "make_desc"]
