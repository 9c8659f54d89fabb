// api.cu -- the extern "C" boundary of librj (include/rj.h) and the host
// orchestration of a query: S0 resolve -> polygon pass (S3 [+ S5]) -> fused
// point pass (S2/S7 + S4) -> S8 finalise.  All device work is in the
// kernels of this library; there is no CPU fallback.
#include <algorithm>
#include <cstdlib>
#include <cmath>
#include <cstring>
#include <new>

#include "rj_internal.cuh"

namespace rj {

rj_status set_error(Ctx *c, rj_status s, const std::string &msg) {
    if (c) c->err = msg;
    return s;
}

rj_status cuda_error(Ctx *c, cudaError_t e, const char *where) {
    if (c) {
        c->poisoned = true;
        c->err = std::string("CUDA error ") + cudaGetErrorName(e) + " (" + cudaGetErrorString(e) + ") at " + where;
    }
    return RJ_ERR_CUDA;
}

cudaError_t dalloc(Ctx *c, Buf &b, size_t bytes) {
    ++c->alloc_gen;
    b.p = nullptr;
    b.bytes = 0;
    if (bytes == 0) bytes = 16;
    if (c->alloc_fn) {
        b.p = c->alloc_fn(bytes, c->alloc_user);
        if (!b.p) return cudaErrorMemoryAllocation;
    } else {
        cudaError_t e = cudaMalloc(&b.p, bytes);
        if (e != cudaSuccess) {
            cudaGetLastError();
            b.p = nullptr;
            return e;
        }
    }
    b.bytes = bytes;
    return cudaSuccess;
}

void dfree(Ctx *c, Buf &b) {
    ++c->alloc_gen;
    if (b.p) {
        if (c->free_fn) c->free_fn(b.p, c->alloc_user);
        else cudaFree(b.p);
    }
    b.p = nullptr;
    b.bytes = 0;
}

cudaError_t dreserve(Ctx *c, Buf &b, size_t bytes) {
    if (b.p && b.bytes >= bytes) return cudaSuccess;
    if (c->capturing) return cudaErrorNotPermitted;          // never grow inside a graph capture
    if (b.p) {
        cudaError_t e = cudaStreamSynchronize(c->stream);    // grow: no kernel may still use it
        if (e != cudaSuccess) return e;
        dfree(c, b);
    }
    return dalloc(c, b, std::max<size_t>(bytes + bytes / 4, 256));
}

cudaError_t dreserve_exact(Ctx *c, Buf &b, size_t bytes) {
    if (b.p && b.bytes >= bytes) return cudaSuccess;
    if (c->capturing) return cudaErrorNotPermitted;
    if (b.p) {
        cudaError_t e = cudaStreamSynchronize(c->stream);
        if (e != cudaSuccess) return e;
        dfree(c, b);
    }
    return dalloc(c, b, bytes);
}

Buf &wsbuf(Ctx *c, int slot) { return c->ws[slot]; }

// S0: canvas resolution from the descriptor (reading Z3: W = ceil(w*sqrt(2)/eps)).
static rj_status resolve(double x0, double y0, double x1, double y1, const rj_query_desc *q, int *W, int *H) {
    double w, h;
    if (q->canvas_w > 0 || q->canvas_h > 0) {
        w = q->canvas_w;
        h = q->canvas_h;
    } else {
        if (!(q->epsilon > 0.0)) return RJ_ERR_RESOLUTION;
        w = std::ceil((x1 - x0) * std::sqrt(2.0) / q->epsilon);
        h = std::ceil((y1 - y0) * std::sqrt(2.0) / q->epsilon);
    }
    if (!(w >= 1.0 && w <= RJ_MAX_CANVAS && h >= 1.0 && h <= RJ_MAX_CANVAS)) return RJ_ERR_RESOLUTION;
    *W = (int)w;
    *H = (int)h;
    return RJ_OK;
}

// Viewport window (reading Z20): all zero = the whole canvas.
static rj_status resolve_view(Ctx *c, const rj_query_desc *q, int W, int H, View &v) {
    v = View{};
    const int32_t *w = q->view;
    if (!w[0] && !w[1] && !w[2] && !w[3]) {
        v.c1 = W;
        v.r1 = H;
        return RJ_OK;
    }
    if (!(0 <= w[0] && w[0] < w[2] && w[2] <= W && 0 <= w[1] && w[1] < w[3] && w[3] <= H))
        return set_error(c, RJ_ERR_INVALID_ARGUMENT, "view must be all zero or 0 <= c0 < c1 <= W, 0 <= r0 < r1 <= H");
    v.c0 = w[0];
    v.r0 = w[1];
    v.c1 = w[2];
    v.r1 = w[3];
    v.full = v.c0 == 0 && v.r0 == 0 && v.c1 == W && v.r1 == H;
    return RJ_OK;
}

// Level-L cell columns [lo, hi] whose pixel extent (cell_pix_lo..hi) meets
// pixels [p0, p1) of a side of n pixels.
static void cell_range(int64_t p0, int64_t p1, int64_t n, int L, uint32_t &lo, uint32_t &hi) {
    const int64_t nc = int64_t(1) << L;
    int64_t a = 0, b = nc - 1;
    while (a < nc - 1 && cell_pix_hi(a, n, L) < p0) ++a;
    while (b > 0 && cell_pix_lo(b, n, L) > p1 - 1) --b;
    lo = (uint32_t)a;
    hi = (uint32_t)b;
}

// Integer predicates become one inclusive int32 range per column:
// t < c <=> t <= ceil(c)-1,  t <= c <=> t <= floor(c),  t > c <=> t >= floor(c)+1,
// t >= c <=> t >= ceil(c),   t == c <=> c integral and t == c  (exact for int32 t).
static void int_range(int op, double c, int64_t &lo, int64_t &hi, int &never) {
    if (std::isnan(c)) { never = 1; return; }
    auto cl = [](double v) -> int64_t {
        if (v < -4294967296.0) return -4294967296ll;
        if (v > 4294967296.0) return 4294967296ll;
        return (int64_t)v;
    };
    switch (op) {
    case RJ_LT: hi = std::min(hi, cl(std::ceil(c)) - 1); break;
    case RJ_LE: hi = std::min(hi, cl(std::floor(c))); break;
    case RJ_GT: lo = std::max(lo, cl(std::floor(c)) + 1); break;
    case RJ_GE: lo = std::max(lo, cl(std::ceil(c))); break;
    default:
        if (std::floor(c) != c) { never = 1; return; }
        lo = std::max(lo, cl(c));
        hi = std::min(hi, cl(c));
    }
}

rj_status build_filter(Ctx *c, const rj_query_desc *q, int n_cols, const int *col_dtype, Filter &f) {
    f = Filter{};
    if (q->n_pred < 0 || q->n_pred > RJ_MAX_PRED) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "n_pred must be in [0, 5]");
    if (q->agg < RJ_COUNT || q->agg > RJ_MAX) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "bad agg");
    if (q->mode < RJ_BOUNDED || q->mode > RJ_EXACT) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "bad mode");
    for (int k = 0; k < q->n_pred; ++k) {
        const rj_pred &p = q->pred[k];
        if (p.column < 0 || p.column >= n_cols) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "predicate column out of range");
        if (p.op < RJ_LT || p.op > RJ_EQ) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "bad predicate op");
    }
    if (q->agg != RJ_COUNT && (q->agg_column < 0 || q->agg_column >= n_cols))
        return set_error(c, RJ_ERR_INVALID_ARGUMENT, "agg_column out of range");
    // slots: the aggregated column first (slot 0: the kernels read it at a
    // fixed index), then the other int-predicate columns, then the other
    // float-predicate columns.  Every slot carries an inclusive int32 range
    // (the whole int32 range unless int predicates narrow it), so the range
    // check of any slot -- float columns included -- is exact.
    int slot_of[RJ_MAX_COLS];
    for (int k = 0; k < RJ_MAX_COLS; ++k) slot_of[k] = -1;
    int64_t lo[6], hi[6];
    for (int s = 0; s < 6; ++s) { lo[s] = INT32_MIN; hi[s] = INT32_MAX; }
    auto slot = [&](int col) {
        if (slot_of[col] < 0) {
            slot_of[col] = f.n_slots;
            f.slot_col[f.n_slots] = col;
            f.slot_is_float[f.n_slots] = col_dtype[col] == RJ_F32;
            f.n_slots++;
        }
        return slot_of[col];
    };
    if (q->agg != RJ_COUNT) {
        f.agg_slot = slot(q->agg_column);
        f.agg_is_float = f.slot_is_float[f.agg_slot];
    }
    for (int k = 0; k < q->n_pred; ++k) {
        const rj_pred &p = q->pred[k];
        if (col_dtype[p.column] != RJ_I32) continue;
        const int s = slot(p.column);
        int_range(p.op, p.value, lo[s], hi[s], f.never);
    }
    for (int k = 0; k < q->n_pred; ++k) {
        const rj_pred &p = q->pred[k];
        if (col_dtype[p.column] != RJ_F32) continue;
        f.f_slot[f.n_fpred] = slot(p.column);
        f.f_op[f.n_fpred] = p.op;
        f.f_val[f.n_fpred] = (float)p.value;
        f.n_fpred++;
    }
    f.n_irange = f.n_slots;
    for (int s = 0; s < 6; ++s) {
        if (lo[s] > hi[s]) { f.never = 1; lo[s] = hi[s] = 0; }
        f.ilo[s] = (int32_t)std::max<int64_t>(lo[s], INT32_MIN);
        f.ihi[s] = (int32_t)std::min<int64_t>(hi[s], INT32_MAX);
    }
    return RJ_OK;
}

// Largest point tile of a W x H canvas at cell level L: (rows, odd row stride).
static void tile_geometry(int W, int H, int L, uint32_t &stride, uint32_t &cap) {
    int64_t mw = 0, mh = 0;
    for (int64_t k = 0; k < (int64_t(1) << L); ++k) {
        mw = std::max(mw, cell_pix_hi(k, W, L) - cell_pix_lo(k, W, L) + 1);
        mh = std::max(mh, cell_pix_hi(k, H, L) - cell_pix_lo(k, H, L) + 1);
    }
    stride = (uint32_t)(mw | 1);
    cap = (uint32_t)((mh * stride + 3) & ~3);    // whole 16-B words: tiles stay aligned, cleared with 16-B stores
}

// Exact-mode chooser (RJ_EXACT).  Both exact variants
// stream every point once; the accurate raster join adds the polygon pass and
// a small per-point cost of its boundary check, and tests only points in
// boundary pixels; the index join tests every point:
//   accurate:   T_poly + N c_acc + f N c_bnd       index join:  N c_idx
// f = estimated boundary-pixel fraction (each edge's supercover touches about
// |dx| W + |dy| H (lattice units / 2^30) + 1 pixels; uniform point density
// assumed), T_poly = floor + crossings + boundary mask.  Constants measured
// on B200 (C2/C3 sweeps, profiles/r1_chooser.md); N = loaded points (the
// filter's selectivity is unknown before the pass).
struct ChooserModel {
    double t_floor_ns = 60e3;      // polygon-pass launch / sync floor
    double t_cross_ns = 0.2;       // per (edge, row) crossing
    double t_mask_ns = 0.002;      // per canvas pixel (boundary mask clear + mark)
    double c_acc_ns = 0.00075;     // per streamed point: boundary-flag check
    double c_bnd_ns = 0.096;       // per boundary point (queued PIP, clustered near edges)
    double c_idx_ns = 0.028;       // per point, index join (full-warp PIP batches)
};

static float boundary_fraction(const Ctx *c, int W, int H) {
    const double px = (double)W * H;
    const double b = (c->edge_len_x * W + c->edge_len_y * H) / 1073741824.0 + (double)c->n_edges;
    return (float)std::min(1.0, b / px);
}

static int choose_exact(const Ctx *c, int W, int H, float f, uint64_t n_points) {
    const ChooserModel m;
    const double n = (double)n_points;
    const double cross = c->edge_len_y * H / 1073741824.0 + (double)c->n_edges;
    const double t_acc = m.t_floor_ns + m.t_cross_ns * cross + m.t_mask_ns * (double)W * H + n * m.c_acc_ns +
                         f * n * m.c_bnd_ns;
    return n * m.c_idx_ns < t_acc ? RJ_INDEX_JOIN : RJ_ACCURATE;
}

struct Prepared {
    bool init_done = false;        // k_pass_init already ran ahead of the polygon pass
    uint32_t poly_launches = 0;    // kernels the polygon pass launched after it
    int W, H, L;
    View view;
    int mode;                      // executed rj_mode (RJ_EXACT resolved)
    bool sum, acc, index;
    PolyPass pp;
    PassArgs a;
};

static rj_status check_ready(Ctx *c, const rj_query_desc *q) {
    if (!c) return RJ_ERR_INVALID_ARGUMENT;
    if (c->poisoned) return set_error(c, RJ_ERR_CUDA, c->err.empty() ? "context poisoned" : c->err);
    if (!q) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL query descriptor");
    if (!c->cell_off.p) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "query before rj_load_points");
    if (!c->n_poly) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "query before rj_load_polygons");
    if (cudaSetDevice(c->device) != cudaSuccess) return set_error(c, RJ_ERR_CUDA, "cudaSetDevice failed");
    return RJ_OK;
}

// Timing events; inside a graph capture they become event-record nodes.
static cudaError_t record_ev(Ctx *c, int i) {
    return cudaEventRecordWithFlags(c->ev[i], c->stream, c->capturing ? cudaEventRecordExternal : cudaEventRecordDefault);
}

// Everything up to (not including) the point-pass launch.
static rj_status prepare(Ctx *c, const rj_query_desc *q, Prepared &P, bool need_polygon_pass = true,
                         bool bands = false, bool need_mask = false, unsigned long long *d_cnt = nullptr,
                         double *d_sum = nullptr) {
    rj_status s = check_ready(c, q);
    if (s != RJ_OK) return s;
    if ((s = resolve(c->x0, c->y0, c->x1, c->y1, q, &P.W, &P.H)) != RJ_OK)
        return set_error(c, s, "canvas resolution outside [1, 131072] or bad epsilon");
    if ((s = resolve_view(c, q, P.W, P.H, P.view)) != RJ_OK) return s;
    Filter f;
    if ((s = build_filter(c, q, c->n_cols, c->col_dtype, f)) != RJ_OK) return s;
    P.sum = q->agg != RJ_COUNT;
    const float f_bnd = boundary_fraction(c, P.W, P.H);
    P.mode = q->mode == RJ_EXACT ? choose_exact(c, P.W, P.H, f_bnd, c->n_pts) : q->mode;
    P.acc = P.mode != RJ_BOUNDED;
    P.index = P.mode == RJ_INDEX_JOIN;
    c->last.mode = P.mode;
    c->last.est_boundary_frac = f_bnd;
    PassArgs &a = P.a;
    memset(&a, 0, sizeof(a));
    a.f = f;
    a.n_poly = c->n_poly;
    // cell level: tiles of ~tile_side pixels, refined while two CTAs with a
    // two-stage ring would not fit in shared memory; per-CTA polygon partials
    // in shared memory unless they crowd out the ring
    P.L = choose_level(P.W, P.H, c->tile_side);
    for (;;) {
        tile_geometry(P.W, P.H, P.L, a.tile_stride, a.tile_cap);
        a.n_stages = 2;
        a.smem_partials = 1;
        if (point_pass_smem(c, a, P.sum, P.acc) > 160 * 1024) a.smem_partials = 0;
        if (point_pass_smem(c, a, P.sum, P.acc) + 3 * 1024 <= 112 * 1024 || P.L >= kMaxLevel) break;
        ++P.L;
    }
    a.n_stages = (uint32_t)point_pass_stages(f.n_slots);
    a.lane_runs = c->lane_runs != 2;
    if ((s = items_for_level(c, P.L)) != RJ_OK) return s;
    c->launches = 0;
    // work counters / pass statistics (cleared per pass)
    Buf &wk = wsbuf(c, kWsWork);
    if (dreserve(c, wk, 64)) return set_error(c, RJ_ERR_OOM, "workspace allocation failed");
    if (c->timing) RJ_CUDA(c, record_ev(c, 0));
    // the index join needs neither spans nor the boundary mask
    P.pp = PolyPass{};
    const bool poly = need_polygon_pass && !P.index;
    if (poly && d_cnt) {
        // the per-query reset runs first, so the point pass's producer warp
        // may start streaming while the polygon pass's last kernel still runs
        // (it reads only the work counter and the static items; PDL: that
        // kernel triggered its dependents after its own wait)
        RJ_CUDA(c, launch_pass_init(c, wsbuf(c, kWsWork).as<uint32_t>(), d_cnt, P.sum ? d_sum : nullptr, c->n_poly));
        P.init_done = true;
    }
    const uint32_t l0 = c->launches;
    if (poly && (s = polygon_pass(c, P.W, P.H, P.L, P.acc || bands, P.pp, P.view, need_mask && P.acc)) != RJ_OK)
        return s;
    P.poly_launches = c->launches - l0;
    if (c->timing) RJ_CUDA(c, record_ev(c, 1));
    a.qx = c->qx.as<uint32_t>();
    a.qy = c->qy.as<uint32_t>();
    for (int k = 0; k < f.n_slots; ++k) a.col[k] = c->col[f.slot_col[k]].as<uint32_t>();
    a.W = P.W;
    a.H = P.H;
    a.items = c->items[P.L].as<int4>();
    a.n_items = c->n_items[P.L];
    a.level = P.L;
    a.cell_off10 = c->cell_off.as<uint32_t>();
    a.piece_off = P.pp.piece_off;
    a.pieces = P.pp.pieces;
    a.mask = P.acc ? P.pp.mask : nullptr;
    a.mask_wpr = P.pp.mask_wpr;
    a.bpiece_off = P.pp.bpiece_off;
    a.bpieces = P.pp.bpieces;
    a.index_join = P.index;
    a.grid_off = c->grid_off.as<uint32_t>();
    a.grid_ent = c->grid_ent.as<uint32_t>();
    a.grid_edge = c->grid_edge.as<int4>();
    a.grid_poly = c->grid_poly.as<uint32_t>();
    a.edges = c->edges.as<int4>();
    a.edge_poly = c->edge_poly.as<uint32_t>();
    Buf &st = wsbuf(c, kWsWork);
    a.work_counter = st.as<uint32_t>();
    a.stats = reinterpret_cast<unsigned long long *>(st.as<uint32_t>() + 2);
    a.view[0] = P.view.c0;
    a.view[1] = P.view.r0;
    a.view[2] = P.view.c1;
    a.view[3] = P.view.r1;
    cell_range(P.view.c0, P.view.c1, P.W, P.L, a.cwin[0], a.cwin[2]);
    cell_range(P.view.r0, P.view.r1, P.H, P.L, a.cwin[1], a.cwin[3]);
    return RJ_OK;
}

// Accurate mode: size the global boundary-point queue (S7).  The capacity
// follows the previous query's boundary count (grow-only), at least twice
// the estimated boundary-pixel fraction of the points and >= 2^22; points
// beyond it are tested inline (always exact).  The index join tests every
// point inline (no queue).
static rj_status setup_bqueue(Ctx *c, Prepared &P) {
    PassArgs &a = P.a;
    a.bq_cap = 0;
    a.bq_count = a.work_counter + 8;
    a.bq_valid = a.work_counter + 9;
    if (!P.acc || P.index || !c->n_pts) return RJ_OK;
    const uint64_t est = (uint64_t)(2.0 * c->last.est_boundary_frac * (double)c->n_pts);
    uint64_t want = std::max<uint64_t>({uint64_t(1) << 22, est, c->h_stats[1] + c->h_stats[1] / 4});
    want = std::min<uint64_t>(want, c->n_pts);
    want = std::min<uint64_t>(want, 0xFFFFFFC0ull);
    Buf &bx = wsbuf(c, kWsBQx), &by = wsbuf(c, kWsBQy), &ba = wsbuf(c, kWsBQa);
    if (dreserve(c, bx, want * 4) || dreserve(c, by, want * 4) || (P.sum && dreserve(c, ba, want * 4)))
        return RJ_OK;                                     // no room: inline tests (exact either way)
    a.bq_x = bx.as<uint32_t>();
    a.bq_y = by.as<uint32_t>();
    a.bq_a = P.sum ? ba.as<uint32_t>() : nullptr;
    a.bq_cap = (uint32_t)want;
    // chunks: a few per consumer warp of a full grid (2 CTAs x 8 warps per SM), 32..512 entries
    const uint64_t warps = (uint64_t)c->num_sms * 16;
    a.bq_chunk = (uint32_t)std::min<uint64_t>(512, std::max<uint64_t>(32, (want / (4 * warps)) & ~uint64_t(31)));
    return RJ_OK;
}

static rj_status run_pass(Ctx *c, Prepared &P, unsigned long long *d_cnt, double *d_sum) {
    PassArgs &a = P.a;
    a.A_cnt = d_cnt;
    a.A_sum = d_sum;
    rj_status s = setup_bqueue(c, P);
    if (s != RJ_OK) return s;
    a.early_stream = P.init_done && P.poly_launches > 0;
    if (!P.init_done) RJ_CUDA(c, launch_pass_init(c, a.work_counter, d_cnt, P.sum ? d_sum : nullptr, c->n_poly));
    s = point_pass(c, a, P.sum, P.acc);
    if (s != RJ_OK) return s;
    if (a.bq_cap && (s = pip_queue_pass(c, a, P.sum)) != RJ_OK) return s;
    c->last_bq = a;
    if (c->timing) RJ_CUDA(c, record_ev(c, 2));
    RJ_CUDA(c, cudaMemcpyAsync(c->h_stats, a.stats, 2 * sizeof(unsigned long long), cudaMemcpyDeviceToHost, c->stream));
    // statistics of this query
    c->stream_stats_pending = 0;
    rj_stats &L = c->last;
    L.W = P.W;
    L.H = P.H;
    L.n_points = c->n_pts;
    L.n_crossings = P.pp.n_cross;
    L.n_spans = P.pp.n_spans;
    L.n_pieces = P.pp.n_pieces;
    L.n_items = c->n_items[P.L];
    L.level = P.L;
    L.stream_bytes = c->n_pts * (8ull + 4ull * (uint64_t)a.f.n_slots);
    return RJ_OK;
}

// Queries served by the label-canvas pass (label_canvas.cu): MIN/MAX,
// several aggregates, streamed points.  ap = the requested aggregates (may be
// empty: COUNT only); values[k * n_poly + i] for each of ap (or the count as
// double when ap is empty).  COUNT entries need no kernel channel.
static rj_status label_query_with_cols(Ctx *c, const rj_query_desc *q, const AggPlan &ap, const LabInput &in,
                                       int n_cols, uint64_t *count, double *values) {
    if (cudaSetDevice(c->device) != cudaSuccess) return set_error(c, RJ_ERR_CUDA, "cudaSetDevice failed");
    int W, H;
    rj_status s = resolve(c->x0, c->y0, c->x1, c->y1, q, &W, &H);
    if (s != RJ_OK) return set_error(c, s, "canvas resolution outside [1, 131072] or bad epsilon");
    View v;
    if ((s = resolve_view(c, q, W, H, v)) != RJ_OK) return s;
    rj_query_desc qf = *q;
    qf.agg = RJ_COUNT;                        // aggregate columns are read by the plan, not the filter
    Filter f;
    if ((s = build_filter(c, &qf, n_cols, in.col_dtype, f)) != RJ_OK) return s;
    const float f_bnd = boundary_fraction(c, W, H);
    const int mode = q->mode == RJ_EXACT ? choose_exact(c, W, H, f_bnd, in.n) : q->mode;
    c->last.mode = mode;
    c->last.est_boundary_frac = f_bnd;
    AggPlan kp;                               // kernel channels: the non-COUNT aggregates
    int slot[kMaxAggs];
    for (int k = 0; k < ap.n; ++k) {
        slot[k] = -1;
        if (ap.kind[k] == RJ_COUNT) continue;
        slot[k] = kp.n;
        kp.kind[kp.n] = ap.kind[k];
        kp.col[kp.n] = ap.col[k];
        ++kp.n;
    }
    const size_t np = c->n_poly;
    const int nv = std::max(1, ap.n);
    if (dreserve(c, c->res_cnt, np * 8) || dreserve(c, c->res_agg, (size_t)std::max(1, kp.n) * np * 8) ||
        dreserve(c, c->res_val, (size_t)nv * np * 8))
        return set_error(c, RJ_ERR_OOM, "result allocation failed");
    if ((s = label_query_impl(c, f, kp, W, H, v, mode, in, c->res_cnt.as<unsigned long long>(), c->res_agg.p)) != RJ_OK)
        return s;
    if (values) {
        for (int k = 0; k < nv; ++k) {
            AggPlan one;
            one.n = 1;
            one.kind[0] = ap.n ? ap.kind[k] : RJ_COUNT;
            one.col[0] = ap.n ? ap.col[k] : 0;
            const void *agg = (ap.n && slot[k] >= 0) ? c->res_agg.as<unsigned char>() + (size_t)slot[k] * np * 8
                                                     : c->res_agg.p;
            RJ_CUDA(c, launch_finalize_aggs(c, one, in.col_dtype, (uint32_t)np, c->res_cnt.as<unsigned long long>(),
                                            agg, c->res_val.as<double>() + (size_t)k * np));
        }
        RJ_CUDA(c, cudaMemcpyAsync(values, c->res_val.p, (size_t)nv * np * 8, cudaMemcpyDeviceToHost, c->stream));
    }
    if (count) RJ_CUDA(c, cudaMemcpyAsync(count, c->res_cnt.p, np * 8, cudaMemcpyDeviceToHost, c->stream));
    if (c->timing) RJ_CUDA(c, record_ev(c, 3));
    RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    return RJ_OK;
}

static LabInput lattice_input(Ctx *c) {
    LabInput in;
    in.lattice = true;
    in.n = c->n_pts;
    in.x = c->qx.p;
    in.y = c->qy.p;
    in.col_dtype = c->col_dtype;
    return in;
}

static AggPlan single_plan(const rj_query_desc *q) {
    AggPlan ap;
    if (q->agg != RJ_COUNT) {
        ap.n = 1;
        ap.kind[0] = q->agg;
        ap.col[0] = q->agg_column;
    }
    return ap;
}

// ---- CUDA-graph replay of repeated queries ---------------------------------
// A query's device work is ~40 launches (the polygon pass's small kernels,
// scans and memsets, the point pass, finalise); at 1/8 of the points per GPU
// the polygon pass becomes launch-bound.  The second consecutive call with
// the same key (descriptor, output pointers, options, loaded data and every
// device allocation) is captured into a CUDA graph, and later calls with
// that key replay it with one cudaGraphLaunch.  Every kernel still runs on
// every query: only the host-side launch sequence is reused.  The capture
// needs a host-sync-free sequence, which the polygon pass's size cache
// (same key => same sizes) provides; if anything would allocate or sync
// during the capture, it is abandoned and the query runs eagerly.
static void key_desc(std::vector<int64_t> &k, const rj_query_desc *q) {
    auto bits = [](double v) { int64_t b; memcpy(&b, &v, 8); return b; };
    k.insert(k.end(), {q->agg, q->agg_column, q->n_pred});
    for (int i = 0; i < q->n_pred && i < RJ_MAX_PRED; ++i)
        k.insert(k.end(), {q->pred[i].column, q->pred[i].op, bits(q->pred[i].value)});
    k.insert(k.end(), {q->canvas_w, q->canvas_h, bits(q->epsilon), q->mode, q->view[0], q->view[1], q->view[2],
                       q->view[3]});
}

static std::vector<int64_t> query_key(Ctx *c, const rj_query_desc *q, int entry, const void *p0, const void *p1) {
    std::vector<int64_t> k = {entry, (int64_t)(uintptr_t)p0, (int64_t)(uintptr_t)p1, (int64_t)c->data_gen,
                              (int64_t)c->alloc_gen, c->timing, c->chunk, c->tile_side, c->force_stages,
                              c->pass_variant, c->lane_runs, (int64_t)(uintptr_t)c->stream};
    key_desc(k, q);
    return k;
}

static void drop_graph(Ctx *c) {
    if (c->graph_exec) cudaGraphExecDestroy(c->graph_exec);
    c->graph_exec = nullptr;
    c->graph_key.clear();
}

template <class F>
static rj_status run_graphed(Ctx *c, std::vector<int64_t> key, F body) {
    // the caller is capturing the context's stream into its own graph: the
    // query's work becomes part of that graph (no internal graph; anything
    // that would allocate or synchronise fails the capture loudly)
    cudaStreamCaptureStatus cs = cudaStreamCaptureStatusNone;
    if (cudaStreamIsCapturing(c->stream, &cs) == cudaSuccess && cs != cudaStreamCaptureStatusNone) {
        c->capturing = true;
        rj_status s = body();
        c->capturing = false;
        return s;
    }
    if (c->use_graphs && c->graph_exec && key == c->graph_key) {
        RJ_CUDA(c, cudaGraphLaunch(c->graph_exec, c->stream));
        c->last = c->graph_last;
        c->launches = c->graph_launches;
        c->last_stages = c->graph_stages;
        c->last_ctas_per_sm = c->graph_ctas;
        c->stream_stats_pending = 0;
        return RJ_OK;
    }
    if (!c->use_graphs || key != c->pending_key) {
        rj_status s = body();
        c->pending_key.clear();
        if (s == RJ_OK) {
            key[4] = (int64_t)c->alloc_gen;      // allocations made by this call are part of the state
            c->pending_key = key;
        }
        return s;
    }
    drop_graph(c);
    c->pending_key.clear();
    if (cudaStreamBeginCapture(c->stream, cudaStreamCaptureModeRelaxed) != cudaSuccess) {
        cudaGetLastError();
        return body();
    }
    c->capturing = true;
    rj_status s = body();
    c->capturing = false;
    cudaGraph_t g = nullptr;
    cudaError_t e = cudaStreamEndCapture(c->stream, &g);
    cudaGraphExec_t ex = nullptr;
    if (s == RJ_OK && e == cudaSuccess && g) e = cudaGraphInstantiate(&ex, g, 0);
    if (g) cudaGraphDestroy(g);
    if (s != RJ_OK || e != cudaSuccess || !ex) {
        // nothing of the capture ran: clear its error and run eagerly
        cudaGetLastError();
        c->poisoned = false;
        c->err.clear();
        return body();
    }
    c->graph_exec = ex;
    key[4] = (int64_t)c->alloc_gen;
    c->graph_key = key;
    c->graph_last = c->last;
    c->graph_launches = c->launches;
    c->graph_stages = c->last_stages;
    c->graph_ctas = c->last_ctas_per_sm;
    RJ_CUDA(c, cudaGraphLaunch(ex, c->stream));
    return RJ_OK;
}

}  // namespace rj

using namespace rj;

struct rj_ctx : rj::Ctx {};

extern "C" {

const char *rj_version(void) { return "rj-b200 0.1 (sm_100a)"; }

const char *rj_status_str(rj_status s) {
    switch (s) {
    case RJ_OK: return "RJ_OK";
    case RJ_ERR_INVALID_ARGUMENT: return "RJ_ERR_INVALID_ARGUMENT";
    case RJ_ERR_OUT_OF_DOMAIN: return "RJ_ERR_OUT_OF_DOMAIN";
    case RJ_ERR_RESOLUTION: return "RJ_ERR_RESOLUTION";
    case RJ_ERR_CAPACITY: return "RJ_ERR_CAPACITY";
    case RJ_ERR_OOM: return "RJ_ERR_OOM";
    case RJ_ERR_CUDA: return "RJ_ERR_CUDA";
    }
    return "RJ_ERR_UNKNOWN";
}

const char *rj_last_error(const rj_ctx *ctx) { return ctx ? ctx->err.c_str() : "NULL context"; }

rj_status rj_resolve_canvas_domain(double x0, double y0, double x1, double y1, const rj_query_desc *q,
                                   int32_t *W, int32_t *H) {
    if (!q || !W || !H) return RJ_ERR_INVALID_ARGUMENT;
    int w, h;
    rj_status s = resolve(x0, y0, x1, y1, q, &w, &h);
    if (s == RJ_OK) { *W = w; *H = h; }
    return s;
}

// Reading Z20: the pixels [p0, p1) of a side of n pixels that hold every
// point with wlo <= v < whi.  O1 is monotone (non-decreasing in v: every op
// is correctly rounded), so such a point has Q(wlo) <= Q(v) <= Q(v'), v' the
// largest double below whi; bounds beyond the domain clamp to it.
static rj_status axis_window(double lo, double hi, int n, double wlo, double whi, int32_t &p0, int32_t &p1) {
    if (std::isnan(wlo) || std::isnan(whi) || !(wlo < whi)) return RJ_ERR_INVALID_ARGUMENT;
    const int64_t top = (int64_t(1) << kLatticeBits) - 1;
    auto q = [&](double v) -> int64_t {
        if (v <= lo) return 0;
        if (v >= hi) return top;
        volatile double d = v - lo;                  // O1, each op rounded, no contraction
        volatile double s = hi - lo;
        volatile double f = d / s;
        volatile double g = f * 1073741824.0;
        return std::min<int64_t>(top, std::max<int64_t>(0, (int64_t)std::floor(g)));
    };
    const int64_t a = (q(wlo) * n) >> kLatticeBits;
    const int64_t b = whi > hi ? n : ((q(std::nextafter(whi, -INFINITY)) * n) >> kLatticeBits) + 1;
    p0 = (int32_t)a;
    p1 = (int32_t)std::max<int64_t>(b, a + 1);
    return RJ_OK;
}

rj_status rj_resolve_window(double x0, double y0, double x1, double y1, const rj_query_desc *q, double wx0,
                            double wy0, double wx1, double wy1, int32_t *view) {
    if (!q || !view) return RJ_ERR_INVALID_ARGUMENT;
    int W, H;
    rj_status s = resolve(x0, y0, x1, y1, q, &W, &H);
    if (s != RJ_OK) return s;
    int32_t v[4];
    if ((s = axis_window(x0, x1, W, wx0, wx1, v[0], v[2])) != RJ_OK) return s;
    if ((s = axis_window(y0, y1, H, wy0, wy1, v[1], v[3])) != RJ_OK) return s;
    std::copy(v, v + 4, view);
    return RJ_OK;
}

rj_status rj_resolve_lod(double x0, double y0, double x1, double y1, double wx0, double wy0, double wx1,
                         double wy1, int32_t w, int32_t h, int32_t *W, int32_t *H, int32_t *view) {
    if (!W || !H || !view || w < 1 || h < 1 || !(wx1 > wx0) || !(wy1 > wy0)) return RJ_ERR_INVALID_ARGUMENT;
    // the finer canvas over the whole domain whose pixels are as large as
    // w x h pixels over the world rectangle
    const double fw = std::nearbyint((double)w * (x1 - x0) / (wx1 - wx0));
    const double fh = std::nearbyint((double)h * (y1 - y0) / (wy1 - wy0));
    if (!(fw >= 1.0 && fh >= 1.0)) return RJ_ERR_RESOLUTION;
    rj_query_desc q{};
    q.canvas_w = (int32_t)std::min(fw, (double)RJ_MAX_CANVAS);
    q.canvas_h = (int32_t)std::min(fh, (double)RJ_MAX_CANVAS);
    rj_status s = rj_resolve_window(x0, y0, x1, y1, &q, wx0, wy0, wx1, wy1, view);
    if (s != RJ_OK) return s;
    *W = q.canvas_w;
    *H = q.canvas_h;
    return RJ_OK;
}

rj_status rj_resolve_canvas(const rj_ctx *ctx, const rj_query_desc *q, int32_t *W, int32_t *H) {
    if (!ctx) return RJ_ERR_INVALID_ARGUMENT;
    return rj_resolve_canvas_domain(ctx->x0, ctx->y0, ctx->x1, ctx->y1, q, W, H);
}

rj_status rj_create(rj_ctx **out, int32_t dev, void *stream, double x0, double y0, double x1, double y1) {
    if (!out) return RJ_ERR_INVALID_ARGUMENT;
    *out = nullptr;
    if (!(std::isfinite(x0) && std::isfinite(x1) && std::isfinite(y0) && std::isfinite(y1) && x1 > x0 && y1 > y0))
        return RJ_ERR_INVALID_ARGUMENT;
    int ndev = 0;
    if (cudaGetDeviceCount(&ndev) != cudaSuccess || dev < 0 || dev >= ndev) {
        cudaGetLastError();
        return RJ_ERR_CUDA;
    }
    if (cudaSetDevice(dev) != cudaSuccess) return RJ_ERR_CUDA;
    cudaDeviceProp prop;
    if (cudaGetDeviceProperties(&prop, dev) != cudaSuccess) return RJ_ERR_CUDA;
    if (prop.major < 10) return RJ_ERR_CUDA;   // built for sm_100a only
    rj_ctx *c = new (std::nothrow) rj_ctx();
    if (!c) return RJ_ERR_OOM;
    c->device = dev;
    c->num_sms = prop.multiProcessorCount;
    c->x0 = x0; c->y0 = y0; c->x1 = x1; c->y1 = y1;
    if (stream) {
        c->stream = (cudaStream_t)stream;
    } else {
        if (cudaStreamCreateWithFlags(&c->stream, cudaStreamNonBlocking) != cudaSuccess) { delete c; return RJ_ERR_CUDA; }
        c->own_stream = true;
    }
    if (cudaMallocHost(&c->h_stats, 64 * sizeof(unsigned long long)) != cudaSuccess) { delete c; return RJ_ERR_CUDA; }
    if (const char *e = std::getenv("RJ_NO_PDL")) c->pdl = (e[0] == '1') ? 0 : 1;
    for (auto &e : c->ev)
        if (cudaEventCreate(&e) != cudaSuccess) { delete c; return RJ_ERR_CUDA; }
    *out = c;
    return RJ_OK;
}

rj_status rj_destroy(rj_ctx *c) {
    if (!c) return RJ_ERR_INVALID_ARGUMENT;
    cudaSetDevice(c->device);
    cudaStreamSynchronize(c->stream);
    drop_graph(c);
    dfree(c, c->qx); dfree(c, c->qy); dfree(c, c->idx);
    for (auto &b : c->col) dfree(c, b);
    free_load_scratch(c);
    dfree(c, c->cell_off); drop_items(c);
    dfree(c, c->edges); dfree(c, c->edge_poly); dfree(c, c->poly_edge_off); dfree(c, c->mbr);
    dfree(c, c->poly_ring_off); dfree(c, c->ring_edge_off); dfree(c, c->edge_sigma);
    dfree(c, c->grid_off); dfree(c, c->grid_ent); dfree(c, c->grid_edge); dfree(c, c->grid_poly);
    for (auto &b : c->ws) dfree(c, b);
    dfree(c, c->res_cnt); dfree(c, c->res_sum); dfree(c, c->res_val); dfree(c, c->res_eps); dfree(c, c->res_agg);
    stream_release(c);
    for (auto &e : c->ev) if (e) cudaEventDestroy(e);
    for (auto &e : c->load_ev) if (e) cudaEventDestroy(e);
    if (c->load_stream) cudaStreamDestroy(c->load_stream);
    if (c->h_stats) cudaFreeHost(c->h_stats);
    if (c->own_stream) cudaStreamDestroy(c->stream);
    delete c;
    return RJ_OK;
}

rj_status rj_set_allocator(rj_ctx *c, void *(*alloc_fn)(size_t, void *), void (*free_fn)(void *, void *), void *user) {
    if (!c || (!alloc_fn) != (!free_fn)) return RJ_ERR_INVALID_ARGUMENT;
    if (c->qx.p || c->edges.p) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "set the allocator before any load");
    c->alloc_fn = alloc_fn;
    c->free_fn = free_fn;
    c->alloc_user = user;
    return RJ_OK;
}

rj_status rj_set_option(rj_ctx *c, int32_t option, int64_t value) {
    if (!c) return RJ_ERR_INVALID_ARGUMENT;
    if (option == RJ_OPT_TIMING) { c->timing = value ? 1 : 0; return RJ_OK; }
    if (option == RJ_OPT_GRAPHS) {
        c->use_graphs = value ? 1 : 0;
        if (!value) { drop_graph(c); c->pending_key.clear(); }
        return RJ_OK;
    }
    if (option == RJ_OPT_PASS) {
        if (value < -1 || value > 1) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "RJ_OPT_PASS must be -1, 0 or 1");
        c->pass_variant = (int)value;
        return RJ_OK;
    }
    if (option == RJ_OPT_STREAM_BATCH) {
        if (value < 1024) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "RJ_OPT_STREAM_BATCH must be >= 1024");
        c->stream_batch = value;
        return RJ_OK;
    }
    if (option == RJ_OPT_STAGES) {
        if (value != 0 && (value < 2 || value > 4)) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "RJ_OPT_STAGES must be 0 or in [2, 4]");
        c->force_stages = (int)value;
        return RJ_OK;
    }
    if (option == RJ_OPT_TILE_SIDE) {
        if (value < 4 || value > 128) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "RJ_OPT_TILE_SIDE must be in [4, 128]");
        c->tile_side = (int)value;
        return RJ_OK;
    }
    if (option == RJ_OPT_KEEP_LOAD_SCRATCH) {
        c->keep_load_scratch = value ? 1 : 0;
        if (!value) free_load_scratch(c);
        return RJ_OK;
    }
    if (option == RJ_OPT_LANE_RUNS) {
        if (value < 0 || value > 2) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "RJ_OPT_LANE_RUNS must be 0, 1 or 2");
        c->lane_runs = (int)value;
        return RJ_OK;
    }
    if (option == RJ_OPT_CHUNK) {
        if (value < 256 || value > (1ll << 30)) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "chunk must be in [256, 2^30]");
        c->chunk = value;
        return RJ_OK;
    }
    return set_error(c, RJ_ERR_INVALID_ARGUMENT, "unknown option");
}

void *rj_get_stream(const rj_ctx *c) { return c ? (void *)c->stream : nullptr; }

uint32_t rj_n_polygons(const rj_ctx *c) { return c ? c->n_poly : 0; }
uint64_t rj_n_points(const rj_ctx *c) { return c ? c->n_pts : 0; }

rj_status rj_load_points(rj_ctx *c, uint64_t n, const void *x, const void *y, int32_t xy_dtype, int32_t n_cols,
                         const void *const *cols, const int32_t *dtypes, uint64_t *n_ood) {
    if (!c) return RJ_ERR_INVALID_ARGUMENT;
    if (c->poisoned) return set_error(c, RJ_ERR_CUDA, c->err);
    if (n && (!x || !y)) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL coordinates");
    if (xy_dtype != RJ_F32 && xy_dtype != RJ_F64) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "coordinates must be RJ_F32 or RJ_F64");
    if (n_cols < 0 || n_cols > RJ_MAX_COLS) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "n_cols must be in [0, 8]");
    if (n_cols && (!cols || !dtypes)) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL attribute columns");
    for (int k = 0; k < n_cols; ++k) {
        if (dtypes[k] != RJ_I32 && dtypes[k] != RJ_F32) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "attributes must be RJ_I32 or RJ_F32");
        if (n && !cols[k]) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL attribute column");
    }
    if (n >= (1ull << 32) - 1) return set_error(c, RJ_ERR_CAPACITY, "at most 2^32 - 2 points per context");
    if (cudaSetDevice(c->device) != cudaSuccess) return set_error(c, RJ_ERR_CUDA, "cudaSetDevice failed");
    return load_points_impl(c, n, x, y, xy_dtype == RJ_F64, n_cols, cols, dtypes, n_ood);
}

rj_status rj_load_polygons(rj_ctx *c, uint32_t n_poly, const uint32_t *pro, const uint32_t *rvo, const double *vx,
                           const double *vy) {
    if (!c) return RJ_ERR_INVALID_ARGUMENT;
    if (c->poisoned) return set_error(c, RJ_ERR_CUDA, c->err);
    if (!n_poly || !pro || !rvo || !vx || !vy) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "empty or NULL polygon arrays");
    if (n_poly >= (1u << 24)) return set_error(c, RJ_ERR_CAPACITY, "at most 2^24 - 1 polygons");
    if (cudaSetDevice(c->device) != cudaSuccess) return set_error(c, RJ_ERR_CUDA, "cudaSetDevice failed");
    return load_polygons_impl(c, n_poly, pro, rvo, vx, vy);
}

rj_status rj_query_device(rj_ctx *c, const rj_query_desc *q, uint64_t *d_count, double *d_sum) {
    if (!d_count) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL d_count");
    if (!q) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL query descriptor");
    if (q->agg > RJ_AVG) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "rj_query_device: COUNT/SUM/AVG partials only");
    if (q->agg != RJ_COUNT && !d_sum) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL d_sum for SUM/AVG");
    rj_status s = check_ready(c, q);
    if (s != RJ_OK) return s;
    return run_graphed(c, query_key(c, q, 1, d_count, d_sum), [&]() -> rj_status {
        Prepared P;
        rj_status s2 = prepare(c, q, P, true, false, false, reinterpret_cast<unsigned long long *>(d_count), d_sum);
        if (s2 != RJ_OK) return s2;
        if ((s2 = run_pass(c, P, reinterpret_cast<unsigned long long *>(d_count), d_sum)) != RJ_OK) return s2;
        if (c->timing) RJ_CUDA(c, record_ev(c, 3));      // ms_total of this query (rj_get_stats)
        return RJ_OK;
    });
}

rj_status rj_finalize_device(rj_ctx *c, int32_t agg, uint32_t n, const uint64_t *d_count, const double *d_sum,
                             double *d_value) {
    if (!c || !d_count || !d_value || (agg != RJ_COUNT && !d_sum)) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "bad finalize arguments");
    if (agg < RJ_COUNT || agg > RJ_AVG) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "bad agg");
    if (c->poisoned) return set_error(c, RJ_ERR_CUDA, c->err);
    RJ_CUDA(c, launch_finalize(c, agg, n, reinterpret_cast<const unsigned long long *>(d_count), d_sum, d_value));
    return RJ_OK;
}

rj_status rj_pack_partials(rj_ctx *c, uint32_t n, const uint64_t *d_count, const double *d_sum, double *d_packed) {
    if (!c || !d_count || !d_packed) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "bad pack arguments");
    if (c->poisoned) return set_error(c, RJ_ERR_CUDA, c->err);
    RJ_CUDA(c, launch_pack(c, n, reinterpret_cast<const unsigned long long *>(d_count), d_sum, d_packed));
    return RJ_OK;
}

rj_status rj_finalize_packed(rj_ctx *c, int32_t agg, uint32_t n, const double *d_packed, uint64_t *d_count,
                             double *d_value) {
    if (!c || !d_packed || !d_count || !d_value) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "bad finalize arguments");
    if (agg < RJ_COUNT || agg > RJ_AVG) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "bad agg");
    if (c->poisoned) return set_error(c, RJ_ERR_CUDA, c->err);
    RJ_CUDA(c, launch_finalize_packed(c, agg, n, d_packed, reinterpret_cast<unsigned long long *>(d_count), d_value));
    return RJ_OK;
}

rj_status rj_query(rj_ctx *c, const rj_query_desc *q, uint64_t *count, double *value) {
    if (q && (q->agg == RJ_MIN || q->agg == RJ_MAX)) {       // distributive, label-canvas pass
        rj_status s = check_ready(c, q);
        if (s != RJ_OK) return s;
        if (q->agg_column < 0 || q->agg_column >= c->n_cols)
            return set_error(c, RJ_ERR_INVALID_ARGUMENT, "agg_column out of range");
        return label_query_with_cols(c, q, single_plan(q), lattice_input(c), c->n_cols, count, value);
    }
    rj_status s = check_ready(c, q);
    if (s != RJ_OK) return s;
    const size_t n = c->n_poly;
    if (dreserve(c, c->res_cnt, n * 8) || dreserve(c, c->res_sum, n * 8) || dreserve(c, c->res_val, n * 8))
        return set_error(c, RJ_ERR_OOM, "result allocation failed");
    s = run_graphed(c, query_key(c, q, 2, nullptr, value ? c->res_val.p : nullptr), [&]() -> rj_status {
        Prepared P;
        rj_status s2 = prepare(c, q, P, true, false, false, c->res_cnt.as<unsigned long long>(), c->res_sum.as<double>());
        if (s2 != RJ_OK) return s2;
        if ((s2 = run_pass(c, P, c->res_cnt.as<unsigned long long>(), c->res_sum.as<double>())) != RJ_OK) return s2;
        if (value) RJ_CUDA(c, launch_finalize(c, q->agg, (uint32_t)n, c->res_cnt.as<unsigned long long>(),
                                              c->res_sum.as<double>(), c->res_val.as<double>()));
        return RJ_OK;
    });
    if (s != RJ_OK) return s;
    if (count) RJ_CUDA(c, cudaMemcpyAsync(count, c->res_cnt.p, n * 8, cudaMemcpyDeviceToHost, c->stream));
    if (value) RJ_CUDA(c, cudaMemcpyAsync(value, c->res_val.p, n * 8, cudaMemcpyDeviceToHost, c->stream));
    if (c->timing) RJ_CUDA(c, record_ev(c, 3));
    RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    return RJ_OK;
}

rj_status rj_query_stream(rj_ctx *c, const rj_query_desc *q, uint64_t n, const void *x, const void *y,
                          int32_t xy_dtype, int32_t n_cols, const void *const *cols, const int32_t *dtypes,
                          uint64_t *count, double *value) {
    if (!c) return RJ_ERR_INVALID_ARGUMENT;
    if (c->poisoned) return set_error(c, RJ_ERR_CUDA, c->err.empty() ? "context poisoned" : c->err);
    if (!q) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL query descriptor");
    if (!c->n_poly) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "query before rj_load_polygons");
    if (n && (!x || !y)) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL coordinates");
    if (xy_dtype != RJ_F32 && xy_dtype != RJ_F64) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "coordinates must be RJ_F32 or RJ_F64");
    if (n_cols < 0 || n_cols > RJ_MAX_COLS) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "n_cols must be in [0, 8]");
    if (n_cols && (!cols || !dtypes)) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL attribute columns");
    int dt[RJ_MAX_COLS];
    for (int k = 0; k < n_cols; ++k) {
        if (dtypes[k] != RJ_I32 && dtypes[k] != RJ_F32) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "attributes must be RJ_I32 or RJ_F32");
        if (n && !cols[k]) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL attribute column");
        dt[k] = dtypes[k];
    }
    if (q->agg < RJ_COUNT || q->agg > RJ_MAX) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "bad agg");
    if (q->agg != RJ_COUNT && (q->agg_column < 0 || q->agg_column >= n_cols))
        return set_error(c, RJ_ERR_INVALID_ARGUMENT, "agg_column out of range");
    LabInput in;
    in.n = n;
    in.x = x;
    in.y = y;
    in.xy_f64 = xy_dtype == RJ_F64;
    in.cols = cols;
    in.col_dtype = dt;
    return label_query_with_cols(c, q, single_plan(q), in, n_cols, count, value);
}

rj_status rj_query_multi(rj_ctx *c, const rj_query_desc *q, int32_t n_aggs, const rj_agg_spec *aggs,
                         uint64_t *count, double *values) {
    rj_status s = check_ready(c, q);
    if (s != RJ_OK) return s;
    if (n_aggs < 1 || n_aggs > RJ_MAX_AGGS || !aggs)
        return set_error(c, RJ_ERR_INVALID_ARGUMENT, "n_aggs must be in [1, 4]");
    AggPlan ap;
    ap.n = n_aggs;
    for (int k = 0; k < n_aggs; ++k) {
        if (aggs[k].agg < RJ_COUNT || aggs[k].agg > RJ_MAX) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "bad agg");
        if (aggs[k].agg != RJ_COUNT && (aggs[k].column < 0 || aggs[k].column >= c->n_cols))
            return set_error(c, RJ_ERR_INVALID_ARGUMENT, "aggregate column out of range");
        ap.kind[k] = aggs[k].agg;
        ap.col[k] = aggs[k].agg == RJ_COUNT ? 0 : aggs[k].column;
    }
    return label_query_with_cols(c, q, ap, lattice_input(c), c->n_cols, count, values);
}

static rj_status query_interval(rj_ctx *c, const rj_query_desc *q, uint64_t *count, double *value,
                                uint64_t *eps_plus, uint64_t *eps_minus, double *exp_plus, double *exp_minus) {
    if (q && q->mode != RJ_BOUNDED) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "result intervals need RJ_BOUNDED");
    if (q && (q->view[0] || q->view[1] || q->view[2] || q->view[3]))
        return set_error(c, RJ_ERR_INVALID_ARGUMENT, "result intervals need the whole canvas (view all zero)");
    Prepared P;
    rj_status s = prepare(c, q, P, true, true);
    if (s != RJ_OK) return s;
    const size_t n = c->n_poly;
    Buf &cv = wsbuf(c, kWsCanvas);
    if (dreserve(c, c->res_cnt, n * 8) || dreserve(c, c->res_sum, n * 8) || dreserve(c, c->res_val, n * 8) ||
        dreserve(c, c->res_eps, n * 32) || dreserve(c, cv, (uint64_t)P.W * P.H * 4))
        return set_error(c, RJ_ERR_OOM, "result allocation failed");
    RJ_CUDA(c, cudaMemsetAsync(cv.p, 0, (uint64_t)P.W * P.H * 4, c->stream));
    P.a.canvas = cv.as<uint32_t>();
    if ((s = run_pass(c, P, c->res_cnt.as<unsigned long long>(), c->res_sum.as<double>())) != RJ_OK) return s;
    unsigned long long *ep = c->res_eps.as<unsigned long long>(), *em = ep + n;
    const bool expected = exp_plus || exp_minus;
    double *xp = expected ? reinterpret_cast<double *>(em + n) : nullptr, *xm = expected ? xp + n : nullptr;
    if ((s = interval_impl(c, P.W, P.H, P.pp, cv.as<uint32_t>(), ep, em, xp, xm)) != RJ_OK) return s;
    if (value) RJ_CUDA(c, launch_finalize(c, q->agg, (uint32_t)n, c->res_cnt.as<unsigned long long>(),
                                          c->res_sum.as<double>(), c->res_val.as<double>()));
    if (count) RJ_CUDA(c, cudaMemcpyAsync(count, c->res_cnt.p, n * 8, cudaMemcpyDeviceToHost, c->stream));
    if (value) RJ_CUDA(c, cudaMemcpyAsync(value, c->res_val.p, n * 8, cudaMemcpyDeviceToHost, c->stream));
    if (eps_plus) RJ_CUDA(c, cudaMemcpyAsync(eps_plus, ep, n * 8, cudaMemcpyDeviceToHost, c->stream));
    if (eps_minus) RJ_CUDA(c, cudaMemcpyAsync(eps_minus, em, n * 8, cudaMemcpyDeviceToHost, c->stream));
    if (exp_plus) RJ_CUDA(c, cudaMemcpyAsync(exp_plus, xp, n * 8, cudaMemcpyDeviceToHost, c->stream));
    if (exp_minus) RJ_CUDA(c, cudaMemcpyAsync(exp_minus, xm, n * 8, cudaMemcpyDeviceToHost, c->stream));
    if (c->timing) RJ_CUDA(c, record_ev(c, 3));
    RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    return RJ_OK;
}

rj_status rj_query_interval(rj_ctx *c, const rj_query_desc *q, uint64_t *count, double *value, uint64_t *eps_plus,
                            uint64_t *eps_minus) {
    return query_interval(c, q, count, value, eps_plus, eps_minus, nullptr, nullptr);
}

rj_status rj_query_interval_ex(rj_ctx *c, const rj_query_desc *q, uint64_t *count, double *value,
                               uint64_t *eps_plus, uint64_t *eps_minus, double *exp_plus, double *exp_minus) {
    return query_interval(c, q, count, value, eps_plus, eps_minus, exp_plus, exp_minus);
}

rj_status rj_debug_point_canvas(rj_ctx *c, const rj_query_desc *q, uint32_t *counts) {
    if (!counts || !q) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL counts or query");
    rj_query_desc qq = *q;
    qq.mode = RJ_BOUNDED;
    qq.view[0] = qq.view[1] = qq.view[2] = qq.view[3] = 0;   // always the whole canvas
    Prepared P;
    rj_status s = prepare(c, &qq, P);
    if (s != RJ_OK) return s;
    const size_t n = c->n_poly;
    Buf &cv = wsbuf(c, kWsCanvas);
    if (dreserve(c, c->res_cnt, n * 8) || dreserve(c, c->res_sum, n * 8) || dreserve(c, cv, (uint64_t)P.W * P.H * 4))
        return set_error(c, RJ_ERR_OOM, "canvas allocation failed");
    RJ_CUDA(c, cudaMemsetAsync(cv.p, 0, (uint64_t)P.W * P.H * 4, c->stream));
    P.a.canvas = cv.as<uint32_t>();
    if ((s = run_pass(c, P, c->res_cnt.as<unsigned long long>(), c->res_sum.as<double>())) != RJ_OK) return s;
    RJ_CUDA(c, cudaMemcpyAsync(counts, cv.p, (uint64_t)P.W * P.H * 4, cudaMemcpyDeviceToHost, c->stream));
    RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    return RJ_OK;
}

rj_status rj_get_stats(const rj_ctx *cc, rj_stats *out) {
    rj_ctx *c = const_cast<rj_ctx *>(cc);
    if (!c || !out) return RJ_ERR_INVALID_ARGUMENT;
    RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    c->last.n_filtered = c->h_stats[0];
    c->last.n_boundary = c->h_stats[1];
    if (c->stream_stats_pending) {
        c->last.n_points -= std::min<uint64_t>(c->last.n_points, c->h_stats[2]);
        c->stream_stats_pending = 0;
    }
    c->last.launches = c->launches;
    c->last.pass_stages = c->last_stages;
    c->last.pass_ctas_per_sm = c->last_ctas_per_sm;
    if (c->timing) {
        float a = 0, b = 0, t = 0;
        cudaEventElapsedTime(&a, c->ev[0], c->ev[1]);
        cudaEventElapsedTime(&b, c->ev[1], c->ev[2]);
        if (cudaEventElapsedTime(&t, c->ev[0], c->ev[3]) != cudaSuccess) { cudaGetLastError(); t = a + b; }
        c->last.ms_polygon = a;
        c->last.ms_point_pass = b;
        c->last.ms_total = t;
    }
    *out = c->last;
    return RJ_OK;
}

rj_status rj_debug_pixel_spans(rj_ctx *c, const rj_query_desc *q, uint64_t cap, uint32_t *out, uint64_t *n_out) {
    if (!q) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL query descriptor");
    rj_query_desc qq = *q;
    qq.mode = RJ_BOUNDED;                  // spans do not depend on the mode
    Prepared P;
    rj_status s = prepare(c, &qq, P);
    if (s != RJ_OK) return s;
    const uint64_t n = P.pp.n_spans;
    if (n_out) *n_out = n;
    if (out && cap) RJ_CUDA(c, cudaMemcpyAsync(out, P.pp.spans, std::min(cap, n) * 16, cudaMemcpyDeviceToHost, c->stream));
    RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    return RJ_OK;
}

rj_status rj_debug_boundary_mask(rj_ctx *c, const rj_query_desc *q, uint32_t *bits) {
    if (!bits || !q) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL bits or query");
    rj_query_desc qq = *q;
    qq.mode = RJ_ACCURATE;
    Prepared P;
    rj_status s = prepare(c, &qq, P, true, false, true);
    if (s != RJ_OK) return s;
    RJ_CUDA(c, cudaMemcpyAsync(bits, P.pp.mask, (uint64_t)P.pp.mask_wpr * P.H * 4, cudaMemcpyDeviceToHost, c->stream));
    RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    return RJ_OK;
}

rj_status rj_debug_boundary_pieces(rj_ctx *c, const rj_query_desc *q, uint32_t *bnd_bits, uint32_t *cover_bits) {
    if (!bnd_bits || !cover_bits || !q) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL bits or query");
    rj_query_desc qq = *q;
    qq.mode = RJ_ACCURATE;
    Prepared P;
    rj_status s = prepare(c, &qq, P);
    if (s != RJ_OK) return s;
    const size_t n = c->n_poly;
    const uint64_t wpr = (uint64_t)(P.W + 31) / 32, words = wpr * P.H;
    Buf d;
    if (dreserve(c, c->res_cnt, n * 8) || dreserve(c, c->res_sum, n * 8) || dalloc(c, d, std::max<uint64_t>(1, 2 * words) * 4))
        return set_error(c, RJ_ERR_OOM, "allocation failed");
    RJ_CUDA(c, cudaMemsetAsync(d.p, 0, 2 * words * 4, c->stream));
    P.a.bnd_bits = d.as<uint32_t>();
    P.a.cover_bits = d.as<uint32_t>() + words;
    P.a.bits_wpr = (uint32_t)wpr;
    if ((s = run_pass(c, P, c->res_cnt.as<unsigned long long>(), c->res_sum.as<double>())) != RJ_OK) return s;
    RJ_CUDA(c, cudaMemcpyAsync(bnd_bits, d.p, words * 4, cudaMemcpyDeviceToHost, c->stream));
    RJ_CUDA(c, cudaMemcpyAsync(cover_bits, d.as<uint32_t>() + words, words * 4, cudaMemcpyDeviceToHost, c->stream));
    RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    dfree(c, d);
    return RJ_OK;
}

rj_status rj_debug_pip_work(rj_ctx *c, uint64_t *n_points, uint64_t *n_edge_tests) {
    if (!c || !n_points || !n_edge_tests) return RJ_ERR_INVALID_ARGUMENT;
    if (c->poisoned) return set_error(c, RJ_ERR_CUDA, c->err);
    return pip_work(c, n_points, n_edge_tests);
}

rj_status rj_debug_point_membership(rj_ctx *c, const rj_query_desc *q, uint64_t *bits) {
    if (!bits) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "NULL bits");
    Prepared P;
    rj_status s = prepare(c, q, P, true, false, true);
    if (s != RJ_OK) return s;
    Buf d;
    if (dalloc(c, d, std::max<uint64_t>(1, c->n_in) * 8)) return set_error(c, RJ_ERR_OOM, "allocation failed");
    RJ_CUDA(c, cudaMemsetAsync(d.p, 0, std::max<uint64_t>(1, c->n_in) * 8, c->stream));
    RJ_CUDA(c, launch_membership(c, P.a, P.acc, d.as<unsigned long long>()));
    RJ_CUDA(c, cudaMemcpyAsync(bits, d.p, c->n_in * 8, cudaMemcpyDeviceToHost, c->stream));
    RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    dfree(c, d);
    return RJ_OK;
}

}  // extern "C"
