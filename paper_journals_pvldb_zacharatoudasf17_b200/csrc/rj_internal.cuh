// rj_internal.cuh -- private context and launcher declarations of librj.
#pragma once
#include <utility>
#include <cuda_runtime.h>
#include <stdint.h>

#include <string>
#include <vector>

#include "../../include/rj.h"
#include "rj_geom.cuh"

namespace rj {

struct Ctx;

// Device buffer owned by a context (grow-only when reused as workspace).
struct Buf {
    void *p = nullptr;
    size_t bytes = 0;
    template <class T> T *as() const { return reinterpret_cast<T *>(p); }
};

// Attribute slot of the point pass: the distinct columns a query reads.
struct Filter {
    int32_t n_slots = 0;          // columns streamed by the point pass (<= 6)
    int32_t slot_col[6];          // slot -> attribute column
    int32_t slot_is_float[6];
    // integer-range predicates: every slot s has its int32 predicates merged
    // into one inclusive range [ilo, ihi] (the whole int32 range when it has
    // none); n_irange == n_slots
    int32_t n_irange = 0;
    int32_t ilo[6], ihi[6];
    // float32 predicates (slot, op, value)
    int32_t n_fpred = 0;
    int32_t f_slot[5], f_op[5];
    float f_val[5];
    int32_t never = 0;            // an int predicate can never hold
    int32_t agg_slot = -1;        // slot of the summed attribute (SUM/AVG): always 0
    int32_t agg_is_float = 0;     // its dtype (avoids a dynamically indexed param)
};

// Viewport window of a query (rj_query_desc.view, reading Z20): pixels
// [c0, c1) x [r0, r1) of the W x H canvas; full = the whole canvas.
struct View {
    int32_t c0 = 0, r0 = 0, c1 = 0, r1 = 0;
    bool full = true;
};

// Device-side parameter block of the fused point pass.
struct PassArgs {
    const uint32_t *qx, *qy;
    const uint32_t *col[6];
    Filter f;
    int32_t W, H;
    const int4 *items;            // (cell_begin, cell_end, point_begin, point_end)
    uint32_t n_items;
    uint32_t *work_counter;
    int32_t level;                // point-cell level L of this query (2^L x 2^L cells)
    const uint32_t *cell_off10;   // [kCells10 + 1] first point of every level-10 cell
    uint32_t tile_stride;         // row stride of a warp's tile (odd: conflict-free row prefix)
    int32_t lane_runs;            // COUNT tile kernel: merge equal-pixel runs inside lanes only
    int32_t early_stream;         // the producer may stream before the predecessor grid completes
                                  // (k_pass_init ran before the polygon pass's PDL kernels)
    const uint32_t *piece_off;    // [4^L + 1]
    const uint2 *pieces;
    const uint32_t *mask;         // accurate: boundary bitmask (diagnostics; the kernels use bpieces)
    uint32_t mask_wpr;
    const uint32_t *bpiece_off;   // accurate: boundary pieces per point cell [4^L + 1]
    const uint32_t *bpieces;      // (local row | lo << 8 | hi << 16)
    const uint32_t *grid_off;     // accurate: edge grid CSR
    const uint32_t *grid_ent;
    const int4 *grid_edge;        // per entry: (xa, ya, xb, yb)
    const uint32_t *grid_poly;    // per entry: polygon
    const int4 *edges;
    const uint32_t *edge_poly;
    unsigned long long *A_cnt;    // per polygon partials (device)
    double *A_sum;
    uint32_t n_poly;
    int32_t smem_partials;        // accumulate per-CTA polygon partials in smem
    uint32_t tile_cap;            // words of the CTA's tile
    uint32_t n_stages;            // depth of the shared-memory stage ring
    int32_t index_join;           // every pixel is a boundary pixel, no span pieces (RJ_INDEX_JOIN)
    uint32_t *canvas;             // tile kernel: dump per-pixel filtered counts (W x H) when set
    uint32_t *bnd_bits;           // diagnostic (accurate): OR the tiles' boundary pixels into [H][bits_wpr]
    uint32_t *cover_bits;         //   and the pixels the tiles covered (cells holding points, in the window)
    uint32_t bits_wpr;
    unsigned long long *stats;    // [0] filtered, [1] boundary
    int32_t view[4];              // viewport pixel window (c0, r0, c1, r1), half-open
    uint32_t cwin[4];             // level-L cells meeting it: columns [cwin0, cwin2], rows [cwin1, cwin3]
    // accurate mode: boundary points are appended to this global queue
    // (SoA, bq_cap entries) and tested by k_pip_queue after the pass;
    // bq_cap == 0 -> tested inline by the consumer warps
    uint32_t *bq_x, *bq_y, *bq_a;
    uint32_t bq_cap;
    uint32_t bq_chunk;            // entries a warp reserves at a time
    uint32_t *bq_count;           // entries reserved
    uint32_t *bq_valid;           // first failed reservation (entries below it are written)
};

struct Ctx {
    int device = 0;
    cudaStream_t stream = nullptr;
    bool own_stream = false;
    double x0, y0, x1, y1;
    bool poisoned = false;
    std::string err;
    void *(*alloc_fn)(size_t, void *) = nullptr;
    void (*free_fn)(void *, void *) = nullptr;
    void *alloc_user = nullptr;
    int num_sms = 148;
    int timing = 0;
    int64_t chunk = 65536;

    // points (S1 output, spatially sorted)
    uint64_t n_in = 0, n_pts = 0;
    int n_cols = 0;
    int col_dtype[RJ_MAX_COLS];
    Buf qx, qy, idx, col[RJ_MAX_COLS];
    Buf load_stage[2 + RJ_MAX_COLS];           // H2D staging (grow-only)
    Buf load_alt[3 + RJ_MAX_COLS];             // the sort's second buffer (grow-only)
    Buf load_qxy;                              // quantised (Qx, Qy) interleaved, before the gather (grow-only)
    int keep_load_scratch = 1;                 // RJ_OPT_KEEP_LOAD_SCRATCH
    Buf cell_off;                 // [kCells10 + 1]
    std::vector<uint32_t> h_cell_off;          // host copy (work-item planning)
    Buf items[kMaxLevel + 1];                  // per level L: int4 work items
    Buf cell_bits[kMaxLevel + 1];              // per level L: bit per point cell, set when it holds points
    uint32_t n_items[kMaxLevel + 1] = {};
    int64_t items_chunk[kMaxLevel + 1] = {};

    // polygons
    uint32_t n_poly = 0;
    uint32_t n_edges = 0;
    double edge_len_x = 0.0, edge_len_y = 0.0;   // sum of |dx|, |dy| over edges (lattice units)
    Buf edges, edge_poly, poly_edge_off, mbr;   // int4 edges/mbr
    Buf poly_ring_off, ring_edge_off;          // rings: [n_poly + 1] first ring, [n_ring + 1] first edge
    Buf edge_sigma;                            // int8 per edge: ring weight orientation * (-1)^depth (Z22)
    uint32_t n_ring = 0;

    // polygon-pass sizes of the last query (host metadata only: every
    // kernel still runs per query).  They are a pure function of the key
    // (canvas, level, mode, window, loaded data), so a repeated key skips the
    // two device->host size reads and the whole query is enqueued without a
    // host round trip.
    uint64_t data_gen = 0;                     // bumped by every load
    int64_t pp_key[9] = {};
    bool pp_key_valid = false;
    uint32_t pp_sizes[6] = {};                 // X, NPR, B, S, NP, NB

    // CUDA-graph replay of a repeated query (api.cu run_graphed): the key
    // covers the descriptor, outputs, options and every allocation
    uint64_t alloc_gen = 0;                    // bumped by every device (re)allocation / free
    bool capturing = false;
    int use_graphs = 1;                        // RJ_OPT_GRAPHS
    int pdl = 1;                               // programmatic dependent launch of the query's kernel chain (env RJ_NO_PDL=1: off)
    std::vector<int64_t> graph_key, pending_key;
    cudaGraphExec_t graph_exec = nullptr;
    rj_stats graph_last{};
    uint32_t graph_launches = 0;
    int graph_stages = 0, graph_ctas = 0;
    Buf grid_off, grid_ent;
    Buf grid_edge, grid_poly;                  // entries inlined: edge endpoints + polygon
    uint64_t n_grid_ent = 0;

    // query workspace (grow-only)
    Buf ws[96];                      // slots: see kWs* in rj_internal.cuh
    Buf res_cnt, res_sum, res_val;   // per-polygon partials / values
    Buf res_eps;                     // result intervals: eps+ [n_poly], eps- [n_poly]
    Buf res_agg;                     // label-pass aggregate partials [n_agg][n_poly] x 8 B
    Buf stats_dev;
    unsigned long long *h_stats = nullptr;   // pinned
    rj_stats last{};
    cudaEvent_t ev[6] = {};
    cudaStream_t load_stream = nullptr;           // load: attribute-column copies beside the sort
    cudaEvent_t load_ev[2] = {};
    uint32_t launches = 0;
    int last_stages = 0, last_ctas_per_sm = 0;   // point-pass launch shape of the last query
    PassArgs last_bq{};                           // last accurate query with a global boundary queue (bq_cap > 0)
    int pass_variant = -1;                        // RJ_OPT_PASS: -1 auto, 0 label, 1 pixel tile
    int force_stages = 0;                         // RJ_OPT_STAGES: 0 = automatic, else 2..4
    int lane_runs = 0;                            // RJ_OPT_LANE_RUNS: 0 auto (= 1), 1 in-lane runs, 2 warp-merged
    int tile_side = 64;                           // RJ_OPT_TILE_SIDE: target point-cell side in pixels

    // streamed query (label_canvas.cu, rj_query_stream)
    int64_t stream_batch = int64_t(1) << 24;      // RJ_OPT_STREAM_BATCH: points per batch
    cudaStream_t copy_stream = nullptr;           // H2D copies of the batches
    cudaEvent_t sev[5] = {};                      // copied[2], consumed[2], start
    Buf sbuf[2][2 + RJ_MAX_COLS];                 // double-buffered device batches
    int stream_stats_pending = 0;                 // last query was streamed: h_stats[2] = out of domain
};

// workspace slot map (Ctx::ws)
enum : int {
    kWsSortCounts = 0,                      // radix-sort digit counts (load_points.cu)
    kWsEdgeRows = 14, kWsEdgeOff, kWsPolyRows, kWsPolyRowOff, kWsCrossPR, kWsCrossT,
    kWsPRCount, kWsPROff, kWsPRCursor, kWsTvals, kWsSpanCount, kWsSpanOff, kWsSpans,
    kWsPieceCount, kWsPieceOff, kWsPieceCursor, kWsPieces, kWsMask, kWsBandCount, kWsBandOff,
    kWsWork, kWsSizes,
    kWsLab, kWsRowCount, kWsRowOff, kWsRowCursor, kWsRowSpans, kWsStream,   // streamed query
    kWsCanvas, kWsBRowCount, kWsBRowOff, kWsBktCount, kWsBktOff, kWsBktCursor, kWsBktRanges,   // intervals
    kWsBQx, kWsBQy, kWsBQa,                 // accurate mode: global boundary-point queue
    kWsBPCount, kWsBPOff, kWsBPCursor, kWsBPieces,   // accurate mode: boundary pieces per point cell
    kWsScan = 72,                           // scan_u32's look-back status words (scan.cu, one slot)
};

// allocation helpers (ctx allocator if set)
cudaError_t dalloc(Ctx *c, Buf &b, size_t bytes);
void dfree(Ctx *c, Buf &b);
cudaError_t dreserve(Ctx *c, Buf &b, size_t bytes);   // grow-only, +25 % slack
cudaError_t dreserve_exact(Ctx *c, Buf &b, size_t bytes);   // grow-only, exact size
Buf &wsbuf(Ctx *c, int slot);

// scan.cu: exclusive scan of n u32 -> out[0..n], out[n] = total.  tmp
// workspace slots base.. are used for block sums.
cudaError_t scan_u32(Ctx *c, const uint32_t *in, uint32_t *out, uint64_t n, int ws_base);
// up to three independent scans in one launch (out[j][n[j]] = total of array j)
struct ScanJobs {
    const uint32_t *in[3];
    uint32_t *out[3];
    uint64_t n[3];
    uint32_t tile0[4];       // first global tile of each array; tile0[nj] = all tiles
    int nj;
};
cudaError_t scan_multi(Ctx *c, int nj, const uint32_t *const *in, uint32_t *const *out, const uint64_t *n,
                       int ws_base);

// load_points.cu
rj_status load_points_impl(Ctx *c, uint64_t n, const void *x, const void *y, int xy_f64,
                           int n_cols, const void *const *cols, const int32_t *dtypes,
                           uint64_t *n_ood);
// work.cu: point-pass work items for level L (cached per level)
rj_status items_for_level(Ctx *c, int L);
void free_load_scratch(Ctx *c);
void drop_items(Ctx *c);
int choose_level(int W, int H, int target_side);

// api.cu
rj_status build_filter(Ctx *c, const rj_query_desc *q, int n_cols, const int *col_dtype, Filter &f);

// label_canvas.cu: the label-canvas point pass -- streamed one-shot queries
// (rj_query_stream), MIN/MAX and multi-aggregate queries (rj_query_multi).
constexpr int kMaxAggs = 4;
struct AggPlan {
    int n = 0;                    // aggregates besides the per-polygon count
    int kind[kMaxAggs];           // rj_agg
    int col[kMaxAggs];            // attribute column (user index)
};
// Inputs: lattice == true: the context's loaded (quantised, sorted) columns;
// else n raw points x/y (f32/f64) + user columns, host or device memory.
struct LabInput {
    bool lattice = false;
    uint64_t n = 0;
    const void *x = nullptr, *y = nullptr;
    bool xy_f64 = false;
    const void *const *cols = nullptr;
    const int *col_dtype = nullptr;
};
// Partials (device, caller-sized): d_cnt[n_poly]; d_agg[k * n_poly ...]:
// binary64 sums for SUM/AVG, orderable u32 keys (in the low half of the
// 8-byte slot array) for MIN/MAX.
rj_status label_query_impl(Ctx *c, const Filter &f, const AggPlan &ap, int W, int H, const View &v, int mode,
                           const LabInput &in, unsigned long long *d_cnt, void *d_agg);
// values[k * n + i] from the partials (NaN for an empty polygon's AVG/MIN/MAX).
cudaError_t launch_finalize_aggs(Ctx *c, const AggPlan &ap, const int *col_dtype, uint32_t n,
                                 const unsigned long long *cnt, const void *d_agg, double *values);
void stream_release(Ctx *c);


// polygons.cu
rj_status load_polygons_impl(Ctx *c, uint32_t n_poly, const uint32_t *pro, const uint32_t *rvo,
                             const double *vx, const double *vy);
struct PolyPass {
    uint64_t n_cross = 0, n_spans = 0, n_pieces = 0, n_bands = 0;
    uint32_t *spans = nullptr;       // 4 x u32 per span (poly,row,lo,hi), (poly,row,lo)-sorted
    uint32_t *piece_off = nullptr;   // [4^L + 1]
    uint2 *pieces = nullptr;
    uint32_t *mask = nullptr;        // accurate only
    uint32_t mask_wpr = 0;
    uint32_t *bpiece_off = nullptr;  // accurate with point cells: [4^L + 1]
    uint32_t *bpieces = nullptr;     // (local row | lo << 8 | hi << 16) of boundary pixels
    uint64_t n_bpieces = 0;
};
// Spans, pieces and the boundary mask are clipped to the viewport window v.
rj_status polygon_pass(Ctx *c, int W, int H, int L, bool accurate, PolyPass &pp, const View &v, bool need_mask);

// interval.cu: bounded-mode worst-case result intervals from the
// per-pixel count canvas, the spans and the S5 bands of the polygon pass.
// With d_exp_plus / d_exp_minus (binary64, may be NULL) also the expected
// interval sums of P:811-827 (reading Z22).
rj_status interval_impl(Ctx *c, int W, int H, const PolyPass &pp, const uint32_t *canvas,
                        unsigned long long *d_eps_plus, unsigned long long *d_eps_minus,
                        double *d_exp_plus = nullptr, double *d_exp_minus = nullptr);
// interval.cu: per-edge ring weights (load time)
rj_status ring_sigma_impl(Ctx *c, uint32_t n_poly, uint32_t n_ring);

// pass.cu
rj_status point_pass(Ctx *c, const PassArgs &a, bool sum, bool accurate);
// accurate mode: exact PIP of the queued boundary points (after point_pass)
rj_status pip_queue_pass(Ctx *c, const PassArgs &a, bool sum);
// diagnostic: points in the last query's boundary queue and the edge-grid
// entries their exact tests walk (SURVEY.md 8(a) S7 note)
rj_status pip_work(Ctx *c, uint64_t *n_points, uint64_t *n_edge_tests);
size_t point_pass_smem(const Ctx *c, const PassArgs &a, bool sum, bool accurate);
int point_pass_stages(int n_slots);

// misc.cu
cudaError_t launch_finalize(Ctx *c, int agg, uint32_t n, const unsigned long long *cnt,
                            const double *sum, double *val);
cudaError_t launch_pass_init(Ctx *c, uint32_t *work, unsigned long long *cnt, double *sum, uint32_t n);
cudaError_t launch_pack(Ctx *c, uint32_t n, const unsigned long long *cnt, const double *sum, double *out);
cudaError_t launch_finalize_packed(Ctx *c, int agg, uint32_t n, const double *in, unsigned long long *cnt,
                                   double *val);
cudaError_t launch_membership(Ctx *c, const PassArgs &a, bool accurate, unsigned long long *bits);

rj_status set_error(Ctx *c, rj_status s, const std::string &msg);
rj_status cuda_error(Ctx *c, cudaError_t e, const char *where);

#define RJ_CUDA(c, expr)                                            \
    do {                                                            \
        cudaError_t _e = (expr);                                    \
        if (_e != cudaSuccess) return ::rj::cuda_error((c), _e, #expr); \
    } while (0)

#define RJ_LAUNCHED(c) do { (c)->launches++; } while (0)

// Device bounds checks (build with RJ_NVCC_EXTRA=-DRJ_CHECKS; off in the
// product build): shared-tile indices, span-piece rows/columns, queue and
// piece slots.  A failed check prints its condition and traps, so the query
// returns RJ_ERR_CUDA.  (compute-sanitizer is closed on this GPU pool.)
#ifdef RJ_CHECKS
#define RJ_DCHECK(c)                                                                              \
    do {                                                                                         \
        if (!(c)) {                                                                              \
            printf("RJ_DCHECK failed %s:%d: %s\n", __FILE__, __LINE__, #c);                      \
            __trap();                                                                            \
        }                                                                                        \
    } while (0)
#else
#define RJ_DCHECK(c) do { } while (0)
#endif

// Programmatic dependent launch: the per-query kernel chain (polygon pass ->
// point pass -> finalisation) is launched with the PDL attribute, so a
// kernel's grid is scheduled while its predecessor drains.  Every such
// kernel first waits for its predecessor's completion and memory
// (griddepcontrol.wait -- a no-op without the attribute), then lets its own
// dependent launch.
__device__ __forceinline__ void pdl_wait() { asm volatile("griddepcontrol.wait;" ::: "memory"); }
__device__ __forceinline__ void pdl_trigger() { asm volatile("griddepcontrol.launch_dependents;" ::: "memory"); }

// the same for a kernel given as a function pointer plus argument array
inline cudaError_t launch_pdl_ptr(Ctx *c, const void *k, dim3 grid, dim3 block, size_t smem, void **args) {
    cudaLaunchConfig_t cfg{};
    cfg.gridDim = grid;
    cfg.blockDim = block;
    cfg.dynamicSmemBytes = smem;
    cfg.stream = c->stream;
    cudaLaunchAttribute at[1];
    at[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    at[0].val.programmaticStreamSerializationAllowed = c->pdl;
    cfg.attrs = at;
    cfg.numAttrs = 1;
    return cudaLaunchKernelExC(&cfg, k, args);
}

template <typename... KArgs, typename... Args>
cudaError_t launch_pdl(Ctx *c, void (*k)(KArgs...), dim3 grid, dim3 block, size_t smem, Args &&...args) {
    cudaLaunchConfig_t cfg{};
    cfg.gridDim = grid;
    cfg.blockDim = block;
    cfg.dynamicSmemBytes = smem;
    cfg.stream = c->stream;
    cudaLaunchAttribute at[1];
    at[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    at[0].val.programmaticStreamSerializationAllowed = c->pdl;
    cfg.attrs = at;
    cfg.numAttrs = 1;
    return cudaLaunchKernelEx(&cfg, k, std::forward<Args>(args)...);
}

inline unsigned blocks_for(uint64_t n, unsigned t) { return (unsigned)((n + t - 1) / t); }

}  // namespace rj
