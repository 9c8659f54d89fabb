// polygons.cu -- the polygon side of Raster Join on the GPU.
//
// Load time (rj_load_polygons):
//   * quantise vertices (host, same O1 formula as the points), build the edge
//     list (closing edges included), per-polygon edge ranges and MBRs;
//   * S6: the uniform edge grid (1024 x 1024 cells over the lattice): per
//     cell, the edges that can toggle the even-odd test of a point in the
//     cell (polygon MBR meets the cell, the edge's y-range meets the cell's
//     rows, the edge reaches right of the cell's left side).  Two passes
//     (count, fill) into one CSR array, as the paper's grid index is built
//     (P:906-917); entries sorted per cell so edges group by polygon.
//
// Per query (polygon_pass):
//   * S3 edge setup: every (edge, pixel row) crossing gets its exact integer
//     column threshold t (rj_geom.cuh threshold()); thresholds are bucketed
//     per (polygon, row) and sorted, so the pixels of row r whose centre is
//     inside polygon P are the spans [t1,t2), [t3,t4), ... (even-odd scanline
//     rasterisation of the polygon = Proc. DrawPolygons' fragments, P:529-554,
//     with the pixel-centre rule).
//   * pieces: every span is cut at the pixel extents of the level-L point
//     cells it crosses and binned per cell; the fused point pass reduces each
//     cell's tile over its pieces (S4).
//   * S5 (accurate): supercover of every edge = the boundary pixels
//     (outline drawn conservatively).
#include <algorithm>
#include <cmath>
#include <vector>

#include "rj_internal.cuh"

namespace rj {

namespace {

__device__ __forceinline__ uint32_t upper_bound_u32(const uint32_t *a, uint32_t n, uint32_t v) {
    // first index k in [0, n] with a[k] > v  (a non-decreasing)
    uint32_t lo = 0, hi = n;
    while (lo < hi) {
        uint32_t m = (lo + hi) >> 1;
        if (a[m] > v) hi = m; else lo = m + 1;
    }
    return lo;
}

// ------------------------------------------------------------- edge grid (S6)
// Cell (gr, gc) lists edge e iff e is not horizontal, gr is one of the grid
// rows its y-extent overlaps, and gc lies between its polygon's MBR left
// side and the edge (the cells where e can toggle the half-open ray).  Each
// edge therefore covers one column run per grid row; the work is cut into
// items of (edge, row, 32-column chunk), so a long edge of a wide polygon is
// spread over many threads instead of one thread walking rows x columns.
constexpr int kGridChunk = 32;

// An edge of polygon P is listed in grid rows [gr0, gr1] (its half-open
// y-extent) and, per row, in two column runs (reading Z25): the cells of P's
// MBR left of the MBR's middle column `split` test a LEFTWARD ray -- the
// edges with min x <= the cell's last column can toggle it -- and the cells
// from `split` on a RIGHTWARD ray -- the edges with max x > the cell's first
// column.  Each cell thus walks only the edges between itself and the nearer
// side of P's MBR.
struct GridRun {
    int gr0, gr1;             // rows [gr0, gr1] (empty: gr1 < gr0)
    int l0, l1, r0, r1;       // leftward-ray columns [l0, l1], rightward-ray columns [r0, r1]
};

__device__ __forceinline__ GridRun grid_run(const int4 E, const int4 M) {
    GridRun g{0, -1, 0, -1, 0, -1};
    if (E.y == E.w || M.z - 1 < M.x) return g;           // horizontal: never toggles; empty MBR
    const int ymin = min(E.y, E.w), ymax = max(E.y, E.w);
    g.gr0 = ymin >> kGridShift;
    g.gr1 = (ymax - 1) >> kGridShift;
    const int m0 = M.x >> kGridShift, m1 = min((M.z - 1) >> kGridShift, kGrid - 1);
    const int split = (int)(((int64_t)M.x + M.z) >> 1) >> kGridShift;
    g.l0 = max(m0, min(E.x, E.z) >> kGridShift);
    g.l1 = min(m1, split - 1);
    g.r0 = max(m0, split);
    g.r1 = min(m1, (max(E.x, E.z) - 1) >> kGridShift);
    if (g.l1 < g.l0 && g.r1 < g.r0) g.gr1 = g.gr0 - 1;
    return g;
}

__device__ __forceinline__ uint32_t grid_chunks(int c0, int c1) {
    return c1 < c0 ? 0u : (uint32_t)(c1 - c0 + kGridChunk) / kGridChunk;
}

// items[e] = rows x chunks of edge e; *total += its entries (64-bit: the u32
// CSR offsets overflow silently otherwise)
__global__ void k_grid_items(const int4 *__restrict__ edges, const uint32_t *__restrict__ edge_poly,
                             const int4 *__restrict__ mbr, uint32_t n_edges, uint32_t *__restrict__ items,
                             unsigned long long *__restrict__ total) {
    const uint32_t e = blockIdx.x * blockDim.x + threadIdx.x;
    unsigned long long ent = 0;
    if (e < n_edges) {
        const GridRun g = grid_run(edges[e], mbr[edge_poly[e]]);
        const uint32_t rows = (uint32_t)max(0, g.gr1 - g.gr0 + 1);
        const uint32_t cols = (uint32_t)max(0, g.l1 - g.l0 + 1) + (uint32_t)max(0, g.r1 - g.r0 + 1);
        items[e] = rows * (grid_chunks(g.l0, g.l1) + grid_chunks(g.r0, g.r1));
        ent = (unsigned long long)rows * cols;
    }
    for (int o = 16; o; o >>= 1) ent += __shfl_xor_sync(0xFFFFFFFFu, ent, o);
    if ((threadIdx.x & 31) == 0 && ent) atomicAdd(total, ent);
}

template <bool FILL>
__global__ void k_grid_edges(const int4 *__restrict__ edges, const uint32_t *__restrict__ edge_poly,
                             const int4 *__restrict__ mbr, uint32_t n_edges, const uint32_t *__restrict__ item_off,
                             uint32_t *__restrict__ cnt, const uint32_t *__restrict__ off,
                             uint32_t *__restrict__ cursor, uint32_t *__restrict__ ent) {
    const uint32_t n_items = item_off[n_edges];
    for (uint32_t j = blockIdx.x * blockDim.x + threadIdx.x; j < n_items; j += gridDim.x * blockDim.x) {
        const uint32_t e = upper_bound_u32(item_off, n_edges + 1, j) - 1;
        const GridRun g = grid_run(edges[e], mbr[edge_poly[e]]);
        const uint32_t nl = grid_chunks(g.l0, g.l1), nch = nl + grid_chunks(g.r0, g.r1), k = j - item_off[e];
        const int gr = g.gr0 + (int)(k / nch);
        const uint32_t q = k % nch;
        const bool left = q < nl;                          // leftward-ray run
        const int c0 = left ? g.l0 + (int)q * kGridChunk : g.r0 + (int)(q - nl) * kGridChunk;
        const int c1 = min(left ? g.l1 : g.r1, c0 + kGridChunk - 1);
        for (int gc = c0; gc <= c1; ++gc) {
            const uint32_t cell = (uint32_t)gr * kGrid + gc;
            // entry = edge id, bit 31 = leftward ray (a cell's entries of one
            // polygon share it, so sorting keeps each polygon contiguous)
            if (FILL) ent[off[cell] + atomicAdd(&cursor[cell], 1u)] = e | (left ? 0x80000000u : 0u);
            else atomicAdd(&cnt[cell], 1u);
        }
    }
}

// Entries inlined for the accurate-mode test: the edge and its polygon next
// to each other, so a boundary point reads one 16-B record and one id per
// entry instead of chasing entry -> edge -> polygon.  The record is the edge
// oriented upwards, (xl, yl, xu - xl, yu) with yl < yu (grid edges are never
// horizontal): the half-open PNPOLY test is symmetric in the endpoints, and
// the orientation leaves one comparison and two 32 x 32 -> 64-bit products
// per entry (pip.cuh).
__global__ void k_grid_inline(const uint32_t *__restrict__ ent, uint32_t n, const int4 *__restrict__ edges,
                              const uint32_t *__restrict__ edge_poly, int4 *__restrict__ gedge,
                              uint32_t *__restrict__ gpoly) {
    const uint32_t i = blockIdx.x * blockDim.x + threadIdx.x;
    if (i >= n) return;
    const uint32_t e = ent[i] & 0x7FFFFFFFu;
    const int4 E = edges[e];
    const bool up = E.w > E.y;
    const int xl = up ? E.x : E.z, yl = up ? E.y : E.w, xu = up ? E.z : E.x, yu = up ? E.w : E.y;
    gedge[i] = make_int4(xl, yl, xu - xl, yu);
    gpoly[i] = edge_poly[e] | (ent[i] & 0x80000000u);   // bit 31: leftward ray
}

// Sort each cell's entries by edge id (so they group by polygon, which the
// walk in pip.cuh relies on): one warp per cell -- a register bitonic sort
// for <= 32 entries, else every entry's rank (distinct ids) into tmp and back.
__global__ void k_grid_sort(const uint32_t *__restrict__ off, uint32_t *__restrict__ ent, uint32_t *__restrict__ tmp) {
    const uint32_t lane = threadIdx.x & 31;
    const uint32_t nw = (gridDim.x * blockDim.x) >> 5;
    for (uint32_t c = (blockIdx.x * blockDim.x + threadIdx.x) >> 5; c < (uint32_t)kGrid * kGrid; c += nw) {
        const uint32_t b = off[c], e = off[c + 1], k = e - b;
        if (k < 2) continue;
        if (k <= 32) {
            uint32_t v = lane < k ? ent[b + lane] : 0xFFFFFFFFu;
            for (uint32_t size = 2; size <= 32; size <<= 1)
                for (uint32_t st = size >> 1; st; st >>= 1) {
                    const uint32_t o = __shfl_xor_sync(0xFFFFFFFFu, v, st);
                    const bool up = (lane & size) == 0, lower = (lane & st) == 0;
                    v = (lower == up) ? min(v, o) : max(v, o);
                }
            if (lane < k) ent[b + lane] = v;
        } else {
            for (uint32_t i = b + lane; i < e; i += 32) {
                const uint32_t v = ent[i];
                uint32_t r = 0;
                for (uint32_t j = b; j < e; ++j) r += ent[j] < v ? 1u : 0u;
                tmp[b + r] = v;
            }
            __syncwarp();
            for (uint32_t i = b + lane; i < e; i += 32) ent[i] = tmp[i];
        }
    }
}

// -------------------------------------------------------- S3 edge setup / spans
// Is polygon P's pixel footprint (its closed lattice MBR: every span and
// every supercover pixel of P lies in it) disjoint from the window?  Then
// the polygon contributes nothing to this query and is culled.
__device__ __forceinline__ bool culled(const int4 M, int W, int H, const int4 view) {
    const int64_t one = (int64_t)1 << kLatticeBits;
    const int64_t c0 = pix(M.x, W), c1 = pix(min((int64_t)M.z, one - 1), W);
    const int64_t r0 = pix(M.y, H), r1 = pix(min((int64_t)M.w, one - 1), H);
    return c1 < view.x || c0 >= view.z || r1 < view.y || r0 >= view.w;
}

__device__ __forceinline__ void edge_rows_body(uint32_t t0, uint32_t ts, const int4 *__restrict__ edges,
                                               const uint32_t *__restrict__ edge_poly, const int4 *__restrict__ mbr,
                                               uint32_t n_edges, int H, uint32_t *__restrict__ rows, int accurate,
                                               int W, uint32_t *__restrict__ bands, int4 view) {
    for (uint32_t e = t0; e < n_edges; e += ts) {
        if (culled(mbr[edge_poly[e]], W, H, view)) {
            rows[e] = 0;
            if (accurate) bands[e] = 0;
            continue;
        }
        const int4 E = edges[e];
        const int64_t ymin = min(E.y, E.w), ymax = max(E.y, E.w);
        rows[e] = (uint32_t)(row_start(ymax, H) - row_start(ymin, H));
        // S5 row bands: pixel rows whose closed lattice extent meets [ymin, ymax]
        if (accurate) bands[e] = (uint32_t)band_rows(ymin, ymax, H);
    }
}

__device__ __forceinline__ void poly_rows_body(uint32_t t0, uint32_t ts, const int4 *__restrict__ mbr,
                                               uint32_t n_poly, int W, int H, uint32_t *__restrict__ rows,
                                               int4 view) {
    for (uint32_t p = t0; p < n_poly; p += ts) {
        const int4 M = mbr[p];
        rows[p] = culled(M, W, H, view) ? 0u : (uint32_t)(row_start(M.w, H) - row_start(M.y, H));
    }
}

__device__ __forceinline__ void crossings_body(uint32_t t0, uint32_t ts, const int4 *__restrict__ edges, const uint32_t *__restrict__ edge_poly,
                            const int4 *__restrict__ mbr, const uint32_t *__restrict__ edge_off,
                            uint32_t n_edges, const uint32_t *__restrict__ prow_off, int W, int H,
                            uint32_t *__restrict__ cx_pr, uint32_t *__restrict__ cx_t,
                            uint32_t *__restrict__ pr_cnt) {
    const uint32_t total = edge_off[n_edges];
    for (uint32_t j = t0; j < total; j += ts) {
        const uint32_t e = upper_bound_u32(edge_off, n_edges + 1, j) - 1;
        const int4 E = edges[e];
        const uint32_t P = edge_poly[e];
        const int64_t ymin = min(E.y, E.w);
        const int64_t r = row_start(ymin, H) + (j - edge_off[e]);
        const uint32_t pr = prow_off[P] + (uint32_t)(r - row_start(mbr[P].y, H));
        const int64_t t = threshold(E.x, E.y, E.z, E.w, centre(r, H), W);
        cx_pr[j] = pr;
        cx_t[j] = (uint32_t)t;
        atomicAdd(&pr_cnt[pr], 1u);
    }
}

__global__ void __launch_bounds__(256) k_crossings(const int4 *__restrict__ edges, const uint32_t *__restrict__ edge_poly,
                            const int4 *__restrict__ mbr, const uint32_t *__restrict__ edge_off,
                            uint32_t n_edges, const uint32_t *__restrict__ prow_off, int W, int H,
                            uint32_t *__restrict__ cx_pr, uint32_t *__restrict__ cx_t,
                            uint32_t *__restrict__ pr_cnt) {
    pdl_wait();
    pdl_trigger();
    crossings_body(blockIdx.x * blockDim.x + threadIdx.x, gridDim.x * blockDim.x, edges, edge_poly, mbr, edge_off, n_edges, prow_off, W, H, cx_pr, cx_t, pr_cnt);
}

__device__ __forceinline__ void scatter_t_body(uint32_t t0, uint32_t ts, const uint32_t *__restrict__ cx_pr, const uint32_t *__restrict__ cx_t,
                            uint32_t total, const uint32_t *__restrict__ pr_off,
                            uint32_t *__restrict__ pr_cur, uint32_t *__restrict__ tv) {
    for (uint32_t j = t0; j < total; j += ts) {
        const uint32_t pr = cx_pr[j];
        tv[pr_off[pr] + atomicAdd(&pr_cur[pr], 1u)] = cx_t[j];
    }
}

__global__ void k_scatter_t(const uint32_t *__restrict__ cx_pr, const uint32_t *__restrict__ cx_t,
                            uint32_t total, const uint32_t *__restrict__ pr_off,
                            uint32_t *__restrict__ pr_cur, uint32_t *__restrict__ tv) {
    pdl_wait();
    pdl_trigger();
    scatter_t_body(blockIdx.x * blockDim.x + threadIdx.x, gridDim.x * blockDim.x, cx_pr, cx_t, total, pr_off, pr_cur, tv);
}

struct SpanGeo {
    int W, H;
    int L;                      // point-cell level of the query
    const uint32_t *prow_off;   // [n_poly + 1]
    uint32_t n_poly;
    const int4 *mbr;
    const uint32_t *cell_bits;  // level-L point cells holding points (pieces of empty cells are skipped)
    int32_t c0, r0, c1, r1;     // viewport window (reading Z20): spans are clipped to it
};

// Clip span [lo, hi) of row r to the viewport window; false if nothing is left.
__device__ __forceinline__ bool clip_span(const SpanGeo &g, int64_t r, int64_t &lo, int64_t &hi) {
    if (r < g.r0 || r >= g.r1) return false;
    lo = max(lo, (int64_t)g.c0);
    hi = min(hi, (int64_t)g.c1);
    return lo < hi;
}

__device__ __forceinline__ void polyrow_of(const SpanGeo &g, uint32_t pr, uint32_t &P, int64_t &r) {
    P = upper_bound_u32(g.prow_off, g.n_poly + 1, pr) - 1;
    r = row_start(g.mbr[P].y, g.H) + (pr - g.prow_off[P]);
}

// Visit the (cell, local row, local lo, local hi) pieces of span [lo, hi) of row r.
template <class F>
__device__ __forceinline__ void for_each_piece(const SpanGeo &g, int64_t r, int64_t lo, int64_t hi, F f) {
    if (g.L < 0) return;                                   // spans only
    const int s = kLatticeBits - g.L;
    const int64_t cr0 = qlo(r, g.H) >> s, cr1 = qhi(r, g.H) >> s;
    const int64_t cc0 = qlo(lo, g.W) >> s, cc1 = qhi(hi - 1, g.W) >> s;
    for (int64_t cr = cr0; cr <= cr1; ++cr) {
        const int64_t r0 = cell_pix_lo(cr, g.H, g.L);
        for (int64_t cc = cc0; cc <= cc1; ++cc) {
            const uint32_t cell = spread16((uint32_t)cc) | (spread16((uint32_t)cr) << 1);
            if (!((__ldg(&g.cell_bits[cell >> 5]) >> (cell & 31)) & 1u)) continue;  // no points
            const int64_t c0 = cell_pix_lo(cc, g.W, g.L), c1 = cell_pix_hi(cc, g.W, g.L);
            const int64_t a = max(lo, c0) - c0, b = min(hi, c1 + 1) - c0;
            f(cell, (uint32_t)(r - r0), (uint32_t)a, (uint32_t)b);
        }
    }
}

// Sort m <= N values in place through registers (compare-exchange insertion
// network, fully unrolled; padding with UINT32_MAX keeps it in place).
template <int N>
__device__ __forceinline__ void sort_small(uint32_t *p, uint32_t m) {
    uint32_t r[N];
#pragma unroll
    for (int i = 0; i < N; ++i) r[i] = (uint32_t)i < m ? p[i] : 0xFFFFFFFFu;
#pragma unroll
    for (int i = 1; i < N; ++i)
#pragma unroll
        for (int j = i; j > 0; --j) {
            const uint32_t lo = min(r[j - 1], r[j]), hi = max(r[j - 1], r[j]);
            r[j - 1] = lo;
            r[j] = hi;
        }
#pragma unroll
    for (int i = 0; i < N; ++i)
        if ((uint32_t)i < m) p[i] = r[i];
}

// Sort each (polygon,row) threshold list, count its spans and their pieces.
__device__ __forceinline__ void prow_count_body(uint32_t t0, uint32_t ts, SpanGeo g, uint32_t n_prow, const uint32_t *__restrict__ pr_off,
                             uint32_t *__restrict__ tv, uint32_t *__restrict__ span_cnt,
                             uint32_t *__restrict__ piece_cnt) {
    for (uint32_t pr = t0; pr < n_prow; pr += ts) {
        const uint32_t b = pr_off[pr], e = pr_off[pr + 1];
        const uint32_t m = e - b;                            // the usual case: sort in registers
        if (m <= 2) {
            if (m == 2) {
                const uint32_t u = tv[b], v = tv[b + 1];
                if (u > v) { tv[b] = v; tv[b + 1] = u; }
            }
        } else if (m <= 4) {
            sort_small<4>(tv + b, m);
        } else if (m <= 16) {
            sort_small<16>(tv + b, m);
        } else {
            for (uint32_t i = b + 1; i < e; ++i) {
                const uint32_t v = tv[i];
                uint32_t j = i;
                while (j > b && tv[j - 1] > v) { tv[j] = tv[j - 1]; --j; }
                tv[j] = v;
            }
        }
        uint32_t P;
        int64_t r;
        polyrow_of(g, pr, P, r);
        uint32_t ns = 0;
        for (uint32_t i = b; i + 1 < e; i += 2) {
            int64_t lo = tv[i], hi = tv[i + 1];
            if (!clip_span(g, r, lo, hi)) continue;
            ++ns;
            for_each_piece(g, r, lo, hi, [&](uint32_t cell, uint32_t, uint32_t, uint32_t) {
                // consecutive threads are consecutive rows of one polygon and
                // mostly walk the same cells: the converged lanes of a cell add
                // their pieces with one atomic
                const unsigned peers = __match_any_sync(__activemask(), cell);
                if ((threadIdx.x & 31) == __ffs(peers) - 1) atomicAdd(&piece_cnt[cell], (uint32_t)__popc(peers));
            });
        }
        span_cnt[pr] = ns;
    }
}

__device__ __forceinline__ void prow_emit_body(uint32_t t0, uint32_t ts, SpanGeo g, uint32_t n_prow, const uint32_t *__restrict__ pr_off,
                            const uint32_t *__restrict__ tv, const uint32_t *__restrict__ span_off,
                            uint32_t *__restrict__ spans, const uint32_t *__restrict__ piece_off,
                            uint32_t *__restrict__ piece_cur, uint2 *__restrict__ pieces) {
    for (uint32_t pr = t0; pr < n_prow; pr += ts) {
        const uint32_t b = pr_off[pr], e = pr_off[pr + 1];
        uint32_t P;
        int64_t r;
        polyrow_of(g, pr, P, r);
        uint32_t k = span_off[pr];
        for (uint32_t i = b; i + 1 < e; i += 2) {
            int64_t lo = tv[i], hi = tv[i + 1];
            if (!clip_span(g, r, lo, hi)) continue;
            uint32_t *s = spans + 4 * (uint64_t)k++;
            s[0] = P; s[1] = (uint32_t)r; s[2] = (uint32_t)lo; s[3] = (uint32_t)hi;
            // the converged lanes of a cell reserve their slots with one atomic
            // (consecutive rows of one polygon mostly walk the same cells)
            const uint32_t pv = P;
            for_each_piece(g, r, lo, hi, [&](uint32_t cell, uint32_t lr, uint32_t a, uint32_t bb) {
                const unsigned peers = __match_any_sync(__activemask(), cell);
                const int lane = threadIdx.x & 31, leader = __ffs(peers) - 1;
                uint32_t base = 0;
                if (lane == leader) base = atomicAdd(&piece_cur[cell], (uint32_t)__popc(peers));
                base = __shfl_sync(peers, base, leader);
                const uint32_t slot = base + __popc(peers & ((1u << lane) - 1u));
                RJ_DCHECK(piece_off[cell] + slot < piece_off[cell + 1]);
                pieces[piece_off[cell] + slot] = make_uint2(pv, lr | (a << 8) | (bb << 16));
            });
        }
    }
}

// -------------------------------------------------------------- S5 supercover
// (marks only inside the viewport window [c0, c1) x [r0, r1))
__global__ void k_mask_mark(const int4 *__restrict__ edges, const uint32_t *__restrict__ band_off,
                            uint32_t n_edges, int W, int H, uint32_t wpr, uint32_t *__restrict__ mask,
                            int4 view) {
    const uint32_t total = band_off[n_edges];
    for (uint32_t j = blockIdx.x * blockDim.x + threadIdx.x; j < total; j += gridDim.x * blockDim.x) {
        const uint32_t e = upper_bound_u32(band_off, n_edges + 1, j) - 1;
        const int4 E = edges[e];
        const int64_t r = pix(min(E.y, E.w), H) + (j - band_off[e]);
        if (r < view.y || r >= view.w) continue;
        int64_t i0, i1;
        if (!supercover_cols(E.x, E.y, E.z, E.w, r, W, H, i0, i1)) continue;
        i0 = max(i0, (int64_t)view.x);
        i1 = min(i1, (int64_t)view.z - 1);
        if (i0 > i1) continue;
        uint32_t *row = mask + (uint64_t)r * wpr;
        for (int64_t w = i0 >> 5; w <= (i1 >> 5); ++w) {
            const int64_t a = max(i0, w << 5) - (w << 5), b = min(i1, (w << 5) + 31) - (w << 5);
            const uint32_t m = (b == 31 ? 0xFFFFFFFFu : ((1u << (b + 1)) - 1u)) & ~((1u << a) - 1u);
            atomicOr(&row[w], m);
        }
    }
}

// S5 as pieces (accurate mode): the supercover column range of every (edge,
// row band) -- the pixels the boundary mask marks -- clipped to the window and
// cut at the level-L point cells, binned per cell as (local row, lo, hi).
// The point-pass kernels paint them into their tiles from this list instead
// of reading the mask rows per cell (a dependent global load between two
// CTA barriers).  A pixel touched by several edges appears several times.
template <bool EMIT>
__device__ __forceinline__ void bnd_pieces_body(uint32_t t0, uint32_t ts, SpanGeo g, const int4 *__restrict__ edges, const uint32_t *__restrict__ band_off,
                             uint32_t n_edges, uint32_t *__restrict__ cnt, const uint32_t *__restrict__ off,
                             uint32_t *__restrict__ cur, uint32_t *__restrict__ out) {
    const uint32_t total = band_off[n_edges];
    for (uint32_t j = t0; j < total; j += ts) {
        const uint32_t e = upper_bound_u32(band_off, n_edges + 1, j) - 1;
        const int4 E = edges[e];
        const int64_t r = pix(min(E.y, E.w), g.H) + (j - band_off[e]);
        int64_t i0, i1;
        if (!supercover_cols(E.x, E.y, E.z, E.w, r, g.W, g.H, i0, i1)) continue;
        int64_t lo = i0, hi = i1 + 1;
        if (!clip_span(g, r, lo, hi)) continue;
        for_each_piece(g, r, lo, hi, [&](uint32_t cell, uint32_t lr, uint32_t a, uint32_t b) {
            if (EMIT) out[off[cell] + atomicAdd(&cur[cell], 1u)] = lr | (a << 8) | (b << 16);
            else atomicAdd(&cnt[cell], 1u);
        });
    }
}

// ---- the polygon pass as a chain of PDL-launched kernels (pdl_wait first)
// rows per edge (+ S5 bands) and per polygon, window-culled
__global__ void k_rows(const int4 *__restrict__ edges, const uint32_t *__restrict__ edge_poly,
                       const int4 *__restrict__ mbr, uint32_t n_edges, uint32_t n_poly, int W, int H, int accurate,
                       uint32_t *__restrict__ erows, uint32_t *__restrict__ bands, uint32_t *__restrict__ prows,
                       int4 view) {
    pdl_wait();
    pdl_trigger();
    const uint32_t t0 = blockIdx.x * blockDim.x + threadIdx.x, ts = gridDim.x * blockDim.x;
    edge_rows_body(t0, ts, edges, edge_poly, mbr, n_edges, H, erows, accurate, W, bands, view);
    poly_rows_body(t0, ts, mbr, n_poly, W, H, prows, view);
}

// zero up to four counter arrays of n[k] + 1 words
struct ZeroJobs {
    uint32_t *p[4];
    uint64_t n[4];
};
__global__ void k_zero(const ZeroJobs z) {
    pdl_wait();
    pdl_trigger();
    const uint64_t t0 = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x, ts = (uint64_t)gridDim.x * blockDim.x;
    for (int k = 0; k < 4; ++k)
        if (z.p[k])
            for (uint64_t i = t0; i <= z.n[k]; i += ts) z.p[k][i] = 0u;
}

// per (polygon, row): sort, count spans and per-cell pieces
__global__ void k_count(SpanGeo g, uint32_t n_prow, const uint32_t *__restrict__ pr_off, uint32_t *__restrict__ tv,
                        uint32_t *__restrict__ span_cnt, uint32_t *__restrict__ piece_cnt) {
    pdl_wait();
    pdl_trigger();
    prow_count_body(blockIdx.x * blockDim.x + threadIdx.x, gridDim.x * blockDim.x, g, n_prow, pr_off, tv, span_cnt,
                    piece_cnt);
}

// spans and their pieces per cell
__global__ void k_emit(SpanGeo g, uint32_t n_prow, const uint32_t *__restrict__ pr_off, const uint32_t *__restrict__ tv,
                       const uint32_t *__restrict__ span_off, uint32_t *__restrict__ spans,
                       const uint32_t *__restrict__ piece_off, uint32_t *__restrict__ piece_cur,
                       uint2 *__restrict__ pieces) {
    pdl_wait();
    pdl_trigger();
    prow_emit_body(blockIdx.x * blockDim.x + threadIdx.x, gridDim.x * blockDim.x, g, n_prow, pr_off, tv, span_off,
                   spans, piece_off, piece_cur, pieces);
}

// accurate mode: boundary pieces per cell (count pass / emit pass)
template <bool EMIT>
__global__ void k_bnd(SpanGeo g, const int4 *__restrict__ edges, const uint32_t *__restrict__ band_off,
                      uint32_t n_edges, uint32_t *__restrict__ cnt, const uint32_t *__restrict__ off,
                      uint32_t *__restrict__ cur, uint32_t *__restrict__ out) {
    pdl_wait();
    pdl_trigger();
    bnd_pieces_body<EMIT>(blockIdx.x * blockDim.x + threadIdx.x, gridDim.x * blockDim.x, g, edges, band_off, n_edges,
                          cnt, off, cur, out);
}

}  // namespace

// ------------------------------------------------------------------- loading
static int64_t host_quantize(double v, double lo, double hi) {
    volatile double d = v - lo;     // no contraction: each op rounded (O1)
    volatile double s = hi - lo;
    volatile double f = d / s;
    volatile double g = f * 1073741824.0;
    double fl = std::floor(g);
    if (!(fl >= -1.0e18 && fl <= 1.0e18)) return INT64_MIN;
    return (int64_t)fl;
}

rj_status load_polygons_impl(Ctx *c, uint32_t n_poly, const uint32_t *pro, const uint32_t *rvo,
                             const double *vx, const double *vy) {
    if (pro[0] != 0) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "poly_ring_off[0] must be 0");
    for (uint32_t p = 0; p < n_poly; ++p)
        if (pro[p + 1] <= pro[p]) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "every polygon needs >= 1 ring");
    const uint32_t n_ring = pro[n_poly];
    if (rvo[0] != 0) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "ring_vert_off[0] must be 0");
    for (uint32_t r = 0; r < n_ring; ++r)
        if (rvo[r + 1] < rvo[r] + 3) return set_error(c, RJ_ERR_INVALID_ARGUMENT, "every ring needs >= 3 vertices");
    const uint64_t n_vert = rvo[n_ring];
    if (n_vert >= (1ull << 31)) return set_error(c, RJ_ERR_CAPACITY, "too many vertices");

    std::vector<int4> edges;
    std::vector<uint32_t> epoly;
    std::vector<uint32_t> peoff(n_poly + 1, 0);
    std::vector<int4> mbr(n_poly);
    edges.reserve(n_vert);
    epoly.reserve(n_vert);
    std::vector<int32_t> qx(n_vert), qy(n_vert);
    for (uint64_t v = 0; v < n_vert; ++v) {
        const int64_t a = host_quantize(vx[v], c->x0, c->x1), b = host_quantize(vy[v], c->y0, c->y1);
        if (a < 0 || a > kOne || b < 0 || b > kOne)
            return set_error(c, RJ_ERR_OUT_OF_DOMAIN, "polygon vertex " + std::to_string(v) + " outside the domain");
        qx[v] = (int32_t)a;
        qy[v] = (int32_t)b;
    }
    for (uint32_t p = 0; p < n_poly; ++p) {
        peoff[p] = (uint32_t)edges.size();
        int4 m = make_int4(INT32_MAX, INT32_MAX, INT32_MIN, INT32_MIN);
        for (uint32_t r = pro[p]; r < pro[p + 1]; ++r)
            for (uint32_t v = rvo[r]; v < rvo[r + 1]; ++v) {
                const uint32_t w = (v + 1 < rvo[r + 1]) ? v + 1 : rvo[r];
                edges.push_back(make_int4(qx[v], qy[v], qx[w], qy[w]));
                epoly.push_back(p);
                m.x = std::min(m.x, qx[v]); m.y = std::min(m.y, qy[v]);
                m.z = std::max(m.z, qx[v]); m.w = std::max(m.w, qy[v]);
            }
        mbr[p] = m;
    }
    peoff[n_poly] = (uint32_t)edges.size();
    const uint32_t ne = (uint32_t)edges.size();
    // total edge extent per axis (lattice units): input of the exact-mode
    // chooser's boundary-pixel estimate
    double lx = 0.0, ly = 0.0;
    for (const int4 &e : edges) {
        lx += std::fabs((double)e.z - (double)e.x);
        ly += std::fabs((double)e.w - (double)e.y);
    }

    dfree(c, c->edges); dfree(c, c->edge_poly); dfree(c, c->poly_edge_off); dfree(c, c->mbr);
    dfree(c, c->poly_ring_off); dfree(c, c->ring_edge_off); dfree(c, c->edge_sigma);
    dfree(c, c->grid_off); dfree(c, c->grid_ent);
    c->n_poly = 0;
    if (dalloc(c, c->edges, ne * sizeof(int4)) || dalloc(c, c->edge_poly, ne * 4) ||
        dalloc(c, c->poly_edge_off, (n_poly + 1) * 4) || dalloc(c, c->mbr, n_poly * sizeof(int4)) ||
        dalloc(c, c->poly_ring_off, (n_poly + 1) * 4) || dalloc(c, c->ring_edge_off, (n_ring + 1) * 4) ||
        dalloc(c, c->edge_sigma, ne))
        return set_error(c, RJ_ERR_OOM, "polygon allocation failed");
    // one edge per vertex, in vertex order: ring r's edges are [rvo[r], rvo[r+1])
    RJ_CUDA(c, cudaMemcpyAsync(c->poly_ring_off.p, pro, (n_poly + 1) * 4, cudaMemcpyHostToDevice, c->stream));
    RJ_CUDA(c, cudaMemcpyAsync(c->ring_edge_off.p, rvo, (n_ring + 1) * 4, cudaMemcpyHostToDevice, c->stream));
    c->n_ring = n_ring;
    ++c->data_gen;
    RJ_CUDA(c, cudaMemcpyAsync(c->edges.p, edges.data(), ne * sizeof(int4), cudaMemcpyHostToDevice, c->stream));
    RJ_CUDA(c, cudaMemcpyAsync(c->edge_poly.p, epoly.data(), ne * 4, cudaMemcpyHostToDevice, c->stream));
    RJ_CUDA(c, cudaMemcpyAsync(c->poly_edge_off.p, peoff.data(), (n_poly + 1) * 4, cudaMemcpyHostToDevice, c->stream));
    RJ_CUDA(c, cudaMemcpyAsync(c->mbr.p, mbr.data(), n_poly * sizeof(int4), cudaMemcpyHostToDevice, c->stream));

    // S6 edge grid: items per edge, count pass, offsets, fill pass, per-cell sort
    const uint64_t ncell = (uint64_t)kGrid * kGrid;
    Buf cnt, cur, items, item_off, tot;
    if (dalloc(c, cnt, ncell * 4) || dalloc(c, cur, ncell * 4) || dalloc(c, c->grid_off, (ncell + 1) * 4) ||
        dalloc(c, items, (uint64_t)(ne + 1) * 4) || dalloc(c, item_off, (uint64_t)(ne + 1) * 4) || dalloc(c, tot, 8))
        return set_error(c, RJ_ERR_OOM, "edge grid allocation failed");
    RJ_CUDA(c, cudaMemsetAsync(cnt.p, 0, ncell * 4, c->stream));
    RJ_CUDA(c, cudaMemsetAsync(cur.p, 0, ncell * 4, c->stream));
    RJ_CUDA(c, cudaMemsetAsync(tot.p, 0, 8, c->stream));
    k_grid_items<<<blocks_for(ne, 256), 256, 0, c->stream>>>(c->edges.as<int4>(), c->edge_poly.as<uint32_t>(),
                                                             c->mbr.as<int4>(), ne, items.as<uint32_t>(),
                                                             reinterpret_cast<unsigned long long *>(tot.p));
    RJ_LAUNCHED(c);
    RJ_CUDA(c, cudaGetLastError());
    RJ_CUDA(c, scan_u32(c, items.as<uint32_t>(), item_off.as<uint32_t>(), ne, kWsScan));
    unsigned long long n_ent64 = 0;
    RJ_CUDA(c, cudaMemcpyAsync(&n_ent64, tot.p, 8, cudaMemcpyDeviceToHost, c->stream));
    RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    // the item count is at most the entry count, so one check covers both u32 offsets
    if (n_ent64 > 0xFFFFFFFFull) {
        dfree(c, cnt); dfree(c, cur); dfree(c, items); dfree(c, item_off); dfree(c, tot);
        return set_error(c, RJ_ERR_CAPACITY, "edge grid: more than 2^32 - 1 (cell, edge) entries");
    }
    const uint32_t n_ent = (uint32_t)n_ent64;
    const unsigned gi = (unsigned)std::max<uint64_t>(1, std::min<uint64_t>(blocks_for(n_ent, 256), c->num_sms * 16ull));
    k_grid_edges<false><<<gi, 256, 0, c->stream>>>(c->edges.as<int4>(), c->edge_poly.as<uint32_t>(),
                                                   c->mbr.as<int4>(), ne, item_off.as<uint32_t>(),
                                                   cnt.as<uint32_t>(), nullptr, nullptr, nullptr);
    RJ_LAUNCHED(c);
    RJ_CUDA(c, cudaGetLastError());
    RJ_CUDA(c, scan_u32(c, cnt.as<uint32_t>(), c->grid_off.as<uint32_t>(), ncell, kWsScan));
    if (dalloc(c, c->grid_ent, std::max<uint64_t>(1, n_ent) * 4))
        return set_error(c, RJ_ERR_OOM, "edge grid allocation failed");
    k_grid_edges<true><<<gi, 256, 0, c->stream>>>(c->edges.as<int4>(), c->edge_poly.as<uint32_t>(),
                                                  c->mbr.as<int4>(), ne, item_off.as<uint32_t>(), nullptr,
                                                  c->grid_off.as<uint32_t>(), cur.as<uint32_t>(),
                                                  c->grid_ent.as<uint32_t>());
    RJ_LAUNCHED(c);
    RJ_CUDA(c, cudaGetLastError());
    {
        Buf tmp;
        if (dalloc(c, tmp, std::max<uint64_t>(1, n_ent) * 4)) return set_error(c, RJ_ERR_OOM, "edge grid allocation failed");
        k_grid_sort<<<(unsigned)(c->num_sms * 16), 256, 0, c->stream>>>(c->grid_off.as<uint32_t>(),
                                                                     c->grid_ent.as<uint32_t>(), tmp.as<uint32_t>());
        RJ_LAUNCHED(c);
        RJ_CUDA(c, cudaGetLastError());
        RJ_CUDA(c, cudaStreamSynchronize(c->stream));
        dfree(c, tmp);
    }
    dfree(c, items);
    dfree(c, item_off);
    dfree(c, tot);
    dfree(c, c->grid_edge);
    dfree(c, c->grid_poly);
    if (dalloc(c, c->grid_edge, std::max<uint64_t>(1, n_ent) * sizeof(int4)) ||
        dalloc(c, c->grid_poly, std::max<uint64_t>(1, n_ent) * 4))
        return set_error(c, RJ_ERR_OOM, "edge grid allocation failed");
    if (n_ent) {
        k_grid_inline<<<blocks_for(n_ent, 256), 256, 0, c->stream>>>(
            c->grid_ent.as<uint32_t>(), n_ent, c->edges.as<int4>(), c->edge_poly.as<uint32_t>(),
            c->grid_edge.as<int4>(), c->grid_poly.as<uint32_t>());
        RJ_LAUNCHED(c);
        RJ_CUDA(c, cudaGetLastError());
    }
    {
        rj_status rs = ring_sigma_impl(c, n_poly, n_ring);
        if (rs != RJ_OK) return rs;
    }
    RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    dfree(c, cnt);
    dfree(c, cur);
    c->n_grid_ent = n_ent;
    c->edge_len_x = lx;
    c->edge_len_y = ly;
    c->n_edges = ne;
    c->n_poly = n_poly;
    return RJ_OK;
}

// ------------------------------------------------------------ per-query pass
rj_status polygon_pass(Ctx *c, int W, int H, int L, bool accurate, PolyPass &pp, const View &v, bool need_mask) {
    // L < 0: spans (and mask) only, no pieces (the streamed query)
    const uint64_t ncell = L >= 0 ? 1ull << (2 * L) : 0;
    const uint32_t ne = c->n_edges, np = c->n_poly;
    cudaStream_t st = c->stream;
    Buf &erows = wsbuf(c, kWsEdgeRows), &eoff = wsbuf(c, kWsEdgeOff);
    Buf &prows = wsbuf(c, kWsPolyRows), &proff = wsbuf(c, kWsPolyRowOff);
    Buf &bcnt = wsbuf(c, kWsBandCount), &boff = wsbuf(c, kWsBandOff);
    Buf &sizes = wsbuf(c, kWsSizes);
    if (dreserve(c, erows, (ne + 1) * 4) || dreserve(c, eoff, (ne + 1) * 4) || dreserve(c, prows, (np + 1) * 4) ||
        dreserve(c, proff, (np + 1) * 4) || dreserve(c, bcnt, (ne + 1) * 4) || dreserve(c, boff, (ne + 1) * 4) ||
        dreserve(c, sizes, 64))
        return set_error(c, RJ_ERR_OOM, "workspace allocation failed");
    const int4 vw = v.full ? make_int4(0, 0, W, H) : make_int4(v.c0, v.r0, v.c1, v.r1);
    const int64_t key[9] = {W, H, L, accurate ? 1 : 0, vw.x, vw.y, vw.z, vw.w, (int64_t)c->data_gen};
    const bool known = c->pp_key_valid && std::equal(key, key + 9, c->pp_key);
    const unsigned gr = (unsigned)std::min<uint64_t>(std::max<uint64_t>(1, blocks_for(std::max(ne, np), 256)),
                                                     c->num_sms * 8ull);
    RJ_CUDA(c, launch_pdl(c, k_rows, dim3(gr), dim3(256), 0, c->edges.as<int4>(), c->edge_poly.as<uint32_t>(),
                          c->mbr.as<int4>(), ne, np, W, H, accurate ? 1 : 0, erows.as<uint32_t>(), bcnt.as<uint32_t>(),
                          prows.as<uint32_t>(), vw));
    RJ_LAUNCHED(c);
    {
        const uint32_t *in[3] = {erows.as<uint32_t>(), prows.as<uint32_t>(), bcnt.as<uint32_t>()};
        uint32_t *out[3] = {eoff.as<uint32_t>(), proff.as<uint32_t>(), boff.as<uint32_t>()};
        const uint64_t n[3] = {ne, np, ne};
        RJ_CUDA(c, scan_multi(c, accurate ? 3 : 2, in, out, n, kWsScan));
    }
    // sync 1: crossing / polygon-row / band totals (skipped for a repeated key)
    uint32_t *hs = reinterpret_cast<uint32_t *>(c->h_stats + 8);
    if (known) {
        std::copy(c->pp_sizes, c->pp_sizes + 6, hs);
    } else {
        c->pp_key_valid = false;
        hs[2] = 0;
        RJ_CUDA(c, cudaMemcpyAsync(hs + 0, eoff.as<uint32_t>() + ne, 4, cudaMemcpyDeviceToHost, st));
        RJ_CUDA(c, cudaMemcpyAsync(hs + 1, proff.as<uint32_t>() + np, 4, cudaMemcpyDeviceToHost, st));
        if (accurate) RJ_CUDA(c, cudaMemcpyAsync(hs + 2, boff.as<uint32_t>() + ne, 4, cudaMemcpyDeviceToHost, st));
        RJ_CUDA(c, cudaStreamSynchronize(st));
    }
    const uint32_t X = hs[0], NPR = hs[1];

    Buf &cpr = wsbuf(c, kWsCrossPR), &ct = wsbuf(c, kWsCrossT), &prc = wsbuf(c, kWsPRCount);
    Buf &pro = wsbuf(c, kWsPROff), &prcur = wsbuf(c, kWsPRCursor), &tv = wsbuf(c, kWsTvals);
    Buf &scnt = wsbuf(c, kWsSpanCount), &soff = wsbuf(c, kWsSpanOff);
    Buf &pcnt = wsbuf(c, kWsPieceCount), &poff = wsbuf(c, kWsPieceOff), &pcur = wsbuf(c, kWsPieceCursor);
    Buf &bpc = wsbuf(c, kWsBPCount), &bpo = wsbuf(c, kWsBPOff), &bpu = wsbuf(c, kWsBPCursor);
    const bool bnd_pieces = accurate && ncell;               // accurate mode with point cells
    if (dreserve(c, cpr, (X + 1) * 4) || dreserve(c, ct, (X + 1) * 4) || dreserve(c, prc, (NPR + 1) * 4) ||
        dreserve(c, pro, (NPR + 1) * 4) || dreserve(c, prcur, (NPR + 1) * 4) || dreserve(c, tv, (X + 1) * 4) ||
        dreserve(c, scnt, (NPR + 1) * 4) || dreserve(c, soff, (NPR + 1) * 4) ||
        dreserve(c, pcnt, (ncell + 1) * 4) || dreserve(c, poff, (ncell + 1) * 4) ||
        dreserve(c, pcur, (ncell + 1) * 4) ||
        (bnd_pieces && (dreserve(c, bpc, (ncell + 1) * 4) || dreserve(c, bpo, (ncell + 1) * 4) ||
                        dreserve(c, bpu, (ncell + 1) * 4))))
        return set_error(c, RJ_ERR_OOM, "workspace allocation failed");
    {
        // counters: (polygon,row) counts + cursors, per-cell piece counts + cursors
        // (cursors follow counts in one allocation-free kernel)
        ZeroJobs z{};
        z.p[0] = prc.as<uint32_t>(); z.n[0] = NPR;
        z.p[1] = prcur.as<uint32_t>(); z.n[1] = NPR;
        z.p[2] = pcnt.as<uint32_t>(); z.n[2] = ncell;
        z.p[3] = pcur.as<uint32_t>(); z.n[3] = ncell;
        const unsigned gz = (unsigned)std::min<uint64_t>(std::max<uint64_t>(1, blocks_for(std::max<uint64_t>(NPR, ncell) + 1, 256)),
                                                         c->num_sms * 8ull);
        RJ_CUDA(c, launch_pdl(c, k_zero, dim3(gz), dim3(256), 0, z));
        RJ_LAUNCHED(c);
        if (bnd_pieces) {
            ZeroJobs zb{};
            zb.p[0] = bpc.as<uint32_t>(); zb.n[0] = ncell;
            zb.p[1] = bpu.as<uint32_t>(); zb.n[1] = ncell;
            RJ_CUDA(c, launch_pdl(c, k_zero, dim3(gz), dim3(256), 0, zb));
            RJ_LAUNCHED(c);
        }
    }
    const unsigned gx = (unsigned)std::min<uint64_t>(std::max<uint64_t>(1, blocks_for(X, 256)), c->num_sms * 8ull);
    RJ_CUDA(c, launch_pdl(c, k_crossings, dim3(gx), dim3(256), 0, c->edges.as<int4>(), c->edge_poly.as<uint32_t>(),
                          c->mbr.as<int4>(), eoff.as<uint32_t>(), ne, proff.as<uint32_t>(), W, H, cpr.as<uint32_t>(),
                          ct.as<uint32_t>(), prc.as<uint32_t>()));
    RJ_LAUNCHED(c);
    RJ_CUDA(c, scan_u32(c, prc.as<uint32_t>(), pro.as<uint32_t>(), NPR, kWsScan));
    RJ_CUDA(c, launch_pdl(c, k_scatter_t, dim3(gx), dim3(256), 0, cpr.as<uint32_t>(), ct.as<uint32_t>(), X,
                          pro.as<uint32_t>(), prcur.as<uint32_t>(), tv.as<uint32_t>()));
    RJ_LAUNCHED(c);
    SpanGeo g{W, H, L, proff.as<uint32_t>(), np, c->mbr.as<int4>(), L >= 0 ? c->cell_bits[L].as<uint32_t>() : nullptr,
              v.full ? 0 : v.c0, v.full ? 0 : v.r0, v.full ? W : v.c1, v.full ? H : v.r1};
    const uint32_t B = accurate ? hs[2] : 0;
    const unsigned gp = (unsigned)std::min<uint64_t>(std::max<uint64_t>(1, blocks_for(NPR, 128)), c->num_sms * 16ull);
    const unsigned gb = (unsigned)std::min<uint64_t>(std::max<uint64_t>(1, blocks_for(B, 256)), c->num_sms * 8ull);
    RJ_CUDA(c, launch_pdl(c, k_count, dim3(gp), dim3(128), 0, g, NPR, pro.as<uint32_t>(), tv.as<uint32_t>(),
                          scnt.as<uint32_t>(), pcnt.as<uint32_t>()));
    RJ_LAUNCHED(c);
    if (bnd_pieces) {
        RJ_CUDA(c, launch_pdl(c, k_bnd<false>, dim3(gb), dim3(256), 0, g, c->edges.as<int4>(), boff.as<uint32_t>(), ne,
                              bpc.as<uint32_t>(), (const uint32_t *)nullptr, (uint32_t *)nullptr, (uint32_t *)nullptr));
        RJ_LAUNCHED(c);
    }
    {
        const uint32_t *in[3] = {scnt.as<uint32_t>(), pcnt.as<uint32_t>(), bpc.as<uint32_t>()};
        uint32_t *out[3] = {soff.as<uint32_t>(), poff.as<uint32_t>(), bpo.as<uint32_t>()};
        const uint64_t n[3] = {NPR, ncell, ncell};
        RJ_CUDA(c, scan_multi(c, ncell ? (bnd_pieces ? 3 : 2) : 1, in, out, n, kWsScan));
    }
    // sync 2: span / piece totals (skipped for a repeated key)
    if (!known) {
        hs[4] = 0;
        hs[5] = 0;
        RJ_CUDA(c, cudaMemcpyAsync(hs + 3, soff.as<uint32_t>() + NPR, 4, cudaMemcpyDeviceToHost, st));
        if (ncell) RJ_CUDA(c, cudaMemcpyAsync(hs + 4, poff.as<uint32_t>() + ncell, 4, cudaMemcpyDeviceToHost, st));
        if (bnd_pieces) RJ_CUDA(c, cudaMemcpyAsync(hs + 5, bpo.as<uint32_t>() + ncell, 4, cudaMemcpyDeviceToHost, st));
        RJ_CUDA(c, cudaStreamSynchronize(st));
        std::copy(hs, hs + 6, c->pp_sizes);
        std::copy(key, key + 9, c->pp_key);
        c->pp_key_valid = true;
    }
    const uint32_t S = hs[3], NP = hs[4], NB = hs[5];
    Buf &spans = wsbuf(c, kWsSpans), &pieces = wsbuf(c, kWsPieces), &bp = wsbuf(c, kWsBPieces);
    if (dreserve(c, spans, (uint64_t)(S + 1) * 16) || dreserve(c, pieces, (uint64_t)(NP + 1) * 8) ||
        (bnd_pieces && dreserve(c, bp, (uint64_t)(NB + 1) * 4)))
        return set_error(c, RJ_ERR_OOM, "workspace allocation failed");
    RJ_CUDA(c, launch_pdl(c, k_emit, dim3(gp), dim3(128), 0, g, NPR, pro.as<uint32_t>(), tv.as<uint32_t>(),
                          soff.as<uint32_t>(), spans.as<uint32_t>(), poff.as<uint32_t>(), pcur.as<uint32_t>(),
                          pieces.as<uint2>()));
    RJ_LAUNCHED(c);
    if (bnd_pieces) {
        RJ_CUDA(c, launch_pdl(c, k_bnd<true>, dim3(gb), dim3(256), 0, g, c->edges.as<int4>(), boff.as<uint32_t>(), ne,
                              (uint32_t *)nullptr, (const uint32_t *)bpo.as<uint32_t>(), bpu.as<uint32_t>(),
                              bp.as<uint32_t>()));
        RJ_LAUNCHED(c);
    }
    if (bnd_pieces) {
        pp.bpiece_off = bpo.as<uint32_t>();
        pp.bpieces = bp.as<uint32_t>();
        pp.n_bpieces = NB;
    }
    pp.n_cross = X;
    pp.n_spans = S;
    pp.n_pieces = NP;
    pp.spans = spans.as<uint32_t>();
    pp.piece_off = poff.as<uint32_t>();
    pp.pieces = pieces.as<uint2>();
    if (accurate) pp.n_bands = B;
    if (accurate && need_mask) {
        // the bitmask is only read by the diagnostics and the streamed
        // (label-canvas) query: the point-pass kernels take bpieces
        const uint32_t wpr = (uint32_t)((W + 31) / 32);
        Buf &mask = wsbuf(c, kWsMask);
        if (dreserve(c, mask, (uint64_t)wpr * H * 4)) return set_error(c, RJ_ERR_OOM, "mask allocation failed");
        RJ_CUDA(c, cudaMemsetAsync(mask.p, 0, (uint64_t)wpr * H * 4, st));
        k_mask_mark<<<gb, 256, 0, st>>>(c->edges.as<int4>(), boff.as<uint32_t>(), ne, W, H, wpr, mask.as<uint32_t>(),
                                        vw);
        RJ_LAUNCHED(c);
        RJ_CUDA(c, cudaGetLastError());
        pp.mask = mask.as<uint32_t>();
        pp.mask_wpr = wpr;
    }
    return RJ_OK;
}

}  // namespace rj
