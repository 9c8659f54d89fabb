// interval.cu -- bounded-mode result intervals.
//
// Paper: for polygon i let P+_i / P-_i be its boundary pixels
// whose points are counted although outside (false positives) / not counted
// although inside (false negatives); eps+_i = sum over P+_i of Fpt,
// eps-_i = sum over P-_i of Fpt, and the exact result lies in
// [A[i] - eps+_i, A[i] + eps-_i] "with 100% confidence".
//
// Reading (O10, Z13): the boundary pixels B_i of polygon i are the S5
// supercover of i's own edges (the conservative outline); a pixel
// of B_i belongs to P+_i when its centre is inside i (it is counted by the
// pixel-centre rule), else to P-_i; Fpt = the pixel's filtered
// point count.  Every pixel of B_i is counted once per polygon.
//
// GPU plan (all exact integer work):
//   1. per polygon, its band rows [pix(ymin), pix(min(ymax, 2^30-1))]
//      -> one bucket per (polygon, row);
//   2. every (edge, row band) of the S5 pass yields one column range
//      (supercover_cols, shared with the mask) -> binned into its bucket;
//   3. one thread per bucket sorts and merges its ranges (a pixel touched by
//      several edges of the polygon counts once), splits them against the
//      polygon's spans of that row (centre inside <=> in a span, lemma L1)
//      and sums the count canvas over each part.
#include <algorithm>

#include "rj_internal.cuh"

namespace rj {

namespace {

inline unsigned blocks_for(uint64_t n, int t) { return (unsigned)std::max<uint64_t>(1, (n + t - 1) / t); }

__device__ __forceinline__ uint32_t ub_u32(const uint32_t *a, uint32_t n, uint32_t v) {
    uint32_t lo = 0, hi = n;                 // first k in [0, n] with a[k] > v
    while (lo < hi) {
        const uint32_t m = (lo + hi) >> 1;
        if (a[m] > v) hi = m; else lo = m + 1;
    }
    return lo;
}

struct IntervalGeo {
    int W, H;
    const int4 *edges;
    const uint32_t *edge_poly;
    const int4 *mbr;
    const uint32_t *band_off;       // [n_edges + 1] S5 row bands per edge
    uint32_t n_edges, n_poly;
    const uint32_t *brow_off;       // [n_poly + 1] buckets (polygon, band row)
    const uint32_t *prow_off;       // [n_poly + 1] span rows (polygon, centre row)
    const uint32_t *span_off;       // [n_prow + 1]
    const uint4 *spans;             // (poly, row, lo, hi), sorted by (poly, row, lo)
    const uint32_t *canvas;         // [H][W] filtered points per pixel
};

__global__ void k_brow_count(const int4 *__restrict__ mbr, uint32_t n_poly, int H, uint32_t *__restrict__ cnt) {
    const uint32_t p = blockIdx.x * blockDim.x + threadIdx.x;
    if (p >= n_poly) return;
    const int4 m = mbr[p];
    cnt[p] = (uint32_t)band_rows(m.y, m.w, H);
}

// (edge, band row) j -> its bucket (polygon, row) and column range
__device__ __forceinline__ bool band_range(const IntervalGeo &g, uint32_t j, uint32_t &bucket, uint32_t &i0,
                                           uint32_t &i1) {
    const uint32_t e = ub_u32(g.band_off, g.n_edges + 1, j) - 1;
    const int4 E = g.edges[e];
    const int64_t r = pix(min(E.y, E.w), g.H) + (j - g.band_off[e]);
    int64_t a, b;
    if (!supercover_cols(E.x, E.y, E.z, E.w, r, g.W, g.H, a, b)) return false;
    const uint32_t P = g.edge_poly[e];
    bucket = g.brow_off[P] + (uint32_t)(r - pix(g.mbr[P].y, g.H));
    i0 = (uint32_t)a;
    i1 = (uint32_t)b;
    return true;
}

__global__ void k_bkt_count(const IntervalGeo g, uint32_t total, uint32_t *__restrict__ cnt) {
    for (uint32_t j = blockIdx.x * blockDim.x + threadIdx.x; j < total; j += gridDim.x * blockDim.x) {
        uint32_t bk, a, b;
        if (band_range(g, j, bk, a, b)) atomicAdd(&cnt[bk], 1u);
    }
}

__global__ void k_bkt_fill(const IntervalGeo g, uint32_t total, const uint32_t *__restrict__ off,
                           uint32_t *__restrict__ cur, uint2 *__restrict__ ranges) {
    for (uint32_t j = blockIdx.x * blockDim.x + threadIdx.x; j < total; j += gridDim.x * blockDim.x) {
        uint32_t bk, a, b;
        if (band_range(g, j, bk, a, b)) ranges[off[bk] + atomicAdd(&cur[bk], 1u)] = make_uint2(a, b);
    }
}

__global__ void k_bkt_eval(const IntervalGeo g, uint32_t n_bkt, const uint32_t *__restrict__ off,
                           uint2 *__restrict__ ranges, unsigned long long *__restrict__ eps_plus,
                           unsigned long long *__restrict__ eps_minus) {
    for (uint32_t bk = blockIdx.x * blockDim.x + threadIdx.x; bk < n_bkt; bk += gridDim.x * blockDim.x) {
        const uint32_t b = off[bk], e = off[bk + 1];
        if (b == e) continue;
        for (uint32_t i = b + 1; i < e; ++i) {               // insertion sort by first column
            const uint2 v = ranges[i];
            uint32_t j = i;
            while (j > b && ranges[j - 1].x > v.x) { ranges[j] = ranges[j - 1]; --j; }
            ranges[j] = v;
        }
        const uint32_t P = ub_u32(g.brow_off, g.n_poly + 1, bk) - 1;
        const int4 m = g.mbr[P];
        const int64_t r = pix(m.y, g.H) + (bk - g.brow_off[P]);
        // the polygon's spans in row r (rows whose centre lies in [ymin, ymax))
        uint32_t s = 0, se = 0;
        const int64_t rs = row_start(m.y, g.H), re = row_start(m.w, g.H);
        if (r >= rs && r < re) {
            const uint32_t pr = g.prow_off[P] + (uint32_t)(r - rs);
            s = g.span_off[pr];
            se = g.span_off[pr + 1];
        }
        const uint32_t *row = g.canvas + (uint64_t)r * g.W;
        unsigned long long ep = 0, em = 0;
        int64_t done = -1;                                   // last column already counted
        for (uint32_t i = b; i < e; ++i) {
            const int64_t lo = max((int64_t)ranges[i].x, done + 1), hi = ranges[i].y;
            for (int64_t x = lo; x <= hi; ++x) {
                while (s < se && (int64_t)g.spans[s].w <= x) ++s;       // spans are sorted, disjoint
                const bool in = s < se && (int64_t)g.spans[s].z <= x;
                const uint32_t cnt = row[x];
                if (in) ep += cnt; else em += cnt;
            }
            done = max(done, hi);
        }
        if (ep) atomicAdd(&eps_plus[P], ep);
        if (em) atomicAdd(&eps_minus[P], em);
    }
}

}  // namespace

rj_status interval_impl(Ctx *c, int W, int H, const PolyPass &pp, const uint32_t *canvas,
                        unsigned long long *d_eps_plus, unsigned long long *d_eps_minus) {
    cudaStream_t st = c->stream;
    const uint32_t np = c->n_poly, ne = c->n_edges;
    Buf &bcnt = wsbuf(c, kWsBRowCount), &boff = wsbuf(c, kWsBRowOff);
    if (dreserve(c, bcnt, (np + 1) * 4) || dreserve(c, boff, (np + 1) * 4))
        return set_error(c, RJ_ERR_OOM, "interval workspace allocation failed");
    k_brow_count<<<blocks_for(np, 256), 256, 0, st>>>(c->mbr.as<int4>(), np, H, bcnt.as<uint32_t>());
    RJ_LAUNCHED(c);
    RJ_CUDA(c, scan_u32(c, bcnt.as<uint32_t>(), boff.as<uint32_t>(), np, kWsScan));
    uint32_t *hs = reinterpret_cast<uint32_t *>(c->h_stats + 8);
    RJ_CUDA(c, cudaMemcpyAsync(hs + 5, boff.as<uint32_t>() + np, 4, cudaMemcpyDeviceToHost, st));
    RJ_CUDA(c, cudaStreamSynchronize(st));
    const uint32_t NB = hs[5];
    Buf &kc = wsbuf(c, kWsBktCount), &ko = wsbuf(c, kWsBktOff), &kcur = wsbuf(c, kWsBktCursor);
    Buf &rg = wsbuf(c, kWsBktRanges);
    const uint64_t NR = pp.n_bands;                         // at most one range per (edge, band row)
    if (dreserve(c, kc, (uint64_t)(NB + 1) * 4) || dreserve(c, ko, (uint64_t)(NB + 1) * 4) ||
        dreserve(c, kcur, (uint64_t)(NB + 1) * 4) || dreserve(c, rg, (NR + 1) * 8))
        return set_error(c, RJ_ERR_OOM, "interval workspace allocation failed");
    RJ_CUDA(c, cudaMemsetAsync(kc.p, 0, (uint64_t)(NB + 1) * 4, st));
    RJ_CUDA(c, cudaMemsetAsync(kcur.p, 0, (uint64_t)(NB + 1) * 4, st));
    RJ_CUDA(c, cudaMemsetAsync(d_eps_plus, 0, (size_t)np * 8, st));
    RJ_CUDA(c, cudaMemsetAsync(d_eps_minus, 0, (size_t)np * 8, st));
    IntervalGeo g;
    g.W = W;
    g.H = H;
    g.edges = c->edges.as<int4>();
    g.edge_poly = c->edge_poly.as<uint32_t>();
    g.mbr = c->mbr.as<int4>();
    g.band_off = wsbuf(c, kWsBandOff).as<uint32_t>();
    g.n_edges = ne;
    g.n_poly = np;
    g.brow_off = boff.as<uint32_t>();
    g.prow_off = wsbuf(c, kWsPolyRowOff).as<uint32_t>();
    g.span_off = wsbuf(c, kWsSpanOff).as<uint32_t>();
    g.spans = reinterpret_cast<const uint4 *>(pp.spans);
    g.canvas = canvas;
    if (NR) {
        const unsigned gr = (unsigned)std::min<uint64_t>(blocks_for(NR, 256), c->num_sms * 8ull);
        k_bkt_count<<<gr, 256, 0, st>>>(g, (uint32_t)NR, kc.as<uint32_t>());
        RJ_LAUNCHED(c);
        RJ_CUDA(c, scan_u32(c, kc.as<uint32_t>(), ko.as<uint32_t>(), NB, kWsScan));
        k_bkt_fill<<<gr, 256, 0, st>>>(g, (uint32_t)NR, ko.as<uint32_t>(), kcur.as<uint32_t>(), rg.as<uint2>());
        RJ_LAUNCHED(c);
        const unsigned gb = (unsigned)std::min<uint64_t>(blocks_for(NB, 128), c->num_sms * 16ull);
        k_bkt_eval<<<gb, 128, 0, st>>>(g, NB, ko.as<uint32_t>(), rg.as<uint2>(), d_eps_plus, d_eps_minus);
        RJ_LAUNCHED(c);
    }
    RJ_CUDA(c, cudaGetLastError());
    return RJ_OK;
}

}  // namespace rj
