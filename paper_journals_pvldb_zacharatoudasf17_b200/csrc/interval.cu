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
//
// Expected interval (reading Z22): with the uniform-in-pixel
// assumption a P+ pixel holds (1 - f) Fpt false positives and a P- pixel
// f Fpt false negatives, f = area(pixel n polygon) / area(pixel).  Step 3
// also evaluates f for every non-empty boundary pixel by Green's theorem:
//   area(P n [X0,X1) x [Y0,Y1)) = sum over P's edges, clipped to the band,
//                                 of sigma_e * int clamp(x(y) - X0, 0, w) dy
// (the integrand is piecewise linear in y; sigma_e = orientation * (-1)^depth
// of the edge's ring makes the ring sum the even-odd area).  The oracle
// clips rings with Sutherland-Hodgman instead -- a different computation of
// the same area.
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
    const uint32_t *poly_edge_off;  // [n_poly + 1]
    const int8_t *edge_sigma;       // [n_edges] ring weights (Z22)
};

// Ring weight sigma = orientation * (-1)^depth for every edge of ring r
// (depth: the polygon's other rings containing the ring's first vertex,
// even-odd PNPOLY).  Twice the signed area is summed exactly in 128 bits.
__global__ void k_ring_sigma(const int4 *__restrict__ edges, const uint32_t *__restrict__ poly_ring_off,
                             const uint32_t *__restrict__ ring_edge_off, uint32_t n_poly, uint32_t n_ring,
                             int8_t *__restrict__ sigma) {
    const uint32_t r = blockIdx.x * blockDim.x + threadIdx.x;
    if (r >= n_ring) return;
    const uint32_t P = ub_u32(poly_ring_off, n_poly + 1, r) - 1;
    const uint32_t e0 = ring_edge_off[r], e1 = ring_edge_off[r + 1];
    __int128 a2 = 0;
    for (uint32_t e = e0; e < e1; ++e) {
        const int4 E = edges[e];
        a2 += (__int128)E.x * E.w - (__int128)E.z * E.y;
    }
    int sg = (a2 > 0) - (a2 < 0);
    const int64_t px = edges[e0].x, py = edges[e0].y;
    for (uint32_t o = poly_ring_off[P]; o < poly_ring_off[P + 1]; ++o) {
        if (o == r) continue;
        bool in = false;
        for (uint32_t e = ring_edge_off[o]; e < ring_edge_off[o + 1]; ++e) {
            const int4 E = edges[e];
            const int64_t xa = E.x, ya = E.y, xb = E.z, yb = E.w;
            if ((ya > py) != (yb > py)) {
                const int64_t lhs = (px - xa) * (yb - ya), rhs = (xb - xa) * (py - ya);
                if (yb > ya ? lhs < rhs : lhs > rhs) in = !in;
            }
        }
        if (in) sg = -sg;
    }
    for (uint32_t e = e0; e < e1; ++e) sigma[e] = (int8_t)sg;
}

// int over the part of edge E inside the band y in [Y0, Y0 + h] of
// clamp(x(y) - X0, 0, w) dy, signed by the edge's direction (pixel-local
// binary64; the clamp is linear between its breakpoints, so the trapezoid
// rule is exact on each piece).
__device__ __forceinline__ double band_integral(const int4 E, int64_t X0, int64_t Y0, double w, double h) {
    const int64_t ya = E.y, yb = E.w;
    if (ya == yb) return 0.0;
    const double lo = fmax((double)(min(ya, yb) - Y0), 0.0), hi = fmin((double)(max(ya, yb) - Y0), h);
    if (!(lo < hi)) return 0.0;
    const double xa = (double)(E.x - X0), ta = (double)(ya - Y0), dx = (double)(E.z - E.x), dy = (double)(yb - ya);
    const double u0 = xa + dx * (lo - ta) / dy, u1 = xa + dx * (hi - ta) / dy;
    double t1 = 1.0, t2 = 1.0;                       // breakpoints where x - X0 crosses 0 and w
    if (u0 != u1) {
        const double a = -u0 / (u1 - u0), b = (w - u0) / (u1 - u0);
        if (a > 0.0 && a < 1.0) t1 = a;
        if (b > 0.0 && b < 1.0) t2 = b;
        if (t2 < t1) { const double t = t1; t1 = t2; t2 = t; }
    }
    auto g = [&](double t) { return fmin(fmax(u0 + (u1 - u0) * t, 0.0), w); };
    const double g0 = g(0.0), g1 = g(t1), g2 = g(t2), g3 = g(1.0);
    const double acc = t1 * (g0 + g1) + (t2 - t1) * (g1 + g2) + (1.0 - t2) * (g2 + g3);
    return (yb > ya ? 0.5 : -0.5) * acc * (hi - lo);
}

// f = area(pixel (i, r) n polygon P) / area(pixel), clamped to [0, 1]
__device__ double area_fraction(const IntervalGeo &g, uint32_t P, int64_t i, int64_t r) {
    const int64_t X0 = qlo(i, g.W), X1 = qlo(i + 1, g.W), Y0 = qlo(r, g.H), Y1 = qlo(r + 1, g.H);
    const double w = (double)(X1 - X0), h = (double)(Y1 - Y0);
    double a = 0.0;
    for (uint32_t e = g.poly_edge_off[P]; e < g.poly_edge_off[P + 1]; ++e) {
        const int4 E = g.edges[e];
        if (max(E.y, E.w) <= Y0 || min(E.y, E.w) >= Y1) continue;      // no dy inside the band
        a += g.edge_sigma[e] * band_integral(E, X0, Y0, w, h);
    }
    const double f = a / (w * h);
    return fmin(fmax(f, 0.0), 1.0);
}

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
                           unsigned long long *__restrict__ eps_minus, double *__restrict__ exp_plus,
                           double *__restrict__ exp_minus) {
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
        double xp = 0.0, xm = 0.0;
        int64_t done = -1;                                   // last column already counted
        for (uint32_t i = b; i < e; ++i) {
            const int64_t lo = max((int64_t)ranges[i].x, done + 1), hi = ranges[i].y;
            for (int64_t x = lo; x <= hi; ++x) {
                while (s < se && (int64_t)g.spans[s].w <= x) ++s;       // spans are sorted, disjoint
                const bool in = s < se && (int64_t)g.spans[s].z <= x;
                const uint32_t cnt = row[x];
                if (in) ep += cnt; else em += cnt;
                if (exp_plus && cnt) {
                    const double f = area_fraction(g, P, x, r);
                    if (in) xp += (1.0 - f) * cnt; else xm += f * cnt;
                }
            }
            done = max(done, hi);
        }
        if (ep) atomicAdd(&eps_plus[P], ep);
        if (em) atomicAdd(&eps_minus[P], em);
        if (xp != 0.0) atomicAdd(&exp_plus[P], xp);
        if (xm != 0.0) atomicAdd(&exp_minus[P], xm);
    }
}

}  // namespace

rj_status ring_sigma_impl(Ctx *c, uint32_t n_poly, uint32_t n_ring) {
    if (!n_ring) return RJ_OK;
    k_ring_sigma<<<blocks_for(n_ring, 128), 128, 0, c->stream>>>(
        c->edges.as<int4>(), c->poly_ring_off.as<uint32_t>(), c->ring_edge_off.as<uint32_t>(), n_poly, n_ring,
        c->edge_sigma.as<int8_t>());
    RJ_LAUNCHED(c);
    RJ_CUDA(c, cudaGetLastError());
    return RJ_OK;
}

rj_status interval_impl(Ctx *c, int W, int H, const PolyPass &pp, const uint32_t *canvas,
                        unsigned long long *d_eps_plus, unsigned long long *d_eps_minus, double *d_exp_plus,
                        double *d_exp_minus) {
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
    if (d_exp_plus) {
        RJ_CUDA(c, cudaMemsetAsync(d_exp_plus, 0, (size_t)np * 8, st));
        RJ_CUDA(c, cudaMemsetAsync(d_exp_minus, 0, (size_t)np * 8, st));
    }
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
    g.poly_edge_off = c->poly_edge_off.as<uint32_t>();
    g.edge_sigma = c->edge_sigma.as<int8_t>();
    if (NR) {
        const unsigned gr = (unsigned)std::min<uint64_t>(blocks_for(NR, 256), c->num_sms * 8ull);
        k_bkt_count<<<gr, 256, 0, st>>>(g, (uint32_t)NR, kc.as<uint32_t>());
        RJ_LAUNCHED(c);
        RJ_CUDA(c, scan_u32(c, kc.as<uint32_t>(), ko.as<uint32_t>(), NB, kWsScan));
        k_bkt_fill<<<gr, 256, 0, st>>>(g, (uint32_t)NR, ko.as<uint32_t>(), kcur.as<uint32_t>(), rg.as<uint2>());
        RJ_LAUNCHED(c);
        const unsigned gb = (unsigned)std::min<uint64_t>(blocks_for(NB, 128), c->num_sms * 16ull);
        k_bkt_eval<<<gb, 128, 0, st>>>(g, NB, ko.as<uint32_t>(), rg.as<uint2>(), d_eps_plus, d_eps_minus,
                                        d_exp_plus, d_exp_minus);
        RJ_LAUNCHED(c);
    }
    RJ_CUDA(c, cudaGetLastError());
    return RJ_OK;
}

}  // namespace rj
