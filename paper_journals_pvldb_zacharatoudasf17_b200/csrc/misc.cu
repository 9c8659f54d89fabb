// misc.cu -- S8 finalisation (AVG = SUM / COUNT) and the
// per-point membership diagnostic used by the parity tests.
#include <algorithm>

#include "rj_internal.cuh"

namespace rj {

namespace {
__global__ void k_finalize(int agg, uint32_t n, const unsigned long long *__restrict__ cnt,
                           const double *__restrict__ sum, double *__restrict__ val) {
    pdl_wait();
    pdl_trigger();
    const uint32_t i = blockIdx.x * blockDim.x + threadIdx.x;
    if (i >= n) return;
    if (agg == RJ_AVG) val[i] = cnt[i] ? __ddiv_rn(sum[i], (double)cnt[i]) : __longlong_as_double(0x7ff8000000000000ll);
    else if (agg == RJ_SUM) val[i] = sum[i];
    else val[i] = (double)cnt[i];
}

// Per-query reset before the point pass (one PDL-chained kernel instead of
// four memset nodes): work counters and statistics, the boundary queue's
// valid mark (all ones), the per-polygon partials.
__global__ void k_pass_init(uint32_t *__restrict__ work, unsigned long long *__restrict__ cnt, double *__restrict__ sum,
                            uint32_t n) {
    pdl_wait();
    pdl_trigger();
    const uint32_t t0 = blockIdx.x * blockDim.x + threadIdx.x, ts = gridDim.x * blockDim.x;
    if (t0 < 16) work[t0] = t0 == 9 ? 0xFFFFFFFFu : 0u;
    for (uint32_t i = t0; i < n; i += ts) {
        cnt[i] = 0ull;
        if (sum) sum[i] = 0.0;
    }
}

// Multi-GPU combine (S8): counts and sums in one binary64 buffer, so one
// all-reduce combines both (counts are exact in binary64 below 2^53).
__global__ void k_pack(uint32_t n, const unsigned long long *__restrict__ cnt, const double *__restrict__ sum,
                       double *__restrict__ out) {
    const uint32_t i = blockIdx.x * blockDim.x + threadIdx.x;
    if (i >= n) return;
    out[i] = (double)cnt[i];
    out[n + i] = sum ? sum[i] : 0.0;
}

__global__ void k_finalize_packed(int agg, uint32_t n, const double *__restrict__ in,
                                  unsigned long long *__restrict__ cnt, double *__restrict__ val) {
    const uint32_t i = blockIdx.x * blockDim.x + threadIdx.x;
    if (i >= n) return;
    const unsigned long long c = (unsigned long long)in[i];
    const double s = in[n + i];
    cnt[i] = c;
    if (agg == RJ_AVG) val[i] = c ? __ddiv_rn(s, (double)c) : __longlong_as_double(0x7ff8000000000000ll);
    else if (agg == RJ_SUM) val[i] = s;
    else val[i] = (double)c;
}

__device__ __forceinline__ bool filter_point(const PassArgs &a, uint64_t i) {
    const Filter &f = a.f;
    if (f.never) return false;
    for (int s = 0; s < f.n_irange; ++s) {
        const int32_t v = (int32_t)a.col[s][i];
        if (v < f.ilo[s] || v > f.ihi[s]) return false;
    }
    for (int p = 0; p < f.n_fpred; ++p) {
        const float v = __uint_as_float(a.col[f.f_slot[p]][i]);
        const float c = f.f_val[p];
        bool ok;
        switch (f.f_op[p]) {
        case RJ_LT: ok = v < c; break;
        case RJ_LE: ok = v <= c; break;
        case RJ_GT: ok = v > c; break;
        case RJ_GE: ok = v >= c; break;
        default: ok = v == c;
        }
        if (!ok) return false;
    }
    return true;
}

// One thread per (sorted) point: membership from the same structures the
// fused pass uses -- the cell's span pieces (pixel-centre rule) and, for
// boundary pixels in accurate mode, the edge-grid PIP.
__global__ void k_membership(const PassArgs a, uint64_t n, int accurate, const uint32_t *__restrict__ idx,
                             unsigned long long *__restrict__ bits) {
    for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n; i += (uint64_t)gridDim.x * blockDim.x) {
        const uint32_t qx = a.qx[i], qy = a.qy[i];
        unsigned long long m = 0;
        const int64_t px = pix(qx, a.W), py = pix(qy, a.H);
        const bool in_view = px >= a.view[0] && px < a.view[2] && py >= a.view[1] && py < a.view[3];
        if (in_view && filter_point(a, i)) {
            bool bnd = false;
            if (accurate) bnd = a.index_join || ((a.mask[(uint64_t)py * a.mask_wpr + (px >> 5)] >> (px & 31)) & 1u);
            if (bnd) {
                const uint32_t cell = (qy >> kGridShift) * kGrid + (qx >> kGridShift);
                uint32_t cur = 0xFFFFFFFFu, par = 0;
                for (uint32_t k = a.grid_off[cell]; k < a.grid_off[cell + 1]; ++k) {
                    const uint32_t ed = a.grid_ent[k] & 0x7FFFFFFFu, P = a.edge_poly[ed];
                    const uint32_t left = a.grid_ent[k] >> 31;   // leftward ray: complement test
                    if (P != cur) {
                        if (par && cur < 64) m |= 1ull << cur;
                        cur = P;
                        par = 0;
                    }
                    const int4 E = a.edges[ed];
                    if ((E.y > (int)qy) != (E.w > (int)qy)) {
                        const int64_t lhs = ((int64_t)qx - E.x) * (int64_t)(E.w - E.y);
                        const int64_t rhs = (int64_t)(E.z - E.x) * ((int64_t)qy - E.y);
                        if (E.w > E.y ? lhs < rhs : lhs > rhs) par ^= 1u ^ left;
                        else par ^= left;
                    }
                }
                if (par && cur < 64) m |= 1ull << cur;
            } else {
                const uint32_t cell = cell_of(qx, qy, a.level);
                const int64_t cc = cell_x(cell), cr = cell_y(cell);
                const int64_t lx = px - cell_pix_lo(cc, a.W, a.level), ly = py - cell_pix_lo(cr, a.H, a.level);
                for (uint32_t k = a.piece_off[cell]; k < a.piece_off[cell + 1]; ++k) {
                    const uint2 pc = a.pieces[k];
                    const int64_t lr = pc.y & 255u, lo = (pc.y >> 8) & 255u, hi = pc.y >> 16;
                    if (lr == ly && lo <= lx && lx < hi && pc.x < 64) m |= 1ull << pc.x;
                }
            }
        }
        bits[idx[i]] = m;
    }
}
}  // namespace

cudaError_t launch_finalize(Ctx *c, int agg, uint32_t n, const unsigned long long *cnt, const double *sum,
                            double *val) {
    if (!n) return cudaSuccess;
    const cudaError_t e = launch_pdl(c, k_finalize, dim3(blocks_for(n, 256)), dim3(256), 0, agg, n, cnt, sum, val);
    RJ_LAUNCHED(c);
    return e;
}

cudaError_t launch_pass_init(Ctx *c, uint32_t *work, unsigned long long *cnt, double *sum, uint32_t n) {
    const unsigned g = std::max(1u, std::min(blocks_for(n, 256), (unsigned)c->num_sms));
    const cudaError_t e = launch_pdl(c, k_pass_init, dim3(g), dim3(256), 0, work, cnt, sum, n);
    RJ_LAUNCHED(c);
    return e;
}

cudaError_t launch_pack(Ctx *c, uint32_t n, const unsigned long long *cnt, const double *sum, double *out) {
    if (!n) return cudaSuccess;
    k_pack<<<blocks_for(n, 256), 256, 0, c->stream>>>(n, cnt, sum, out);
    RJ_LAUNCHED(c);
    return cudaGetLastError();
}

cudaError_t launch_finalize_packed(Ctx *c, int agg, uint32_t n, const double *in, unsigned long long *cnt,
                                   double *val) {
    if (!n) return cudaSuccess;
    k_finalize_packed<<<blocks_for(n, 256), 256, 0, c->stream>>>(agg, n, in, cnt, val);
    RJ_LAUNCHED(c);
    return cudaGetLastError();
}

cudaError_t launch_membership(Ctx *c, const PassArgs &a, bool accurate, unsigned long long *bits) {
    if (!c->n_pts) return cudaSuccess;
    const unsigned g = (unsigned)std::min<uint64_t>(blocks_for(c->n_pts, 256), (uint64_t)c->num_sms * 8);
    k_membership<<<g, 256, 0, c->stream>>>(a, c->n_pts, accurate ? 1 : 0, c->idx.as<uint32_t>(), bits);
    RJ_LAUNCHED(c);
    return cudaGetLastError();
}

}  // namespace rj
