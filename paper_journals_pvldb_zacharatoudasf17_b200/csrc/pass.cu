// pass.cu -- the fused point pass (S2 / S7 + S4), one persistent kernel.
//
// Paper: Proc. DrawPoints adds every point into the pixel it
// projects to; Proc. DrawPolygons then adds each polygon
// fragment's pixel value into A[i].  Accurate mode (Procs. AccuratePoints /
// JoinPoint / AccuratePolygons) sends the points of boundary
// pixels to an exact point-in-polygon test instead and leaves those pixels
// empty.  Filters are evaluated per point before projection.
//
// B200 design: the canvas never touches HBM.  The
// points are stored sorted by 256x256 lattice cell (load time), so a work
// item = (cell, point range) whose pixels form a small tile (<= 129 x 129)
// that lives in shared memory:
//   1. clear the tile (count u32 [+ sum f64]);
//   2. stream the item's columns with 256-bit non-allocating loads
//      (8 points per lane), filter, project to pixels, reduce runs of equal
//      pixels across the warp (the points are Morton-sorted, so dense pixels
//      arrive as runs) and add each run with one shared-memory atomic;
//      accurate mode: points in boundary pixels go to a per-warp queue and
//      are tested 32 at a time (one point per lane) against the edge grid;
//   3. inclusive row prefix of the tile (in shared memory);
//   4. every span piece of this cell (polygon P, row, [lo, hi)) adds
//      prefix[hi-1] - prefix[lo-1] to A[P] -- an O(1) scanline span sum.
// Per-polygon partials accumulate in shared memory per CTA and are flushed
// once with 64-bit global reductions.  Linearity of the sums makes the
// per-item partial tiles add up to the full canvas exactly.
#include <algorithm>

#include "rj_internal.cuh"

namespace rj {

namespace {
constexpr int kThreads = 256;
constexpr int kWarps = kThreads / 32;
constexpr int kIPL = 8;                      // points per lane per window (256-bit loads)
constexpr int kWin = 32 * kIPL;              // 256 points per warp window
constexpr int kQ = 32 + kWin;                // per-warp boundary queue capacity
constexpr uint32_t kNoKey = 0xFFFFFFFFu;
constexpr unsigned kFull = 0xFFFFFFFFu;

struct V8 { uint32_t v[8]; };

__device__ __forceinline__ V8 ld_stream8(const uint32_t *p) {
    V8 r;
    asm volatile("ld.global.nc.L1::no_allocate.L2::evict_first.v8.b32 {%0,%1,%2,%3,%4,%5,%6,%7}, [%8];"
                 : "=r"(r.v[0]), "=r"(r.v[1]), "=r"(r.v[2]), "=r"(r.v[3]), "=r"(r.v[4]), "=r"(r.v[5]),
                   "=r"(r.v[6]), "=r"(r.v[7])
                 : "l"(p));
    return r;
}

__device__ __forceinline__ bool cmp_f(float v, int op, float c) {
    switch (op) {
    case RJ_LT: return v < c;
    case RJ_LE: return v <= c;
    case RJ_GT: return v > c;
    case RJ_GE: return v >= c;
    default: return v == c;
    }
}

template <int NS>
__device__ __forceinline__ uint32_t slot_val(const uint32_t (&v)[NS > 0 ? NS : 1][kIPL], int s, int j) {
    uint32_t r = 0;
#pragma unroll
    for (int k = 0; k < NS; ++k)
        if (k == s) r = v[k][j];
    return r;
}

template <int NS>
__device__ __forceinline__ bool pass_filter(const Filter &f, const uint32_t (&v)[NS > 0 ? NS : 1][kIPL], int j) {
    bool ok = !f.never;
#pragma unroll
    for (int s = 0; s < NS; ++s)
        if (s < f.n_irange)   // (uint32)(v - lo) <= (uint32)(hi - lo)  <=>  lo <= v <= hi
            ok &= (v[s][j] - (uint32_t)f.ilo[s]) <= (uint32_t)(f.ihi[s] - f.ilo[s]);
    for (int p = 0; p < f.n_fpred; ++p)
        ok &= cmp_f(__uint_as_float(slot_val<NS>(v, f.f_slot[p], j)), f.f_op[p], f.f_val[p]);
    return ok;
}

__device__ __forceinline__ double attr_val(uint32_t bits, int is_float) {
    return is_float ? (double)__uint_as_float(bits) : (double)(int32_t)bits;
}

struct Smem {
    uint32_t *tcnt;
    double *tsum;
    uint32_t *pcnt;
    double *psum;
    uint32_t *qx, *qy, *qa;   // per-warp boundary queues [kWarps][kQ]
};

template <bool SUM>
__device__ __forceinline__ void emit_poly(const PassArgs &a, const Smem &sm, uint32_t P, uint32_t cnt, double s) {
    if (a.smem_partials) {
        atomicAdd(&sm.pcnt[P], cnt);
        if (SUM) atomicAdd(&sm.psum[P], s);
    } else {
        atomicAdd(&a.A_cnt[P], (unsigned long long)cnt);
        if (SUM) atomicAdd(&a.A_sum[P], s);
    }
}

// JoinPoint: exact even-odd test of lattice point (px, py)
// against every polygon through the edge-grid cell; each containing polygon
// gets (1, v).  Entries are sorted by edge id, so edges group by polygon.
template <bool SUM>
__device__ __forceinline__ void join_point(const PassArgs &a, const Smem &sm, uint32_t px, uint32_t py, double v) {
    const uint32_t cell = (py >> kGridShift) * kGrid + (px >> kGridShift);
    const uint32_t b = __ldg(&a.grid_off[cell]), e = __ldg(&a.grid_off[cell + 1]);
    uint32_t cur = kNoKey, par = 0;
    const int64_t X = px, Y = py;
    for (uint32_t k = b; k < e; ++k) {
        const uint32_t ed = __ldg(&a.grid_ent[k]);
        const uint32_t P = __ldg(&a.edge_poly[ed]);
        if (P != cur) {
            if (par) emit_poly<SUM>(a, sm, cur, 1u, v);
            cur = P;
            par = 0;
        }
        const int4 E = __ldg(&a.edges[ed]);
        if ((E.y > (int)py) != (E.w > (int)py)) {
            const int64_t lhs = (X - E.x) * (int64_t)(E.w - E.y);
            const int64_t rhs = (int64_t)(E.z - E.x) * (Y - E.y);
            if (E.w > E.y ? lhs < rhs : lhs > rhs) par ^= 1u;
        }
    }
    if (par) emit_poly<SUM>(a, sm, cur, 1u, v);
}

// Process the <= 8 points a lane holds (act[j] false = no point).
template <bool SUM, bool ACC, int NS>
__device__ __forceinline__ void process_lane(const PassArgs &a, const Smem &sm, uint32_t &qn,
                                             const uint32_t (&qx)[kIPL], const uint32_t (&qy)[kIPL],
                                             const uint32_t (&v)[NS > 0 ? NS : 1][kIPL], const bool (&act)[kIPL],
                                             int64_t c0, int64_t r0, uint32_t tw, uint32_t &n_pass,
                                             uint32_t &n_bnd) {
    const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
    uint32_t key[kIPL], cnt[kIPL];
    double val[kIPL];
#pragma unroll
    for (int j = 0; j < kIPL; ++j) {
        const bool pass = act[j] && pass_filter<NS>(a.f, v, j);
        const uint32_t px = (uint32_t)(((uint64_t)qx[j] * (uint32_t)a.W) >> kLatticeBits);
        const uint32_t py = (uint32_t)(((uint64_t)qy[j] * (uint32_t)a.H) >> kLatticeBits);
        key[j] = act[j] ? (uint32_t)((py - (uint32_t)r0) * tw + (px - (uint32_t)c0)) : kNoKey;
        bool bnd = false;
        if (ACC && pass)
            bnd = (__ldg(&a.mask[(uint64_t)py * a.mask_wpr + (px >> 5)]) >> (px & 31)) & 1u;
        cnt[j] = (pass && !bnd) ? 1u : 0u;
        val[j] = 0.0;
        if (SUM && pass && !bnd) val[j] = attr_val(slot_val<NS>(v, a.f.agg_slot, j), a.f.slot_is_float[a.f.agg_slot]);
        const unsigned bp = __ballot_sync(kFull, pass);
        if (lane == 0) n_pass += __popc(bp);
        if (ACC) {
            const unsigned bb = __ballot_sync(kFull, bnd);
            if (bb) {
                if (lane == 0) n_bnd += __popc(bb);
                if (bnd) {
                    const uint32_t pos = qn + __popc(bb & ((1u << lane) - 1u));
                    sm.qx[w * kQ + pos] = qx[j];
                    sm.qy[w * kQ + pos] = qy[j];
                    sm.qa[w * kQ + pos] = SUM ? slot_val<NS>(v, a.f.agg_slot, j) : 0u;
                }
                qn += __popc(bb);
            }
        }
    }
    // --- warp segmented reduction of equal consecutive keys (run-length add)
    bool head[kIPL];
    const uint32_t kprev = __shfl_up_sync(kFull, key[kIPL - 1], 1);
    head[0] = lane == 0 || key[0] != kprev;
#pragma unroll
    for (int j = 1; j < kIPL; ++j) head[j] = key[j] != key[j - 1];
    uint32_t s[kIPL];
    double d[kIPL];
    bool anyh = head[0];
    s[0] = cnt[0];
    d[0] = val[0];
#pragma unroll
    for (int j = 1; j < kIPL; ++j) {
        s[j] = head[j] ? cnt[j] : s[j - 1] + cnt[j];
        if (SUM) d[j] = head[j] ? val[j] : d[j - 1] + val[j];
        anyh |= head[j];
    }
    uint32_t packed = s[kIPL - 1] | (anyh ? 0x80000000u : 0u);
    double dv = SUM ? d[kIPL - 1] : 0.0;
#pragma unroll
    for (int dd = 1; dd < 32; dd <<= 1) {
        const uint32_t o = __shfl_up_sync(kFull, packed, dd);
        double od = 0.0;
        if (SUM) od = __shfl_up_sync(kFull, dv, dd);
        if (lane >= dd && !(packed & 0x80000000u)) {
            packed = (packed + (o & 0x7FFFFFFFu)) | (o & 0x80000000u);
            if (SUM) dv += od;
        }
    }
    uint32_t pre = __shfl_up_sync(kFull, packed, 1) & 0x7FFFFFFFu;
    double dpre = 0.0;
    if (SUM) dpre = __shfl_up_sync(kFull, dv, 1);
    if (lane == 0) { pre = 0; dpre = 0.0; }
    const uint32_t knext = __shfl_down_sync(kFull, key[0], 1);
    bool seen = false;
#pragma unroll
    for (int j = 0; j < kIPL; ++j) {
        seen |= head[j];
        const uint32_t t = s[j] + (seen ? 0u : pre);
        const bool tail = (j + 1 < kIPL) ? head[j + 1] : (lane == 31 || key[j] != knext);
        if (tail && t && key[j] != kNoKey) {
            atomicAdd(&sm.tcnt[key[j]], t);
            if (SUM) atomicAdd(&sm.tsum[key[j]], d[j] + (seen ? 0.0 : dpre));
        }
    }
    // --- accurate: test queued boundary points, one per lane
    if (ACC) {
        while (qn >= 32) {
            __syncwarp();
            const uint32_t pos = qn - 32 + lane;
            const uint32_t x = sm.qx[w * kQ + pos], y = sm.qy[w * kQ + pos], ab = sm.qa[w * kQ + pos];
            __syncwarp();
            join_point<SUM>(a, sm, x, y, SUM ? attr_val(ab, a.f.slot_is_float[a.f.agg_slot]) : 0.0);
            qn -= 32;
        }
    }
}

template <bool SUM, bool ACC, int NS>
__global__ void __launch_bounds__(kThreads) k_point_pass(const PassArgs a) {
    extern __shared__ __align__(16) unsigned char smem_raw[];
    __shared__ int4 s_item;
    __shared__ uint32_t s_pass, s_bnd;
    const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
    // carve shared memory: [tsum f64][psum f64][tcnt u32][pcnt u32][queues]
    Smem sm;
    unsigned char *p = smem_raw;
    sm.tsum = reinterpret_cast<double *>(p);
    if (SUM) p += sizeof(double) * a.tile_cap;
    sm.psum = reinterpret_cast<double *>(p);
    if (SUM && a.smem_partials) p += sizeof(double) * a.n_poly;
    sm.tcnt = reinterpret_cast<uint32_t *>(p);
    p += sizeof(uint32_t) * a.tile_cap;
    sm.pcnt = reinterpret_cast<uint32_t *>(p);
    if (a.smem_partials) p += sizeof(uint32_t) * a.n_poly;
    sm.qx = reinterpret_cast<uint32_t *>(p);
    sm.qy = sm.qx + kWarps * kQ;
    sm.qa = sm.qy + kWarps * kQ;

    if (a.smem_partials)
        for (uint32_t k = threadIdx.x; k < a.n_poly; k += kThreads) {
            sm.pcnt[k] = 0;
            if (SUM) sm.psum[k] = 0.0;
        }
    if (threadIdx.x == 0) { s_pass = 0; s_bnd = 0; }
    uint32_t n_pass = 0, n_bnd = 0, qn = 0;

    for (;;) {
        if (threadIdx.x == 0) {
            const uint32_t it = atomicAdd(a.work_counter, 1u);
            s_item = it < a.n_items ? a.items[it] : make_int4(-1, 0, 0, 0);
        }
        __syncthreads();
        const int4 item = s_item;
        if (item.x < 0) break;
        const uint32_t cell = (uint32_t)item.x;
        const int64_t cc = cell_x(cell), cr = cell_y(cell);
        const int64_t c0 = cell_pix_lo(cc, a.W), r0 = cell_pix_lo(cr, a.H);
        const uint32_t tw = (uint32_t)(cell_pix_hi(cc, a.W) - c0 + 1);
        const uint32_t th = (uint32_t)(cell_pix_hi(cr, a.H) - r0 + 1);
        const uint32_t npx = tw * th;
        for (uint32_t k = threadIdx.x; k < npx; k += kThreads) {
            sm.tcnt[k] = 0;
            if (SUM) sm.tsum[k] = 0.0;
        }
        __syncthreads();

        // ---- stream the item's points [b, e)
        const uint32_t b = (uint32_t)item.y, e = (uint32_t)item.z;
        const uint32_t b8 = (b + 7u) & ~7u, e8 = e & ~7u;
        const bool body = b8 < e8;
        const uint32_t he = body ? b8 : e;           // head [b, he), tail [te, e)
        const uint32_t te = body ? e8 : e;
        if (w == 0) {                                // head and tail (<= 14 points), one per lane
            const uint32_t nh = he - b, nt = e - te;
            uint32_t qxv[kIPL], qyv[kIPL], vv[NS > 0 ? NS : 1][kIPL];
            bool act[kIPL];
            const uint32_t i = lane < nh ? b + lane : te + (lane - nh);
            const bool on = lane < nh + nt;
#pragma unroll
            for (int j = 0; j < kIPL; ++j) {
                act[j] = (j == 0) && on;
                qxv[j] = act[j] ? a.qx[i] : 0u;
                qyv[j] = act[j] ? a.qy[i] : 0u;
#pragma unroll
                for (int s = 0; s < NS; ++s) vv[s][j] = act[j] ? a.col[s][i] : 0u;
            }
            process_lane<SUM, ACC, NS>(a, sm, qn, qxv, qyv, vv, act, c0, r0, tw, n_pass, n_bnd);
        }
        if (body) {
            const uint32_t nwin = (e8 - b8 + kWin - 1) / kWin;
            for (uint32_t wi = w; wi < nwin; wi += kWarps) {
                const uint32_t base = b8 + wi * kWin + lane * kIPL;
                const bool on = base < e8;
                uint32_t qxv[kIPL], qyv[kIPL], vv[NS > 0 ? NS : 1][kIPL];
                bool act[kIPL];
                if (on) {
                    const V8 X = ld_stream8(a.qx + base), Y = ld_stream8(a.qy + base);
#pragma unroll
                    for (int j = 0; j < kIPL; ++j) { qxv[j] = X.v[j]; qyv[j] = Y.v[j]; }
#pragma unroll
                    for (int s = 0; s < NS; ++s) {
                        const V8 C = ld_stream8(a.col[s] + base);
#pragma unroll
                        for (int j = 0; j < kIPL; ++j) vv[s][j] = C.v[j];
                    }
                } else {
#pragma unroll
                    for (int j = 0; j < kIPL; ++j) {
                        qxv[j] = qyv[j] = 0u;
#pragma unroll
                        for (int s = 0; s < NS; ++s) vv[s][j] = 0u;
                    }
                }
#pragma unroll
                for (int j = 0; j < kIPL; ++j) act[j] = on;
                process_lane<SUM, ACC, NS>(a, sm, qn, qxv, qyv, vv, act, c0, r0, tw, n_pass, n_bnd);
            }
        }
        if (ACC && qn) {                              // drain this warp's queue
            __syncwarp();
            if ((uint32_t)lane < qn) {
                const uint32_t x = sm.qx[w * kQ + lane], y = sm.qy[w * kQ + lane], ab = sm.qa[w * kQ + lane];
                join_point<SUM>(a, sm, x, y, SUM ? attr_val(ab, a.f.slot_is_float[a.f.agg_slot]) : 0.0);
            }
            __syncwarp();
            qn = 0;
        }
        __syncthreads();

        // ---- inclusive row prefix of the tile (one warp per row)
        for (uint32_t row = w; row < th; row += kWarps) {
            uint32_t carry = 0;
            double dcarry = 0.0;
            uint32_t *rc = sm.tcnt + row * tw;
            double *rs = sm.tsum + row * tw;
            for (uint32_t x0 = 0; x0 < tw; x0 += 32) {
                const uint32_t i = x0 + lane;
                uint32_t v = i < tw ? rc[i] : 0u;
                double dv = (SUM && i < tw) ? rs[i] : 0.0;
#pragma unroll
                for (int dd = 1; dd < 32; dd <<= 1) {
                    const uint32_t o = __shfl_up_sync(kFull, v, dd);
                    double od = 0.0;
                    if (SUM) od = __shfl_up_sync(kFull, dv, dd);
                    if (lane >= dd) { v += o; if (SUM) dv += od; }
                }
                v += carry;
                if (SUM) dv += dcarry;
                if (i < tw) { rc[i] = v; if (SUM) rs[i] = dv; }
                carry = __shfl_sync(kFull, v, 31);
                if (SUM) dcarry = __shfl_sync(kFull, dv, 31);
            }
        }
        __syncthreads();

        // ---- span pieces of this cell: O(1) prefix differences (S4)
        const uint32_t pb = __ldg(&a.piece_off[cell]), pe = __ldg(&a.piece_off[cell + 1]);
        for (uint32_t k = pb + threadIdx.x; k < pe; k += kThreads) {
            const uint2 pc = __ldg(&a.pieces[k]);
            const uint32_t lr = pc.y & 255u, lo = (pc.y >> 8) & 255u, hi = pc.y >> 16;
            const uint32_t base = lr * tw;
            const uint32_t cnt = sm.tcnt[base + hi - 1] - (lo ? sm.tcnt[base + lo - 1] : 0u);
            if (cnt) {
                double s = 0.0;
                if (SUM) s = sm.tsum[base + hi - 1] - (lo ? sm.tsum[base + lo - 1] : 0.0);
                emit_poly<SUM>(a, sm, pc.x, cnt, s);
            }
        }
        // the next item's __syncthreads (after the fetch) orders these reads
        // before the tile is cleared again
    }

    // ---- flush per-CTA partials and statistics
    atomicAdd(&s_pass, n_pass);
    if (ACC) atomicAdd(&s_bnd, n_bnd);
    __syncthreads();
    if (a.smem_partials)
        for (uint32_t k = threadIdx.x; k < a.n_poly; k += kThreads) {
            const uint32_t c = sm.pcnt[k];
            if (c) {
                atomicAdd(&a.A_cnt[k], (unsigned long long)c);
                if (SUM) atomicAdd(&a.A_sum[k], sm.psum[k]);
            }
        }
    if (threadIdx.x == 0) {
        atomicAdd(&a.stats[0], (unsigned long long)s_pass);
        if (ACC) atomicAdd(&a.stats[1], (unsigned long long)s_bnd);
    }
    (void)lane;
}

template <bool SUM, bool ACC, int NS>
void *kernel_ptr() { return (void *)k_point_pass<SUM, ACC, NS>; }

void *select_kernel(bool sum, bool acc, int ns) {
#define RJ_K(S, A)                                               \
    switch (ns) {                                                \
    case 0: return kernel_ptr<S, A, 0>();                        \
    case 1: return kernel_ptr<S, A, 1>();                        \
    case 2: return kernel_ptr<S, A, 2>();                        \
    case 3: return kernel_ptr<S, A, 3>();                        \
    case 4: return kernel_ptr<S, A, 4>();                        \
    case 5: return kernel_ptr<S, A, 5>();                        \
    default: return kernel_ptr<S, A, 6>();                       \
    }
    if (sum) { if (acc) { RJ_K(true, true) } else { RJ_K(true, false) } }
    else { if (acc) { RJ_K(false, true) } else { RJ_K(false, false) } }
#undef RJ_K
}
}  // namespace

size_t point_pass_smem(const PassArgs &a, bool sum, bool accurate) {
    size_t b = (size_t)a.tile_cap * (4 + (sum ? 8 : 0));
    if (a.smem_partials) b += (size_t)a.n_poly * (4 + (sum ? 8 : 0));
    if (accurate) b += (size_t)3 * kWarps * kQ * 4;
    return b;
}

rj_status point_pass(Ctx *c, const PassArgs &a, bool sum, bool accurate) {
    void *k = select_kernel(sum, accurate, a.f.n_slots);
    const size_t smem = point_pass_smem(a, sum, accurate);
    RJ_CUDA(c, cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
    int per_sm = 0;
    RJ_CUDA(c, cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k, kThreads, smem));
    if (per_sm < 1) return set_error(c, RJ_ERR_RESOLUTION, "point-pass tile does not fit in shared memory");
    const unsigned grid = (unsigned)std::max<uint64_t>(1, std::min<uint64_t>((uint64_t)per_sm * c->num_sms,
                                                                             std::max<uint32_t>(1, a.n_items)));
    void *args[] = {(void *)&a};
    RJ_CUDA(c, cudaLaunchKernel(k, dim3(grid), dim3(kThreads), args, smem, c->stream));
    RJ_LAUNCHED(c);
    return RJ_OK;
}

}  // namespace rj
