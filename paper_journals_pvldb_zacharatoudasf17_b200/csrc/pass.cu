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
// points are sorted by Morton key at load time, so the points of a level-L
// lattice cell are contiguous and project into a small pixel tile (~16-33
// pixels a side) -- one tile per warp, in shared memory.  Each warp pulls
// work items (a run of light cells, or one chunk of a heavy cell) from a
// global counter and, per cell:
//   1. clears its tile (count u32 [+ sum f64]);
//   2. streams the cell's columns with 256-bit non-allocating loads (8 points
//      per lane, next window prefetched), filters, projects to pixels
//      (pix = umulhi(q, 4W)), reduces runs of equal pixels across the warp
//      (Morton order makes dense pixels arrive as runs) and adds each run to
//      the tile with one shared-memory atomic;  accurate mode: points in
//      boundary pixels go to a per-warp queue and are tested 32 at a time
//      (one per lane) against the edge grid (Proc. JoinPoint);
//   3. row-prefixes the tile (one lane per row, odd row stride);
//   4. for every span piece of the cell (polygon P, row, [lo, hi)) adds
//      prefix[hi-1] - prefix[lo-1] to A[P]: an O(1) scanline span sum (S4).
// There is no __syncthreads in the work loop.  Per-polygon partials
// accumulate per CTA in shared memory and are flushed once with 64-bit
// global reductions.  Linearity of the sums makes the per-cell partial tiles
// add up to the full canvas exactly.
#include <algorithm>

#include "rj_internal.cuh"

namespace rj {

namespace {
constexpr int kThreads = 256;
constexpr int kWarps = kThreads / 32;
constexpr int kIPL = 8;                      // points per lane per window (256-bit loads)
constexpr int kWin = 32 * kIPL;              // 256 points per warp window
constexpr int kQ = 64;                       // per-warp boundary queue capacity (drained at >= 32)
constexpr uint32_t kNoKey = 0xFFFFFFFFu;
constexpr unsigned kFull = 0xFFFFFFFFu;
constexpr uint32_t kFlag = 0x80000000u;
constexpr int kMaxTileW = 33;                // widest tile row of the chosen cell levels
constexpr int kMaxStages = 4;

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

__device__ __forceinline__ double attr_val(uint32_t bits, int is_float) {
    return is_float ? (double)__uint_as_float(bits) : (double)(int32_t)bits;
}

template <int NS> struct Win {
    uint32_t x[kIPL], y[kIPL];
    uint32_t v[NS > 0 ? NS : 1][kIPL];
};

template <int NS>
__device__ __forceinline__ void load_win(Win<NS> &w, const PassArgs &a, uint32_t base) {
    const V8 X = ld_stream8(a.qx + base), Y = ld_stream8(a.qy + base);
#pragma unroll
    for (int j = 0; j < kIPL; ++j) { w.x[j] = X.v[j]; w.y[j] = Y.v[j]; }
#pragma unroll
    for (int s = 0; s < NS; ++s) {
        const V8 C = ld_stream8(a.col[s] + base);
#pragma unroll
        for (int j = 0; j < kIPL; ++j) w.v[s][j] = C.v[j];
    }
}

// per-warp view of one cell's tile
struct Tile {
    uint32_t *cnt;
    double *sum;
    uint32_t base;         // r0 * stride + c0: key = py * stride + px - base
    uint32_t stride, tw, th;
};

struct Shared {
    uint32_t *pcnt;        // CTA partials [n_poly]
    double *psum;
    uint32_t *qx, *qy, *qa;  // this warp's boundary queue [kQ]
};

template <bool SUM>
__device__ __forceinline__ void emit_poly(const PassArgs &a, const Shared &sh, uint32_t P, uint32_t cnt, double s) {
    if (a.smem_partials) {
        atomicAdd(&sh.pcnt[P], cnt);
        if (SUM) atomicAdd(&sh.psum[P], s);
    } else {
        atomicAdd(&a.A_cnt[P], (unsigned long long)cnt);
        if (SUM) atomicAdd(&a.A_sum[P], s);
    }
}

// Proc. JoinPoint: exact even-odd test of lattice point (px, py)
// against every polygon through the edge-grid cell; each containing polygon
// gets (1, v).  Cell entries are sorted by edge id, so they group by polygon.
template <bool SUM>
__device__ __forceinline__ void join_point(const PassArgs &a, const Shared &sh, uint32_t px, uint32_t py, double v) {
    const uint32_t cell = (py >> kGridShift) * kGrid + (px >> kGridShift);
    const uint32_t b = __ldg(&a.grid_off[cell]), e = __ldg(&a.grid_off[cell + 1]);
    uint32_t cur = kNoKey, par = 0;
    const int64_t X = px, Y = py;
    for (uint32_t k = b; k < e; ++k) {
        const uint32_t ed = __ldg(&a.grid_ent[k]);
        const uint32_t P = __ldg(&a.edge_poly[ed]);
        if (P != cur) {
            if (par) emit_poly<SUM>(a, sh, cur, 1u, v);
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
    if (par) emit_poly<SUM>(a, sh, cur, 1u, v);
}

template <bool SUM>
__device__ __forceinline__ void drain_queue(const PassArgs &a, const Shared &sh, uint32_t &qn, bool all) {
    const int lane = threadIdx.x & 31;
    while (qn >= 32 || (all && qn > 0)) {
        __syncwarp();
        const uint32_t take = qn >= 32 ? 32u : qn;
        if ((uint32_t)lane < take) {
            const uint32_t pos = qn - take + lane;
            const uint32_t x = sh.qx[pos], y = sh.qy[pos], ab = sh.qa[pos];
            join_point<SUM>(a, sh, x, y, SUM ? attr_val(ab, a.f.agg_is_float) : 0.0);
        }
        __syncwarp();
        qn -= take;
    }
}

// Per-query constants held in registers by every warp.
template <int NS>
struct Consts {
    uint32_t ilo[NS > 0 ? NS : 1], span[NS > 0 ? NS : 1];   // int ranges: (v - ilo) <= span
    uint32_t W4, H4;                                        // pix(q) = umulhi(q, 4W)
};

// Opaque to the optimiser (keeps the compiler from folding the tile offset
// into a 64-bit IMAD.HI addend).
__device__ __forceinline__ uint32_t mulhi(uint32_t a, uint32_t b) {
    uint32_t r;
    asm("mul.hi.u32 %0, %1, %2;" : "=r"(r) : "r"(a), "r"(b));
    return r;
}
// shared-memory add of v at byte address addr, skipped when v == 0
__device__ __forceinline__ void red_add_nz(uint32_t addr, uint32_t v) {
    asm volatile("{\n\t.reg .pred p;\n\tsetp.ne.u32 p, %1, 0;\n\t@p red.shared.add.u32 [%0], %1;\n\t}"
                 :: "r"(addr), "r"(v) : "memory");
}
// ... and only when `when` != 0 (branch-free: one predicated RED)
__device__ __forceinline__ void red_add_nz_if(uint32_t addr, uint32_t v, uint32_t when) {
    asm volatile("{\n\t.reg .pred p, q;\n\tsetp.ne.u32 p, %1, 0;\n\tsetp.ne.and.u32 q, %2, 0, p;\n\t"
                 "@q red.shared.add.u32 [%0], %1;\n\t}"
                 :: "r"(addr), "r"(v), "r"(when) : "memory");
}
__device__ __forceinline__ uint32_t atom_add(uint32_t addr, uint32_t v) {
    uint32_t old;
    asm volatile("atom.shared.add.u32 %0, [%1], %2;" : "=r"(old) : "r"(addr), "r"(v) : "memory");
    return old;
}

template <int NS, bool FP>
__device__ __forceinline__ bool pass_point(const PassArgs &a, const Consts<NS> &k, const Win<NS> &w, int j) {
    bool ok = true;
#pragma unroll
    for (int q = 0; q < NS; ++q) ok &= (w.v[q][j] - k.ilo[q]) <= k.span[q];
    if (FP) {
#pragma unroll
        for (int p = 0; p < RJ_MAX_PRED; ++p) {
            if (p < a.f.n_fpred) {
                uint32_t bits = 0;
#pragma unroll
                for (int q = 0; q < NS; ++q)
                    if (q == a.f.f_slot[p]) bits = w.v[q][j];
                ok &= cmp_f(__uint_as_float(bits), a.f.f_op[p], a.f.f_val[p]);
            }
        }
    }
    return ok;
}

template <int NS>
__device__ __forceinline__ double agg_of(const PassArgs &a, const Win<NS> &w, int j) {
    uint32_t ab = 0;
#pragma unroll
    for (int q = 0; q < NS; ++q)
        if (q == a.f.agg_slot) ab = w.v[q][j];
    return attr_val(ab, a.f.agg_is_float);
}

template <bool SUM, int NS>
__device__ __forceinline__ void enqueue(const PassArgs &a, const Shared &sh, const Win<NS> &w, int j, bool bnd,
                                        uint32_t &qn, uint32_t &n_bnd) {
    const unsigned bb = __ballot_sync(kFull, bnd);
    if (bb) {
        const int lane = threadIdx.x & 31;
        if (bnd) {
            const uint32_t pos = qn + __popc(bb & ((1u << lane) - 1u));
            sh.qx[pos] = w.x[j];
            sh.qy[pos] = w.y[j];
            uint32_t ab = 0;
            if (SUM) {
#pragma unroll
                for (int q = 0; q < NS; ++q)
                    if (q == a.f.agg_slot) ab = w.v[q][j];
            }
            sh.qa[pos] = ab;
            ++n_bnd;
        }
        qn += __popc(bb);
    }
}

template <bool SUM>
__device__ __forceinline__ void emit_run(const Tile &t, uint32_t tbase, uint32_t key, uint32_t cnt, double sum,
                                         bool when) {
    red_add_nz_if(tbase + key * 4u, cnt, when ? 1u : 0u);
    if (SUM && when && cnt) atomicAdd(&t.sum[key - t.base], sum);
}

// Process one window of kIPL points per lane (`on`: the lane holds points).
// Morton order makes points of one pixel arrive as runs, inside a lane and
// across lanes.  Runs inside a lane are merged in registers; runs crossing
// lane boundaries are merged by a warp segmented scan, so each run costs
// one shared reduction (same-address atomics from many lanes would
// serialise).  Accurate mode: boundary pixels carry kFlag in the tile; their
// points skip the tile and go to the warp queue for the exact test.
// tbase = shared byte address of tile word 0 minus 4 * (r0 * stride + c0).
template <bool SUM, bool ACC, int NS, bool FP>
__device__ __forceinline__ void process(const PassArgs &a, const Shared &sh, const Tile &t, const Consts<NS> &k,
                                        const Win<NS> &w, uint32_t first, uint32_t count, uint32_t tbase,
                                        uint32_t &qn, uint32_t &n_pass, uint32_t &n_bnd) {
    // point j of this lane is active iff (lane index + j - first) < count
    const int lane = threadIdx.x & 31;
    bool ok[kIPL];
    uint32_t key[kIPL];
#pragma unroll
    for (int j = 0; j < kIPL; ++j) {
        ok[j] = ((uint32_t)(lane * kIPL + j) - first) < count && pass_point<NS, FP>(a, k, w, j);
        key[j] = mulhi(w.y[j], k.H4) * t.stride + mulhi(w.x[j], k.W4);
        n_pass += ok[j] ? 1u : 0u;
    }
    if (ACC) {
        uint32_t bm = 0;
#pragma unroll
        for (int j = 0; j < kIPL; ++j) {
            if (ok[j]) {
                uint32_t v;
                asm volatile("ld.shared.u32 %0, [%1];" : "=r"(v) : "r"(tbase + key[j] * 4u) : "memory");
                if (v & kFlag) bm |= 1u << j;
            }
        }
        if (__any_sync(kFull, bm != 0u)) {
#pragma unroll
            for (int j = 0; j < kIPL; ++j) {
                enqueue<SUM, NS>(a, sh, w, j, (bm >> j) & 1u, qn, n_bnd);   // adds <= 32
                drain_queue<SUM>(a, sh, qn, false);                          // leaves < 32
            }
#pragma unroll
            for (int j = 0; j < kIPL; ++j) ok[j] = ok[j] && !((bm >> j) & 1u);
        }
    }
    const uint32_t kprev = __shfl_up_sync(kFull, key[kIPL - 1], 1);
    const uint32_t knext = __shfl_down_sync(kFull, key[0], 1);
    const bool cin = lane > 0 && key[0] == kprev;           // first run may continue from lane - 1
    const bool cout = lane < 31 && key[kIPL - 1] == knext;  // last run continues into lane + 1
    // phase 1: runs closed inside the lane are added now, except the first
    // one when it continues from the previous lane (it needs the carry)
    uint32_t run = 0, fcnt = 0, fkey = 0;
    double dsum = 0.0, fsum = 0.0;
    bool seen = false;                                      // an internal run end was passed
#pragma unroll
    for (int j = 0; j + 1 < kIPL; ++j) {
        run += ok[j] ? 1u : 0u;
        if (SUM && ok[j]) dsum += agg_of<NS>(a, w, j);
        const bool tail = key[j + 1] != key[j];
        const bool defer = tail && !seen && cin;
        if (defer) { fcnt = run; fsum = dsum; fkey = key[j]; }
        emit_run<SUM>(t, tbase, key[j], run, dsum, tail && !defer);
        seen = seen || tail;
        run = tail ? 0u : run;
        if (SUM) dsum = tail ? 0.0 : dsum;
    }
    run += ok[kIPL - 1] ? 1u : 0u;
    if (SUM && ok[kIPL - 1]) dsum += agg_of<NS>(a, w, kIPL - 1);
    // phase 2: segmented scan of the last runs' partials across lanes
    const bool starts = seen || !cin;                        // this lane's last run starts here
    uint32_t packed = run | (starts ? kFlag : 0u);
    double dv = SUM ? dsum : 0.0;
#pragma unroll
    for (int dd = 1; dd < 32; dd <<= 1) {
        const uint32_t o = __shfl_up_sync(kFull, packed, dd);
        double od = 0.0;
        if (SUM) od = __shfl_up_sync(kFull, dv, dd);
        if (lane >= dd && !(packed & kFlag)) {
            packed = (packed + (o & ~kFlag)) | (o & kFlag);
            if (SUM) dv += od;
        }
    }
    const uint32_t pre = __shfl_up_sync(kFull, packed, 1) & ~kFlag;    // carry into this lane
    double dpre = 0.0;
    if (SUM) dpre = __shfl_up_sync(kFull, dv, 1);
    // phase 3: the deferred first run and the last run (unless it continues)
    if (cin && seen) emit_run<SUM>(t, tbase, fkey, fcnt + pre, fsum + dpre, true);
    const bool add_pre = cin && !seen;
    emit_run<SUM>(t, tbase, key[kIPL - 1], run + (add_pre ? pre : 0u), dsum + (add_pre ? dpre : 0.0), !cout);
}

// ---------------------------------------------------------------- pipeline
// mbarrier / bulk-copy primitives (PTX ISA: mbarrier, cp.async.bulk)
__device__ __forceinline__ void mbar_init(uint32_t bar, uint32_t count) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" :: "r"(bar), "r"(count) : "memory");
}
__device__ __forceinline__ void mbar_expect_tx(uint32_t bar, uint32_t bytes) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" :: "r"(bar), "r"(bytes) : "memory");
}
__device__ __forceinline__ void mbar_arrive(uint32_t bar) {
    asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" :: "r"(bar) : "memory");
}
__device__ __forceinline__ void mbar_wait(uint32_t bar, uint32_t parity) {
    asm volatile("{\n\t.reg .pred p;\n"
                 "WAIT_%=:\n\t"
                 "mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n\t"
                 "@!p bra WAIT_%=;\n\t}"
                 :: "r"(bar), "r"(parity) : "memory");
}
__device__ __forceinline__ void bulk_g2s(uint32_t dst, const void *src, uint32_t bytes, uint32_t bar,
                                         uint64_t policy) {
    asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes.L2::cache_hint"
                 " [%0], [%1], %2, [%3], %4;"
                 :: "r"(dst), "l"(src), "r"(bytes), "r"(bar), "l"(policy) : "memory");
}
__device__ __forceinline__ void consumers_sync() {      // named barrier: the 8 consumer warps only
    asm volatile("bar.sync 1, %0;" :: "n"(kThreads) : "memory");
}

constexpr int kStagePts = kWarps * kWin;     // 2048 points per stage: one window per consumer warp
constexpr uint32_t kDone = 0xFFFFFFFFu;

// Stage descriptor written by the producer before it arms the stage.
struct StageMeta {
    uint32_t cell;     // level-L cell (kDone: no more work)
    uint32_t sb, se;   // points [sb, se) of the cell processed from this stage
    uint32_t cb;       // first point copied (sb rounded down to 4: 16-B aligned)
    uint32_t flags;    // bit 0: first stage of the cell, bit 1: last stage of the cell
};

template <int NS>
__device__ __forceinline__ void load_win_smem(Win<NS> &w, const uint32_t *stage, uint32_t off) {
    // stage = [col][kStagePts] u32; off is a multiple of 8 points (32 B)
    const uint4 *px = reinterpret_cast<const uint4 *>(stage + off);
    const uint4 *py = reinterpret_cast<const uint4 *>(stage + kStagePts + off);
    uint4 a0 = px[0], a1 = px[1], b0 = py[0], b1 = py[1];
    w.x[0] = a0.x; w.x[1] = a0.y; w.x[2] = a0.z; w.x[3] = a0.w; w.x[4] = a1.x; w.x[5] = a1.y; w.x[6] = a1.z; w.x[7] = a1.w;
    w.y[0] = b0.x; w.y[1] = b0.y; w.y[2] = b0.z; w.y[3] = b0.w; w.y[4] = b1.x; w.y[5] = b1.y; w.y[6] = b1.z; w.y[7] = b1.w;
#pragma unroll
    for (int q = 0; q < NS; ++q) {
        const uint4 *pc = reinterpret_cast<const uint4 *>(stage + (2 + q) * kStagePts + off);
        const uint4 c0 = pc[0], c1 = pc[1];
        w.v[q][0] = c0.x; w.v[q][1] = c0.y; w.v[q][2] = c0.z; w.v[q][3] = c0.w;
        w.v[q][4] = c1.x; w.v[q][5] = c1.y; w.v[q][6] = c1.z; w.v[q][7] = c1.w;
    }
}

// Block = 8 consumer warps + 1 producer warp.  The producer streams the
// points of its CTA's work items, cell by cell, into a ring of shared-memory
// stages with bulk async copies (TMA engine, mbarrier completion); the
// consumers process each stage (one 256-point window per warp) into the
// cell's tile, and at a cell's last stage row-prefix the tile and reduce
// its span pieces.  The copy engine keeps streaming during those phases.
template <bool SUM, bool ACC, int NS, bool FP>
__global__ void __launch_bounds__(kThreads + 32, 1) k_point_pass(const PassArgs a) {
    extern __shared__ __align__(128) unsigned char smem_raw[];
    __shared__ __align__(8) uint64_t s_full[kMaxStages], s_empty[kMaxStages];
    __shared__ StageMeta s_meta[kMaxStages];
    __shared__ uint32_t s_pass, s_bnd;
    const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5;
    const uint32_t nstage = a.n_stages;
    const int ncol = 2 + NS;
    // carve: [ring stages][tile sums f64][partial sums f64][tile counts u32][partial counts u32][queues]
    unsigned char *p = smem_raw;
    uint32_t *ring = reinterpret_cast<uint32_t *>(p);
    p += (size_t)nstage * ncol * kStagePts * 4;
    double *tsum = reinterpret_cast<double *>(p);          // [2][tile_cap]: tiles alternate per cell
    if (SUM) p += sizeof(double) * a.tile_cap * 2;
    Shared sh;
    sh.psum = reinterpret_cast<double *>(p);
    if (SUM && a.smem_partials) p += sizeof(double) * a.n_poly;
    uint32_t *tcnt = reinterpret_cast<uint32_t *>(p);
    p += sizeof(uint32_t) * a.tile_cap * 2;
    sh.pcnt = reinterpret_cast<uint32_t *>(p);
    if (a.smem_partials) p += sizeof(uint32_t) * a.n_poly;
    uint32_t *q = reinterpret_cast<uint32_t *>(p) + (wid < kWarps ? wid : 0) * 3 * kQ;
    sh.qx = q;
    sh.qy = q + kQ;
    sh.qa = q + 2 * kQ;

    if (threadIdx.x == 0) {
        for (uint32_t st = 0; st < nstage; ++st) {
            mbar_init((uint32_t)__cvta_generic_to_shared(&s_full[st]), 1);
            mbar_init((uint32_t)__cvta_generic_to_shared(&s_empty[st]), kWarps);
        }
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
        s_pass = 0;
        s_bnd = 0;
    }
    if (a.smem_partials)
        for (uint32_t k = threadIdx.x; k < a.n_poly; k += blockDim.x) {
            sh.pcnt[k] = 0;
            if (SUM) sh.psum[k] = 0.0;
        }
    __syncthreads();

    const int L = a.level, s_lat = kLatticeBits - L, sh2 = 2 * (kMaxLevel - L);

    if (wid == kWarps) {
        // ================================================= producer warp
        if (lane == 0) {
            uint64_t policy;
            asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(policy));
            const uint32_t *src[2 + 6] = {a.qx, a.qy, a.col[0], a.col[1], a.col[2], a.col[3], a.col[4], a.col[5]};
            uint32_t st = 0, ph = 0;
            for (;;) {
                const uint32_t it = atomicAdd(a.work_counter, 1u);
                if (it >= a.n_items) break;
                const int4 I = a.items[it];
                for (uint32_t c = (uint32_t)I.x; c < (uint32_t)I.y; ++c) {
                    const uint32_t b = max((uint32_t)I.z, a.cell_off10[(uint64_t)c << sh2]);
                    const uint32_t e = min((uint32_t)I.w, a.cell_off10[(uint64_t)(c + 1) << sh2]);
                    if (b >= e) continue;
                    for (uint32_t sb = b; sb < e;) {
                        const uint32_t cb = sb & ~3u;
                        const uint32_t ce = min((e + 3u) & ~3u, cb + (uint32_t)kStagePts);
                        const uint32_t se = min(e, ce);
                        mbar_wait((uint32_t)__cvta_generic_to_shared(&s_empty[st]), ph ^ 1u);
                        s_meta[st] = StageMeta{c, sb, se, cb, (sb == b ? 1u : 0u) | (se == e ? 2u : 0u)};
                        const uint32_t full = (uint32_t)__cvta_generic_to_shared(&s_full[st]);
                        const uint32_t bytes = (ce - cb) * 4u;
                        mbar_expect_tx(full, bytes * ncol);
                        const uint32_t dst = (uint32_t)__cvta_generic_to_shared(ring + (size_t)st * ncol * kStagePts);
                        for (int cc = 0; cc < ncol; ++cc)
                            bulk_g2s(dst + cc * kStagePts * 4, src[cc] + cb, bytes, full, policy);
                        sb = se;
                        if (++st == nstage) { st = 0; ph ^= 1u; }
                    }
                }
            }
            mbar_wait((uint32_t)__cvta_generic_to_shared(&s_empty[st]), ph ^ 1u);
            s_meta[st].cell = kDone;
            mbar_arrive((uint32_t)__cvta_generic_to_shared(&s_full[st]));
        }
    } else {
        // ================================================= consumer warps
        Consts<NS> k;
#pragma unroll
        for (int qq = 0; qq < NS; ++qq) {
            k.ilo[qq] = (uint32_t)a.f.ilo[qq];
            k.span[qq] = (uint32_t)a.f.ihi[qq] - (uint32_t)a.f.ilo[qq];
        }
        k.W4 = (uint32_t)a.W << 2;
        k.H4 = (uint32_t)a.H << 2;
        const bool never = a.f.never != 0;
        Tile t;
        t.stride = a.tile_stride;
        uint32_t tbase = 0, c0 = 0, r0 = 0, tsel = 0, pb = 0, pe = 0;
        uint2 pc0 = make_uint2(0u, 0u);
        uint32_t n_pass = 0, n_bnd = 0, qn = 0;
        uint32_t st = 0, ph = 0;
        for (;;) {
            mbar_wait((uint32_t)__cvta_generic_to_shared(&s_full[st]), ph);
            const StageMeta m = s_meta[st];
            if (m.cell == kDone) break;
            if (m.flags & 1u) {                           // first stage of a cell: set up its tile
                // the two tiles alternate between consecutive cells, so the
                // previous cell's span reads never race with this clear
                t.cnt = tcnt + tsel * a.tile_cap;
                t.sum = tsum + tsel * a.tile_cap;
                tsel ^= 1u;
                pb = __ldg(&a.piece_off[m.cell]);          // consumed at the cell's last stage
                pe = __ldg(&a.piece_off[m.cell + 1]);
                const int64_t cx = cell_x(m.cell), cy = cell_y(m.cell);
                c0 = (uint32_t)pix(cx << s_lat, a.W);
                r0 = (uint32_t)pix(cy << s_lat, a.H);
                t.tw = (uint32_t)pix(((cx + 1) << s_lat) - 1, a.W) - c0 + 1;
                t.th = (uint32_t)pix(((cy + 1) << s_lat) - 1, a.H) - r0 + 1;
                t.base = r0 * t.stride + c0;
                tbase = (uint32_t)__cvta_generic_to_shared(t.cnt) - 4u * t.base;
                const uint32_t words = t.th * t.stride;
                for (uint32_t i = threadIdx.x; i < words; i += kThreads) {
                    uint32_t v = 0u;
                    if (ACC) {
                        const uint32_t r = i / t.stride, x = i - r * t.stride;
                        if (x < t.tw) {
                            const uint32_t px = c0 + x;
                            v = ((__ldg(&a.mask[(uint64_t)(r0 + r) * a.mask_wpr + (px >> 5)]) >> (px & 31)) & 1u) ? kFlag
                                                                                                             : 0u;
                        }
                    }
                    t.cnt[i] = v;
                    if (SUM) t.sum[i] = 0.0;
                }
                consumers_sync();
            }
            if ((m.flags & 2u) && pb + threadIdx.x < pe) pc0 = __ldg(&a.pieces[pb + threadIdx.x]);  // in flight
            // ---- this warp's window of the stage
            const uint32_t woff = (uint32_t)wid * kWin;                 // window offset in the stage
            const uint32_t ncopy = ((m.se + 3u) & ~3u) - m.cb;
            if (woff < ncopy && !never) {
                Win<NS> w;
                load_win_smem<NS>(w, ring + (size_t)st * ncol * kStagePts, woff + lane * kIPL);
                // active points: stage index in [sb - cb, se - cb)
                const uint32_t first = (m.sb - m.cb) - woff;   // may wrap: handled as unsigned range
                const uint32_t count = m.se - m.sb;
                process<SUM, ACC, NS, FP>(a, sh, t, k, w, first, count, tbase, qn, n_pass, n_bnd);
            }
            __syncwarp();
            if (lane == 0) mbar_arrive((uint32_t)__cvta_generic_to_shared(&s_empty[st]));
            if (m.flags & 2u) {                           // last stage of the cell: reduce the tile
                if (ACC) drain_queue<SUM>(a, sh, qn, true);
                consumers_sync();                          // every point of the cell is in the tile
                // span pieces (S4): each thread sums its pieces' pixels straight
                // from the tile (<= 33 words each), no separate prefix phase
                for (uint32_t kk = pb + threadIdx.x; kk < pe; kk += kThreads) {
                    const uint2 pc = (kk == pb + threadIdx.x) ? pc0 : __ldg(&a.pieces[kk]);
                    const uint32_t lr = pc.y & 255u, lo = (pc.y >> 8) & 255u, hi = pc.y >> 16;
                    const uint32_t *rc = t.cnt + lr * t.stride;
                    uint32_t cnt = 0;
                    for (uint32_t i = lo; i < hi; ++i) cnt += rc[i];
                    // boundary pixels hold only kFlag (2^31): their sum only
                    // touches bit 31, and a piece's count is < 2^31
                    if (ACC) cnt &= ~kFlag;
                    if (cnt) {
                        double sm = 0.0;
                        if (SUM) {
                            const double *rs = t.sum + lr * t.stride;
                            for (uint32_t i = lo; i < hi; ++i) sm += rs[i];
                        }
                        emit_poly<SUM>(a, sh, pc.x, cnt, sm);
                    }
                }
            }
            if (++st == nstage) { st = 0; ph ^= 1u; }
        }
        for (int o = 16; o; o >>= 1) {
            n_pass += __shfl_xor_sync(kFull, n_pass, o);
            if (ACC) n_bnd += __shfl_xor_sync(kFull, n_bnd, o);
        }
        if (lane == 0) {
            atomicAdd(&s_pass, n_pass);
            if (ACC) atomicAdd(&s_bnd, n_bnd);
        }
    }
    __syncthreads();
    if (a.smem_partials)
        for (uint32_t kk = threadIdx.x; kk < a.n_poly; kk += blockDim.x) {
            const uint32_t cc = sh.pcnt[kk];
            if (cc) {
                atomicAdd(&a.A_cnt[kk], (unsigned long long)cc);
                if (SUM) atomicAdd(&a.A_sum[kk], sh.psum[kk]);
            }
        }
    if (threadIdx.x == 0) {
        atomicAdd(&a.stats[0], (unsigned long long)s_pass);
        if (ACC) atomicAdd(&a.stats[1], (unsigned long long)s_bnd);
    }
}

template <bool SUM, bool ACC, bool FP>
void *select_ns(int ns) {
    switch (ns) {
    case 0: return (void *)k_point_pass<SUM, ACC, 0, FP>;
    case 1: return (void *)k_point_pass<SUM, ACC, 1, FP>;
    case 2: return (void *)k_point_pass<SUM, ACC, 2, FP>;
    case 3: return (void *)k_point_pass<SUM, ACC, 3, FP>;
    case 4: return (void *)k_point_pass<SUM, ACC, 4, FP>;
    case 5: return (void *)k_point_pass<SUM, ACC, 5, FP>;
    default: return (void *)k_point_pass<SUM, ACC, 6, FP>;
    }
}

void *select_kernel(bool sum, bool acc, int ns, bool fp) {
    if (sum) {
        if (acc) return fp ? select_ns<true, true, true>(ns) : select_ns<true, true, false>(ns);
        return fp ? select_ns<true, false, true>(ns) : select_ns<true, false, false>(ns);
    }
    if (acc) return fp ? select_ns<false, true, true>(ns) : select_ns<false, true, false>(ns);
    return fp ? select_ns<false, false, true>(ns) : select_ns<false, false, false>(ns);
}
}  // namespace

size_t point_pass_smem(const PassArgs &a, bool sum, bool accurate) {
    size_t b = (size_t)a.n_stages * (2 + a.f.n_slots) * kStagePts * 4;
    b += (size_t)a.tile_cap * 2 * (4 + (sum ? 8 : 0));
    if (a.smem_partials) b += (size_t)a.n_poly * (4 + (sum ? 8 : 0));
    if (accurate) b += (size_t)3 * kWarps * kQ * 4;
    return b;
}

int point_pass_stages(int n_slots) { return (2 + n_slots) <= 4 ? 3 : 2; }

rj_status point_pass(Ctx *c, const PassArgs &a_in, bool sum, bool accurate) {
    void *k = select_kernel(sum, accurate, a_in.f.n_slots, a_in.f.n_fpred > 0);
    // ring depth: the deepest ring that keeps two CTAs (16 consumer warps) per
    // SM, else the deepest that fits one CTA
    PassArgs a = a_in;
    const size_t budget = 227 * 1024 - 1024;
    int best = 0, best_score = -1;
    for (int st = 2; st <= kMaxStages; ++st) {
        a.n_stages = st;
        const size_t need = point_pass_smem(a, sum, accurate) + 2048;
        const int ctas = (int)std::min<size_t>(2, (228 * 1024) / (need + 1024));
        if (need > budget || ctas < 1) continue;
        const int score = ctas * 8 + st;
        if (score > best_score) { best_score = score; best = st; }
    }
    if (!best) return set_error(c, RJ_ERR_RESOLUTION, "point-pass tiles do not fit in shared memory");
    a.n_stages = best;
    const size_t smem = point_pass_smem(a, sum, accurate);
    RJ_CUDA(c, cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
    int per_sm = 0;
    RJ_CUDA(c, cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k, kThreads + 32, smem));
    if (per_sm < 1) return set_error(c, RJ_ERR_RESOLUTION, "point-pass tiles do not fit in shared memory");
    const unsigned grid = (unsigned)std::max<uint64_t>(
        1, std::min<uint64_t>((uint64_t)per_sm * c->num_sms, std::max<uint32_t>(1, a.n_items)));
    void *args[] = {(void *)&a};
    RJ_CUDA(c, cudaLaunchKernel(k, dim3(grid), dim3(kThreads + 32), args, smem, c->stream));
    c->last_stages = best;
    c->last_ctas_per_sm = per_sm;
    RJ_LAUNCHED(c);
    return RJ_OK;
}

}  // namespace rj
