// pass.cu -- the fused point pass (S2 / S7 + S4), one persistent kernel,
// canvas tiles of per-pixel partial aggregates.  (pass_label.cu holds the
// label variant used for bounded SUM/AVG; point_pass() below picks.)
//
// Paper: Proc. DrawPoints adds every point into the pixel it
// projects to; Proc. DrawPolygons then adds each polygon
// fragment's pixel value into A[i].  Accurate mode (Procs. AccuratePoints /
// JoinPoint / AccuratePolygons) sends the points of boundary
// pixels to an exact point-in-polygon test and leaves those pixels empty.
// Filters are evaluated per point before projection.
//
// B200 design: the canvas never exists in HBM.
// Points are sorted by Morton key at load time, so the points of a level-L
// lattice cell (~32 pixels a side at the query's resolution) are
// contiguous and project into a small pixel tile in shared memory.  Per CTA:
//   * producer warp (pass_common.cuh produce()): streams the CTA's work
//     items, cell by cell, into a ring of shared-memory stages with bulk
//     async copies (TMA engine, cp.async.bulk, L2 evict-first) completing
//     on mbarriers -- the stream keeps flowing during the per-cell phases;
//   * 8 consumer warps, per cell:
//       1. clear the tile (accurate mode: boundary pixels carry kFlag);
//       2. per stage, one 256-point window per warp (8 points per lane):
//          filter, project (pix = umulhi(q, 4W)), merge runs of equal pixels
//          (Morton order: inside a lane in registers -- process_lane_runs,
//          the default; or also across lanes with a warp segmented scan --
//          process, RJ_OPT_LANE_RUNS = 2) and add each run with one shared
//          reduction; accurate mode: boundary points go to the global queue
//          (k_pip_queue tests them after the pass);
//       3. at the cell's last stage, every span piece (polygon P, row,
//          [lo, hi)) sums its pixels straight from the tile into P's
//          per-CTA partial (S4).
// Tiles alternate between consecutive cells (two CTA barriers per cell).
// Linearity of the sums makes the per-cell partial tiles add up to the
// full canvas exactly.  Per-CTA partials are flushed once with 64-bit
// global reductions.
#include <algorithm>

#include "pass_common.cuh"

namespace rj {

rj_status point_pass_label(Ctx *c, const PassArgs &a, bool accurate);   // pass_label.cu
size_t point_pass_label_smem(const PassArgs &a, bool accurate);

namespace {
using namespace pass;

// per-cell view of the CTA's pixel tile
struct Tile {
    uint32_t *cnt;
    double *sum;
    uint32_t base;         // r0 * stride + c0
    uint32_t tbase;        // shared byte address of word 0 minus 4 * base
    uint32_t stride, tw, th;
};

template <bool SUM>
__device__ __forceinline__ void emit_pixel_run(const Tile &t, uint32_t key, uint32_t cnt, double sum, bool when) {
    RJ_DCHECK(!(when && cnt) || (key - t.base < t.th * t.stride && (key - t.base) % t.stride < t.tw));
    red_add_if(t.tbase + key * 4u, cnt, when ? 1u : 0u);
    if (SUM && when && cnt) atomicAdd(&t.sum[key - t.base], sum);
}

// One 256-point window: point j of this lane is active iff
// (lane*8 + j - first) < count.  Runs of equal pixels inside the lane are
// merged in registers; runs crossing lane boundaries by a warp segmented
// scan, so each run costs one shared reduction (same-address atomics from
// many lanes would serialise).  Accurate mode: boundary pixels carry kFlag;
// their points skip the tile and go to the warp queue.
template <bool SUM, bool ACC, int NS, bool FP>
__device__ __forceinline__ void process(const PassArgs &a, const Shared &sh, const Tile &t, const Consts<NS> &k,
                                        const Win<NS> &w, const uint32_t *sp, uint32_t first, uint32_t count,
                                        BQ &bq, uint32_t &n_pass, uint32_t &n_bnd) {
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
            if (ok[j]) RJ_DCHECK(key[j] - t.base < t.th * t.stride && (key[j] - t.base) % t.stride < t.tw);
            if (ok[j] && (lds(t.tbase + key[j] * 4u) & kFlag)) bm |= 1u << j;
        }
        if (__any_sync(kFull, bm != 0u)) {
            enqueue_window<SUM>(a, sh, sp, kStagePts, bm, bq, n_bnd);
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
        if (SUM && ok[j]) dsum += attr_val(agg_bits<NS>(a, w, j), a.f.agg_is_float);
        const bool tail = key[j + 1] != key[j];
        const bool defer = tail && !seen && cin;
        if (defer) { fcnt = run; fsum = dsum; fkey = key[j]; }
        emit_pixel_run<SUM>(t, key[j], run, dsum, tail && !defer);
        seen = seen || tail;
        run = tail ? 0u : run;
        if (SUM) dsum = tail ? 0.0 : dsum;
    }
    run += ok[kIPL - 1] ? 1u : 0u;
    if (SUM && ok[kIPL - 1]) dsum += attr_val(agg_bits<NS>(a, w, kIPL - 1), a.f.agg_is_float);
    // phase 2: carry of runs crossing lanes; phase 3: the deferred first run
    // and the last run (unless it continues into the next lane)
    uint32_t pre;
    double dpre;
    run_carry<SUM>(run, dsum, seen || !cin, pre, dpre);
    if (cin && seen) emit_pixel_run<SUM>(t, fkey, fcnt + pre, fsum + dpre, true);
    const bool add_pre = cin && !seen;
    emit_pixel_run<SUM>(t, key[kIPL - 1], run + (add_pre ? pre : 0u), dsum + (add_pre ? dpre : 0.0), !cout);
}

// COUNT window with runs merged inside each lane only: a run of equal pixels
// among a lane's 8 Morton-consecutive points takes one shared reduction; a
// run crossing lanes takes one per lane.  Cheaper than process()'s warp
// segmented scan at every canvas size measured on B200 (r2 sweep: C2
// 1.93 -> 1.66 ms, C5 32768^2 2.95 -> 2.25 ms, C5 1024^2 1.70 -> 1.25 ms):
// the few extra same-address shared reductions of hot pixels cost less than
// the scan's shuffles in every window.  Accurate mode: boundary points go to
// the queue first, as in process().
template <bool ACC, int NS, bool FP>
__device__ __forceinline__ void process_lane_runs(const PassArgs &a, const Shared &sh, const Tile &t,
                                                  const Consts<NS> &k, const Win<NS> &w, const uint32_t *sp,
                                                  uint32_t first, uint32_t count, BQ &bq, uint32_t &n_pass,
                                                  uint32_t &n_bnd) {
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
            if (ok[j]) RJ_DCHECK(key[j] - t.base < t.th * t.stride && (key[j] - t.base) % t.stride < t.tw);
            if (ok[j] && (lds(t.tbase + key[j] * 4u) & kFlag)) bm |= 1u << j;
        }
        if (__any_sync(kFull, bm != 0u)) {
            enqueue_window<false>(a, sh, sp, kStagePts, bm, bq, n_bnd);
#pragma unroll
            for (int j = 0; j < kIPL; ++j) ok[j] = ok[j] && !((bm >> j) & 1u);
        }
    }
    uint32_t run = 0;
#pragma unroll
    for (int j = 0; j + 1 < kIPL; ++j) {
        run += ok[j] ? 1u : 0u;
        const bool tail = key[j + 1] != key[j];
        emit_pixel_run<false>(t, key[j], run, 0.0, tail);
        run = tail ? 0u : run;
    }
    run += ok[kIPL - 1] ? 1u : 0u;
    emit_pixel_run<false>(t, key[kIPL - 1], run, 0.0, true);
}

// Result intervals: add the cell's per-pixel filtered counts to the global
// count canvas (a heavy cell split over several work items adds partials).
__device__ __forceinline__ void dump_canvas(const PassArgs &a, const Tile &t, uint32_t cell, int s_lat) {
    const int64_t cx = cell_x(cell), cy = cell_y(cell);
    const uint32_t c0 = (uint32_t)pix(cx << s_lat, a.W), r0 = (uint32_t)pix(cy << s_lat, a.H);
    for (uint32_t i = threadIdx.x; i < t.th * t.stride; i += kThreads) {
        const uint32_t r = i / t.stride, x = i - r * t.stride;
        const uint32_t v = t.cnt[i] & ~kFlag;
        if (x < t.tw && v) atomicAdd(&a.canvas[(uint64_t)(r0 + r) * a.W + c0 + x], v);
    }
}

template <bool SUM, bool ACC, int NS, bool FP>
__global__ void __maxnreg__(96) k_point_pass(const __grid_constant__ PassArgs a) {
    extern __shared__ __align__(128) unsigned char smem_raw[];
    __shared__ __align__(8) Ring rg;
    __shared__ uint32_t s_pass, s_bnd;
    const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5;
    const uint32_t nstage = a.n_stages;
    const int ncol = 2 + NS;
    // carve: [ring][tile sums f64 x2][tile counts u32 x2][partial counts u32][queues]
    unsigned char *p = smem_raw;
    uint32_t *ring = reinterpret_cast<uint32_t *>(p);
    p += ring_bytes(nstage, NS);
    double *tsum = reinterpret_cast<double *>(p);
    if (SUM) p += sizeof(double) * a.tile_cap * 2;
    Shared sh;
    sh.psum = nullptr;                                      // fp64 sums reduce in global memory
    uint32_t *tcnt = reinterpret_cast<uint32_t *>(p);
    p += sizeof(uint32_t) * a.tile_cap * 2;
    sh.pcnt = reinterpret_cast<uint32_t *>(p);
    if (a.smem_partials) p += sizeof(uint32_t) * a.n_poly;
    uint32_t *q = reinterpret_cast<uint32_t *>(p) + (wid < kWarps ? wid : 0) * 3 * kQ;
    sh.qx = q;
    sh.qy = q + kQ;
    sh.qa = q + 2 * kQ;

    if (threadIdx.x == 0) {
        ring_init(rg, nstage);
        s_pass = 0;
        s_bnd = 0;
    }
    if (a.smem_partials)
        for (uint32_t kk = threadIdx.x; kk < a.n_poly; kk += blockDim.x) {
            sh.pcnt[kk] = 0;
        }
    // everything above is CTA-local setup; the work counter, the polygon
    // pass's pieces and the partial vectors are the predecessors' output.
    // early_stream: the work counter was zeroed before the polygon pass, so
    // the producer streams at once while the last polygon kernel finishes;
    // only the consumers wait for the pieces
    if (!a.early_stream) pdl_wait();
    pdl_trigger();
    __syncthreads();

    if (wid == kWarps) {
        if (lane == 0) produce(a, rg, ring, nstage, ncol);
        __syncwarp();                                      // reconverge before the CTA barrier
    } else {
        if (a.early_stream) pdl_wait();
        const Consts<NS> k = make_consts<NS>(a);
        const int s_lat = kLatticeBits - a.level;
        const bool never = a.f.never != 0;
        Tile t;
        t.stride = a.tile_stride;
        uint32_t tsel = 0, pb = 0, pe = 0;
        uint32_t n_pass = 0, n_bnd = 0;
        BQ bq = bq_init(a);
        uint32_t st = 0, ph = 0;
        for (;;) {
            mbar_wait(smem_u32(&rg.full[st]), ph);
            const StageMeta m = rg.meta[st];
            if (m.cell == kDone) break;
            if (m.flags & 1u) {
                // ---- first stage of a cell: clear its tile.  Tiles alternate
                // between consecutive cells, so this never races with the
                // previous cell's span reads.
                t.cnt = tcnt + tsel * a.tile_cap;
                t.sum = tsum + tsel * a.tile_cap;
                tsel ^= 1u;
                pb = pe = 0u;                              // consumed at the cell's last stage
                if (!ACC || !a.index_join) {
                    pb = __ldg(&a.piece_off[m.cell]);
                    pe = __ldg(&a.piece_off[m.cell + 1]);
                }
                const int64_t cx = cell_x(m.cell), cy = cell_y(m.cell);
                const uint32_t c0 = (uint32_t)pix(cx << s_lat, a.W), r0 = (uint32_t)pix(cy << s_lat, a.H);
                t.tw = (uint32_t)pix(((cx + 1) << s_lat) - 1, a.W) - c0 + 1;
                t.th = (uint32_t)pix(((cy + 1) << s_lat) - 1, a.H) - r0 + 1;
                t.base = r0 * t.stride + c0;
                t.tbase = smem_u32(t.cnt) - 4u * t.base;
                const uint32_t words = t.th * t.stride;
                if (ACC) {
                    clear_tile_acc(t.cnt, t.stride, t.th, t.tw, r0, c0, a.index_join, kFlag, 0u, a.view);
                } else {
                    fill_tile(t.cnt, words, 0u);
                }
                if (SUM)
                    for (uint32_t i = threadIdx.x; i < words; i += kThreads) t.sum[i] = 0.0;
                consumers_sync();
                if (ACC && !a.index_join) {
                    // flag the cell's boundary pixels (cell-uniform branch: the barrier is safe)
                    const uint32_t bb = __ldg(&a.bpiece_off[m.cell]), be = __ldg(&a.bpiece_off[m.cell + 1]);
                    if (bb < be) {
                        paint_bnd(t.cnt, t.stride, a.bpieces, bb, be, kFlag);
                        consumers_sync();
                    }
                }
            }
            uint2 pc0 = make_uint2(0u, 0u);
            if ((m.flags & 2u) && pb + threadIdx.x < pe) pc0 = __ldg(&a.pieces[pb + threadIdx.x]);  // in flight
            // ---- this warp's window of the stage
            const uint32_t woff = (uint32_t)wid * kWin;
            const uint32_t ncopy = ((m.se + 3u) & ~3u) - m.cb;
            if (woff < ncopy && !never) {
                Win<NS> w;
                const uint32_t *sp = ring + (size_t)st * ncol * kStagePts + woff + lane * kIPL;
                load_win_smem<NS>(w, sp, 0);
                const uint32_t first = (m.sb - m.cb) - woff;    // may wrap: unsigned range test
                if (!SUM && a.lane_runs)
                    process_lane_runs<ACC, NS, FP>(a, sh, t, k, w, sp, first, m.se - m.sb, bq, n_pass, n_bnd);
                else
                    process<SUM, ACC, NS, FP>(a, sh, t, k, w, sp, first, m.se - m.sb, bq, n_pass, n_bnd);
            }
            stage_release(smem_u32(&rg.empty[st]));
            if (m.flags & 2u) {
                // ---- last stage of the cell: reduce the tile over the span pieces (S4)
                consumers_sync();                          // every point of the cell is in the tile
                if (a.canvas) dump_canvas(a, t, m.cell, s_lat);
                if (ACC && a.bnd_bits)
                    dump_bnd(a, t.cnt, t.stride, t.th, t.tw, (uint32_t)pix(cell_y(m.cell) << s_lat, a.H),
                             (uint32_t)pix(cell_x(m.cell) << s_lat, a.W), kFlag, kFlag);
                for (uint32_t kk = pb + threadIdx.x; kk < pe; kk += kThreads) {
                    const uint2 pc = (kk == pb + threadIdx.x) ? pc0 : __ldg(&a.pieces[kk]);
                    const uint32_t lr = pc.y & 255u, lo = (pc.y >> 8) & 255u, hi = pc.y >> 16;
                    RJ_DCHECK(lr < t.th && lo < hi && hi <= t.tw);
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
        if (ACC) bq_finish<SUM>(a, sh, bq);                 // boundary points are independent of the tiles
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
            if (cc) atomicAdd(&a.A_cnt[kk], (unsigned long long)cc);
        }
    if (threadIdx.x == 0) {
        atomicAdd(&a.stats[0], (unsigned long long)s_pass);
        if (ACC) atomicAdd(&a.stats[1], (unsigned long long)s_bnd);
    }
}

// Accurate mode, after the point pass: the exact test (Proc. JoinPoint,
// P:718-726) of every queued boundary point, one per thread, at full
// occupancy.  The queue holds the points in the order the consumer warps met
// them -- batches of 32 from one cell, Morton-ordered -- so neighbouring
// threads walk the same grid cells (L1 hits) and mostly land in the same
// polygon (one partial update per distinct polygon of a warp).
template <bool SUM>
__global__ void __launch_bounds__(256) k_pip_queue(const __grid_constant__ PassArgs a) {
    extern __shared__ __align__(16) unsigned char smem_raw[];
    Shared sh{};
    sh.pcnt = reinterpret_cast<uint32_t *>(smem_raw);
    if (a.smem_partials)
        for (uint32_t k = threadIdx.x; k < a.n_poly; k += blockDim.x) sh.pcnt[k] = 0;
    pdl_wait();
    pdl_trigger();
    __syncthreads();
    const uint32_t n = min(*a.bq_count, *a.bq_valid);
    const int lane = threadIdx.x & 31;
    const uint32_t step = gridDim.x * blockDim.x;
    for (uint32_t base = blockIdx.x * blockDim.x + (threadIdx.x & ~31u); base < n; base += step) {
        const uint32_t i = base + lane;
        uint32_t P = kNoPoly;
        double v = 0.0;
        const uint32_t x = i < n ? __ldcs(&a.bq_x[i]) : kDone;
        if (x != kDone) {                                   // kDone: padding of a chunk
            const uint32_t y = __ldcs(&a.bq_y[i]);
            if (SUM) v = attr_val(__ldcs(&a.bq_a[i]), a.f.agg_is_float);
            P = join_point<SUM>(a, sh, x, y, v);
        }
        unsigned active = __ballot_sync(kFull, P != kNoPoly);
        while (active) {
            const int leader = __ffs(active) - 1;
            const uint32_t PL = __shfl_sync(kFull, P, leader);
            const unsigned m = __ballot_sync(kFull, P == PL);
            double s = (SUM && P == PL) ? v : 0.0;
            if (SUM)
                for (int o = 16; o; o >>= 1) s += __shfl_xor_sync(kFull, s, o);
            if (lane == leader) emit_poly<SUM>(a, sh, PL, __popc(m), s);
            active &= ~m;
        }
    }
    __syncthreads();
    if (a.smem_partials)
        for (uint32_t k = threadIdx.x; k < a.n_poly; k += blockDim.x) {
            const uint32_t cc = sh.pcnt[k];
            if (cc) atomicAdd(&a.A_cnt[k], (unsigned long long)cc);
        }
}

// Diagnostic: the grid entries (edge tests) the exact test of every queued
// boundary point walks -- the cell's list in pip.cuh.
__global__ void k_pip_work(const __grid_constant__ PassArgs a, unsigned long long *out) {
    const uint32_t n = min(*a.bq_count, *a.bq_valid);
    unsigned long long pts = 0, tests = 0;
    for (uint32_t i = blockIdx.x * blockDim.x + threadIdx.x; i < n; i += gridDim.x * blockDim.x) {
        const uint32_t x = a.bq_x[i];
        if (x == kDone) continue;
        const uint32_t y = a.bq_y[i];
        const uint32_t cell = (y >> kGridShift) * kGrid + (x >> kGridShift);
        ++pts;
        tests += a.grid_off[cell + 1] - a.grid_off[cell];
    }
    for (int o = 16; o; o >>= 1) {
        pts += __shfl_xor_sync(kFull, pts, o);
        tests += __shfl_xor_sync(kFull, tests, o);
    }
    if ((threadIdx.x & 31) == 0 && pts) {
        atomicAdd(&out[0], pts);
        atomicAdd(&out[1], tests);
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

size_t tile_pass_smem(const PassArgs &a, bool sum, bool accurate) {
    size_t b = ring_bytes(a.n_stages, a.f.n_slots);
    b += (size_t)a.tile_cap * 2 * (4 + (sum ? 8 : 0));
    if (a.smem_partials) b += (size_t)a.n_poly * 4;
    return b + queue_bytes(accurate);
}
}  // namespace

// Static shared memory of the point-pass kernels (ptxas -v: 256 B) plus margin.
constexpr size_t kStaticSmem = 512;

// Largest ring that keeps two CTAs (16 consumer warps) per SM, else the
// largest that fits one CTA; 0 if nothing fits.
int choose_stages(PassArgs a, size_t (*smem)(const PassArgs &, bool, bool), bool sum, bool accurate, int force) {
    const size_t budget = 227 * 1024 - 1024;
    if (force >= 2 && force <= kMaxStages) {
        a.n_stages = force;
        if (smem(a, sum, accurate) + kStaticSmem <= budget) return force;
    }
    int best = 0, best_score = -1;
    for (int st = 2; st <= kMaxStages; ++st) {
        a.n_stages = st;
        const size_t need = smem(a, sum, accurate) + kStaticSmem;
        if (need > budget) continue;
        const int ctas = (int)std::min<size_t>(2, (228 * 1024) / (need + 1024));
        const int score = ctas * 8 + st;
        if (score > best_score) { best_score = score; best = st; }
    }
    return best;
}

rj_status launch_pass(Ctx *c, void *k, const PassArgs &a, size_t smem) {
    RJ_CUDA(c, cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
    int per_sm = 0;
    RJ_CUDA(c, cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k, kThreads + 32, smem));
    if (per_sm < 1) return set_error(c, RJ_ERR_RESOLUTION, "point-pass tiles do not fit in shared memory");
    const unsigned grid = (unsigned)std::max<uint64_t>(
        1, std::min<uint64_t>((uint64_t)per_sm * c->num_sms, std::max<uint32_t>(1, a.n_items)));
    void *args[] = {(void *)&a};
    RJ_CUDA(c, launch_pdl_ptr(c, k, dim3(grid), dim3(kThreads + 32), smem, args));
    RJ_LAUNCHED(c);
    c->last_stages = (int)a.n_stages;
    c->last_ctas_per_sm = per_sm;
    return RJ_OK;
}

// Kernel choice: COUNT always uses the pixel tile (cheapest per cell); SUM/AVG
// use polygon labels (no per-pixel fp64 shared atomics, which are CAS loops
// on sm_100; measured faster at C3 and C4 in both modes); RJ_OPT_PASS
// overrides.
static bool use_label(const Ctx *c, const PassArgs &a, bool sum, bool accurate) {
    (void)accurate;
    if (!sum || a.canvas) return false;              // the count canvas comes from the pixel tiles
    if (c->pass_variant >= 0) return c->pass_variant == 0;
    return true;
}

size_t point_pass_smem(const Ctx *c, const PassArgs &a, bool sum, bool accurate) {
    return use_label(c, a, sum, accurate) ? point_pass_label_smem(a, accurate) : tile_pass_smem(a, sum, accurate);
}

rj_status pip_queue_pass(Ctx *c, const PassArgs &a_in, bool sum) {
    PassArgs a = a_in;
    a.smem_partials = (size_t)a.n_poly * 4 <= 64 * 1024;
    const size_t smem = a.smem_partials ? (size_t)a.n_poly * 4 : 0;
    void *k = sum ? (void *)k_pip_queue<true> : (void *)k_pip_queue<false>;
    RJ_CUDA(c, cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
    int per_sm = 0;
    RJ_CUDA(c, cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k, 256, smem));
    const unsigned grid = (unsigned)std::max(1, per_sm) * (unsigned)c->num_sms;
    void *args[] = {(void *)&a};
    RJ_CUDA(c, launch_pdl_ptr(c, k, dim3(grid), dim3(256), smem, args));
    RJ_LAUNCHED(c);
    return RJ_OK;
}

rj_status pip_work(Ctx *c, uint64_t *n_points, uint64_t *n_edge_tests) {
    *n_points = *n_edge_tests = 0;
    if (!c->last_bq.bq_cap) return RJ_OK;
    Buf d;
    if (dalloc(c, d, 16)) return set_error(c, RJ_ERR_OOM, "allocation failed");
    RJ_CUDA(c, cudaMemsetAsync(d.p, 0, 16, c->stream));
    k_pip_work<<<c->num_sms * 4, 256, 0, c->stream>>>(c->last_bq, reinterpret_cast<unsigned long long *>(d.p));
    RJ_CUDA(c, cudaGetLastError());
    unsigned long long h[2];
    RJ_CUDA(c, cudaMemcpyAsync(h, d.p, 16, cudaMemcpyDeviceToHost, c->stream));
    RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    dfree(c, d);
    *n_points = h[0];
    *n_edge_tests = h[1];
    return RJ_OK;
}

int point_pass_stages(int n_slots) { return (2 + n_slots) <= 4 ? 3 : 2; }

rj_status point_pass(Ctx *c, const PassArgs &a_in, bool sum, bool accurate) {
    if (use_label(c, a_in, sum, accurate)) return point_pass_label(c, a_in, accurate);
    PassArgs a = a_in;
    a.n_stages = (uint32_t)choose_stages(a, tile_pass_smem, sum, accurate, c->force_stages);
    // a fp64 pixel tile that does not fit (canvases beyond 2^16) -> polygon labels
    if (!a.n_stages && sum && !a.canvas) return point_pass_label(c, a_in, accurate);
    if (!a.n_stages) return set_error(c, RJ_ERR_RESOLUTION, "point-pass tiles do not fit in shared memory");
    return launch_pass(c, select_kernel(sum, accurate, a.f.n_slots, a.f.n_fpred > 0), a,
                       tile_pass_smem(a, sum, accurate));
}

}  // namespace rj
