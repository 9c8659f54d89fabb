// pass_label.cu -- fused point pass, label variant (SUM / AVG).
//
// A[i] = sum over the fragments of polygon i of the aggregate of its pixels
// (Proc. DrawPolygons).  Swapping the draw order gives the same
// sums: paint every pixel of a cell's tile with the id of the polygon whose
// span piece covers it (S3 pieces; MULTI where pieces of several polygons
// overlap), then give each point the label of its pixel and add (1, attr)
// per label.  Morton order makes equal labels arrive in long runs, so the
// per-polygon partials (count u32, sum f64) take one shared atomic per run
// instead of one fp64 shared CAS loop per pixel run in pass.cu's tile.
// Accurate mode: boundary pixels are labelled BND and their points go to the
// exact test (Proc. JoinPoint) through the per-warp queue.  The stream
// (producer warp, stage ring) is pass_common.cuh's.
#include <algorithm>

#include "pass_common.cuh"

namespace rj {

int choose_stages(PassArgs a, size_t (*smem)(const PassArgs &, bool, bool), bool sum, bool accurate, int force);  // pass.cu
rj_status launch_pass(Ctx *c, void *k, const PassArgs &a, size_t smem);

namespace {
using namespace pass;

constexpr uint32_t kNone = 0xFFFFFFFFu;      // label: no polygon covers the pixel
constexpr uint32_t kMulti = 0xFFFFFFFEu;     // label: several polygons cover the pixel
constexpr uint32_t kBnd = 0xFFFFFFFDu;       // label: boundary pixel (accurate mode)

struct LabTile {
    uint32_t lab_base;       // shared byte address of label word 0 minus 4 * (r0 * stride + c0)
    uint32_t stride, c0, r0;
    uint32_t pb, pe;         // the cell's span pieces
    uint32_t th, tw;         // the cell's pixel rows and columns
};

// Emit a label run (skipped when !when, cnt == 0 or the label is not a polygon).
__device__ __forceinline__ void emit_lab_run(const PassArgs &a, const Shared &sh, uint32_t lab, uint32_t cnt,
                                             double sum, bool when) {
    if (when && lab < kBnd && cnt) emit_poly<true>(a, sh, lab, cnt, sum);
}

// A second polygon claims an already-labelled pixel (accurate mode): turn
// it into MULTI unless a concurrent boundary store made it BND.  Out of line:
// an inlined CAS loop inside the painting loop slows the common path.
__device__ __noinline__ void make_multi(uint32_t *px, uint32_t o) {
    while (o < kBnd) {
        const uint32_t o2 = atomicCAS(px, o, kMulti);
        if (o2 == o) break;
        o = o2;
    }
}

// Points whose pixel several polygons cover: look up every covering piece.
__device__ __noinline__ void multi_point(const PassArgs &a, const Shared &sh, const LabTile &t, uint32_t px,
                                            uint32_t py, double v) {
    const uint32_t lx = px - t.c0, ly = py - t.r0;
    for (uint32_t k = t.pb; k < t.pe; ++k) {
        const uint2 pc = __ldg(&a.pieces[k]);
        const uint32_t lr = pc.y & 255u, lo = (pc.y >> 8) & 255u, hi = pc.y >> 16;
        if (lr == ly && lo <= lx && lx < hi) emit_poly<true>(a, sh, pc.x, 1u, v);
    }
}

// Warp-uniform run carried from window to window: (label, count, sum).
struct Carry {
    uint32_t lab = kNone, cnt = 0;
    double sum = 0.0;
};

// Per-lane partials of the carry's label, filled by windows whose points all
// carry that label (the common case: Morton order keeps a warp inside one
// polygon for long stretches), folded into the carry when a window holds
// another label.
struct LaneAcc {
    uint32_t cnt = 0;
    double sum = 0.0;
};

// the aggregated attribute as binary64: AF = float32 column, else int32 (exact)
template <bool AF>
__device__ __forceinline__ double attr_d(uint32_t bits) {
    return AF ? (double)__uint_as_float(bits) : (double)(int32_t)bits;
}

__device__ __forceinline__ void fold(LaneAcc &acc, Carry &cy) {
    if (__any_sync(kFull, acc.cnt != 0u)) {
        uint32_t c = acc.cnt;
        double s = acc.sum;
#pragma unroll
        for (int o = 16; o; o >>= 1) {
            c += __shfl_xor_sync(kFull, c, o);
            s += __shfl_xor_sync(kFull, s, o);
        }
        cy.cnt += c;
        cy.sum += s;
        acc.cnt = 0;
        acc.sum = 0.0;
    }
}

template <bool ACC, int NS, bool FP, bool AF>
__device__ __forceinline__ void process_lab(const PassArgs &a, const Shared &sh, const LabTile &t,
                                            const Consts<NS> &k, const Win<NS> &w, const uint32_t *sp,
                                            uint32_t first, uint32_t count, Carry &cy, LaneAcc &acc, BQ &bq,
                                            uint32_t &n_pass, uint32_t &n_bnd) {
    const int lane = threadIdx.x & 31;
    uint32_t lab[kIPL];
    bool spec = false, uni = true;
    uint32_t okm = 0;
#pragma unroll
    for (int j = 0; j < kIPL; ++j) {
        const bool ok = ((uint32_t)(lane * kIPL + j) - first) < count && pass_point<NS, FP>(a, k, w, j);
        n_pass += ok ? 1u : 0u;
        okm |= ok ? 1u << j : 0u;
        const uint32_t px = mulhi(w.x[j], k.W4), py = mulhi(w.y[j], k.H4);
        if (ok) RJ_DCHECK(py - t.r0 < t.th && px - t.c0 < t.tw);
        lab[j] = ok ? lds(t.lab_base + (py * t.stride + px) * 4u) : kNone;
        spec |= lab[j] == kMulti || lab[j] == kBnd;
        uni &= !ok || lab[j] == cy.lab;
    }
    // fast path: every point of the window carries the carry's label (never
    // MULTI / BND: the carry's label is a polygon or NONE)
    if (__all_sync(kFull, uni)) {
        // pairwise: three dependent binary64 adds per window instead of eight
        // (any order is within the 1e-9 bound; integer sums stay exact)
        double v[kIPL];
#pragma unroll
        for (int j = 0; j < kIPL; ++j) v[j] = ((okm >> j) & 1u) ? attr_d<AF>(agg_bits<NS>(a, w, j)) : 0.0;
        acc.cnt += __popc(okm);
        acc.sum += ((v[0] + v[1]) + (v[2] + v[3])) + ((v[4] + v[5]) + (v[6] + v[7]));
        return;
    }
    fold(acc, cy);
    if (__any_sync(kFull, spec)) {                            // rare: overlaps, boundary pixels
        uint32_t bm = 0;
#pragma unroll
        for (int j = 0; j < kIPL; ++j) {
            if (lab[j] == kMulti)
                multi_point(a, sh, t, mulhi(w.x[j], k.W4), mulhi(w.y[j], k.H4),
                            attr_d<AF>(agg_bits<NS>(a, w, j)));
            if (ACC && lab[j] == kBnd) bm |= 1u << j;
            if (lab[j] >= kBnd) lab[j] = kNone;
        }
        if (ACC) enqueue_window<true>(a, sh, sp, kStagePts, bm, bq, n_bnd);
    }
    // Runs of equal labels: inside the lane in registers, across lanes by a
    // segmented scan, and across windows through the warp's carry (Morton
    // order keeps a warp inside one polygon for long stretches, so a
    // polygon's partial is typically emitted once per stretch, not per window).
    uint32_t kprev = __shfl_up_sync(kFull, lab[kIPL - 1], 1);
    if (lane == 0) kprev = cy.lab;
    const uint32_t knext = __shfl_down_sync(kFull, lab[0], 1);
    const bool cin = lab[0] == kprev;                       // first run continues from before
    const bool cout = lane == 31 || lab[kIPL - 1] == knext; // last run continues (lane 31: into the carry)
    if (lane == 0 && !cin) emit_lab_run(a, sh, cy.lab, cy.cnt, cy.sum, true);   // carry ends here
    uint32_t run = 0, fcnt = 0, flab = kNone;
    double dsum = 0.0, fsum = 0.0;
    bool seen = false;
#pragma unroll
    for (int j = 0; j + 1 < kIPL; ++j) {
        const bool c = lab[j] != kNone;
        run += c ? 1u : 0u;
        if (c) dsum += attr_d<AF>(agg_bits<NS>(a, w, j));
        const bool tail = lab[j + 1] != lab[j];
        const bool defer = tail && !seen && cin;
        if (defer) { fcnt = run; fsum = dsum; flab = lab[j]; }
        emit_lab_run(a, sh, lab[j], run, dsum, tail && !defer);
        seen = seen || tail;
        run = tail ? 0u : run;
        dsum = tail ? 0.0 : dsum;
    }
    if (lab[kIPL - 1] != kNone) {
        run += 1u;
        dsum += attr_d<AF>(agg_bits<NS>(a, w, kIPL - 1));
    }
    // lane 0 takes the carry as its incoming partial
    const bool lane0_in = lane == 0 && cin;
    uint32_t scan_run = run + ((lane0_in && !seen) ? cy.cnt : 0u);
    double scan_sum = dsum + ((lane0_in && !seen) ? cy.sum : 0.0);
    uint32_t pre;
    double dpre;
    run_carry<true>(scan_run, scan_sum, seen || !cin || lane == 0, pre, dpre);
    if (lane == 0) { pre = cin ? cy.cnt : 0u; dpre = cin ? cy.sum : 0.0; }
    if (cin && seen) emit_lab_run(a, sh, flab, fcnt + pre, fsum + dpre, true);
    const bool add_pre = cin && !seen;
    const uint32_t last_cnt = (lane == 0) ? scan_run : run + (add_pre ? pre : 0u);
    const double last_sum = (lane == 0) ? scan_sum : dsum + (add_pre ? dpre : 0.0);
    emit_lab_run(a, sh, lab[kIPL - 1], last_cnt, last_sum, !cout);
    // the window's last run becomes the carry
    cy.lab = __shfl_sync(kFull, lab[kIPL - 1], 31);
    cy.cnt = __shfl_sync(kFull, last_cnt, 31);
    cy.sum = __shfl_sync(kFull, last_sum, 31);
}

template <bool ACC, int NS, bool FP, bool AF>
__global__ void __maxnreg__(96) k_point_pass_label(const __grid_constant__ PassArgs a) {
    extern __shared__ __align__(128) unsigned char smem_raw[];
    __shared__ __align__(8) Ring rg;
    __shared__ uint32_t s_pass, s_bnd;
    const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5;
    const uint32_t nstage = a.n_stages;
    const int ncol = 2 + NS;
    // carve: [ring][label tiles u32 x2][partial counts u32][queues]
    unsigned char *p = smem_raw;
    uint32_t *ring = reinterpret_cast<uint32_t *>(p);
    p += ring_bytes(nstage, NS);
    Shared sh;
    sh.psum = nullptr;                                      // fp64 sums reduce in global memory
    uint32_t *labels = reinterpret_cast<uint32_t *>(p);
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
    // predecessors' output from here on (early_stream: the producer streams
    // at once, see pass.cu)
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
        LabTile t;
        t.stride = a.tile_stride;
        uint32_t tsel = 0, n_pass = 0, n_bnd = 0;
        BQ bq = bq_init(a);
        Carry cy;
        LaneAcc acc;
        uint32_t st = 0, ph = 0;
        for (;;) {
            mbar_wait(smem_u32(&rg.full[st]), ph);
            const StageMeta m = rg.meta[st];
            if (m.cell == kDone) break;
            if (m.flags & 1u) {
                // ---- first stage of a cell: paint its label tile (tiles
                // alternate between consecutive cells)
                uint32_t *lt = labels + tsel * a.tile_cap;
                tsel ^= 1u;
                const int64_t cx = cell_x(m.cell), cy = cell_y(m.cell);
                t.c0 = (uint32_t)pix(cx << s_lat, a.W);
                t.r0 = (uint32_t)pix(cy << s_lat, a.H);
                const uint32_t th = (uint32_t)pix(((cy + 1) << s_lat) - 1, a.H) - t.r0 + 1;
                const uint32_t tw = (uint32_t)pix(((cx + 1) << s_lat) - 1, a.W) - t.c0 + 1;
                t.lab_base = smem_u32(lt) - 4u * (t.r0 * t.stride + t.c0);
                t.th = th;
                t.tw = tw;
                t.pb = t.pe = 0u;
                if (!ACC || !a.index_join) {
                    t.pb = __ldg(&a.piece_off[m.cell]);
                    t.pe = __ldg(&a.piece_off[m.cell + 1]);
                }
                if (ACC) {
                    clear_tile_acc(lt, t.stride, th, tw, t.r0, t.c0, a.index_join, kBnd, kNone, a.view);
                } else {
                    fill_tile(lt, th * t.stride, kNone);
                }
                consumers_sync();
                // one thread per piece.  Labels only move up the order
                // polygon < MULTI < BND: a polygon claims NONE, a second
                // polygon turns a polygon into MULTI (CAS, so a concurrent
                // BND is never overwritten), boundary pixels become BND.
                // With fewer pieces than threads, G = kThreads / pieces
                // threads paint one piece's column range together (a cell's
                // ~60 row pieces would otherwise leave 3/4 of the CTA idle
                // at the barrier while 64-pixel CAS runs complete).
                const uint32_t npc = t.pe - t.pb;
                const uint32_t G = npc ? max(1u, (uint32_t)kThreads / npc) : 1u;
                const uint32_t part = threadIdx.x % G;
                for (uint32_t kk = t.pb + threadIdx.x / G; kk < t.pe; kk += kThreads / G) {
                    const uint2 pc = __ldg(&a.pieces[kk]);
                    uint32_t *row = lt + (pc.y & 255u) * t.stride;
                    const uint32_t plo = (pc.y >> 8) & 255u, phi = pc.y >> 16;
                    RJ_DCHECK((pc.y & 255u) < th && plo < phi && phi <= tw);
                    const uint32_t lo = plo + (phi - plo) * part / G, hi = plo + (phi - plo) * (part + 1) / G;
                    for (uint32_t x = lo; x < hi; ++x) {
                        uint32_t o = atomicCAS(&row[x], kNone, pc.x);
                        if (!ACC) {
                            // no BND labels: any other claimant makes it MULTI.
                            // (The CAS loop below costs the bounded kernel ~15 %
                            // -- C4 2.01 vs 2.35 ms -- measured on B200.)
                            if (o != kNone) atomicExch(&row[x], kMulti);
                        } else if (o < kBnd) {
                            make_multi(&row[x], o);         // rare: overlapping polygons
                        }
                    }
                }
                if (ACC && !a.index_join) {
                    const uint32_t bb = __ldg(&a.bpiece_off[m.cell]), be = __ldg(&a.bpiece_off[m.cell + 1]);
                    for (uint32_t kk = bb + threadIdx.x; kk < be; kk += kThreads) {
                        const uint32_t v = __ldg(&a.bpieces[kk]);
                        RJ_DCHECK((v & 255u) < th && (v >> 16) <= tw);
                        uint32_t *row = lt + (v & 255u) * t.stride;
                        // plain stores: a polygon's CAS never overwrites BND, and BND
                        // landing after a CAS wins either way
                        for (uint32_t x = (v >> 8) & 255u, hi = v >> 16; x < hi; ++x) row[x] = kBnd;
                    }
                }
                consumers_sync();
                if (ACC && a.bnd_bits) dump_bnd(a, lt, t.stride, th, tw, t.r0, t.c0, 0xFFFFFFFFu, kBnd);
            }
            const uint32_t woff = (uint32_t)wid * kWin;
            const uint32_t ncopy = ((m.se + 3u) & ~3u) - m.cb;
            if (woff < ncopy && !never) {
                Win<NS> w;
                const uint32_t *sp = ring + (size_t)st * ncol * kStagePts + woff + lane * kIPL;
                load_win_smem<NS>(w, sp, 0);
                process_lab<ACC, NS, FP, AF>(a, sh, t, k, w, sp, (m.sb - m.cb) - woff, m.se - m.sb, cy, acc, bq,
                                             n_pass, n_bnd);
            }
            stage_release(smem_u32(&rg.empty[st]));
            if (++st == nstage) { st = 0; ph ^= 1u; }
        }
        if (ACC) bq_finish<true>(a, sh, bq);
        fold(acc, cy);
        if (lane == 0) emit_lab_run(a, sh, cy.lab, cy.cnt, cy.sum, true);
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

// SUM/AVG always stream the aggregated column (slot 0): NS >= 1
template <bool ACC, bool FP, bool AF>
void *select_ns(int ns) {
    switch (ns) {
    case 1: return (void *)k_point_pass_label<ACC, 1, FP, AF>;
    case 2: return (void *)k_point_pass_label<ACC, 2, FP, AF>;
    case 3: return (void *)k_point_pass_label<ACC, 3, FP, AF>;
    case 4: return (void *)k_point_pass_label<ACC, 4, FP, AF>;
    case 5: return (void *)k_point_pass_label<ACC, 5, FP, AF>;
    default: return (void *)k_point_pass_label<ACC, 6, FP, AF>;
    }
}

template <bool ACC, bool FP>
void *select_af(int ns, bool af) { return af ? select_ns<ACC, FP, true>(ns) : select_ns<ACC, FP, false>(ns); }

size_t label_smem(const PassArgs &a, bool, bool accurate) {
    size_t b = ring_bytes(a.n_stages, a.f.n_slots) + (size_t)a.tile_cap * 2 * 4;
    if (a.smem_partials) b += (size_t)a.n_poly * 4;
    return b + queue_bytes(accurate);
}
}  // namespace

size_t point_pass_label_smem(const PassArgs &a, bool accurate) { return label_smem(a, true, accurate); }

rj_status point_pass_label(Ctx *c, const PassArgs &a_in, bool accurate) {
    PassArgs a = a_in;
    a.n_stages = (uint32_t)choose_stages(a, label_smem, true, accurate, c->force_stages);
    if (a.smem_partials && a.n_stages < 3 && !c->force_stages) {
        // A deeper ring beats shared-memory count partials: the sums already
        // reduce in global memory, and Morton-ordered label runs make the
        // count reductions rare.  Two stages of 2048 points leave too few
        // bytes in flight per SM to cover HBM latency.
        PassArgs b = a;
        b.smem_partials = 0;
        b.n_stages = (uint32_t)choose_stages(b, label_smem, true, accurate, 0);
        if (b.n_stages >= 3) a = b;
    }
    if (!a.n_stages) return set_error(c, RJ_ERR_RESOLUTION, "point-pass tiles do not fit in shared memory");
    const bool fp = a.f.n_fpred > 0;
    const bool af = a.f.agg_is_float != 0;
    void *k = accurate ? (fp ? select_af<true, true>(a.f.n_slots, af) : select_af<true, false>(a.f.n_slots, af))
                       : (fp ? select_af<false, true>(a.f.n_slots, af) : select_af<false, false>(a.f.n_slots, af));
    return launch_pass(c, k, a, label_smem(a, true, accurate));
}

}  // namespace rj
