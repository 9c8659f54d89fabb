// stream.cu -- the streamed one-shot query.
//
// Paper: when the points do not fit in GPU memory they are transferred and
// drawn in batches; COUNT/SUM partials of the batches add (P:786-790,
// P:754-761).  Here the points of rj_query_stream are never loaded into the
// context: no spatial sort, each point is read exactly once, batch by batch,
// with the host->device copy of batch k+1 (copy stream, pinned host memory:
// DMA) overlapping the kernel on batch k.
//
// Per query the polygons are rasterized ONCE into a label canvas lab[H][W]:
//   polygon id   -- exactly one polygon holds the pixel centre (Proc.
//                   DrawPolygons' pixel-centre rule, reading Z3),
//   LAB_NONE     -- none,
//   LAB_MULTI    -- several (overlapping polygons): resolved per point from
//                   the row's spans,
//   LAB_BND      -- accurate mode: a boundary pixel (S5 supercover mask);
//                   its points get the exact grid PIP (Proc. JoinPoint,
//                   P:718-726); the index join marks every pixel.
// Each point then costs its quantisation (S1 arithmetic), the filter, one
// 4-byte label read and a warp-aggregated partial update: the kernel keeps up
// with PCIe/C2C by a wide margin, so the streamed query is transfer-bound.
#include <algorithm>

#include "pip.cuh"
#include "rj_internal.cuh"

namespace rj {

namespace {

constexpr uint32_t kLabNone = 0xFFFFFFFFu, kLabMulti = 0xFFFFFFFEu, kLabBnd = 0xFFFFFFFDu;
constexpr unsigned kAll = 0xFFFFFFFFu;
constexpr int kStreamThreads = 512;

inline unsigned blocks_for(uint64_t n, int t) { return (unsigned)std::max<uint64_t>(1, (n + t - 1) / t); }

// lab = LAB_BND on boundary pixels (or everywhere: index join), else LAB_NONE.
__global__ void k_lab_init(uint32_t *__restrict__ lab, int W, const uint32_t *__restrict__ mask, uint32_t wpr,
                           int all_bnd) {
    const uint64_t r = blockIdx.y;
    for (uint32_t x = blockIdx.x * blockDim.x + threadIdx.x; x < (uint32_t)W; x += gridDim.x * blockDim.x) {
        const bool b = all_bnd || (mask && ((mask[r * wpr + (x >> 5)] >> (x & 31)) & 1u));
        lab[r * W + x] = b ? kLabBnd : kLabNone;
    }
}

// One warp per pixel span (polygon, row, lo, hi): claim its pixels; a pixel
// claimed twice becomes LAB_MULTI; boundary pixels stay LAB_BND.
__global__ void k_lab_paint(const uint4 *__restrict__ spans, uint64_t S, uint32_t *__restrict__ lab, int W) {
    const uint32_t lane = threadIdx.x & 31;
    const uint64_t nw = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    for (uint64_t s = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5; s < S; s += nw) {
        const uint4 sp = spans[s];
        uint32_t *row = lab + (uint64_t)sp.y * W;
        for (uint32_t x = sp.z + lane; x < sp.w; x += 32) {
            const uint32_t o = atomicCAS(&row[x], kLabNone, sp.x);
            if (o != kLabNone && o < kLabBnd) atomicExch(&row[x], kLabMulti);
        }
    }
}

// Row index of the spans (CSR by row), read only for LAB_MULTI pixels.
__global__ void k_row_count(const uint4 *__restrict__ spans, uint64_t S, uint32_t *__restrict__ cnt) {
    for (uint64_t s = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; s < S; s += (uint64_t)gridDim.x * blockDim.x)
        atomicAdd(&cnt[spans[s].y], 1u);
}
__global__ void k_row_fill(const uint4 *__restrict__ spans, uint64_t S, const uint32_t *__restrict__ off,
                           uint32_t *__restrict__ cur, uint4 *__restrict__ rs) {
    for (uint64_t s = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; s < S; s += (uint64_t)gridDim.x * blockDim.x) {
        const uint4 sp = spans[s];
        rs[off[sp.y] + atomicAdd(&cur[sp.y], 1u)] = sp;
    }
}

struct StreamArgs {
    const void *x, *y;
    const uint32_t *col[6];          // filter / aggregate slots of this batch
    Filter f;
    double x0, sx, y0, sy;           // lattice transform (S1, reading Z1)
    uint32_t W, W4, H4;
    const uint32_t *lab;
    const uint32_t *row_off;
    const uint4 *row_spans;
    const uint32_t *grid_off, *grid_poly;
    const int4 *grid_edge;
    unsigned long long *A_cnt;
    double *A_sum;
    uint32_t n_poly;
    int smem_partials;
    unsigned long long *stats;       // [0] filtered, [1] boundary, [2] out of domain
};

__device__ __forceinline__ bool stream_filter(const StreamArgs &s, uint64_t i) {
    const Filter &f = s.f;
    if (f.never) return false;
    for (int k = 0; k < f.n_irange; ++k) {
        const int32_t v = (int32_t)__ldg(&s.col[k][i]);
        if (v < f.ilo[k] || v > f.ihi[k]) return false;
    }
    for (int p = 0; p < f.n_fpred; ++p) {
        const float v = __uint_as_float(__ldg(&s.col[f.f_slot[p]][i]));
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

template <bool SUM, bool XY64>
__global__ void __launch_bounds__(kStreamThreads) k_stream(const __grid_constant__ StreamArgs s, uint64_t n) {
    extern __shared__ __align__(16) unsigned char smem[];
    double *psum = reinterpret_cast<double *>(smem);
    uint32_t *pcnt = reinterpret_cast<uint32_t *>(smem + (SUM ? sizeof(double) * s.n_poly : 0));
    if (s.smem_partials)
        for (uint32_t k = threadIdx.x; k < s.n_poly; k += blockDim.x) {
            pcnt[k] = 0;
            if (SUM) psum[k] = 0.0;
        }
    __syncthreads();
    auto emit = [&](uint32_t P, uint32_t cnt, double v) {
        if (s.smem_partials) {
            atomicAdd(&pcnt[P], cnt);
            if (SUM) atomicAdd(&psum[P], v);
        } else {
            atomicAdd(&s.A_cnt[P], (unsigned long long)cnt);
            if (SUM) atomicAdd(&s.A_sum[P], v);
        }
    };
    const uint32_t lane = threadIdx.x & 31;
    uint32_t n_pass = 0, n_bnd = 0, n_ood = 0;
    const uint64_t step = (uint64_t)gridDim.x * blockDim.x;
    // whole warps iterate together: the aggregation below shuffles
    for (uint64_t base = (uint64_t)blockIdx.x * blockDim.x + (threadIdx.x & ~31u); base < n; base += step) {
        const uint64_t i = base + lane;
        uint32_t P = kPipNone;
        double v = 0.0;
        if (i < n) {
            double fx, fy;
            if (XY64) {
                fx = __ldcs(reinterpret_cast<const double *>(s.x) + i);
                fy = __ldcs(reinterpret_cast<const double *>(s.y) + i);
            } else {
                fx = (double)__ldcs(reinterpret_cast<const float *>(s.x) + i);
                fy = (double)__ldcs(reinterpret_cast<const float *>(s.y) + i);
            }
            // S1: Q = floor(((x - x0) / (x1 - x0)) * 2^30), binary64 (reading Z1)
            const double qxd = floor(__dmul_rn(__ddiv_rn(__dsub_rn(fx, s.x0), s.sx), 1073741824.0));
            const double qyd = floor(__dmul_rn(__ddiv_rn(__dsub_rn(fy, s.y0), s.sy), 1073741824.0));
            if (!(qxd >= 0.0 && qxd < 1073741824.0 && qyd >= 0.0 && qyd < 1073741824.0)) {
                ++n_ood;                                  // dropped (reading Z11)
            } else if (stream_filter(s, i)) {
                ++n_pass;
                const uint32_t qx = (uint32_t)qxd, qy = (uint32_t)qyd;
                const uint32_t px = __umulhi(qx, s.W4), py = __umulhi(qy, s.H4);   // (q W) >> 30
                const uint32_t L = __ldg(&s.lab[(uint64_t)py * s.W + px]);
                if (SUM) v = s.f.agg_is_float ? (double)__uint_as_float(__ldg(&s.col[s.f.agg_slot][i]))
                                              : (double)(int32_t)__ldg(&s.col[s.f.agg_slot][i]);
                if (L < kLabBnd) {
                    P = L;
                } else if (L == kLabMulti) {
                    for (uint32_t k = __ldg(&s.row_off[py]), e = __ldg(&s.row_off[py + 1]); k < e; ++k) {
                        const uint4 sp = __ldg(&s.row_spans[k]);
                        if (sp.z <= px && px < sp.w) emit(sp.x, 1u, v);
                    }
                } else if (L == kLabBnd) {
                    ++n_bnd;
                    P = grid_pip(s.grid_off, s.grid_poly, s.grid_edge, qx, qy,
                                 [&](uint32_t Q) { emit(Q, 1u, v); });
                }
            }
        }
        // one partial update per distinct polygon of the warp's 32 points
        unsigned active = __ballot_sync(kAll, P != kPipNone);
        while (active) {
            const int leader = __ffs(active) - 1;
            const uint32_t PL = __shfl_sync(kAll, P, leader);
            const unsigned m = __ballot_sync(kAll, P == PL);
            double sm = 0.0;
            if (SUM) {
                sm = P == PL ? v : 0.0;
                for (int o = 16; o; o >>= 1) sm += __shfl_xor_sync(kAll, sm, o);
            }
            if ((int)lane == leader) emit(PL, __popc(m), sm);
            active &= ~m;
        }
    }
    for (int o = 16; o; o >>= 1) {
        n_pass += __shfl_xor_sync(kAll, n_pass, o);
        n_bnd += __shfl_xor_sync(kAll, n_bnd, o);
        n_ood += __shfl_xor_sync(kAll, n_ood, o);
    }
    if (lane == 0) {
        if (n_pass) atomicAdd(&s.stats[0], (unsigned long long)n_pass);
        if (n_bnd) atomicAdd(&s.stats[1], (unsigned long long)n_bnd);
        if (n_ood) atomicAdd(&s.stats[2], (unsigned long long)n_ood);
    }
    __syncthreads();
    if (s.smem_partials)
        for (uint32_t k = threadIdx.x; k < s.n_poly; k += blockDim.x)
            if (pcnt[k]) {
                atomicAdd(&s.A_cnt[k], (unsigned long long)pcnt[k]);
                if (SUM) atomicAdd(&s.A_sum[k], psum[k]);
            }
}

bool on_device(const void *p) {
    cudaPointerAttributes a;
    if (cudaPointerGetAttributes(&a, p) != cudaSuccess) {
        cudaGetLastError();
        return false;
    }
    return a.type == cudaMemoryTypeDevice || a.type == cudaMemoryTypeManaged;
}

void *stream_kernel(bool sum, bool xy64) {
    if (sum) return xy64 ? (void *)k_stream<true, true> : (void *)k_stream<true, false>;
    return xy64 ? (void *)k_stream<false, true> : (void *)k_stream<false, false>;
}

}  // namespace

void stream_release(Ctx *c) {
    for (auto &bb : c->sbuf)
        for (auto &b : bb) dfree(c, b);
    for (auto &e : c->sev)
        if (e) { cudaEventDestroy(e); e = nullptr; }
    if (c->copy_stream) { cudaStreamDestroy(c->copy_stream); c->copy_stream = nullptr; }
}

rj_status stream_query_impl(Ctx *c, const Filter &f, bool sum, int W, int H, int mode, uint64_t n,
                            const void *x, const void *y, bool xy_f64, const void *const *cols,
                            unsigned long long *d_cnt, double *d_sum) {
    cudaStream_t st = c->stream;
    const bool acc = mode != RJ_BOUNDED, index = mode == RJ_INDEX_JOIN;
    c->launches = 0;
    if (c->timing) RJ_CUDA(c, cudaEventRecord(c->ev[0], st));

    // ---- label canvas (S3 spans painted, S5 mask) + row index of the spans
    PolyPass pp;
    rj_status s;
    if (!index && (s = polygon_pass(c, W, H, -1, acc, pp)) != RJ_OK) return s;
    const uint64_t S = pp.n_spans;
    Buf &lab = wsbuf(c, kWsLab), &rcnt = wsbuf(c, kWsRowCount), &roff = wsbuf(c, kWsRowOff);
    Buf &rcur = wsbuf(c, kWsRowCursor), &rsp = wsbuf(c, kWsRowSpans), &sts = wsbuf(c, kWsStream);
    if (dreserve(c, lab, (uint64_t)W * H * 4) || dreserve(c, rcnt, (uint64_t)(H + 1) * 4) ||
        dreserve(c, roff, (uint64_t)(H + 1) * 4) || dreserve(c, rcur, (uint64_t)(H + 1) * 4) ||
        dreserve(c, rsp, (S + 1) * 16) || dreserve(c, sts, 64))
        return set_error(c, RJ_ERR_OOM, "streamed-query workspace allocation failed");
    k_lab_init<<<dim3(blocks_for(W, 256), H), 256, 0, st>>>(lab.as<uint32_t>(), W, acc && !index ? pp.mask : nullptr,
                                                           pp.mask_wpr, index);
    RJ_LAUNCHED(c);
    RJ_CUDA(c, cudaMemsetAsync(rcnt.p, 0, (uint64_t)(H + 1) * 4, st));
    RJ_CUDA(c, cudaMemsetAsync(rcur.p, 0, (uint64_t)(H + 1) * 4, st));
    if (S) {
        const unsigned g = (unsigned)std::min<uint64_t>(blocks_for(S * 32, 256), c->num_sms * 16ull);
        k_lab_paint<<<g, 256, 0, st>>>(reinterpret_cast<const uint4 *>(pp.spans), S, lab.as<uint32_t>(), W);
        RJ_LAUNCHED(c);
        const unsigned g2 = (unsigned)std::min<uint64_t>(blocks_for(S, 256), c->num_sms * 8ull);
        k_row_count<<<g2, 256, 0, st>>>(reinterpret_cast<const uint4 *>(pp.spans), S, rcnt.as<uint32_t>());
        RJ_LAUNCHED(c);
        RJ_CUDA(c, scan_u32(c, rcnt.as<uint32_t>(), roff.as<uint32_t>(), (uint64_t)H, kWsScan));
        k_row_fill<<<g2, 256, 0, st>>>(reinterpret_cast<const uint4 *>(pp.spans), S, roff.as<uint32_t>(),
                                       rcur.as<uint32_t>(), rsp.as<uint4>());
        RJ_LAUNCHED(c);
    } else {
        RJ_CUDA(c, cudaMemsetAsync(roff.p, 0, (uint64_t)(H + 1) * 4, st));
    }
    RJ_CUDA(c, cudaGetLastError());
    if (c->timing) RJ_CUDA(c, cudaEventRecord(c->ev[1], st));

    // ---- kernel arguments
    StreamArgs a;
    memset(&a, 0, sizeof(a));
    a.f = f;
    a.x0 = c->x0;
    a.sx = c->x1 - c->x0;
    a.y0 = c->y0;
    a.sy = c->y1 - c->y0;
    a.W = (uint32_t)W;
    a.W4 = (uint32_t)W << 2;
    a.H4 = (uint32_t)H << 2;
    a.lab = lab.as<uint32_t>();
    a.row_off = roff.as<uint32_t>();
    a.row_spans = rsp.as<uint4>();
    a.grid_off = c->grid_off.as<uint32_t>();
    a.grid_poly = c->grid_poly.as<uint32_t>();
    a.grid_edge = c->grid_edge.as<int4>();
    a.A_cnt = d_cnt;
    a.A_sum = d_sum;
    a.n_poly = c->n_poly;
    a.stats = sts.as<unsigned long long>();
    const size_t part = (size_t)c->n_poly * (4 + (sum ? 8 : 0));
    a.smem_partials = part <= 96 * 1024;
    const size_t smem = a.smem_partials ? part : 0;
    void *k = stream_kernel(sum, xy_f64);
    RJ_CUDA(c, cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
    int per_sm = 0;
    RJ_CUDA(c, cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k, kStreamThreads, smem));
    if (per_sm < 1) return set_error(c, RJ_ERR_RESOLUTION, "streamed-query partials do not fit in shared memory");
    const unsigned grid = (unsigned)(c->num_sms * per_sm);
    RJ_CUDA(c, cudaMemsetAsync(d_cnt, 0, (size_t)c->n_poly * 8, st));
    if (sum) RJ_CUDA(c, cudaMemsetAsync(d_sum, 0, (size_t)c->n_poly * 8, st));
    RJ_CUDA(c, cudaMemsetAsync(sts.p, 0, 64, st));

    // ---- inputs: device pointers are read in place; host columns stream
    // through two device batch buffers
    const int ncol = 2 + f.n_slots;
    const void *src[2 + 6];
    size_t esz[2 + 6];
    src[0] = x;
    src[1] = y;
    esz[0] = esz[1] = xy_f64 ? 8 : 4;
    for (int k2 = 0; k2 < f.n_slots; ++k2) {
        src[2 + k2] = cols[f.slot_col[k2]];
        esz[2 + k2] = 4;
    }
    bool host[2 + 6], any_host = false;
    for (int k2 = 0; k2 < ncol; ++k2) any_host |= (host[k2] = n && !on_device(src[k2]));
    auto launch = [&](uint64_t off, uint64_t cnt, const void *const *p) -> rj_status {
        StreamArgs b = a;
        b.x = p[0];
        b.y = p[1];
        for (int k2 = 0; k2 < f.n_slots; ++k2) b.col[k2] = reinterpret_cast<const uint32_t *>(p[2 + k2]);
        (void)off;
        void *args[] = {&b, &cnt};
        RJ_CUDA(c, cudaLaunchKernel(k, dim3(grid), dim3(kStreamThreads), args, smem, st));
        RJ_LAUNCHED(c);
        return RJ_OK;
    };
    if (n && !any_host) {
        if ((s = launch(0, n, src)) != RJ_OK) return s;
    } else if (n) {
        if (!c->copy_stream) {
            RJ_CUDA(c, cudaStreamCreateWithFlags(&c->copy_stream, cudaStreamNonBlocking));
            for (auto &e : c->sev) RJ_CUDA(c, cudaEventCreateWithFlags(&e, cudaEventDisableTiming));
        }
        const uint64_t B = (uint64_t)std::max<int64_t>(1, c->stream_batch);
        const uint64_t nb = (n + B - 1) / B;
        const uint64_t bcap = std::min(B, n);
        for (int b = 0; b < (nb > 1 ? 2 : 1); ++b)
            for (int k2 = 0; k2 < ncol; ++k2)
                if (host[k2] && dreserve_exact(c, c->sbuf[b][k2], bcap * esz[k2]))
                    return set_error(c, RJ_ERR_OOM, "stream batch allocation failed");
        // earlier work on the query stream (previous users of the buffers)
        // precedes every copy
        RJ_CUDA(c, cudaEventRecord(c->sev[4], st));
        RJ_CUDA(c, cudaStreamWaitEvent(c->copy_stream, c->sev[4], 0));
        for (uint64_t bi = 0; bi < nb; ++bi) {
            const int b = (int)(bi & 1);
            const uint64_t off = bi * B, cnt = std::min(B, n - off);
            if (bi >= 2) RJ_CUDA(c, cudaStreamWaitEvent(c->copy_stream, c->sev[2 + b], 0));
            const void *p[2 + 6];
            for (int k2 = 0; k2 < ncol; ++k2) {
                const unsigned char *h = reinterpret_cast<const unsigned char *>(src[k2]) + off * esz[k2];
                if (host[k2]) {
                    RJ_CUDA(c, cudaMemcpyAsync(c->sbuf[b][k2].p, h, cnt * esz[k2], cudaMemcpyHostToDevice,
                                               c->copy_stream));
                    p[k2] = c->sbuf[b][k2].p;
                } else {
                    p[k2] = h;
                }
            }
            RJ_CUDA(c, cudaEventRecord(c->sev[b], c->copy_stream));
            RJ_CUDA(c, cudaStreamWaitEvent(st, c->sev[b], 0));
            if ((s = launch(off, cnt, p)) != RJ_OK) return s;
            RJ_CUDA(c, cudaEventRecord(c->sev[2 + b], st));
        }
    }
    RJ_CUDA(c, cudaGetLastError());
    if (c->timing) RJ_CUDA(c, cudaEventRecord(c->ev[2], st));
    RJ_CUDA(c, cudaMemcpyAsync(c->h_stats, sts.p, 3 * sizeof(unsigned long long), cudaMemcpyDeviceToHost, st));

    rj_stats &L = c->last;
    L.W = W;
    L.H = H;
    L.n_points = n;                 // corrected for out-of-domain points in rj_get_stats
    L.n_crossings = pp.n_cross;
    L.n_spans = pp.n_spans;
    L.n_pieces = 0;
    L.n_items = 0;
    L.level = -1;
    L.stream_bytes = 0;
    for (int k2 = 0; k2 < ncol; ++k2) L.stream_bytes += n * esz[k2];
    c->last_stages = 0;
    c->last_ctas_per_sm = per_sm;
    c->stream_stats_pending = 1;
    return RJ_OK;
}

}  // namespace rj
