// label_canvas.cu -- the label-canvas point pass: streamed one-shot queries
// and MIN/MAX + multi-aggregate queries (NEXT-4).
//
// Paper: when the points do not fit in GPU memory they are transferred and
// drawn in batches; COUNT/SUM partials of the batches add (P:786-790,
// P:754-761).  Distributive aggregates other than COUNT/SUM (MIN, MAX) and
// several aggregates per query use more canvas channels / FBO attachments
// (P:754-766).
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
// Each point then costs the filter, one 4-byte label read and a
// warp-aggregated update of the per-polygon partials (count + up to
// kMaxAggs aggregates: binary64 sums, orderable-u32 MIN/MAX keys).
//
// Inputs: (a) the context's loaded lattice columns (spatially sorted: label
// reads hit L1/L2) -- rj_query with MIN/MAX and rj_query_multi; (b) raw
// points of rj_query_stream, never loaded: read exactly once, batch by
// batch, with the host->device copy of batch k+1 (copy stream, pinned host
// memory: DMA) overlapping the kernel on batch k; each point is quantised
// with the S1 arithmetic.  The streamed query is transfer-bound.
#include <algorithm>

#include "pip.cuh"
#include "rj_internal.cuh"

namespace rj {

namespace {

constexpr uint32_t kLabNone = 0xFFFFFFFFu, kLabMulti = 0xFFFFFFFEu, kLabBnd = 0xFFFFFFFDu;
constexpr unsigned kAll = 0xFFFFFFFFu;
constexpr int kLabThreads = 512;

inline unsigned blocks_for(uint64_t n, int t) { return (unsigned)std::max<uint64_t>(1, (n + t - 1) / t); }

// The label canvas covers the viewport window only (reading Z20): pixel
// (c0 + x, r0 + r) of the W x H canvas is lab[r * vw + x], r < vh, x < vw.

// lab = LAB_BND on boundary pixels (or everywhere: index join), else LAB_NONE.
__global__ void k_lab_init(uint32_t *__restrict__ lab, uint32_t vw, uint32_t vh, uint32_t c0, uint32_t r0,
                           const uint32_t *__restrict__ mask, uint32_t wpr, int all_bnd) {
    // rows stride over gridDim.y (<= 65535: a window may be 131072 rows high)
    for (uint64_t r = blockIdx.y; r < vh; r += gridDim.y)
        for (uint32_t x = blockIdx.x * blockDim.x + threadIdx.x; x < vw; x += gridDim.x * blockDim.x) {
            const uint32_t px = c0 + x;
            const bool b = all_bnd || (mask && ((mask[(r0 + r) * wpr + (px >> 5)] >> (px & 31)) & 1u));
            lab[r * vw + x] = b ? kLabBnd : kLabNone;
        }
}

// One warp per pixel span (polygon, row, lo, hi) -- clipped to the window by
// the polygon pass: claim its pixels; a pixel claimed twice becomes
// LAB_MULTI; boundary pixels stay LAB_BND.
__global__ void k_lab_paint(const uint4 *__restrict__ spans, uint64_t S, uint32_t *__restrict__ lab, uint32_t vw,
                            uint32_t c0, uint32_t r0) {
    const uint32_t lane = threadIdx.x & 31;
    const uint64_t nw = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    for (uint64_t s = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5; s < S; s += nw) {
        const uint4 sp = spans[s];
        uint32_t *row = lab + (uint64_t)(sp.y - r0) * vw - c0;
        for (uint32_t x = sp.z + lane; x < sp.w; x += 32) {
            const uint32_t o = atomicCAS(&row[x], kLabNone, sp.x);
            if (o != kLabNone && o < kLabBnd) atomicExch(&row[x], kLabMulti);
        }
    }
}

// Row index of the spans (CSR by window row), read only for LAB_MULTI pixels.
__global__ void k_row_count(const uint4 *__restrict__ spans, uint64_t S, uint32_t r0, uint32_t *__restrict__ cnt) {
    for (uint64_t s = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; s < S; s += (uint64_t)gridDim.x * blockDim.x)
        atomicAdd(&cnt[spans[s].y - r0], 1u);
}
__global__ void k_row_fill(const uint4 *__restrict__ spans, uint64_t S, uint32_t r0, const uint32_t *__restrict__ off,
                           uint32_t *__restrict__ cur, uint4 *__restrict__ rs) {
    for (uint64_t s = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; s < S; s += (uint64_t)gridDim.x * blockDim.x) {
        const uint4 sp = spans[s];
        rs[off[sp.y - r0] + atomicAdd(&cur[sp.y - r0], 1u)] = sp;
    }
}

struct LabArgs {
    const void *x, *y;               // f32 / f64 world coordinates, or u32 lattice (XY == 2)
    const uint32_t *col[6];          // filter slots
    Filter f;
    double x0, sx, y0, sy;           // lattice transform (S1, reading Z1)
    uint32_t W4, H4;
    uint32_t vc0, vr0, vw, vh;       // viewport window: the label canvas's extent
    const uint32_t *lab;
    const uint32_t *row_off;
    const uint4 *row_spans;
    const uint32_t *grid_off, *grid_poly;
    const int4 *grid_edge;
    unsigned long long *A_cnt;
    int32_t n_agg;
    int32_t agg_kind[kMaxAggs], agg_float[kMaxAggs];
    const uint32_t *agg_col[kMaxAggs];
    void *A_agg[kMaxAggs];           // double sums (SUM/AVG) or u32 keys (MIN/MAX)
    uint32_t smem_agg[kMaxAggs];     // byte offsets of the per-CTA aggregate partials
    uint32_t smem_cnt;
    uint32_t n_poly;
    int smem_partials;
    unsigned long long *stats;       // [0] filtered, [1] boundary, [2] out of domain
};

__device__ __forceinline__ bool lab_filter(const LabArgs &s, uint64_t i) {
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

// Orderable key: unsigned order of the key = IEEE totalOrder of the float32
// (reading Z16) / signed order of the int32.
__device__ __forceinline__ uint32_t order_key(uint32_t bits, int is_float) {
    if (!is_float) return bits ^ 0x80000000u;
    return (bits & 0x80000000u) ? ~bits : (bits | 0x80000000u);
}

template <int XY>
__global__ void __launch_bounds__(kLabThreads) k_label_pass(const __grid_constant__ LabArgs s, uint64_t n) {
    extern __shared__ __align__(16) unsigned char smem[];
    uint32_t *pcnt = reinterpret_cast<uint32_t *>(smem + s.smem_cnt);
    const int na = s.n_agg;
    if (s.smem_partials)
        for (uint32_t k = threadIdx.x; k < s.n_poly; k += blockDim.x) {
            pcnt[k] = 0;
            for (int a = 0; a < na; ++a) {
                const int kind = s.agg_kind[a];
                if (kind == RJ_SUM || kind == RJ_AVG) reinterpret_cast<double *>(smem + s.smem_agg[a])[k] = 0.0;
                else if (kind == RJ_MIN) reinterpret_cast<uint32_t *>(smem + s.smem_agg[a])[k] = 0xFFFFFFFFu;
                else if (kind == RJ_MAX) reinterpret_cast<uint32_t *>(smem + s.smem_agg[a])[k] = 0u;
            }
        }
    __syncthreads();
    double v[kMaxAggs];
    uint32_t key[kMaxAggs];
    // add (cnt, v/key) to polygon P's partials
    auto emit = [&](uint32_t P, uint32_t cnt, const double *vv, const uint32_t *kk) {
        if (s.smem_partials) atomicAdd(&pcnt[P], cnt);
        else atomicAdd(&s.A_cnt[P], (unsigned long long)cnt);
        for (int a = 0; a < na; ++a) {
            const int kind = s.agg_kind[a];
            if (s.smem_partials) {
                unsigned char *base = smem + s.smem_agg[a];
                if (kind == RJ_SUM || kind == RJ_AVG) atomicAdd(&reinterpret_cast<double *>(base)[P], vv[a]);
                else if (kind == RJ_MIN) atomicMin(&reinterpret_cast<uint32_t *>(base)[P], kk[a]);
                else if (kind == RJ_MAX) atomicMax(&reinterpret_cast<uint32_t *>(base)[P], kk[a]);
            } else {
                if (kind == RJ_SUM || kind == RJ_AVG) atomicAdd(&reinterpret_cast<double *>(s.A_agg[a])[P], vv[a]);
                else if (kind == RJ_MIN) atomicMin(&reinterpret_cast<uint32_t *>(s.A_agg[a])[P], kk[a]);
                else if (kind == RJ_MAX) atomicMax(&reinterpret_cast<uint32_t *>(s.A_agg[a])[P], kk[a]);
            }
        }
    };
    const uint32_t lane = threadIdx.x & 31;
    uint32_t n_pass = 0, n_bnd = 0, n_ood = 0;
    const uint64_t step = (uint64_t)gridDim.x * blockDim.x;
    // whole warps iterate together: the aggregation below shuffles
    for (uint64_t base = (uint64_t)blockIdx.x * blockDim.x + (threadIdx.x & ~31u); base < n; base += step) {
        const uint64_t i = base + lane;
        uint32_t P = kPipNone;
        if (i < n) {
            uint32_t qx = 0, qy = 0;
            bool in = true;
            if (XY == 2) {
                qx = __ldcs(reinterpret_cast<const uint32_t *>(s.x) + i);
                qy = __ldcs(reinterpret_cast<const uint32_t *>(s.y) + i);
            } else {
                double fx, fy;
                if (XY == 1) {
                    fx = __ldcs(reinterpret_cast<const double *>(s.x) + i);
                    fy = __ldcs(reinterpret_cast<const double *>(s.y) + i);
                } else {
                    fx = (double)__ldcs(reinterpret_cast<const float *>(s.x) + i);
                    fy = (double)__ldcs(reinterpret_cast<const float *>(s.y) + i);
                }
                // S1: Q = floor(((x - x0) / (x1 - x0)) * 2^30), binary64 (reading Z1)
                const double qxd = floor(__dmul_rn(__ddiv_rn(__dsub_rn(fx, s.x0), s.sx), 1073741824.0));
                const double qyd = floor(__dmul_rn(__ddiv_rn(__dsub_rn(fy, s.y0), s.sy), 1073741824.0));
                in = qxd >= 0.0 && qxd < 1073741824.0 && qyd >= 0.0 && qyd < 1073741824.0;
                if (in) {
                    qx = (uint32_t)qxd;
                    qy = (uint32_t)qyd;
                }
            }
            const uint32_t px = __umulhi(qx, s.W4), py = __umulhi(qy, s.H4);   // (q W) >> 30
            const uint32_t lx = px - s.vc0, ly = py - s.vr0;                     // window-relative
            if (!in) {
                ++n_ood;                                  // dropped (reading Z11)
            } else if (lx < s.vw && ly < s.vh && lab_filter(s, i)) {   // clipped to the window (Z20)
                ++n_pass;
                const uint32_t L = __ldg(&s.lab[(uint64_t)ly * s.vw + lx]);
                for (int a = 0; a < na; ++a) {
                    const uint32_t bits = __ldg(&s.agg_col[a][i]);
                    const int kind = s.agg_kind[a];
                    if (kind == RJ_SUM || kind == RJ_AVG)
                        v[a] = s.agg_float[a] ? (double)__uint_as_float(bits) : (double)(int32_t)bits;
                    else
                        key[a] = order_key(bits, s.agg_float[a]);
                }
                if (L < kLabBnd) {
                    P = L;
                } else if (L == kLabMulti) {
                    for (uint32_t k = __ldg(&s.row_off[ly]), e = __ldg(&s.row_off[ly + 1]); k < e; ++k) {
                        const uint4 sp = __ldg(&s.row_spans[k]);
                        if (sp.z <= px && px < sp.w) emit(sp.x, 1u, v, key);
                    }
                } else if (L == kLabBnd) {
                    ++n_bnd;
                    P = grid_pip(s.grid_off, s.grid_poly, s.grid_edge, qx, qy,
                                 [&](uint32_t Q) { emit(Q, 1u, v, key); });
                }
            }
        }
        // one partial update per distinct polygon of the warp's 32 points
        unsigned active = __ballot_sync(kAll, P != kPipNone);
        while (active) {
            const int leader = __ffs(active) - 1;
            const uint32_t PL = __shfl_sync(kAll, P, leader);
            const unsigned m = __ballot_sync(kAll, P == PL);
            const bool mine = P == PL;
            double rv[kMaxAggs];
            uint32_t rk[kMaxAggs];
            for (int a = 0; a < na; ++a) {
                const int kind = s.agg_kind[a];
                if (kind == RJ_SUM || kind == RJ_AVG) {
                    double t = mine ? v[a] : 0.0;
                    for (int o = 16; o; o >>= 1) t += __shfl_xor_sync(kAll, t, o);
                    rv[a] = t;
                } else if (kind == RJ_MIN) {
                    rk[a] = __reduce_min_sync(kAll, mine ? key[a] : 0xFFFFFFFFu);
                } else if (kind == RJ_MAX) {
                    rk[a] = __reduce_max_sync(kAll, mine ? key[a] : 0u);
                }
            }
            if ((int)lane == leader) emit(PL, __popc(m), rv, rk);
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
        for (uint32_t k = threadIdx.x; k < s.n_poly; k += blockDim.x) {
            if (!pcnt[k]) continue;
            atomicAdd(&s.A_cnt[k], (unsigned long long)pcnt[k]);
            for (int a = 0; a < na; ++a) {
                const int kind = s.agg_kind[a];
                const unsigned char *b = smem + s.smem_agg[a];
                if (kind == RJ_SUM || kind == RJ_AVG)
                    atomicAdd(&reinterpret_cast<double *>(s.A_agg[a])[k], reinterpret_cast<const double *>(b)[k]);
                else if (kind == RJ_MIN)
                    atomicMin(&reinterpret_cast<uint32_t *>(s.A_agg[a])[k], reinterpret_cast<const uint32_t *>(b)[k]);
                else if (kind == RJ_MAX)
                    atomicMax(&reinterpret_cast<uint32_t *>(s.A_agg[a])[k], reinterpret_cast<const uint32_t *>(b)[k]);
            }
        }
}

// values[k * n + i]: COUNT, SUM, AVG = SUM / COUNT, MIN / MAX
// decoded from the orderable key; NaN for an empty polygon's AVG / MIN / MAX.
__global__ void k_finalize_aggs(int kind, int is_float, uint32_t n, const unsigned long long *__restrict__ cnt,
                                const void *__restrict__ agg, double *__restrict__ out) {
    const uint32_t i = blockIdx.x * blockDim.x + threadIdx.x;
    if (i >= n) return;
    const double qnan = __longlong_as_double(0x7ff8000000000000ll);
    const unsigned long long c = cnt[i];
    double r;
    if (kind == RJ_COUNT) {
        r = (double)c;
    } else if (kind == RJ_SUM) {
        r = reinterpret_cast<const double *>(agg)[i];
    } else if (kind == RJ_AVG) {
        r = c ? __ddiv_rn(reinterpret_cast<const double *>(agg)[i], (double)c) : qnan;
    } else {
        const uint32_t k = reinterpret_cast<const uint32_t *>(agg)[i];
        if (!c) {
            r = qnan;
        } else if (is_float) {
            const uint32_t bits = (k & 0x80000000u) ? (k & 0x7FFFFFFFu) : ~k;
            r = (double)__uint_as_float(bits);
        } else {
            r = (double)(int32_t)(k ^ 0x80000000u);
        }
    }
    out[i] = r;
}

bool on_device(const void *p) {
    cudaPointerAttributes a;
    if (cudaPointerGetAttributes(&a, p) != cudaSuccess) {
        cudaGetLastError();
        return false;
    }
    return a.type == cudaMemoryTypeDevice || a.type == cudaMemoryTypeManaged;
}

void *label_kernel(int xy) {
    if (xy == 2) return (void *)k_label_pass<2>;
    return xy == 1 ? (void *)k_label_pass<1> : (void *)k_label_pass<0>;
}

}  // namespace

void stream_release(Ctx *c) {
    for (auto &bb : c->sbuf)
        for (auto &b : bb) dfree(c, b);
    for (auto &e : c->sev)
        if (e) { cudaEventDestroy(e); e = nullptr; }
    if (c->copy_stream) { cudaStreamDestroy(c->copy_stream); c->copy_stream = nullptr; }
}

cudaError_t launch_finalize_aggs(Ctx *c, const AggPlan &ap, const int *col_dtype, uint32_t n,
                                 const unsigned long long *cnt, const void *d_agg, double *values) {
    for (int a = 0; a < ap.n; ++a) {
        const int is_float = ap.kind[a] == RJ_COUNT ? 0 : col_dtype[ap.col[a]] == RJ_F32;
        k_finalize_aggs<<<blocks_for(n, 256), 256, 0, c->stream>>>(
            ap.kind[a], is_float, n, cnt, reinterpret_cast<const unsigned char *>(d_agg) + (size_t)a * n * 8,
            values + (size_t)a * n);
        RJ_LAUNCHED(c);
    }
    return cudaGetLastError();
}

rj_status label_query_impl(Ctx *c, const Filter &f, const AggPlan &ap, int W, int H, const View &v, int mode,
                           const LabInput &in, unsigned long long *d_cnt, void *d_agg) {
    cudaStream_t st = c->stream;
    const bool acc = mode != RJ_BOUNDED, index = mode == RJ_INDEX_JOIN;
    const uint64_t n = in.n;
    c->launches = 0;
    if (c->timing) RJ_CUDA(c, cudaEventRecord(c->ev[0], st));

    // ---- label canvas (S3 spans painted, S5 mask) + row index of the spans
    PolyPass pp;
    rj_status s;
    if (!index && (s = polygon_pass(c, W, H, -1, acc, pp, v, acc)) != RJ_OK) return s;
    const uint64_t S = pp.n_spans;
    const uint32_t vc0 = v.full ? 0u : (uint32_t)v.c0, vr0 = v.full ? 0u : (uint32_t)v.r0;
    const uint32_t vw = v.full ? (uint32_t)W : (uint32_t)(v.c1 - v.c0), vh = v.full ? (uint32_t)H : (uint32_t)(v.r1 - v.r0);
    Buf &lab = wsbuf(c, kWsLab), &rcnt = wsbuf(c, kWsRowCount), &roff = wsbuf(c, kWsRowOff);
    Buf &rcur = wsbuf(c, kWsRowCursor), &rsp = wsbuf(c, kWsRowSpans), &sts = wsbuf(c, kWsStream);
    if (dreserve(c, lab, (uint64_t)vw * vh * 4) || dreserve(c, rcnt, (uint64_t)(vh + 1) * 4) ||
        dreserve(c, roff, (uint64_t)(vh + 1) * 4) || dreserve(c, rcur, (uint64_t)(vh + 1) * 4) ||
        dreserve(c, rsp, (S + 1) * 16) || dreserve(c, sts, 64))
        return set_error(c, RJ_ERR_OOM, "label-canvas workspace allocation failed");
    k_lab_init<<<dim3(blocks_for(vw, 256), std::min<uint32_t>(vh, 65535u)), 256, 0, st>>>(lab.as<uint32_t>(), vw, vh, vc0, vr0,
                                                             acc && !index ? pp.mask : nullptr, pp.mask_wpr, index);
    RJ_LAUNCHED(c);
    RJ_CUDA(c, cudaMemsetAsync(rcnt.p, 0, (uint64_t)(vh + 1) * 4, st));
    RJ_CUDA(c, cudaMemsetAsync(rcur.p, 0, (uint64_t)(vh + 1) * 4, st));
    if (S) {
        const unsigned g = (unsigned)std::min<uint64_t>(blocks_for(S * 32, 256), c->num_sms * 16ull);
        k_lab_paint<<<g, 256, 0, st>>>(reinterpret_cast<const uint4 *>(pp.spans), S, lab.as<uint32_t>(), vw, vc0, vr0);
        RJ_LAUNCHED(c);
        const unsigned g2 = (unsigned)std::min<uint64_t>(blocks_for(S, 256), c->num_sms * 8ull);
        k_row_count<<<g2, 256, 0, st>>>(reinterpret_cast<const uint4 *>(pp.spans), S, vr0, rcnt.as<uint32_t>());
        RJ_LAUNCHED(c);
        RJ_CUDA(c, scan_u32(c, rcnt.as<uint32_t>(), roff.as<uint32_t>(), (uint64_t)vh, kWsScan));
        k_row_fill<<<g2, 256, 0, st>>>(reinterpret_cast<const uint4 *>(pp.spans), S, vr0, roff.as<uint32_t>(),
                                       rcur.as<uint32_t>(), rsp.as<uint4>());
        RJ_LAUNCHED(c);
    } else {
        RJ_CUDA(c, cudaMemsetAsync(roff.p, 0, (uint64_t)(vh + 1) * 4, st));
    }
    RJ_CUDA(c, cudaGetLastError());
    if (c->timing) RJ_CUDA(c, cudaEventRecord(c->ev[1], st));

    // ---- kernel arguments
    const uint32_t np = c->n_poly;
    LabArgs a;
    memset(&a, 0, sizeof(a));
    a.f = f;
    a.x0 = c->x0;
    a.sx = c->x1 - c->x0;
    a.y0 = c->y0;
    a.sy = c->y1 - c->y0;
    a.vc0 = vc0;
    a.vr0 = vr0;
    a.vw = vw;
    a.vh = vh;
    a.W4 = (uint32_t)W << 2;
    a.H4 = (uint32_t)H << 2;
    a.lab = lab.as<uint32_t>();
    a.row_off = roff.as<uint32_t>();
    a.row_spans = rsp.as<uint4>();
    a.grid_off = c->grid_off.as<uint32_t>();
    a.grid_poly = c->grid_poly.as<uint32_t>();
    a.grid_edge = c->grid_edge.as<int4>();
    a.A_cnt = d_cnt;
    a.n_poly = np;
    a.stats = sts.as<unsigned long long>();
    a.n_agg = ap.n;
    // shared partials: [sums f64 ...][count u32][keys u32 ...]
    size_t off = 0;
    for (int k = 0; k < ap.n; ++k) {
        a.agg_kind[k] = ap.kind[k];
        a.agg_float[k] = in.col_dtype[ap.col[k]] == RJ_F32;
        a.A_agg[k] = reinterpret_cast<unsigned char *>(d_agg) + (size_t)k * np * 8;
        if (ap.kind[k] == RJ_SUM || ap.kind[k] == RJ_AVG) { a.smem_agg[k] = (uint32_t)off; off += (size_t)np * 8; }
    }
    a.smem_cnt = (uint32_t)off;
    off += (size_t)np * 4;
    for (int k = 0; k < ap.n; ++k)
        if (ap.kind[k] == RJ_MIN || ap.kind[k] == RJ_MAX) { a.smem_agg[k] = (uint32_t)off; off += (size_t)np * 4; }
    a.smem_partials = off <= 96 * 1024;
    const size_t smem = a.smem_partials ? off : 0;
    const int xy = in.lattice ? 2 : (in.xy_f64 ? 1 : 0);
    void *kern = label_kernel(xy);
    RJ_CUDA(c, cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
    int per_sm = 0;
    RJ_CUDA(c, cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, kern, kLabThreads, smem));
    if (per_sm < 1) return set_error(c, RJ_ERR_RESOLUTION, "label-pass partials do not fit in shared memory");
    const unsigned grid = (unsigned)(c->num_sms * per_sm);
    RJ_CUDA(c, cudaMemsetAsync(d_cnt, 0, (size_t)np * 8, st));
    for (int k = 0; k < ap.n; ++k)   // MIN starts at the largest key, SUM / MAX at 0
        RJ_CUDA(c, cudaMemsetAsync(a.A_agg[k], ap.kind[k] == RJ_MIN ? 0xFF : 0, (size_t)np * 8, st));
    RJ_CUDA(c, cudaMemsetAsync(sts.p, 0, 64, st));

    // ---- inputs: the distinct columns this query reads (x, y, filter slots,
    // aggregate columns).  Device pointers are read in place; host columns
    // stream through two device batch buffers.
    const void *src[2 + 6 + kMaxAggs];
    size_t esz[2 + 6 + kMaxAggs];
    int ucol[2 + 6 + kMaxAggs];
    int ncol = 2;
    src[0] = in.x;
    src[1] = in.y;
    esz[0] = esz[1] = in.lattice ? 4 : (in.xy_f64 ? 8 : 4);
    ucol[0] = ucol[1] = -1;
    auto need = [&](int uc) -> int {
        for (int k = 2; k < ncol; ++k)
            if (ucol[k] == uc) return k;
        src[ncol] = in.lattice ? c->col[uc].p : in.cols[uc];
        esz[ncol] = 4;
        ucol[ncol] = uc;
        return ncol++;
    };
    int slot_idx[6], agg_idx[kMaxAggs];
    for (int k = 0; k < f.n_slots; ++k) slot_idx[k] = need(f.slot_col[k]);
    for (int k = 0; k < ap.n; ++k) agg_idx[k] = need(ap.col[k]);
    bool host[2 + 6 + kMaxAggs], any_host = false;
    for (int k = 0; k < ncol; ++k) any_host |= (host[k] = n && !in.lattice && !on_device(src[k]));
    auto launch = [&](uint64_t cnt, const void *const *p) -> rj_status {
        LabArgs b = a;
        b.x = p[0];
        b.y = p[1];
        for (int k = 0; k < f.n_slots; ++k) b.col[k] = reinterpret_cast<const uint32_t *>(p[slot_idx[k]]);
        for (int k = 0; k < ap.n; ++k) b.agg_col[k] = reinterpret_cast<const uint32_t *>(p[agg_idx[k]]);
        void *args[] = {&b, &cnt};
        RJ_CUDA(c, cudaLaunchKernel(kern, dim3(grid), dim3(kLabThreads), args, smem, st));
        RJ_LAUNCHED(c);
        return RJ_OK;
    };
    if (n && !any_host) {
        if ((s = launch(n, src)) != RJ_OK) return s;
    } else if (n) {
        if (!c->copy_stream) {
            RJ_CUDA(c, cudaStreamCreateWithFlags(&c->copy_stream, cudaStreamNonBlocking));
            for (auto &e : c->sev) RJ_CUDA(c, cudaEventCreateWithFlags(&e, cudaEventDisableTiming));
        }
        const uint64_t B = (uint64_t)std::max<int64_t>(1, c->stream_batch);
        const uint64_t nb = (n + B - 1) / B;
        const uint64_t bcap = std::min(B, n);
        for (int b = 0; b < (nb > 1 ? 2 : 1); ++b)
            for (int k = 0; k < ncol; ++k)
                if (host[k] && dreserve_exact(c, c->sbuf[b][k], bcap * esz[k]))
                    return set_error(c, RJ_ERR_OOM, "stream batch allocation failed");
        // earlier work on the query stream (previous users of the buffers)
        // precedes every copy
        RJ_CUDA(c, cudaEventRecord(c->sev[4], st));
        RJ_CUDA(c, cudaStreamWaitEvent(c->copy_stream, c->sev[4], 0));
        for (uint64_t bi = 0; bi < nb; ++bi) {
            const int b = (int)(bi & 1);
            const uint64_t o = bi * B, cnt = std::min(B, n - o);
            if (bi >= 2) RJ_CUDA(c, cudaStreamWaitEvent(c->copy_stream, c->sev[2 + b], 0));
            const void *p[2 + 6 + kMaxAggs];
            for (int k = 0; k < ncol; ++k) {
                const unsigned char *h = reinterpret_cast<const unsigned char *>(src[k]) + o * esz[k];
                if (host[k]) {
                    RJ_CUDA(c, cudaMemcpyAsync(c->sbuf[b][k].p, h, cnt * esz[k], cudaMemcpyHostToDevice,
                                               c->copy_stream));
                    p[k] = c->sbuf[b][k].p;
                } else {
                    p[k] = h;
                }
            }
            RJ_CUDA(c, cudaEventRecord(c->sev[b], c->copy_stream));
            RJ_CUDA(c, cudaStreamWaitEvent(st, c->sev[b], 0));
            if ((s = launch(cnt, p)) != RJ_OK) return s;
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
    for (int k = 0; k < ncol; ++k) L.stream_bytes += n * esz[k];
    c->last_stages = 0;
    c->last_ctas_per_sm = per_sm;
    c->stream_stats_pending = 1;
    return RJ_OK;
}

}  // namespace rj
