// load_points.cu -- S1: quantise + spatial layout of the point set (once per
// load, the paper's "transformed into the screen space",
// P:507-508, and its transfer-once rule).
//
//  1. k_quantize: Q(x) = floor(((x - x0) / (x1 - x0)) * 2^30) in binary64 with
//     explicitly rounded ops (__dsub_rn, __ddiv_rn, exact *2^30), points with
//     Q outside [0, 2^30) or NaN marked out-of-domain (reading Z11).
//  2. Stable LSD radix sort (4 passes x 8 bits) of (key, original index)
//     pairs, key = the 32-bit Morton key of (Qx >> 14, Qy >> 14) capped at
//     0xFFFFFFFE, or 0xFFFFFFFF for an out-of-domain point (it sinks to the
//     end); then one
//     gather puts Qx, Qy and the attribute columns in sorted order, so the
//     point pass streams contiguous columns.
//  3. cell_off: start of every level-10 (1024x1024) Morton cell; a cell of
//     any coarser level L is the union of 4^(10-L) consecutive level-10
//     cells, so the point tiles of every query resolution are contiguous
//     ranges (work items: work.cu).
#include <algorithm>

#include "rj_internal.cuh"

namespace rj {

namespace {
constexpr uint32_t kInvalid = 0xFFFFFFFFu;
constexpr int kSortThreads = 256;
constexpr int kSortItems = 8;                        // per thread
constexpr int kSortTile = kSortThreads * kSortItems; // 2048
constexpr int kDigits = 257;                         // 256 + out-of-domain
constexpr int kMaxPayload = 3 + RJ_MAX_COLS;

template <typename T>
__global__ void k_quantize(const T *__restrict__ x, const T *__restrict__ y, uint64_t n, double x0,
                           double sx, double y0, double sy, uint2 *__restrict__ qxy) {
    for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n;
         i += (uint64_t)gridDim.x * blockDim.x) {
        const double fx = floor(__dmul_rn(__ddiv_rn(__dsub_rn((double)x[i], x0), sx), 1073741824.0));
        const double fy = floor(__dmul_rn(__ddiv_rn(__dsub_rn((double)y[i], y0), sy), 1073741824.0));
        const bool ok = fx >= 0.0 && fx < 1073741824.0 && fy >= 0.0 && fy < 1073741824.0;
        // (Qx, Qy) interleaved: the final gather reads both with one 8-B access
        qxy[i] = ok ? make_uint2((uint32_t)fx, (uint32_t)fy) : make_uint2(kInvalid, kInvalid);
    }
}

// Sort key: the 32-bit Morton key of (Qx >> 14, Qy >> 14) (level-16 order),
// capped at 0xFFFFFFFE; out-of-domain points get 0xFFFFFFFF, so they sort
// last by the key alone (the cap only merges two level-16 cells inside the
// last level-10 cell, whose order within a cell is free).
__global__ void k_keys(const uint2 *__restrict__ qxy, uint64_t n, uint32_t *__restrict__ key) {
    for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n; i += (uint64_t)gridDim.x * blockDim.x) {
        const uint2 q = qxy[i];
        key[i] = q.x == kInvalid ? 0xFFFFFFFFu : min(morton_key(q.x, q.y), 0xFFFFFFFEu);
    }
}

__device__ __forceinline__ uint32_t sort_digit(uint32_t key, int shift) { return (key >> shift) & 255u; }

// After the (key, index) sort: every column in sorted order, gathered once
// (Qx, Qy and the attribute columns of point idx[i] go to position i).
struct Gather {
    const uint2 *qxy;
    uint32_t *qx, *qy;
    const uint32_t *src[RJ_MAX_COLS];
    uint32_t *dst[RJ_MAX_COLS];
    int n;
};
__global__ void k_gather(const uint32_t *__restrict__ idx, uint64_t n, const Gather g) {
    for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n; i += (uint64_t)gridDim.x * blockDim.x) {
        const uint32_t j = idx[i];
        const uint2 q = __ldg(&g.qxy[j]);
        g.qx[i] = q.x;
        g.qy[i] = q.y;
        for (int k = 0; k < g.n; ++k) g.dst[k][i] = __ldg(&g.src[k][j]);
    }
}

struct Payload {
    const uint32_t *src[kMaxPayload];
    uint32_t *dst[kMaxPayload];
    int n;
};

__global__ void __launch_bounds__(kSortThreads) k_radix_hist(const uint32_t *__restrict__ key,
                                                             uint64_t n, int shift,
                                                             uint32_t *__restrict__ counts,
                                                             uint32_t ntiles) {
    __shared__ uint32_t hist[kDigits];
    for (int d = threadIdx.x; d < kDigits; d += kSortThreads) hist[d] = 0;
    __syncthreads();
    const uint64_t base = (uint64_t)blockIdx.x * kSortTile;
    // all of the thread's keys in flight at once, then the per-key matching
    uint32_t kv[kSortItems];
#pragma unroll
    for (int j = 0; j < kSortItems; ++j) {
        const uint64_t i = base + threadIdx.x + j * kSortThreads;
        kv[j] = i < n ? key[i] : 0u;
    }
#pragma unroll
    for (int j = 0; j < kSortItems; ++j) {
        const uint64_t i = base + threadIdx.x + j * kSortThreads;
        const uint32_t d = i < n ? sort_digit(kv[j], shift) : 511u;   // 511: past the end, not counted
        const unsigned peers = __match_any_sync(0xFFFFFFFFu, d);
        if (d < (uint32_t)kDigits && (threadIdx.x & 31) == __ffs(peers) - 1) atomicAdd(&hist[d], __popc(peers));
    }
    __syncthreads();
    for (int d = threadIdx.x; d < kDigits; d += kSortThreads)
        counts[(uint64_t)d * ntiles + blockIdx.x] = hist[d];
}

// Stable scatter, staged through shared memory so that global writes are
// coalesced runs per digit: items are first ranked stably inside the tile
// (warp w owns items [w*512, w*512+512), ranked round by round), placed in
// tile-sorted order in shared memory, then written out sequentially -- item
// i of the sorted tile goes to goff[d] + (i - toff[d]).
__global__ void __launch_bounds__(kSortThreads) k_radix_scatter(Payload pl, uint64_t n, int shift,
                                                                const uint32_t *__restrict__ offs,
                                                                uint32_t ntiles) {
    __shared__ uint32_t wcount[kSortThreads / 32][kDigits];
    __shared__ uint32_t toff[kDigits + 1], goff[kDigits];
    __shared__ uint32_t wsum[kSortThreads / 32];
    __shared__ uint16_t sdig[kSortTile];
    __shared__ uint32_t buf[kSortTile];
    const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
    const uint64_t tile0 = (uint64_t)blockIdx.x * kSortTile;
    const uint64_t seg = tile0 + (uint64_t)w * 32 * kSortItems;
    for (int d = lane; d < kDigits; d += 32) wcount[w][d] = 0;
    __syncwarp();
    uint32_t dig[kSortItems], peers[kSortItems];
#pragma unroll
    for (int j = 0; j < kSortItems; ++j) {                // keys in flight together
        const uint64_t i = seg + j * 32 + lane;
        dig[j] = i < n ? pl.src[0][i] : 0u;
    }
#pragma unroll
    for (int j = 0; j < kSortItems; ++j) {
        const uint64_t i = seg + j * 32 + lane;
        dig[j] = i < n ? sort_digit(dig[j], shift) : 511u;
        peers[j] = __match_any_sync(0xffffffffu, dig[j]);
        if (dig[j] < kDigits && lane == __ffs(peers[j]) - 1) wcount[w][dig[j]] += __popc(peers[j]);
        __syncwarp();
    }
    __syncthreads();
    // tile-local digit offsets: toff = exclusive scan of the tile's digit counts
    const int d0 = threadIdx.x;                 // thread t owns digit t (thread 0 also digit 256)
    // block exclusive scan of `tot` in digit order (thread t holds digit t; thread 0 also 256)
    uint32_t mine = 0;
    for (int ww = 0; ww < kSortThreads / 32; ++ww) mine += (d0 < kDigits) ? wcount[ww][d0] : 0u;
    uint32_t incl = mine;
#pragma unroll
    for (int dd = 1; dd < 32; dd <<= 1) {
        const uint32_t o = __shfl_up_sync(0xffffffffu, incl, dd);
        if (lane >= dd) incl += o;
    }
    if (lane == 31) wsum[w] = incl;
    __syncthreads();
    uint32_t wpre = 0;
    for (int ww = 0; ww < w; ++ww) wpre += wsum[ww];
    toff[d0] = wpre + incl - mine;
    if (d0 == kSortThreads - 1) {
        uint32_t c256 = 0;
        for (int ww = 0; ww < kSortThreads / 32; ++ww) c256 += wcount[ww][256];
        toff[256] = wpre + incl;
        toff[257] = wpre + incl + c256;
    }
    for (int d = d0; d < kDigits; d += kSortThreads) goff[d] = offs[(uint64_t)d * ntiles + blockIdx.x];
    __syncthreads();
    // per (warp, digit) running tile positions
    for (int d = d0; d < kDigits; d += kSortThreads) {
        uint32_t run = toff[d];
#pragma unroll
        for (int ww = 0; ww < kSortThreads / 32; ++ww) {
            const uint32_t t = wcount[ww][d];
            wcount[ww][d] = run;
            run += t;
        }
    }
    __syncthreads();
    const unsigned lt = (1u << lane) - 1u;
    uint32_t lpos[kSortItems];
#pragma unroll
    for (int j = 0; j < kSortItems; ++j) {
        const uint32_t d = dig[j];
        uint32_t pos = 0xFFFFFFFFu;
        if (d < kDigits) pos = wcount[w][d] + __popc(peers[j] & lt);
        __syncwarp();
        if (d < kDigits && lane == __ffs(peers[j]) - 1) wcount[w][d] += __popc(peers[j]);
        __syncwarp();
        lpos[j] = pos;
        if (d < kDigits) sdig[pos] = (uint16_t)d;
    }
    const uint32_t tile_n = (uint32_t)((n - tile0) < (uint64_t)kSortTile ? (n - tile0) : (uint64_t)kSortTile);
    for (int k = 0; k < pl.n; ++k) {
        __syncthreads();                        // buf free (previous column written out)
#pragma unroll
        for (int j = 0; j < kSortItems; ++j) {
            const uint64_t i = seg + j * 32 + lane;
            if (lpos[j] != 0xFFFFFFFFu) buf[lpos[j]] = pl.src[k] ? pl.src[k][i] : (uint32_t)i;
        }
        __syncthreads();
        uint32_t *dst = pl.dst[k];
        for (uint32_t i = threadIdx.x; i < tile_n; i += kSortThreads) {
            const uint32_t d = sdig[i];
            dst[goff[d] + (i - toff[d])] = buf[i];
        }
    }
}

// cell_off[c] = first sorted point of level-10 cell c (Morton order);
// out-of-domain points (sorted last) count as cell kCells10.
__global__ void k_cell_bounds(const uint32_t *__restrict__ qx, const uint32_t *__restrict__ qy,
                              uint64_t n, uint32_t *__restrict__ cell_off) {
    for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i <= n;
         i += (uint64_t)gridDim.x * blockDim.x) {
        const int64_t c = (i < n && qx[i] != kInvalid) ? (int64_t)cell_of(qx[i], qy[i], kMaxLevel)
                                                       : (int64_t)kCells10;
        const int64_t p = i == 0 ? -1
                                 : ((qx[i - 1] != kInvalid) ? (int64_t)cell_of(qx[i - 1], qy[i - 1], kMaxLevel)
                                                            : (int64_t)kCells10);
        for (int64_t cc = p + 1; cc <= c; ++cc) cell_off[cc] = (uint32_t)i;
    }
}

bool is_device_ptr(const void *p) {
    cudaPointerAttributes a;
    if (cudaPointerGetAttributes(&a, p) != cudaSuccess) {
        cudaGetLastError();
        return false;
    }
    return a.type == cudaMemoryTypeDevice || a.type == cudaMemoryTypeManaged;
}
}  // namespace

// Stage a column on the device (copy if host memory). Returns the device pointer.
// Stage a column on the device (copy if host memory) into a grow-only
// context buffer. Returns the device pointer.
static rj_status stage(Ctx *c, const void *p, size_t bytes, Buf &tmp, const void **out, cudaStream_t st = nullptr) {
    if (is_device_ptr(p)) {
        *out = p;
        return RJ_OK;
    }
    if (dreserve_exact(c, tmp, bytes) != cudaSuccess) return set_error(c, RJ_ERR_OOM, "staging allocation failed");
    RJ_CUDA(c, cudaMemcpyAsync(tmp.p, p, bytes, cudaMemcpyHostToDevice, st ? st : c->stream));
    *out = tmp.p;
    return RJ_OK;
}

// Release the load-time scratch (staging and the sort's second buffer).
void free_load_scratch(Ctx *c) {
    for (auto &b : c->load_stage) dfree(c, b);
    for (auto &b : c->load_alt) dfree(c, b);
    dfree(c, c->load_qxy);
}

rj_status load_points_impl(Ctx *c, uint64_t n, const void *x, const void *y, int xy_f64, int n_cols,
                           const void *const *cols, const int32_t *dtypes, uint64_t *n_ood) {
    // the previous point set's columns are reused as the sort's output buffers
    // (grow-only), so reloading same-sized data allocates nothing
    dfree(c, c->cell_off);
    drop_items(c);
    c->n_in = c->n_pts = 0; c->n_cols = 0;
    ++c->data_gen;

    const size_t esz = xy_f64 ? 8 : 4;
    const void *dx = nullptr, *dy = nullptr, *dcol[RJ_MAX_COLS] = {};
    const uint64_t nn = std::max<uint64_t>(n, 1);
    rj_status s;
    if (n) {
        if ((s = stage(c, x, n * esz, c->load_stage[0], &dx)) != RJ_OK) return s;
        if ((s = stage(c, y, n * esz, c->load_stage[1], &dy)) != RJ_OK) return s;
        // the attribute columns are needed only by the final gather: their
        // host-to-device copies run on a second stream beside the sort
        if (n_cols) {
            if (!c->load_stream) {
                RJ_CUDA(c, cudaStreamCreateWithFlags(&c->load_stream, cudaStreamNonBlocking));
                for (auto &e : c->load_ev) RJ_CUDA(c, cudaEventCreateWithFlags(&e, cudaEventDisableTiming));
            }
            RJ_CUDA(c, cudaEventRecord(c->load_ev[0], c->stream));        // staging buffers free
            RJ_CUDA(c, cudaStreamWaitEvent(c->load_stream, c->load_ev[0], 0));
        }
        for (int k = 0; k < n_cols; ++k)
            if ((s = stage(c, cols[k], n * 4, c->load_stage[2 + k], &dcol[k], c->load_stream)) != RJ_OK) return s;
        if (n_cols) RJ_CUDA(c, cudaEventRecord(c->load_ev[1], c->load_stream));
    }
    const int P = 3 + n_cols;
    Buf *B[kMaxPayload] = {&c->qx, &c->qy, &c->idx};
    for (int k = 0; k < n_cols; ++k) B[3 + k] = &c->col[k];
    for (int k = n_cols; k < RJ_MAX_COLS; ++k) dfree(c, c->col[k]);
    Buf *A[kMaxPayload];
    for (int k = 0; k < P; ++k) {
        A[k] = &c->load_alt[k];
        // +8 points of padding: the point pass copies 16-B aligned supersets of ranges
        if (dreserve_exact(c, *A[k], (nn + 8) * 4) != cudaSuccess || dreserve_exact(c, *B[k], (nn + 8) * 4) != cudaSuccess)
            return set_error(c, RJ_ERR_OOM, "point buffers allocation failed");
    }

    if (n) {
        const unsigned qb = (unsigned)std::min<uint64_t>(blocks_for(n, 256), (uint64_t)c->num_sms * 16);
        if (dreserve_exact(c, c->load_qxy, n * 8) != cudaSuccess)
            return set_error(c, RJ_ERR_OOM, "point buffers allocation failed");
        uint2 *qxy = c->load_qxy.as<uint2>();
        if (xy_f64)
            k_quantize<double><<<qb, 256, 0, c->stream>>>((const double *)dx, (const double *)dy, n, c->x0,
                                                          c->x1 - c->x0, c->y0, c->y1 - c->y0, qxy);
        else
            k_quantize<float><<<qb, 256, 0, c->stream>>>((const float *)dx, (const float *)dy, n, c->x0,
                                                         c->x1 - c->x0, c->y0, c->y1 - c->y0, qxy);
        RJ_LAUNCHED(c);
        RJ_CUDA(c, cudaGetLastError());

        const uint32_t ntiles = (uint32_t)((n + kSortTile - 1) / kSortTile);
        Buf &counts = wsbuf(c, kWsSortCounts);
        if (dreserve(c, counts, ((uint64_t)kDigits * ntiles + 1) * 4) != cudaSuccess)
            return set_error(c, RJ_ERR_OOM, "sort counts allocation failed");
        // Sort (key, index) pairs only -- 8 B per point per pass instead of
        // every column -- then gather the columns once.  Buffers: keys
        // ping-pong A[0] <-> A[1], indices B[2] <-> A[2]; pass 0 reads the
        // implicit index.
        k_keys<<<qb, 256, 0, c->stream>>>(qxy, n, A[0]->as<uint32_t>());
        RJ_LAUNCHED(c);
        RJ_CUDA(c, cudaGetLastError());
        uint32_t *key[2] = {A[0]->as<uint32_t>(), A[1]->as<uint32_t>()};
        uint32_t *ix[2] = {A[2]->as<uint32_t>(), B[2]->as<uint32_t>()};
        for (int pass = 0; pass < 4; ++pass) {
            Payload pl;
            pl.n = 2;
            pl.src[0] = key[pass & 1];
            pl.src[1] = pass == 0 ? nullptr : ix[pass & 1];
            pl.dst[0] = key[(pass + 1) & 1];
            pl.dst[1] = ix[(pass + 1) & 1];
            k_radix_hist<<<ntiles, kSortThreads, 0, c->stream>>>(pl.src[0], n, 8 * pass, counts.as<uint32_t>(),
                                                                 ntiles);
            RJ_LAUNCHED(c);
            RJ_CUDA(c, cudaGetLastError());
            RJ_CUDA(c, scan_u32(c, counts.as<uint32_t>(), counts.as<uint32_t>(), (uint64_t)kDigits * ntiles, kWsScan));
            k_radix_scatter<<<ntiles, kSortThreads, 0, c->stream>>>(pl, n, 8 * pass, counts.as<uint32_t>(), ntiles);
            RJ_LAUNCHED(c);
            RJ_CUDA(c, cudaGetLastError());
        }
        // sorted indices in A[2] (pass 3 wrote ix[0]); keys are dead.  Gather
        // qx -> A[0], qy -> A[1], attributes -> B[3 + k], then the context
        // takes A[0..2] as its qx, qy, idx.
        Gather g;
        g.n = n_cols;
        g.qxy = qxy;
        g.qx = A[0]->as<uint32_t>();
        g.qy = A[1]->as<uint32_t>();
        for (int k = 0; k < n_cols; ++k) {
            g.src[k] = (const uint32_t *)dcol[k];
            g.dst[k] = B[3 + k]->as<uint32_t>();
        }
        if (n_cols) RJ_CUDA(c, cudaStreamWaitEvent(c->stream, c->load_ev[1], 0));
        k_gather<<<qb, 256, 0, c->stream>>>(A[2]->as<uint32_t>(), n, g);
        RJ_LAUNCHED(c);
        RJ_CUDA(c, cudaGetLastError());
        std::swap(c->qx, c->load_alt[0]);
        std::swap(c->qy, c->load_alt[1]);
        std::swap(c->idx, c->load_alt[2]);
    }
    for (int k = 0; k < n_cols; ++k) c->col_dtype[k] = dtypes[k];
    c->n_cols = n_cols;
    c->n_in = n;

    if (dalloc(c, c->cell_off, ((uint64_t)kCells10 + 1) * 4) != cudaSuccess)
        return set_error(c, RJ_ERR_OOM, "cell offsets allocation failed");
    {
        const unsigned cb = (unsigned)std::min<uint64_t>(blocks_for(n + 1, 256), (uint64_t)c->num_sms * 16);
        k_cell_bounds<<<cb, 256, 0, c->stream>>>(c->qx.as<uint32_t>(), c->qy.as<uint32_t>(), n,
                                                 c->cell_off.as<uint32_t>());
        RJ_LAUNCHED(c);
        RJ_CUDA(c, cudaGetLastError());
    }
    uint32_t n_valid = 0;
    RJ_CUDA(c, cudaMemcpyAsync(&n_valid, c->cell_off.as<uint32_t>() + kCells10, 4, cudaMemcpyDeviceToHost, c->stream));
    RJ_CUDA(c, cudaStreamSynchronize(c->stream));
    c->n_pts = n_valid;
    ++c->data_gen;
    if (n_ood) *n_ood = n - n_valid;
    if (!c->keep_load_scratch) free_load_scratch(c);
    return RJ_OK;
}

}  // namespace rj
