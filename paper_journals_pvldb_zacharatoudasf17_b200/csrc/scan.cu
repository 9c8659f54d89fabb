// scan.cu -- device exclusive prefix sum (u32) used by every CSR build of
// the path (radix-sort digit offsets, crossings, spans, pieces, edge grid).
// Three-phase: per-block scan of 4096 elements with block totals, recursive
// scan of the totals, add-back.  256 threads x 16 elements per block.
// out[n] receives the total; in == out (in place) is allowed.
#include "rj_internal.cuh"

namespace rj {

namespace {
constexpr int kScanThreads = 256;
constexpr int kScanItems = 16;
constexpr int kScanTile = kScanThreads * kScanItems;

__device__ __forceinline__ uint32_t warp_incl_scan(uint32_t v) {
    const int lane = threadIdx.x & 31;
#pragma unroll
    for (int d = 1; d < 32; d <<= 1) {
        uint32_t o = __shfl_up_sync(0xffffffffu, v, d);
        if (lane >= d) v += o;
    }
    return v;
}

// block-wide exclusive scan of one value per thread; returns the block total
__device__ __forceinline__ uint32_t block_excl_scan(uint32_t v, uint32_t &total) {
    __shared__ uint32_t warp_tot[kScanThreads / 32];
    __shared__ uint32_t tot_s;
    const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
    uint32_t inc = warp_incl_scan(v);
    if (lane == 31) warp_tot[w] = inc;
    __syncthreads();
    if (w == 0) {
        uint32_t t = lane < kScanThreads / 32 ? warp_tot[lane] : 0u;
        uint32_t ti = warp_incl_scan(t);
        if (lane < kScanThreads / 32) warp_tot[lane] = ti - t;
        if (lane == kScanThreads / 32 - 1) tot_s = ti;
    }
    __syncthreads();
    total = tot_s;
    return warp_tot[w] + inc - v;
}

__global__ void __launch_bounds__(kScanThreads) k_scan_tiles(const uint32_t *in,
                                                             uint32_t *out, uint64_t n,
                                                             uint32_t *__restrict__ tile_sums) {
    const uint64_t base = (uint64_t)blockIdx.x * kScanTile + (uint64_t)threadIdx.x * kScanItems;
    uint32_t v[kScanItems];
    uint32_t s = 0;
#pragma unroll
    for (int k = 0; k < kScanItems; ++k) {
        uint64_t i = base + k;
        v[k] = i < n ? in[i] : 0u;
        s += v[k];
    }
    uint32_t total;
    uint32_t pre = block_excl_scan(s, total);
#pragma unroll
    for (int k = 0; k < kScanItems; ++k) {
        uint64_t i = base + k;
        if (i < n) out[i] = pre;
        pre += v[k];
        if (i + 1 == n) out[n] = pre;
    }
    if (threadIdx.x == 0) tile_sums[blockIdx.x] = total;
}

__global__ void __launch_bounds__(kScanThreads) k_scan_add(uint32_t *out, uint64_t n,
                                                           const uint32_t *__restrict__ tile_pre) {
    const uint32_t add = tile_pre[blockIdx.x];
    if (add == 0) return;
    const uint64_t base = (uint64_t)blockIdx.x * kScanTile;
    for (int k = threadIdx.x; k < kScanTile; k += kScanThreads) {
        uint64_t i = base + k;
        if (i < n) out[i] += add;
    }
    if (blockIdx.x == gridDim.x - 1 && threadIdx.x == 0) out[n] += add;
}

__global__ void k_scan_zero(uint32_t *out) { out[0] = 0u; }
}  // namespace

cudaError_t scan_u32(Ctx *c, const uint32_t *in, uint32_t *out, uint64_t n, int ws_base) {
    if (n == 0) {
        k_scan_zero<<<1, 1, 0, c->stream>>>(out);
        RJ_LAUNCHED(c);
        return cudaGetLastError();
    }
    const uint64_t tiles = (n + kScanTile - 1) / kScanTile;
    Buf &sums = wsbuf(c, ws_base);
    cudaError_t e = dreserve(c, sums, (tiles + 1) * sizeof(uint32_t));
    if (e != cudaSuccess) return e;
    k_scan_tiles<<<(unsigned)tiles, kScanThreads, 0, c->stream>>>(in, out, n, sums.as<uint32_t>());
    RJ_LAUNCHED(c);
    if (tiles > 1) {
        Buf &pre = wsbuf(c, ws_base + 1);
        e = dreserve(c, pre, (tiles + 1) * sizeof(uint32_t));
        if (e != cudaSuccess) return e;
        e = scan_u32(c, sums.as<uint32_t>(), pre.as<uint32_t>(), tiles, ws_base + 2);
        if (e != cudaSuccess) return e;
        k_scan_add<<<(unsigned)tiles, kScanThreads, 0, c->stream>>>(out, n, pre.as<uint32_t>());
        RJ_LAUNCHED(c);
    }
    return cudaGetLastError();
}

}  // namespace rj
