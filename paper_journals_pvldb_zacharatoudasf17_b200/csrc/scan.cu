// scan.cu -- device exclusive prefix sum (u32) used by every CSR build of
// the path (radix-sort digit offsets, crossings, spans, pieces, edge grid).
// Single pass with decoupled look-back, 256 threads x 16 elements per block.
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

// Single-pass scan with decoupled look-back: every block takes a ticket (so
// all its predecessors are already resident), scans its 4096-element tile,
// publishes the tile aggregate, then warp 0 walks back over the predecessors'
// status words 32 at a time until it meets an inclusive prefix, and
// publishes its own.  One memset + one launch per scan instead of a
// recursive three-phase scan (the polygon pass runs six of them per query).
constexpr unsigned long long kFlagAgg = 1ull << 32, kFlagInc = 2ull << 32;

__device__ __forceinline__ unsigned long long ld_volatile(const unsigned long long *p) {
    return *reinterpret_cast<const volatile unsigned long long *>(p);
}

__global__ void __launch_bounds__(kScanThreads) k_scan_lb(const uint32_t *in, uint32_t *out, uint64_t n,
                                                          unsigned long long *__restrict__ ws) {
    __shared__ uint32_t s_tile, s_excl;
    unsigned long long *status = ws + 1;                  // ws[0]: ticket
    if (threadIdx.x == 0) s_tile = (uint32_t)atomicAdd(ws, 1ull);
    __syncthreads();
    const uint32_t tile = s_tile;
    const uint64_t base = (uint64_t)tile * kScanTile + (uint64_t)threadIdx.x * kScanItems;
    uint32_t v[kScanItems];
    uint32_t sum = 0;
#pragma unroll
    for (int k = 0; k < kScanItems; ++k) {
        const uint64_t i = base + k;
        v[k] = i < n ? in[i] : 0u;
        sum += v[k];
    }
    uint32_t total;
    uint32_t pre = block_excl_scan(sum, total);
    if (tile == 0) {
        if (threadIdx.x == 0) {
            atomicExch(&status[0], kFlagInc | total);
            s_excl = 0;
        }
    } else if (threadIdx.x < 32) {
        const int lane = threadIdx.x;
        if (lane == 0) atomicExch(&status[tile], kFlagAgg | total);
        uint32_t excl = 0;
        int64_t j = (int64_t)tile - 1;
        for (;;) {
            const int64_t k = j - lane;
            unsigned long long st = k >= 0 ? ld_volatile(&status[k]) : kFlagInc;
            while (__any_sync(0xffffffffu, (st >> 32) == 0))
                if ((st >> 32) == 0) st = ld_volatile(&status[k]);
            const unsigned inc = __ballot_sync(0xffffffffu, (st >> 32) == 2);
            const int first = inc ? __ffs(inc) - 1 : 32;
            uint32_t c = lane <= first ? (uint32_t)st : 0u;
#pragma unroll
            for (int o = 16; o; o >>= 1) c += __shfl_xor_sync(0xffffffffu, c, o);
            excl += c;
            if (inc) break;
            j -= 32;
        }
        if (lane == 0) {
            atomicExch(&status[tile], kFlagInc | (excl + total));
            s_excl = excl;
        }
    }
    __syncthreads();
    pre += s_excl;
#pragma unroll
    for (int k = 0; k < kScanItems; ++k) {
        const uint64_t i = base + k;
        if (i < n) out[i] = pre;
        pre += v[k];
        if (i + 1 == n) out[n] = pre;
    }
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
    Buf &ws = wsbuf(c, ws_base);
    cudaError_t e = dreserve(c, ws, (tiles + 1) * sizeof(unsigned long long));
    if (e != cudaSuccess) return e;
    e = cudaMemsetAsync(ws.p, 0, (tiles + 1) * sizeof(unsigned long long), c->stream);
    if (e != cudaSuccess) return e;
    k_scan_lb<<<(unsigned)tiles, kScanThreads, 0, c->stream>>>(in, out, n, ws.as<unsigned long long>());
    RJ_LAUNCHED(c);
    return cudaGetLastError();
}

}  // namespace rj
