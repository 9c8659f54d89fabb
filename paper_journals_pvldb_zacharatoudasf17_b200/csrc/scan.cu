// scan.cu -- device exclusive prefix sum (u32) used by every CSR build of
// the path (radix-sort digit offsets, crossings, spans, pieces, edge grid).
// Single pass with decoupled look-back, 256 threads x 16 elements per block.
// out[n] receives the total; in == out (in place) is allowed.
#include <algorithm>

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

// Single-pass scan with decoupled look-back over up to three arrays in ONE
// launch: every block takes a ticket (so all its predecessors are already
// resident), maps it to (array, tile), scans its 4096-element tile,
// publishes the tile aggregate, then warp 0 walks back over the
// predecessors' status words of the same array 32 at a time until it meets
// an inclusive prefix, and publishes its own.  The status words reset
// themselves: the last block to finish (a second counter) zeroes them, so a
// scan needs no memset node -- consecutive polygon-pass kernels chain with
// programmatic dependent launch (pdl_wait / pdl_trigger).
constexpr unsigned long long kFlagAgg = 1ull << 32, kFlagInc = 2ull << 32;

__device__ __forceinline__ unsigned long long ld_volatile(const unsigned long long *p) {
    return *reinterpret_cast<const volatile unsigned long long *>(p);
}

__global__ void __launch_bounds__(kScanThreads) k_scan_lb(const ScanJobs J, unsigned long long *__restrict__ ws) {
    pdl_wait();
    pdl_trigger();
    __shared__ uint32_t s_tile, s_excl;
    __shared__ int s_last;
    unsigned long long *status = ws + 2;                  // ws[0]: ticket, ws[1]: blocks done
    if (threadIdx.x == 0) s_tile = (uint32_t)atomicAdd(ws, 1ull);
    __syncthreads();
    const uint32_t gt = s_tile;
    int j = 0;
    while (j + 1 < J.nj && gt >= J.tile0[j + 1]) ++j;
    const uint32_t tile = gt - J.tile0[j], ntiles = J.tile0[j + 1] - J.tile0[j];
    const uint32_t *in = J.in[j];
    uint32_t *out = J.out[j];
    const uint64_t n = J.n[j];
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
    unsigned long long *st_j = status + J.tile0[j];
    if (tile == 0) {
        if (threadIdx.x == 0) {
            atomicExch(&st_j[0], kFlagInc | total);
            s_excl = 0;
        }
    } else if (threadIdx.x < 32) {
        const int lane = threadIdx.x;
        if (lane == 0) atomicExch(&st_j[tile], kFlagAgg | total);
        uint32_t excl = 0;
        int64_t jj = (int64_t)tile - 1;
        for (;;) {
            const int64_t k = jj - lane;
            unsigned long long st = k >= 0 ? ld_volatile(&st_j[k]) : kFlagInc;
            while (__any_sync(0xffffffffu, (st >> 32) == 0))
                if ((st >> 32) == 0) st = ld_volatile(&st_j[k]);
            const unsigned inc = __ballot_sync(0xffffffffu, (st >> 32) == 2);
            const int first = inc ? __ffs(inc) - 1 : 32;
            uint32_t c = lane <= first ? (uint32_t)st : 0u;
#pragma unroll
            for (int o = 16; o; o >>= 1) c += __shfl_xor_sync(0xffffffffu, c, o);
            excl += c;
            if (inc) break;
            jj -= 32;
        }
        if (lane == 0) {
            atomicExch(&st_j[tile], kFlagInc | (excl + total));
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
    }
    if (tile == ntiles - 1 && threadIdx.x == 0) out[n] = s_excl + total;
    // the last block to finish (every look-back done) resets the status words
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        s_last = atomicAdd(&ws[1], 1ull) == (unsigned long long)J.tile0[J.nj] - 1;
    }
    __syncthreads();
    if (s_last) {
        __threadfence();
        for (uint32_t k = threadIdx.x; k < J.tile0[J.nj]; k += kScanThreads) status[k] = 0ull;
        if (threadIdx.x == 0) {
            ws[0] = 0ull;
            ws[1] = 0ull;
        }
    }
}
}  // namespace

cudaError_t scan_multi(Ctx *c, int nj, const uint32_t *const *in, uint32_t *const *out, const uint64_t *n,
                       int ws_base) {
    ScanJobs J{};
    J.nj = nj;
    J.tile0[0] = 0;
    for (int j = 0; j < nj; ++j) {
        J.in[j] = in[j];
        J.out[j] = out[j];
        J.n[j] = n[j];
        J.tile0[j + 1] = J.tile0[j] + (uint32_t)std::max<uint64_t>(1, (n[j] + kScanTile - 1) / kScanTile);
    }
    const uint32_t tiles = J.tile0[nj];
    Buf &ws = wsbuf(c, ws_base);
    const size_t need = (tiles + 2) * sizeof(unsigned long long);
    if (ws.bytes < need) {
        // (re)allocated status words start at zero; from then on the scans
        // leave them zero themselves
        cudaError_t e = dreserve(c, ws, need);
        if (e != cudaSuccess) return e;
        e = cudaMemsetAsync(ws.p, 0, ws.bytes, c->stream);
        if (e != cudaSuccess) return e;
    }
    cudaError_t e = launch_pdl(c, k_scan_lb, dim3(tiles), dim3(kScanThreads), 0, J, ws.as<unsigned long long>());
    RJ_LAUNCHED(c);
    return e;
}

cudaError_t scan_u32(Ctx *c, const uint32_t *in, uint32_t *out, uint64_t n, int ws_base) {
    return scan_multi(c, 1, &in, &out, &n, ws_base);
}

}  // namespace rj
