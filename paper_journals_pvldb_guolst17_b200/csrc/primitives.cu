// primitives.cu -- LSD radix sort of (u64, u32) pairs and u32->u64 exclusive
// scan, written for sm_100a without library calls.
//
// Sort pass (8-bit digit, 256 buckets), three kernels:
//   rs_hist     per-CTA digit histogram of a 4096-key tile (shared atomics)
//   rs_scan     one CTA per digit: exclusive scan of that digit's per-tile
//               counts (digit-major, tile-minor) + digit total
//   rs_scatter  per CTA: stable rank of each key inside the tile with
//               __match_any_sync / popc per warp and per-warp digit offsets in
//               shared memory, then a scatter to
//               digit_base + tile_offset + rank.
// Small sorts (n <= 2^18) use 512-key tiles and, with at most 64 tiles,
// fold the offset scan into the scatter (two kernels per pass).
// Keys are read striped (item r of thread t is tile_base + r*256 + t) so
// loads are coalesced and the (round, thread) order is the input order,
// which keeps the sort stable.
#include "primitives.cuh"

#include <map>
#include <mutex>
#include <utility>
#include "block_scan.cuh"

namespace ppr {

// ---------------------------------------------------------------- radix sort

// Lanes of the warp holding the same 8-bit digit d (valid lanes; an invalid
// lane is its own group).  Eight ballots (PPR_RS_MATCH=1: one MATCH.ANY).
__device__ __forceinline__ unsigned digit_peers(uint32_t d, bool valid) {
#if defined(PPR_RS_MATCH) && PPR_RS_MATCH
    (void)valid;
    return __match_any_sync(0xffffffffu, d);
#else
    unsigned peers = __ballot_sync(0xffffffffu, valid);
#pragma unroll
    for (int bit = 0; bit < 8; bit++) {
        const bool x = (d >> bit) & 1u;
        const unsigned b = __ballot_sync(0xffffffffu, x);
        peers &= x ? b : ~b;
    }
    return valid ? peers : (1u << (threadIdx.x & 31u));
#endif
}

template <int ITEMS>
__global__ void __launch_bounds__(RS_THREADS) k_rs_hist(const uint64_t* __restrict__ keys,
                                                        uint64_t n, int shift,
                                                        uint32_t* __restrict__ hist,
                                                        uint32_t ntiles,
                                                        uint32_t* __restrict__ hist_zero = nullptr) {
    __shared__ uint32_t s_h[256];
    if (hist_zero)
        for (uint32_t i = blockIdx.x * RS_THREADS + threadIdx.x; i < 256u * ntiles; i += gridDim.x * RS_THREADS)
            hist_zero[i] = 0u;
    s_h[threadIdx.x] = 0;
    __syncthreads();
    const uint64_t base = (uint64_t)blockIdx.x * RS_THREADS * ITEMS;
#pragma unroll
    for (int r = 0; r < ITEMS; r++) {
        uint64_t i = base + (uint64_t)r * RS_THREADS + threadIdx.x;
        if (i < n) atomicAdd(&s_h[(keys[i] >> shift) & 255u], 1u);
    }
    __syncthreads();
    hist[(uint64_t)threadIdx.x * ntiles + blockIdx.x] = s_h[threadIdx.x];
}

// one CTA per digit: exclusive scan over tiles, digit total in hist[256*ntiles + d]
__global__ void __launch_bounds__(RS_THREADS) k_rs_scan(uint32_t* __restrict__ hist,
                                                        uint32_t ntiles) {
    __shared__ uint32_t s_warp[RS_THREADS / 32 + 1];
    const uint32_t d = blockIdx.x;
    uint32_t* row = hist + (uint64_t)d * ntiles;
    uint32_t carry = 0;
    for (uint32_t b = 0; b < ntiles; b += RS_THREADS) {
        uint32_t i = b + threadIdx.x;
        uint32_t x = i < ntiles ? row[i] : 0u;
        uint32_t tot;
        uint32_t ex = block_exclusive_scan_u32<RS_THREADS>(x, s_warp, &tot);
        if (i < ntiles) row[i] = carry + ex;
        carry += tot;
    }
    if (threadIdx.x == 0) hist[(uint64_t)256 * ntiles + d] = carry;
}

// FUSED: the tile offsets are summed here from the raw per-tile counts
// (ntiles <= RS_FUSED_MAX_TILES), otherwise k_rs_scan has prepared them.
// CHAIN (small sorts, FUSED): the scatter also builds the NEXT pass's per-tile
// histogram -- each key it writes to position pos adds 1 to (next digit, pos's
// tile) of hist_next -- and zeroes hist_zero (the buffer the pass after next will
// fill), so only the first pass needs a histogram kernel.  Three buffers rotate:
// pass p reads H[p % 3], fills H[(p + 1) % 3], zeroes H[(p + 2) % 3].
template <int ITEMS, bool FUSED, bool CHAIN = false>
__global__ void __launch_bounds__(RS_THREADS) k_rs_scatter(
    const uint64_t* __restrict__ kin, const uint32_t* __restrict__ vin,
    uint64_t* __restrict__ kout, uint32_t* __restrict__ vout, uint64_t n, int shift,
    const uint32_t* __restrict__ hist, uint32_t ntiles, int next_shift = -1,
    uint32_t* __restrict__ hist_next = nullptr, uint32_t* __restrict__ hist_zero = nullptr) {
    constexpr int NW = RS_THREADS / 32;
    __shared__ uint32_t s_warp[NW + 1];
    __shared__ uint32_t s_run[256];      // next output position per digit
    __shared__ uint32_t s_wc[NW][256];   // per-warp digit counts this round
    __shared__ uint32_t s_wo[NW][256];   // per-warp digit offsets this round
    const unsigned t = threadIdx.x, lane = t & 31u, warp = t >> 5;
    uint32_t tot_t, pre_t;
    if (FUSED) {
        const uint32_t* row = hist + (uint64_t)t * ntiles;
        tot_t = pre_t = 0;
        for (uint32_t b = 0; b < ntiles; b++) {
            const uint32_t x = row[b];
            tot_t += x;
            pre_t += b < blockIdx.x ? x : 0u;
        }
    } else {
        tot_t = hist[(uint64_t)256 * ntiles + t];
        pre_t = hist[(uint64_t)t * ntiles + blockIdx.x];
    }
    // digit base = exclusive scan of digit totals (thread t owns digit t)
    uint32_t dbase = block_exclusive_scan_u32<RS_THREADS>(tot_t, s_warp, nullptr);
    s_run[t] = dbase + pre_t;
#pragma unroll
    for (int w = 0; w < NW; w++) s_wc[w][t] = 0;
    __syncthreads();
    const uint64_t base = (uint64_t)blockIdx.x * RS_THREADS * ITEMS;
    for (int r = 0; r < ITEMS; r++) {
        uint64_t i = base + (uint64_t)r * RS_THREADS + t;
        bool valid = i < n;
        uint64_t k = valid ? kin[i] : 0ull;
        uint32_t v = valid ? vin[i] : 0u;
        uint32_t d = valid ? (uint32_t)((k >> shift) & 255u) : 256u + lane;  // invalid: unique
        unsigned peers = digit_peers(d, valid);
        unsigned rank = __popc(peers & ((1u << lane) - 1u));
        if (valid && rank == 0) s_wc[warp][d] = __popc(peers);
        __syncthreads();
        {  // thread t: digit t, prefix over warps in order
            uint32_t run = s_run[t];
#pragma unroll
            for (int w = 0; w < NW; w++) {
                uint32_t c = s_wc[w][t];
                s_wo[w][t] = run;
                run += c;
                s_wc[w][t] = 0;
            }
            s_run[t] = run;
        }
        __syncthreads();
        if (valid) {
            uint32_t pos = s_wo[warp][d] + rank;
            kout[pos] = k;
            vout[pos] = v;
            if (CHAIN && next_shift >= 0)
                atomicAdd(&hist_next[(uint64_t)((k >> next_shift) & 255u) * ntiles +
                                     pos / (RS_THREADS * ITEMS)], 1u);
        }
    }
    if (CHAIN && hist_zero)
        for (uint32_t i = blockIdx.x * RS_THREADS + t; i < 256u * ntiles; i += gridDim.x * RS_THREADS)
            hist_zero[i] = 0u;
}

int radix_sort_pairs(uint64_t* k0, uint32_t* v0, uint64_t* k1, uint32_t* v1, uint64_t n,
                     const int* shifts, int npasses, uint32_t* hist, cudaStream_t st,
                     uint32_t* launches) {
    if (n <= 1 || npasses == 0) return 0;
    const uint32_t ntiles = (uint32_t)rs_tiles(n);
    const bool small = rs_items(n) == 2;
    const bool fused = ntiles <= RS_FUSED_MAX_TILES;
    uint64_t *ki = k0, *ko = k1;
    uint32_t *vi = v0, *vo = v1;
    int where = 0;
    if (small && fused) {  // chained passes: one histogram kernel, then one scatter per pass
        const uint64_t stride = 256ull * (ntiles + 1);
        uint32_t* H[3] = {hist, hist + stride, hist + 2 * stride};
        k_rs_hist<2><<<ntiles, RS_THREADS, 0, st>>>(ki, n, shifts[0], H[0], ntiles, H[1]);
        ++*launches;
        for (int p = 0; p < npasses; p++) {
            const bool last = p + 1 == npasses;
            k_rs_scatter<2, true, true><<<ntiles, RS_THREADS, 0, st>>>(
                ki, vi, ko, vo, n, shifts[p], H[p % 3], ntiles, last ? -1 : shifts[p + 1],
                H[(p + 1) % 3], last ? nullptr : H[(p + 2) % 3]);
            ++*launches;
            uint64_t* tk = ki;
            ki = ko;
            ko = tk;
            uint32_t* tv = vi;
            vi = vo;
            vo = tv;
            where ^= 1;
        }
        return where;
    }
    for (int p = 0; p < npasses; p++) {
        if (small) {
            k_rs_hist<2><<<ntiles, RS_THREADS, 0, st>>>(ki, n, shifts[p], hist, ntiles);
            if (fused) {
                k_rs_scatter<2, true><<<ntiles, RS_THREADS, 0, st>>>(ki, vi, ko, vo, n, shifts[p],
                                                                     hist, ntiles);
            } else {
                k_rs_scan<<<256, RS_THREADS, 0, st>>>(hist, ntiles);
                k_rs_scatter<2, false><<<ntiles, RS_THREADS, 0, st>>>(ki, vi, ko, vo, n,
                                                                      shifts[p], hist, ntiles);
                ++*launches;
            }
        } else {
            k_rs_hist<16><<<ntiles, RS_THREADS, 0, st>>>(ki, n, shifts[p], hist, ntiles);
            k_rs_scan<<<256, RS_THREADS, 0, st>>>(hist, ntiles);
            k_rs_scatter<16, false><<<ntiles, RS_THREADS, 0, st>>>(ki, vi, ko, vo, n, shifts[p],
                                                                   hist, ntiles);
            ++*launches;
        }
        *launches += 2;
        uint64_t* tk = ki;
        ki = ko;
        ko = tk;
        uint32_t* tv = vi;
        vi = vo;
        vo = tv;
        where ^= 1;
    }
    return where;
}

int key_shifts(int bits, int* shifts) {
    int np = 0;
    for (int s = 0; s < bits; s += 8) shifts[np++] = s;
    for (int s = 0; s < bits; s += 8) shifts[np++] = 32 + s;
    return np;
}

// ---------------------------------------------------------------- scan

__global__ void __launch_bounds__(SCAN_THREADS) k_scan_reduce(const uint32_t* __restrict__ in,
                                                              uint64_t n,
                                                              unsigned long long* __restrict__ part) {
    __shared__ unsigned long long s_warp[SCAN_THREADS / 32 + 1];
    const uint64_t base = (uint64_t)blockIdx.x * SCAN_TILE;
    unsigned long long s = 0;
#pragma unroll
    for (int r = 0; r < SCAN_ITEMS; r++) {
        uint64_t i = base + (uint64_t)r * SCAN_THREADS + threadIdx.x;
        if (i < n) s += in[i];
    }
    unsigned long long tot;
    block_exclusive_scan_u64<SCAN_THREADS>(s, s_warp, &tot);
    if (threadIdx.x == 0) part[blockIdx.x] = tot;
}

__global__ void __launch_bounds__(SCAN_THREADS) k_scan_part(unsigned long long* __restrict__ part,
                                                            uint64_t np,
                                                            unsigned long long* __restrict__ total) {
    __shared__ unsigned long long s_warp[SCAN_THREADS / 32 + 1];
    unsigned long long carry = 0;
    for (uint64_t b = 0; b < np; b += SCAN_THREADS) {
        uint64_t i = b + threadIdx.x;
        unsigned long long x = i < np ? part[i] : 0ull;
        unsigned long long tot;
        unsigned long long ex = block_exclusive_scan_u64<SCAN_THREADS>(x, s_warp, &tot);
        if (i < np) part[i] = carry + ex;
        carry += tot;
    }
    if (threadIdx.x == 0) *total = carry;
}

__global__ void __launch_bounds__(SCAN_THREADS) k_scan_down(const uint32_t* __restrict__ in,
                                                            uint64_t n,
                                                            const unsigned long long* __restrict__ part,
                                                            unsigned long long* __restrict__ out) {
    __shared__ unsigned long long s_warp[SCAN_THREADS / 32 + 1];
    const uint64_t base = (uint64_t)blockIdx.x * SCAN_TILE + (uint64_t)threadIdx.x * SCAN_ITEMS;
    uint32_t x[SCAN_ITEMS];
    unsigned long long s = 0;
#pragma unroll
    for (int r = 0; r < SCAN_ITEMS; r++) {
        uint64_t i = base + r;
        x[r] = i < n ? in[i] : 0u;
        s += x[r];
    }
    unsigned long long ex = block_exclusive_scan_u64<SCAN_THREADS>(s, s_warp, nullptr);
    unsigned long long run = part[blockIdx.x] + ex;
#pragma unroll
    for (int r = 0; r < SCAN_ITEMS; r++) {
        uint64_t i = base + r;
        if (i < n) out[i] = run;
        run += x[r];
    }
}

void exclusive_scan_u32(const uint32_t* in, unsigned long long* out, uint64_t n,
                        unsigned long long* part, unsigned long long* total, cudaStream_t st,
                        uint32_t* launches) {
    uint64_t np = scan_parts(n);
    if (np == 0) {
        cudaMemsetAsync(total, 0, sizeof(unsigned long long), st);
        return;
    }
    k_scan_reduce<<<(unsigned)np, SCAN_THREADS, 0, st>>>(in, n, part);
    k_scan_part<<<1, SCAN_THREADS, 0, st>>>(part, np, total);
    k_scan_down<<<(unsigned)np, SCAN_THREADS, 0, st>>>(in, n, part, out);
    *launches += 3;
}

cudaError_t blocks_per_sm(const void* fn, int threads, int cap, int* out) {
    static std::mutex mu;
    static std::map<std::pair<int, const void*>, int> cache;
    int dev = 0;
    cudaError_t e = cudaGetDevice(&dev);
    if (e != cudaSuccess) return e;
    const auto key = std::make_pair(dev, fn);
    {
        std::lock_guard<std::mutex> lk(mu);
        auto it = cache.find(key);
        if (it != cache.end()) {
            *out = it->second;
            return cudaSuccess;
        }
    }
    int b = 0;
    e = cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, fn, threads, 0);
    if (e != cudaSuccess) return e;
    if (b < 1) return cudaErrorInvalidConfiguration;
    if (b > cap) b = cap;
    std::lock_guard<std::mutex> lk(mu);
    cache[key] = b;
    *out = b;
    return cudaSuccess;
}

}  // namespace ppr
