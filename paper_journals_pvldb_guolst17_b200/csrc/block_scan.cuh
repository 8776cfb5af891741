// block_scan.cuh -- CTA-wide exclusive scans (warp shuffles + one shared
// array of per-warp totals).  s_warp needs NT/32 + 1 entries.
#pragma once
#include <cstdint>

namespace ppr {

template <int NT>
__device__ __forceinline__ uint32_t block_exclusive_scan_u32(uint32_t x, uint32_t* s_warp,
                                                             uint32_t* total) {
    const unsigned lane = threadIdx.x & 31u, warp = threadIdx.x >> 5;
    uint32_t inc = x;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
        uint32_t y = __shfl_up_sync(0xffffffffu, inc, o);
        if (lane >= (unsigned)o) inc += y;
    }
    if (lane == 31) s_warp[warp] = inc;
    __syncthreads();
    if (warp == 0) {
        constexpr int NW = NT / 32;
        uint32_t w = lane < NW ? s_warp[lane] : 0u;
        uint32_t wi = w;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            uint32_t y = __shfl_up_sync(0xffffffffu, wi, o);
            if (lane >= (unsigned)o) wi += y;
        }
        if (lane < NW) s_warp[lane] = wi - w;
        if (lane == NW - 1) s_warp[NW] = wi;
    }
    __syncthreads();
    uint32_t res = s_warp[warp] + inc - x;
    if (total) *total = s_warp[NT / 32];
    __syncthreads();
    return res;
}

template <int NT>
__device__ __forceinline__ unsigned long long block_exclusive_scan_u64(unsigned long long x,
                                                                       unsigned long long* s_warp,
                                                                       unsigned long long* total) {
    const unsigned lane = threadIdx.x & 31u, warp = threadIdx.x >> 5;
    unsigned long long inc = x;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
        unsigned long long y = __shfl_up_sync(0xffffffffu, inc, o);
        if (lane >= (unsigned)o) inc += y;
    }
    if (lane == 31) s_warp[warp] = inc;
    __syncthreads();
    if (warp == 0) {
        constexpr int NW = NT / 32;
        unsigned long long w = lane < NW ? s_warp[lane] : 0ull;
        unsigned long long wi = w;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            unsigned long long y = __shfl_up_sync(0xffffffffu, wi, o);
            if (lane >= (unsigned)o) wi += y;
        }
        if (lane < NW) s_warp[lane] = wi - w;
        if (lane == NW - 1) s_warp[NW] = wi;
    }
    __syncthreads();
    unsigned long long res = s_warp[warp] + inc - x;
    if (total) *total = s_warp[NT / 32];
    __syncthreads();
    return res;
}

}  // namespace ppr
