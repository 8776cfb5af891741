// Microbenchmark (dev tool): warp-coalesced fp64 reductions into a vertex-major
// [n][S] residual array, the access pattern of the shared-adjacency
// multi-source push (one warp = 32 sources of one group, one red per lane).
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o ms_atomic_bench ms_atomic_bench.cu
#include <cstdint>
#include <cstdio>
#include <cuda_runtime.h>

__device__ __forceinline__ uint32_t hash(uint32_t x) {
    x ^= x >> 16; x *= 0x7feb352d; x ^= x >> 15; x *= 0x846ca68b; x ^= x >> 16; return x;
}
// ACTIVE lanes of 32 issue a red per warp-op; rows are random (uniform over n,
// or over the first `hot` rows with probability 1/2 to mimic hub reuse)
template <int ACTIVE>
__global__ void k(double* a, uint32_t n, uint32_t S, uint32_t hot, uint64_t iters) {
    const uint32_t lane = threadIdx.x & 31;
    const uint64_t wid = (blockIdx.x * (uint64_t)blockDim.x + threadIdx.x) >> 5;
    const uint32_t G = S / 32;
    for (uint64_t i = 0; i < iters; i++) {
        const uint32_t h = hash((uint32_t)(wid * 2654435761u + i * 40503u + 17));
        uint32_t v = h % n;
        if (hot && (h & 1)) v = (h >> 1) % hot;
        const uint32_t g = (h >> 7) % G;
        const bool on = ACTIVE == 32 || ((hash(h ^ lane) & 31) < ACTIVE);
        if (on) atomicAdd(a + (size_t)v * S + g * 32 + lane, 1e-9);
    }
}
int main() {
    const uint32_t n = 4847571;
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    for (uint32_t S : {32u, 256u}) {
        double* a;
        if (cudaMalloc(&a, (size_t)n * S * 8) != cudaSuccess) return 1;
        cudaMemset(a, 0, (size_t)n * S * 8);
        for (uint32_t hot : {0u, 100000u})
            for (int act : {32, 8, 1}) {
                const int blocks = 148 * 8, threads = 256;
                const uint64_t iters = 256;
                auto launch = [&]() {
                    if (act == 32) k<32><<<blocks, threads>>>(a, n, S, hot, iters);
                    if (act == 8) k<8><<<blocks, threads>>>(a, n, S, hot, iters);
                    if (act == 1) k<1><<<blocks, threads>>>(a, n, S, hot, iters);
                };
                launch();
                cudaDeviceSynchronize();
                cudaEventRecord(e0);
                for (int r = 0; r < 3; r++) launch();
                cudaEventRecord(e1);
                cudaEventSynchronize(e1);
                float ms;
                cudaEventElapsedTime(&ms, e0, e1);
                const double wops = 3.0 * blocks * (threads / 32) * iters;
                printf("S %3u (%6.0f MB) hot %6u active %2d : %7.2f G warp-red/s  %7.1f G lane-red/s\n", S,
                       n * (double)S * 8 / 1e6, hot, act, wops / (ms * 1e-3) / 1e9,
                       wops * act / (ms * 1e-3) / 1e9);
            }
        cudaFree(a);
    }
    return 0;
}
