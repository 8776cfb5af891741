// Microbenchmark: random fp64 atomicAdd throughput on the B200 (dev tool).
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o atomic_bench atomic_bench.cu
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

__device__ __forceinline__ uint32_t hash(uint32_t x) {
    x ^= x >> 16; x *= 0x7feb352d; x ^= x >> 15; x *= 0x846ca68b; x ^= x >> 16; return x;
}
template <int MODE>  // 0: atomicAdd with return, 1: red (no return), 2: plain load, 3: load + atomic (2 deps)
__global__ void k(double* a, uint32_t n, uint32_t stride, uint64_t iters, double* sink) {
    uint64_t tid = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x;
    double acc = 0;
    for (uint64_t i = 0; i < iters; i++) {
        uint32_t idx = hash((uint32_t)(tid * 1315423911u + i * 2654435761u)) % n;
        double* p = a + (size_t)idx * stride;
        if (MODE == 0) acc += atomicAdd(p, 1e-9);
        else if (MODE == 1) atomicAdd(p, 1e-9);
        else if (MODE == 2) acc += __ldcg(p);
        else { double x = __ldcg(p + 1); acc += atomicAdd(p, x * 1e-9); }
    }
    if (acc == 12345.0) *sink = acc;
}
int main() {
    const uint32_t n = 4847571;
    double* a; double* sink;
    cudaMalloc(&a, (size_t)n * 4 * sizeof(double));
    cudaMalloc(&sink, 8);
    cudaMemset(a, 0, (size_t)n * 4 * sizeof(double));
    cudaEvent_t e0, e1; cudaEventCreate(&e0); cudaEventCreate(&e1);
    for (int stride : {1, 4}) for (int mode = 0; mode < 4; mode++) for (int threads : {256 * 148 * 4, 256 * 148 * 8}) {
        uint64_t iters = 64;
        auto launch = [&]() {
            int blocks = threads / 256;
            if (mode == 0) k<0><<<blocks, 256>>>(a, n, stride, iters, sink);
            if (mode == 1) k<1><<<blocks, 256>>>(a, n, stride, iters, sink);
            if (mode == 2) k<2><<<blocks, 256>>>(a, n, stride, iters, sink);
            if (mode == 3) k<3><<<blocks, 256>>>(a, n, stride, iters, sink);
        };
        launch(); cudaDeviceSynchronize();
        cudaEventRecord(e0); for (int r = 0; r < 5; r++) launch(); cudaEventRecord(e1); cudaEventSynchronize(e1);
        float ms; cudaEventElapsedTime(&ms, e0, e1);
        double ops = 5.0 * threads * iters;
        printf("stride %d (%5.0f MB) mode %d threads %7d : %6.1f Gop/s\n", stride, n * stride * 8 / 1e6, mode, threads, ops / (ms * 1e-3) / 1e9);
    }
    return 0;
}
