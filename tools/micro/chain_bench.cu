// Microbenchmark of the push's per-edge chain on the B200 (dev tool):
//   v = pool[e] (streamed u32) -> d = dout[v] (random u32, 19 MB)
//   -> inc = w / d -> pre = atomicAdd(&R[v], inc) (random f64, 39 MB) -> test pre
// U independent chains per thread; grid = 148 SMs x BLOCKS x 256 threads.
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>
__host__ __device__ __forceinline__ uint32_t hash(uint32_t x) {
    x ^= x >> 16; x *= 0x7feb352d; x ^= x >> 15; x *= 0x846ca68b; x ^= x >> 16; return x;
}
template <int U>
__global__ void __launch_bounds__(256) k(const uint32_t* pool, const uint32_t* dout, double* R,
                                         uint64_t npool, uint64_t iters, unsigned* cnt) {
    const uint64_t tid = blockIdx.x * 256ull + threadIdx.x, nt = gridDim.x * 256ull;
    unsigned c = 0;
    for (uint64_t i = 0; i < iters; i++) {
        uint32_t v[U], d[U];
        double pre[U], inc[U];
#pragma unroll
        for (int k = 0; k < U; k++) v[k] = __ldg(&pool[(tid + (i * U + k) * nt) % npool]);
#pragma unroll
        for (int k = 0; k < U; k++) d[k] = __ldg(&dout[v[k]]);
#pragma unroll
        for (int k = 0; k < U; k++) { inc[k] = 1e-9 / (double)d[k]; pre[k] = atomicAdd(&R[v[k]], inc[k]); }
#pragma unroll
        for (int k = 0; k < U; k++) c += (pre[k] <= 1e-3 && pre[k] + inc[k] > 1e-3);
    }
    if (c) atomicAdd(cnt, c);
}
int main() {
    const uint32_t n = 4847571; const uint64_t npool = 64ull << 20;
    uint32_t *pool, *dout; double* R; unsigned* cnt;
    cudaMalloc(&pool, npool * 4); cudaMalloc(&dout, n * 4); cudaMalloc(&R, n * 8); cudaMalloc(&cnt, 4);
    uint32_t* h = (uint32_t*)malloc(npool * 4);
    for (uint64_t i = 0; i < npool; i++) h[i] = (uint32_t)((i * 2654435761ull + (i >> 7) * 97) % n);
    cudaMemcpy(pool, h, npool * 4, cudaMemcpyHostToDevice);
    for (uint32_t i = 0; i < n; i++) h[i] = 1 + (hash(i) & 7);
    cudaMemcpy(dout, h, n * 4, cudaMemcpyHostToDevice);
    cudaMemset(R, 0, n * 8);
    cudaEvent_t e0, e1; cudaEventCreate(&e0); cudaEventCreate(&e1);
    for (int blocks : {4, 8}) for (int U : {1, 2, 4, 8}) {
        int grid = 148 * blocks; uint64_t iters = 32 / U;
        auto launch = [&]() {
            if (U == 1) k<1><<<grid, 256>>>(pool, dout, R, npool, iters, cnt);
            if (U == 2) k<2><<<grid, 256>>>(pool, dout, R, npool, iters, cnt);
            if (U == 4) k<4><<<grid, 256>>>(pool, dout, R, npool, iters, cnt);
            if (U == 8) k<8><<<grid, 256>>>(pool, dout, R, npool, iters, cnt);
        };
        launch(); cudaDeviceSynchronize();
        cudaEventRecord(e0); for (int r = 0; r < 10; r++) launch(); cudaEventRecord(e1); cudaEventSynchronize(e1);
        float ms; cudaEventElapsedTime(&ms, e0, e1);
        double edges = 10.0 * grid * 256 * iters * U;
        printf("blocks/SM %d U %d : %6.1f G edges/s\n", blocks, U, edges / (ms * 1e-3) / 1e9);
    }
    return 0;
}
