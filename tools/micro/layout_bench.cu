// Microbenchmark (dev tool, B200): the push's per-edge chain
//   v = pool[e] -> d = d_out(v) -> pre = atomicAdd(&R(v), w / d) -> crossing test
// with R and d_out as two arrays (SoA: two random sectors per edge) or
// interleaved as 16-byte {R, d_out} records (one random sector per edge), for
// an LJ-sized (4.8M) and a Twitter-sized (41.6M) vertex set, uniform or
// skewed (v = n * x^3) targets.
// Build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o layout_bench tools/layout_bench.cu
#include <cstdint>
#include <cstdio>
#include <cuda_runtime.h>

__host__ __device__ __forceinline__ uint32_t hash(uint32_t x) {
    x ^= x >> 16; x *= 0x7feb352d; x ^= x >> 15; x *= 0x846ca68b; x ^= x >> 16; return x;
}

template <bool AOS, int U>
__global__ void __launch_bounds__(256, 4) k(const uint32_t* pool, const uint32_t* dout, double* R, uint64_t npool,
                                            uint64_t iters, unsigned* cnt) {
    const uint64_t tid = blockIdx.x * 256ull + threadIdx.x, nt = gridDim.x * 256ull;
    unsigned c = 0;
    for (uint64_t i = 0; i < iters; i++) {
        uint32_t v[U], d[U];
        double pre[U], inc[U];
#pragma unroll
        for (int j = 0; j < U; j++) v[j] = __ldcs(&pool[(tid + (i * U + j) * nt) % npool]);
#pragma unroll
        for (int j = 0; j < U; j++)
            d[j] = AOS ? __ldcg(reinterpret_cast<const uint32_t*>(R + 2ull * v[j]) + 2) : __ldcg(&dout[v[j]]);
#pragma unroll
        for (int j = 0; j < U; j++) {
            inc[j] = __ddiv_rn(1e-9, (double)d[j]);
            pre[j] = atomicAdd(AOS ? R + 2ull * v[j] : R + v[j], inc[j]);
        }
#pragma unroll
        for (int j = 0; j < U; j++) c += (pre[j] <= 1e-3 && __dadd_rn(pre[j], inc[j]) > 1e-3);
    }
    if (c) atomicAdd(cnt, c);
}

int main() {
    const uint64_t npool = 128ull << 20;
    uint32_t* h = (uint32_t*)malloc(npool * 4);
    uint32_t *pool, *dout;
    double* R;
    unsigned* cnt;
    cudaMalloc(&pool, npool * 4);
    cudaMalloc(&cnt, 4);
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    for (uint32_t n : {4847571u, 41652230u}) {
        cudaMalloc(&dout, n * 4ull);
        cudaMalloc(&R, n * 16ull);
        for (uint32_t i = 0; i < n && i < npool; i++) h[i] = 1 + (hash(i) & 7);
        cudaMemcpy(dout, h, n * 4ull, cudaMemcpyHostToDevice);
        for (int skew = 0; skew < 2; skew++) {
            for (uint64_t i = 0; i < npool; i++) {
                const double x = (hash((uint32_t)i * 2654435761u + 12345u) + 0.5) / 4294967296.0;
                h[i] = skew ? (uint32_t)(n * x * x * x) : (uint32_t)(n * x);
                if (h[i] >= n) h[i] = n - 1;
            }
            cudaMemcpy(pool, h, npool * 4, cudaMemcpyHostToDevice);
            for (int aos = 0; aos < 2; aos++) {
                cudaMemset(R, 0, n * 16ull);
                if (aos) {  // d_out into the records
                    for (uint32_t i = 0; i < n; i++) h[i] = 1 + (hash(i) & 7);
                    uint32_t* rec = (uint32_t*)malloc(n * 16ull);
                    for (uint32_t i = 0; i < n; i++) rec[4ull * i] = rec[4ull * i + 1] = 0, rec[4ull * i + 2] = h[i], rec[4ull * i + 3] = 0;
                    cudaMemcpy(R, rec, n * 16ull, cudaMemcpyHostToDevice);
                    free(rec);
                    // restore the pool host copy for the next skew
                    for (uint64_t i = 0; i < npool; i++) {
                        const double x = (hash((uint32_t)i * 2654435761u + 12345u) + 0.5) / 4294967296.0;
                        h[i] = skew ? (uint32_t)(n * x * x * x) : (uint32_t)(n * x);
                        if (h[i] >= n) h[i] = n - 1;
                    }
                }
                const int grid = 148 * 4;
                const uint64_t iters = 64;
                auto launch = [&]() {
                    if (aos) k<true, 2><<<grid, 256>>>(pool, dout, R, npool, iters / 2, cnt);
                    else k<false, 2><<<grid, 256>>>(pool, dout, R, npool, iters / 2, cnt);
                };
                launch();
                cudaDeviceSynchronize();
                cudaEventRecord(e0);
                for (int r = 0; r < 5; r++) launch();
                cudaEventRecord(e1);
                cudaEventSynchronize(e1);
                float ms;
                cudaEventElapsedTime(&ms, e0, e1);
                const double edges = 5.0 * grid * 256 * iters;
                printf("n %9u %-7s %-18s: %6.1f G edges/s\n", n, skew ? "skewed" : "uniform",
                       aos ? "{R,dout} records" : "R[], dout[] (SoA)", edges / (ms * 1e-3) / 1e9);
            }
        }
        cudaFree(dout);
        cudaFree(R);
    }
    printf("status: %s\n", cudaGetErrorString(cudaDeviceSynchronize()));
    return 0;
}
