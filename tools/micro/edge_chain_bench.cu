// Microbenchmark (dev tool): the push's per-edge access chain in isolation, on
// LJ-shaped arrays, to bound what the edge walk of k_push can reach on a B200.
//
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o edge_chain_bench edge_chain_bench.cu
//
// Each warp walks a coalesced stream of in-list entries (u32 vertex ids, like
// the slab pool) in steps of U x 32 edges; per edge: pool entry -> d_out(v)
// gather -> atomicAdd(&R(v), w / d) with return -> crossing test on the
// returned value (the k_push<OPT> chain, push.cu walk_edges).  Variants:
//   chain 3: pool -> d_out -> atomic (narrow entries, LJ default)
//   chain 2: pool entry carries d_out -> atomic (wide entries)
//   chain 1: atomic only (ids precomputed in registers)
// Target ids are uniform over n, or drawn from the R-MAT-shaped (0.5,0.2,0.2)
// column distribution with the hubs at low ids (the relabelled layout), which
// is what the push sees.  Persistent grid of SMs x 4 CTAs x 256 threads (the
// push's occupancy), R + d_out in the persisting L2 set-aside, pool streamed.
// Prints G edges/s per variant; compare with the push's in-round rate (trace).
#include <cstdio>
#include <cstdint>
#include <vector>
#include <cuda_runtime.h>

__host__ __device__ __forceinline__ uint32_t hash32(uint32_t x) {
    x ^= x >> 16; x *= 0x7feb352du; x ^= x >> 15; x *= 0x846ca68bu; x ^= x >> 16; return x;
}

template <int CHAIN, int U>
__global__ void __launch_bounds__(256, 4) k_walk(const uint32_t* __restrict__ pool, const uint64_t* __restrict__ wpool,
                                                 uint64_t m, const uint32_t* __restrict__ dout, double* R,
                                                 double eps, unsigned long long* hits) {
    const unsigned lane = threadIdx.x & 31u;
    const uint64_t warp = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const uint64_t nwarps = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    unsigned long long h = 0;
    const double w = 1.7e-9;
    for (uint64_t base = warp * 32 * U; base < m; base += nwarps * 32 * U) {
        uint32_t v[U], d[U];
#pragma unroll
        for (int k = 0; k < U; k++) {
            const uint64_t e = base + k * 32 + lane;
            if (CHAIN == 2) {
                const uint64_t x = e < m ? __ldcs(&wpool[e]) : 0ull;
                v[k] = (uint32_t)x;
                d[k] = (uint32_t)(x >> 32);
            } else if (CHAIN == 3) {
                v[k] = e < m ? __ldcs(&pool[e]) : 0u;
            } else {
                v[k] = hash32((uint32_t)e) % 4847571u;
                d[k] = 1u + (v[k] & 7u);
            }
        }
        if (CHAIN == 3) {
#pragma unroll
            for (int k = 0; k < U; k++) d[k] = __ldg(&dout[v[k]]);
        }
        double pre[U], inc[U];
#pragma unroll
        for (int k = 0; k < U; k++) {
            inc[k] = __ddiv_rn(w, (double)d[k]);
            pre[k] = atomicAdd(&R[v[k]], inc[k]);
        }
#pragma unroll
        for (int k = 0; k < U; k++) {
            const double cur = __dadd_rn(pre[k], inc[k]);
            h += (pre[k] <= eps && cur > eps) ? 1u : 0u;
        }
    }
    if (h) atomicAdd(hits, h);
}

int main() {
    const uint32_t n = 4847571;           // LJ-shaped vertex count
    const uint64_t m = 1ull << 27;        // 134 M edges per launch (one batch's pushed edges)
    const uint64_t pool_len = 8u << 20;   // an 8 M-entry pool (LJ window ~6.9 M arcs), walked 16x
    std::vector<uint32_t> hp(pool_len), hd(n);
    std::vector<uint64_t> hw(pool_len);
    for (uint32_t v = 0; v < n; v++) hd[v] = 1u + hash32(v * 7u + 1u) % 8u;
    double* R; uint32_t* dout; uint32_t* pool; uint64_t* wpool; unsigned long long* hits;
    cudaMalloc(&R, sizeof(double) * n);
    cudaMalloc(&dout, sizeof(uint32_t) * n);
    cudaMalloc(&pool, sizeof(uint32_t) * m);
    cudaMalloc(&wpool, sizeof(uint64_t) * m);
    cudaMalloc(&hits, 8);
    cudaMemcpy(dout, hd.data(), sizeof(uint32_t) * n, cudaMemcpyHostToDevice);
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    for (int dist = 0; dist < 2; dist++) {
        // dist 0: uniform ids; dist 1: R-MAT (a+c = 0.7 per bit) column ids, hubs at low ids
        for (uint64_t i = 0; i < pool_len; i++) {
            uint32_t x = hash32((uint32_t)i * 2654435761u + 12345u), v = 0;
            if (dist == 0) {
                v = x % n;
            } else {
                for (int b = 0; b < 23; b++) {
                    const uint32_t r = hash32(x + b * 0x9e3779b9u) % 10u;
                    v = (v << 1) | (r >= 7u ? 1u : 0u);
                }
                v %= n;
            }
            hp[i] = v;
            hw[i] = ((uint64_t)hd[v] << 32) | v;
        }
        for (uint64_t off = 0; off < m; off += pool_len) {
            cudaMemcpy(pool + off, hp.data(), sizeof(uint32_t) * pool_len, cudaMemcpyHostToDevice);
            cudaMemcpy(wpool + off, hw.data(), sizeof(uint64_t) * pool_len, cudaMemcpyHostToDevice);
        }
        cudaMemset(R, 0, sizeof(double) * n);
        auto run = [&](auto kern, const char* name) {
            const int grid = sms * 4;
            kern<<<grid, 256>>>(pool, wpool, m, dout, R, 1e-9, hits);
            cudaDeviceSynchronize();
            cudaEventRecord(e0);
            for (int r = 0; r < 5; r++) kern<<<grid, 256>>>(pool, wpool, m, dout, R, 1e-9, hits);
            cudaEventRecord(e1);
            cudaEventSynchronize(e1);
            float ms = 0;
            cudaEventElapsedTime(&ms, e0, e1);
            printf("%-8s %-28s %6.1f G edges/s (%.3f ms per 2^27 edges)\n", dist ? "rmat" : "uniform", name,
                   5.0 * m / (ms * 1e-3) / 1e9, ms / 5);
        };
        run(k_walk<3, 1>, "pool->dout->atomic U=1");
        run(k_walk<3, 2>, "pool->dout->atomic U=2");
        run(k_walk<3, 4>, "pool->dout->atomic U=4");
        run(k_walk<2, 2>, "wide pool->atomic U=2");
        run(k_walk<2, 4>, "wide pool->atomic U=4");
        run(k_walk<1, 2>, "atomic only U=2");
        run(k_walk<1, 4>, "atomic only U=4");
    }
    cudaError_t e = cudaGetLastError();
    if (e != cudaSuccess) printf("CUDA error: %s\n", cudaGetErrorString(e));
    return 0;
}
