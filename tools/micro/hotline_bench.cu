// Microbenchmark (dev tool, B200): costs of the push kernel's hot lines.
//   1. grid barrier over a persistent cooperative grid (148 SMs x 4 CTAs x 256
//      threads): the generation barrier of ppr_internal.cuh with several poll
//      back-offs, and a two-level (group) variant;
//   2. same-address atomicAdd with return issued by one thread per CTA / per
//      warp (the tile-claim and frontier-flush counters);
//   3. same-address loads by one thread per warp (polling).
// Build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o hotline_bench tools/hotline_bench.cu
#include <cooperative_groups.h>
#include <cstdint>
#include <cstdio>
#include <cuda_runtime.h>

struct __align__(128) Line { unsigned int v; unsigned int pad[31]; };
struct Ctl { Line count, gen, grp_count[64], grp_gen[64]; unsigned long long ctr[16]; };

__device__ __forceinline__ unsigned ld_acq(const unsigned* p) {
    unsigned v;
    asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ void st_rel(unsigned* p, unsigned v) {
    asm volatile("st.release.gpu.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}

template <int SLEEP>
__device__ __forceinline__ void bar_flat(Ctl* c) {
    __syncthreads();
    if (threadIdx.x == 0) {
        unsigned gen = ld_acq(&c->gen.v);
        __threadfence();
        if (atomicAdd(&c->count.v, 1u) + 1u == gridDim.x) {
            c->count.v = 0;
            __threadfence();
            st_rel(&c->gen.v, gen + 1u);
        } else {
            while (ld_acq(&c->gen.v) == gen)
                if (SLEEP) __nanosleep(SLEEP);
        }
        __threadfence();
    }
    __syncthreads();
}

// two levels: groups of G CTAs arrive on their own line; the last of a group
// arrives at the top; every CTA polls the global generation
template <int G>
__device__ __forceinline__ void bar_tree(Ctl* c) {
    __syncthreads();
    if (threadIdx.x == 0) {
        const unsigned g = blockIdx.x / G, ng = (gridDim.x + G - 1) / G;
        const unsigned gsz = (g + 1) * G <= gridDim.x ? G : gridDim.x - g * G;
        unsigned gen = ld_acq(&c->gen.v);
        __threadfence();
        bool top = false;
        if (atomicAdd(&c->grp_count[g].v, 1u) + 1u == gsz) {
            c->grp_count[g].v = 0;
            if (atomicAdd(&c->count.v, 1u) + 1u == ng) {
                c->count.v = 0;
                __threadfence();
                st_rel(&c->gen.v, gen + 1u);
                top = true;
            }
        }
        if (!top)
            while (ld_acq(&c->gen.v) == gen) __nanosleep(32);
        __threadfence();
    }
    __syncthreads();
}

template <int V>
__global__ void __launch_bounds__(256, 4) k_bar(Ctl* c, int iters) {
    for (int i = 0; i < iters; i++) {
        if (V == 0) bar_flat<32>(c);
        if (V == 1) bar_flat<0>(c);
        if (V == 2) bar_flat<256>(c);
        if (V == 3) bar_tree<8>(c);
        if (V == 4) bar_tree<16>(c);
    }
}

// same-address atomics: `who` = 0: thread 0 of each CTA, 1: lane 0 of each warp;
// each issuer does `iters` dependent atomicAdd-with-return on one counter
__global__ void __launch_bounds__(256, 4) k_atom(Ctl* c, int iters, int who, int nctr) {
    const bool me = who == 0 ? threadIdx.x == 0 : (threadIdx.x & 31) == 0;
    if (!me) return;
    const unsigned id = blockIdx.x * 8 + threadIdx.x / 32;
    unsigned long long* p = &c->ctr[(id % nctr) * 1];  // 8-byte stride: same line when nctr small
    unsigned long long acc = 0;
    for (int i = 0; i < iters; i++) acc += atomicAdd(p + (acc & 0), 1ull);
    if (acc == 42) c->ctr[15] = acc;
}

// same-address polling loads: lane 0 of each warp, `iters` dependent volatile loads
__global__ void __launch_bounds__(256, 4) k_poll(Ctl* c, int iters) {
    if (threadIdx.x & 31) return;
    unsigned acc = 0;
    for (int i = 0; i < iters; i++) acc += *(volatile unsigned*)(&c->gen.v + (acc & 0));
    if (acc == 12345) c->count.pad[0] = acc;
}

int main() {
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    const int grid = sms * 4;
    Ctl* c;
    cudaMalloc(&c, sizeof(Ctl));
    cudaMemset(c, 0, sizeof(Ctl));
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    const char* names[] = {"flat poll sleep32", "flat poll spin", "flat poll sleep256", "tree G=8", "tree G=16"};
    void* fns[] = {(void*)k_bar<0>, (void*)k_bar<1>, (void*)k_bar<2>, (void*)k_bar<3>, (void*)k_bar<4>};
    for (int v = 0; v < 5; v++) {
        for (int rep = 0; rep < 2; rep++) {
            int iters = 2000;
            void* args[] = {&c, &iters};
            cudaEventRecord(e0);
            cudaLaunchCooperativeKernel(fns[v], grid, 256, args, 0, 0);
            cudaEventRecord(e1);
            cudaEventSynchronize(e1);
            float ms;
            cudaEventElapsedTime(&ms, e0, e1);
            if (rep) printf("barrier %-20s grid %d: %.3f us per barrier\n", names[v], grid, ms * 1e3 / iters);
        }
    }
    for (int who = 0; who < 2; who++) {
        for (int nctr : {1, 8}) {
            int iters = 200;
            k_atom<<<grid, 256>>>(c, iters, who, nctr);
            cudaEventRecord(e0);
            k_atom<<<grid, 256>>>(c, iters, who, nctr);
            cudaEventRecord(e1);
            cudaEventSynchronize(e1);
            float ms;
            cudaEventElapsedTime(&ms, e0, e1);
            const double ops = (double)iters * grid * (who ? 8 : 1);
            printf("same-address atomicAdd, issuers = %s, %d counter(s) on one line: %.0f ops in %.3f ms = %.2f ns/op (%.1f M/s)\n",
                   who ? "lane 0 of every warp" : "thread 0 of every CTA", nctr, ops, ms, ms * 1e6 / ops, ops / ms / 1e3);
        }
    }
    {
        int iters = 200;
        k_poll<<<grid, 256>>>(c, iters);
        cudaEventRecord(e0);
        k_poll<<<grid, 256>>>(c, iters);
        cudaEventRecord(e1);
        cudaEventSynchronize(e1);
        float ms;
        cudaEventElapsedTime(&ms, e0, e1);
        const double ops = (double)iters * grid * 8;
        printf("same-address volatile loads, lane 0 of every warp: %.0f loads in %.3f ms = %.2f ns/load (%.1f M/s)\n", ops, ms,
               ms * 1e6 / ops, ops / ms / 1e3);
    }
    cudaError_t e = cudaDeviceSynchronize();
    printf("status: %s\n", cudaGetErrorString(e));
    return 0;
}
