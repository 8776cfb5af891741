// push.cuh -- host interface of the persistent frontier-push kernel.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

#include "ppr_internal.cuh"

namespace ppr {

#ifndef PPR_PUSH_THREADS
#define PPR_PUSH_THREADS 256
#endif
constexpr int PUSH_THREADS = PPR_PUSH_THREADS;  // one frontier tile = up to PUSH_THREADS entries
#ifndef PPR_PUSH_MIN_BLOCKS
#define PPR_PUSH_MIN_BLOCKS 4
#endif
constexpr int PUSH_MIN_BLOCKS = PPR_PUSH_MIN_BLOCKS;  // resident CTAs per SM (persistent grid = SMs x this)

struct PushArgs {
    DevGraph g;
    void* l2_base;             // persisting L2 window (R and d_out), l2_bytes = 0: none
    size_t l2_bytes;
    float l2_hit;
    DevCtl* ctl;
    unsigned long long* F[2];  // frontier buffers, capacity S*n each
    double* W;                 // Alg 3 snapshot / Alg 4 r_u, aligned with F
    uint32_t* bitmap;          // UniqueEnqueue bits, S*n
    // seeds of each phase's initial frontier (exactly one kind is used)
    const uint32_t* seed_v;    // vertices, crossed with all S sources
    const unsigned int* n_seed_v_dev;  // device count of seed_v (touched list)
    const unsigned long long* seed_e;  // explicit (sidx << 32 | v) entries
    uint64_t n_seed_e;
    int seed_all;              // 1: scan all S*n (Alg 3 lines 1 and 4)
    int phases;                // bit 0: POS, bit 1: NEG
    uint32_t max_iters;        // 0: unlimited (run to eps)
    uint32_t iter_cap;         // safety cap -> KERR_NOCONV
    unsigned long long* ring;  // async mode: ring queue of ring_cap slots, all EMPTY between calls
    unsigned long long ring_cap;
    int hyb_all;               // Opt: every phase runs on the ring from its seeds (dense graphs)
    uint64_t hyb_thresh;       // Opt: a phase whose frontier is <= this many entries finishes on the ring (0: off)
    uint32_t g_lo, g_hi;       // SHARED: source groups [g_lo, g_hi) of this launch (a wave); 0, 0: all
    unsigned long long* trace; // optional: 4 words per round {C | phase<<63, t_ns, edges, -}
    uint32_t trace_cap;        // rounds the trace buffer holds
};

// Launches the cooperative persistent push kernel for `mode` (PPR_MODE_*).
cudaError_t launch_push(int mode, const PushArgs& a, int num_sms, cudaStream_t st);

// The Opt push with 3 edge chains per lane (push_u3.cu; dense graphs).
cudaError_t launch_push_u3(int mode, const PushArgs& a, int num_sms, cudaStream_t st);

// The Opt push with the exactly-once enqueue check (push_chk.cu; PPR_OPT_CHECK_ENQUEUE).
cudaError_t launch_push_chk(int mode, const PushArgs& a, int num_sms, cudaStream_t st);

// PPR_MODE_SHARED: shared-adjacency multi-source push (push_ms.cu).
cudaError_t launch_push_ms(const PushArgs& a, int num_sms, cudaStream_t st);

// PPR_MODE_SORTAGG: host-driven Alg 3 rounds with sort-and-aggregate propagation
// (push_sortagg.cu).  Synchronises the stream once or twice per round.
struct SortAgg;  // scratch owned by the handle, grown on demand
struct SortAggStats {
    unsigned long long pushes = 0, edges = 0, max_frontier = 0;
    unsigned iters[2] = {0, 0};
    int noconv = 0;
    unsigned active_pool = 0;  // in: which slab pool is active
};
cudaError_t sortagg_push(SortAgg** s, const PushArgs& a, uint64_t n_seed_v, cudaStream_t st,
                         SortAggStats* out, uint32_t* launches);
uint64_t sortagg_bytes(const SortAgg* s);
void sortagg_free(SortAgg* s);

}  // namespace ppr
