// store.cuh -- dynamic graph store (step a1) and invariant restore (step a2):
// kernel launchers used by the orchestrator in ppr_api.cu.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

#include "ppr_internal.cuh"

namespace ppr {

constexpr uint32_t NONE = 0xFFFFFFFFu;

// Scratch for one batch of N sort entries (arcs after undirected expansion).
struct BatchBufs {
    uint64_t* kv[2];   // keys (v << 32 | u), sorted for the store
    uint32_t* ov[2];   // op code (0: delete, 1: no-op, 2: insert)
    uint64_t* ku[2];   // keys (u << 32 | v), sorted for the restore
    uint32_t* ou[2];
    uint32_t* hist;    // radix-sort scratch (store order)
    uint32_t* hist2;   // radix-sort scratch (restore order, sorted concurrently)
    int32_t* rnv;      // net multiplicity change at each run head (v-sorted)
    int32_t* rnu;      // same, u-sorted
    uint32_t* vheads;  // v-segment heads
    uint32_t* uheads;  // u-segment heads
    uint32_t* claim;   // deletion claims per run head
    uint32_t* delpos;  // slab positions of claimed deletions, per segment
    uint32_t* seg_end; // per v-segment head: end index
    uint32_t* seg_D;   // deletions claimed
    uint32_t* seg_I;   // insertions
};

// Per-vertex scratch (size n) for rebuild and create.
struct VertexBufs {
    uint32_t* vseg;    // v -> its segment head in the current batch, NONE otherwise
    uint32_t* newcap;  // rebuild / build capacities
    unsigned long long* newoff;
    unsigned long long* part;  // scan partials
    uint32_t* big;     // vertices copied warp-wide in a rebuild
    uint32_t* touched; // distinct u restored this batch
};

struct StoreParams {
    double slack;
    uint32_t min_cap;
    uint64_t cap0, cap1;  // pool capacities; the rebuild targets the one not active on the device
};

void launch_ctl_reset(DevCtl* ctl, cudaStream_t st, uint32_t* launches);

// a0: keys of both sort orders + id range check
void launch_batch_keys(const uint32_t* is, const uint32_t* id, uint64_t n_ins, const uint32_t* ds,
                       const uint32_t* dd, uint64_t n_del, int undirected, uint32_t n,
                       const BatchBufs& b, int slot, DevCtl* ctl, const uint32_t* perm,
                       cudaStream_t st, uint32_t* launches);

// run nets + segment heads of a sorted key array
void launch_heads(const uint64_t* keys, const uint32_t* ops, uint64_t N, int32_t* run_net,
                  uint32_t* heads, unsigned int* nheads, cudaStream_t st, uint32_t* launches);

// a1: validate deletions (claims), decide in-place vs rebuild
void launch_store_validate(const DevGraph& g, const uint64_t* kv, uint64_t N, const BatchBufs& b,
                           const VertexBufs& vb, DevCtl* ctl, int force_rebuild, cudaStream_t st,
                           uint32_t* launches);
// a1: in-place slab update (skipped on error or rebuild)
void launch_store_apply(const DevGraph& g, const uint64_t* kv, uint64_t N, const BatchBufs& b,
                        DevCtl* ctl, cudaStream_t st, uint32_t* launches);
// a1: sort/merge rebuild into the other pool (skipped unless DevCtl::rebuild)
// (finish: also reset the v -> segment map and refresh the degrees cached in the
// pool entries after the restore -- the last launch of every batch's store pipeline)
cudaError_t launch_store_rebuild(const DevGraph& g, const uint64_t* kv, uint64_t N, const BatchBufs& b,
                                 const VertexBufs& vb, const StoreParams& sp, DevCtl* ctl,
                                 cudaStream_t st, uint32_t* launches, bool finish);
// Degree refresh of wide pool entries through a shared-memory filter of the
// batch's touched vertices (no-op for u32 pools).
void launch_refresh_degrees(const DevGraph& g, const VertexBufs& vb, DevCtl* ctl, cudaStream_t st,
                            uint32_t* launches);
cudaError_t prepare_refresh_degrees();  // once per device before the first launch
void launch_seg_cleanup(const uint64_t* kv, uint64_t N, const BatchBufs& b, const VertexBufs& vb,
                        DevCtl* ctl, cudaStream_t st, uint32_t* launches);

// small-batch path: a1 in-place apply and a2 restore in one launch (after validation)
void launch_apply_restore(const DevGraph& g, const uint64_t* kv, const uint64_t* ku, uint64_t N,
                          const BatchBufs& b, const VertexBufs& vb, DevCtl* ctl, cudaStream_t st,
                          uint32_t* launches);
// a2: Lemma 3 closed-form restore per touched u (and d_out update)
void launch_restore(const DevGraph& g, const uint64_t* ku, uint64_t N, const BatchBufs& b,
                    const VertexBufs& vb, DevCtl* ctl, cudaStream_t st, uint32_t* launches);

// create: count / capacities / fill from an arc list on the device
void launch_build_count(const uint32_t* src, const uint32_t* dst, uint64_t m, int undirected,
                        const DevGraph& g, uint32_t n, cudaStream_t st, uint32_t* launches);
void launch_caps_from_len(const DevGraph& g, const VertexBufs& vb, double slack, uint32_t min_cap,
                          cudaStream_t st, uint32_t* launches);
void launch_build_fill(const uint32_t* src, const uint32_t* dst, uint64_t m, int undirected,
                       const DevGraph& g, const VertexBufs& vb, cudaStream_t st,
                       uint32_t* launches);
void launch_init_state(const DevGraph& g, cudaStream_t st, uint32_t* launches);

// export: (v << 32 | u) keys of every arc into keys[0..m)
void launch_export(const DevGraph& g, int active, const unsigned long long* off, uint64_t* keys,
                   const uint32_t* inv, cudaStream_t st, uint32_t* launches);
// degree-ordered relabelling: perm (external -> internal), inv (internal -> external)
void launch_relabel(const uint32_t* src, const uint32_t* dst, uint64_t m, int undirected, uint32_t n,
                    uint32_t* deg, uint64_t* k0, uint32_t* v0, uint64_t* k1, uint32_t* v1,
                    uint32_t* hist, uint32_t* perm, uint32_t* inv, cudaStream_t st,
                    uint32_t* launches);
void launch_map_ids(uint32_t* a, uint64_t m, const uint32_t* perm, cudaStream_t st,
                    uint32_t* launches);
void launch_gather_u32(const uint32_t* src, const uint32_t* perm, uint32_t n, uint32_t* dst,
                       cudaStream_t st, uint32_t* launches);
void launch_len_to_u32(const DevGraph& g, uint32_t* out, cudaStream_t st, uint32_t* launches);
// arrays layout: dst[v] = src[v * S + sidx]
void launch_gather_col(const double* src, uint32_t S, uint32_t sidx, uint32_t n, double* dst,
                       const uint32_t* perm, cudaStream_t st, uint32_t* launches);
// packed layout: copy P / R / d_out (any may be null) out of the records; zero_pr clears P and R
void launch_gather_rec(const DevGraph& g, double* P, double* R, uint32_t* dout, int zero_pr,
                       const uint32_t* perm, cudaStream_t st, uint32_t* launches);

}  // namespace ppr
