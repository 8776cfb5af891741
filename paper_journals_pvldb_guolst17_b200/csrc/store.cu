// store.cu -- dynamic graph store (hot-path step a1), invariant restore
// (step a2) and the build/export utilities.
//
// Store layout: per-vertex slabs of N_in(v) (Table 1) in a u32
// pool with slack; d_out in a separate u32 array.  A batch of arc updates
// (u, v, op) is sorted twice with the in-house radix sort:
//   by (v, u) -> the store: one warp per v-segment validates deletions
//                (claims matching slab entries), then edits the slab in place
//                (fill holes from the tail, append insertions) -- or, when a
//                slab would overflow, the whole store is rebuilt into the
//                other pool (capacities re-derived, scanned, copied, merged).
//   by (u, v) -> the restore: one thread per u-segment evaluates the batch
//                closed form of Alg 1 (Lemma 3 proof):
//                  R(u) = r0 + [S1 + S0 (a 1[u=s] - P(u) - a r0)] / (a d_k)
//                with S1 = (1-a) sum_j op_j P(v_j), S0 = sum_j op_j,
//                d_k = d_0 + S0 (the post-batch out-degree, R3);
//                d_k = 0 gives R(u) = 1[u=s] - P(u)/a (reading R4).
// Identical (u, v) updates are first reduced to their net multiplicity so an
// insertion and a deletion of the same arc in one batch cancel exactly.
#include "block_scan.cuh"
#include "primitives.cuh"
#include <algorithm>
#include <cstdlib>

#include "store.cuh"

#ifndef PPR_REFRESH_FILTER
#define PPR_REFRESH_FILTER 1
#endif

namespace ppr {

namespace {

__device__ __forceinline__ void set_err(DevCtl* ctl, int code) { atomicCAS(&ctl->st.err, KERR_OK, code); }

__device__ __forceinline__ uint32_t warp_sum_u32(uint32_t x) {
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) x += __shfl_xor_sync(0xffffffffu, x, o);
    return x;
}

__device__ __forceinline__ uint32_t warp_excl_scan_u32(uint32_t x, uint32_t& total) {
    const unsigned lane = threadIdx.x & 31u;
    uint32_t inc = x;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
        uint32_t y = __shfl_up_sync(0xffffffffu, inc, o);
        if (lane >= (unsigned)o) inc += y;
    }
    total = __shfl_sync(0xffffffffu, inc, 31);
    return inc - x;
}

// first index in [lo, hi) with keys[i] >= key
__device__ __forceinline__ uint64_t lower_bound_u64(const uint64_t* keys, uint64_t lo, uint64_t hi,
                                                    uint64_t key) {
    while (lo < hi) {
        uint64_t mid = (lo + hi) >> 1;
        if (keys[mid] < key) lo = mid + 1; else hi = mid;
    }
    return lo;
}

__device__ __forceinline__ bool contains_u32(const uint32_t* a, uint32_t n, uint32_t x) {
    uint32_t lo = 0, hi = n;
    while (lo < hi) {
        uint32_t mid = (lo + hi) >> 1;
        if (a[mid] < x) lo = mid + 1; else hi = mid;
    }
    return lo < n && a[lo] == x;
}

// end of the segment starting at i0 (all keys with the same high word)
__device__ __forceinline__ uint64_t warp_segment_end(const uint64_t* keys, uint64_t N, uint64_t i0) {
    const unsigned lane = threadIdx.x & 31u;
    const uint64_t hi = keys[i0] >> 32;
    uint64_t i1 = i0;
    while (true) {
        const uint64_t j = i1 + lane;
        const bool same = j < N && (keys[j] >> 32) == hi;
        const unsigned b = __ballot_sync(0xffffffffu, same);
        if (b == 0xffffffffu) {
            i1 += 32;
            continue;
        }
        i1 += (uint64_t)(__ffs(~b) - 1);
        return i1;
    }
}

__device__ __forceinline__ bool is_run_head(const uint64_t* keys, uint64_t j, uint64_t i0) {
    return j == i0 || keys[j] != keys[j - 1];
}

// ---------------------------------------------------------------- a0 keys

__global__ void k_ctl_reset(DevCtl* ctl) {
    ctl->st.pushes = ctl->st.pushed_edges = ctl->st.max_frontier = 0;
    ctl->st.iters[0] = ctl->st.iters[1] = 0;
    ctl->st.err = KERR_OK;
    ctl->st.rebuild = 0;
    ctl->st.n_vheads = ctl->st.n_uheads = ctl->st.n_touched = 0;
    ctl->st.arc_delta = 0;
    ctl->st.n_big = 0;
    ctl->st.ns_push[0] = ctl->st.ns_push[1] = 0;
    ctl->st.walk_edges = ctl->st.entries = 0;
    ctl->st.dup_enq = 0;
    ctl->st.t_restore[0] = ~0ull;
    ctl->st.t_restore[1] = 0;
}

__global__ void k_batch_keys(const uint32_t* __restrict__ is, const uint32_t* __restrict__ id,
                             uint64_t n_ins, const uint32_t* __restrict__ ds,
                             const uint32_t* __restrict__ dd, uint64_t n_del, int undirected,
                             uint32_t n, uint64_t* __restrict__ kv, uint32_t* __restrict__ ov,
                             uint64_t* __restrict__ ku, uint32_t* __restrict__ ou, DevCtl* ctl,
                             const uint32_t* __restrict__ perm) {
    const uint64_t tot = n_ins + n_del;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < tot;
         i += (uint64_t)gridDim.x * blockDim.x) {
        const bool ins = i < n_ins;
        uint32_t u = ins ? is[i] : ds[i - n_ins];
        uint32_t v = ins ? id[i] : dd[i - n_ins];
        uint32_t op = ins ? 2u : 0u;  // op + 1
        if (u >= n || v >= n) {
            set_err(ctl, KERR_RANGE);
            u = v = 0;
            op = 1u;
        } else if (perm) {  // internal (degree-ordered) vertex ids
            u = perm[u];
            v = perm[v];
        }
        if (!undirected) {
            kv[i] = ((uint64_t)v << 32) | u;
            ku[i] = ((uint64_t)u << 32) | v;
            ov[i] = ou[i] = op;
        } else {  // {u,v} -> u->v and v->u; a self-loop is one arc
            kv[2 * i] = ((uint64_t)v << 32) | u;
            ku[2 * i] = ((uint64_t)u << 32) | v;
            ov[2 * i] = ou[2 * i] = op;
            kv[2 * i + 1] = ((uint64_t)u << 32) | v;
            ku[2 * i + 1] = ((uint64_t)v << 32) | u;
            ov[2 * i + 1] = ou[2 * i + 1] = (u == v) ? 1u : op;
        }
    }
}

// run nets at run heads; segment heads appended to `heads`
__global__ void k_heads(const uint64_t* __restrict__ keys, const uint32_t* __restrict__ ops,
                        uint64_t N, int32_t* __restrict__ run_net, uint32_t* __restrict__ heads,
                        unsigned int* nheads) {
    const unsigned lane = threadIdx.x & 31u;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t b = (uint64_t)blockIdx.x * blockDim.x; b < N; b += stride) {
        const uint64_t i = b + threadIdx.x;
        bool seg = false;
        if (i < N) {
            const uint64_t k = keys[i];
            if (i == 0 || keys[i - 1] != k) {
                int32_t net = 0;
                for (uint64_t j = i; j < N && keys[j] == k; j++) net += (int32_t)ops[j] - 1;
                run_net[i] = net;
            }
            seg = (i == 0) || ((keys[i - 1] >> 32) != (k >> 32));
        }
        const unsigned m = __ballot_sync(0xffffffffu, seg);
        if (m) {
            unsigned base = 0;
            if (lane == 0) base = atomicAdd(nheads, (unsigned)__popc(m));
            base = __shfl_sync(0xffffffffu, base, 0);
            if (seg) heads[base + __popc(m & ((1u << lane) - 1u))] = (uint32_t)i;
        }
    }
}

// ---------------------------------------------------------------- a1 store

// One warp per v-segment of the (v, u)-sorted batch: run nets -> insertions I
// and deletions Dn of v, then (Dn > 0) a scan of v's slab that claims one
// matching slab entry per deleted copy.  The scan reads VQ consecutive slab
// entries per lane per step (32 * VQ in flight per warp, so a hub's long
// in-list costs len / 256 dependent steps, not len / 32) and stops once Dn
// copies are claimed; the claimed positions are written in ascending order
// (per-lane blocks + a warp scan), which k_store_apply relies on.
constexpr int VQ = 8;

template <bool PK>
__global__ void k_store_validate(const __grid_constant__ DevGraph g, const uint64_t* __restrict__ kv, uint64_t N,
                                 BatchBufs b, uint32_t* __restrict__ vseg, DevCtl* ctl,
                                 int force_rebuild) {
    __shared__ long long s_delta;  // the CTA's net arc-count change (one global atomic per CTA)
    if (threadIdx.x == 0) s_delta = 0;
    __syncthreads();
    const unsigned lane = threadIdx.x & 31u;
    const uint32_t nseg = *(volatile unsigned*)&ctl->st.n_vheads;
    const PoolEnt* pool = g.pool[*(volatile unsigned*)&ctl->st.active_pool];
    const uint64_t warp = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const uint64_t nwarps = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    if (force_rebuild && blockIdx.x == 0 && threadIdx.x == 0) ctl->st.rebuild = 1;
    for (uint64_t w = warp; w < nseg; w += nwarps) {
        const uint64_t i0 = b.vheads[w];
        const uint32_t v = (uint32_t)(kv[i0] >> 32);
        const Slab sl = get_slab<PK>(g, v);  // issued before the segment walk (independent)
        const uint64_t i1 = warp_segment_end(kv, N, i0);
        uint32_t I = 0, Dn = 0;
        for (uint64_t j = i0 + lane; j < i1; j += 32) {
            if (is_run_head(kv, j, i0)) {
                const int32_t net = b.rnv[j];
                if (net > 0) I += (uint32_t)net; else Dn += (uint32_t)(-net);
            }
        }
        I = warp_sum_u32(I);
        Dn = warp_sum_u32(Dn);
        uint32_t found = 0;
        for (uint32_t p0 = 0; Dn > 0 && p0 < sl.len && found < Dn; p0 += 32 * VQ) {
            const uint32_t pb = p0 + lane * VQ;  // this lane's block of VQ positions
            uint32_t x[VQ];
#pragma unroll
            for (int q = 0; q < VQ; q++) x[q] = pb + q < sl.len ? pool_id(g, pool, sl.off + pb + q) : 0u;
            uint32_t cl = 0;  // claimed positions of the block (bit q)
#pragma unroll
            for (int q = 0; q < VQ; q++) {
                if (pb + q < sl.len) {
                    const uint64_t key = ((uint64_t)v << 32) | x[q];
                    const uint64_t r = lower_bound_u64(kv, i0, i1, key);
                    if (r < i1 && kv[r] == key) {
                        const int32_t net = b.rnv[r];
                        if (net < 0 && atomicAdd(&b.claim[r], 1u) < (uint32_t)(-net)) cl |= 1u << q;
                    }
                }
            }
            uint32_t tot;
            uint32_t pos = i0 + found + warp_excl_scan_u32((uint32_t)__popc(cl), tot);
#pragma unroll
            for (int q = 0; q < VQ; q++)
                if (cl & (1u << q)) b.delpos[pos++] = pb + q;
            found += tot;
        }
        if (lane == 0) {
            b.seg_end[i0] = (uint32_t)i1;
            b.seg_D[i0] = found;
            b.seg_I[i0] = I;
            vseg[v] = (uint32_t)i0;
            if (found < Dn) set_err(ctl, KERR_NOENT);  // deletion of an absent arc
            if ((uint64_t)sl.len - found + I > sl.cap) ctl->st.rebuild = 1;
            atomicAdd((unsigned long long*)&s_delta, (unsigned long long)((long long)I - (long long)Dn));
        }
    }
    __syncthreads();
    if (threadIdx.x == 0 && s_delta)
        atomicAdd((unsigned long long*)&ctl->st.arc_delta, (unsigned long long)s_delta);
}

// in-place slab edit of every v-segment (warps `warp` + k * nwarps)
template <bool PK>
__device__ __forceinline__ void apply_segments(const DevGraph& g, const uint64_t* __restrict__ kv,
                                               const BatchBufs& b, DevCtl* ctl, uint64_t warp,
                                               uint64_t nwarps) {
    const unsigned lane = threadIdx.x & 31u;
    const uint32_t nseg = *(volatile unsigned*)&ctl->st.n_vheads;
    PoolEnt* pool = g.pool[*(volatile unsigned*)&ctl->st.active_pool];
    for (uint64_t w = warp; w < nseg; w += nwarps) {
        const uint64_t i0 = b.vheads[w];
        const uint32_t v = (uint32_t)(kv[i0] >> 32);
        const uint64_t i1 = b.seg_end[i0];
        const uint32_t D = b.seg_D[i0], I = b.seg_I[i0];
        const Slab sl = get_slab<PK>(g, v);
        const uint32_t keep = sl.len - D;
        const uint32_t* dp = b.delpos + i0;
        // fill the holes (deleted positions < keep) with the surviving tail entries
        uint32_t filled = 0;
        for (uint32_t t0 = keep; t0 < sl.len; t0 += 32) {
            const uint32_t t = t0 + lane;
            const bool filler = t < sl.len && !contains_u32(dp, D, t);
            const unsigned m = __ballot_sync(0xffffffffu, filler);
            if (filler) {
                const uint32_t hole = dp[filled + __popc(m & ((1u << lane) - 1u))];
                pool_copy(g, pool, sl.off + hole, pool, sl.off + t);
            }
            filled += __popc(m);
        }
        __syncwarp();
        // append insertions (net multiplicity copies of u) at [keep, keep + I)
        uint32_t pos = keep;
        for (uint64_t j0 = i0; j0 < i1; j0 += 32) {
            const uint64_t j = j0 + lane;
            uint32_t c = 0, x = 0;
            if (j < i1 && is_run_head(kv, j, i0)) {
                const int32_t net = b.rnv[j];
                if (net > 0) {
                    c = (uint32_t)net;
                    x = (uint32_t)kv[j];
                }
            }
            uint32_t tot;
            const uint32_t ex = warp_excl_scan_u32(c, tot);
            // d_out(x) is filled in by the degree refresh after the restore (k_rebuild)
            for (uint32_t k = 0; k < c; k++) pool_put(g, pool, sl.off + pos + ex + k, x, 0);
            pos += tot;
        }
        // slots vacated when more copies were deleted than inserted become empty
        for (uint32_t t = keep + I + lane; t < sl.len; t += 32) pool_clear(g, pool, sl.off + t);
        if (lane == 0) *lenp<PK>(g, v) = keep + I;
    }
}

template <bool PK>
__global__ void k_store_apply(const __grid_constant__ DevGraph g, const uint64_t* __restrict__ kv,
                              BatchBufs b, DevCtl* ctl) {
    if (*(volatile int*)&ctl->st.err != KERR_OK || *(volatile int*)&ctl->st.rebuild) return;
    apply_segments<PK>(g, kv, b, ctl, ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5,
                       ((uint64_t)gridDim.x * blockDim.x) >> 5);
}

// ---------------------------------------------------------------- a1 rebuild
//
// One cooperative kernel (it exits at once unless DevCtl::rebuild is set, so
// the common no-overflow batch pays one short launch): capacities of every
// slab with the batch merged -> exclusive scan -> stable copy of each slab
// into the other pool with its deletions dropped and insertions appended ->
// flip the active pool.  Phases are separated by grid barriers.

constexpr int RB_THREADS = 256;

// new length of v after this batch (the batch's segment for v, if any)
template <bool PK>
__device__ __forceinline__ uint32_t merged_len(const DevGraph& g, const BatchBufs& b,
                                               const VertexBufs& vb, uint64_t v) {
    uint32_t len = *lenp<PK>(g, (uint32_t)v);
    const uint32_t sg = vb.vseg[v];
    if (sg != NONE) len = len - b.seg_D[sg] + b.seg_I[sg];
    return len;
}

__device__ __forceinline__ uint32_t cap_for(uint32_t len, double slack, uint32_t min_cap) {
    const uint32_t extra = (uint32_t)ceil((double)len * slack);
    return len + (extra > min_cap ? extra : min_cap);
}

// warp-wide stable copy of slab v into dst[no ..] without its claimed
// deletions, followed by its net insertions; returns the new length
__device__ uint32_t copy_merged_warp(const DevGraph& g, const PoolEnt* src, PoolEnt* dst, const Slab sl,
                                     unsigned long long no, uint32_t cap, const uint64_t* kv,
                                     const BatchBufs& b, uint32_t sg) {
    const unsigned lane = threadIdx.x & 31u;
    const uint32_t D = sg != NONE ? b.seg_D[sg] : 0u;
    const uint32_t* dp = sg != NONE ? b.delpos + sg : nullptr;
    uint32_t pos = 0;
    for (uint32_t p0 = 0; p0 < sl.len; p0 += 32) {
        const uint32_t p = p0 + lane;
        const bool keep = p < sl.len && !(D && contains_u32(dp, D, p));
        const unsigned m = __ballot_sync(0xffffffffu, keep);
        if (keep) pool_copy(g, dst, no + pos + __popc(m & ((1u << lane) - 1u)), src, sl.off + p);
        pos += __popc(m);
    }
    if (sg != NONE) {
        const uint64_t i0 = sg, i1 = b.seg_end[sg];
        for (uint64_t j0 = i0; j0 < i1; j0 += 32) {
            const uint64_t j = j0 + lane;
            uint32_t c = 0, x = 0;
            if (j < i1 && is_run_head(kv, j, i0)) {
                const int32_t net = b.rnv[j];
                if (net > 0) {
                    c = (uint32_t)net;
                    x = (uint32_t)kv[j];
                }
            }
            uint32_t tot;
            const uint32_t ex = warp_excl_scan_u32(c, tot);
            for (uint32_t k = 0; k < c; k++) pool_put(g, dst, no + pos + ex + k, x, 0);  // degree: refresh
            pos += tot;
        }
    }
    for (uint32_t t = pos + lane; t < cap; t += 32) pool_clear(g, dst, no + t);  // the slab's slack
    return pos;
}

template <bool PK>
__device__ __forceinline__ unsigned long long rebuild_body(const DevGraph& g, const uint64_t* __restrict__ kv,
                                             const BatchBufs& b, const VertexBufs& vb, double slack,
                                             uint32_t min_cap, uint64_t cap0, uint64_t cap1,
                                             DevCtl* ctl) {
    __shared__ uint32_t s_warp[RB_THREADS / 32 + 1];
    __shared__ unsigned long long s_warp64[RB_THREADS / 32 + 1];
    const unsigned act = *(volatile unsigned*)&ctl->st.active_pool;
    // the spare pool's capacity, read with the device-side active flag (a replayed
    // batch graph must not bake in the pool that was spare when it was captured)
    const uint64_t alt_cap = act ? cap0 : cap1;
    const PoolEnt* src = act ? g.pool[1] : g.pool[0];
    PoolEnt* dst = act ? g.pool[0] : g.pool[1];
    const unsigned lane = threadIdx.x & 31u;
    // contiguous vertex range of this CTA
    const uint64_t chunk = ((uint64_t)g.n + gridDim.x - 1) / gridDim.x;
    const uint64_t v0 = (uint64_t)blockIdx.x * chunk;
    const uint64_t v1 = v0 + chunk < g.n ? v0 + chunk : g.n;
    // phase 1: capacities and the CTA's sum
    unsigned long long mysum = 0;
    for (uint64_t v = v0 + threadIdx.x; v < v1; v += RB_THREADS) {
        const uint32_t nc = cap_for(merged_len<PK>(g, b, vb, v), slack, min_cap);
        vb.newcap[v] = nc;
        mysum += nc;
    }
    unsigned long long cta_sum;
    block_exclusive_scan_u64<RB_THREADS>(mysum, s_warp64, &cta_sum);
    if (threadIdx.x == 0) vb.part[blockIdx.x] = cta_sum;
    grid_sync(ctl);
    // phase 2: CTA bases (every CTA scans the partials itself)
    unsigned long long base = 0, total = 0;
    for (uint32_t i = threadIdx.x; i < gridDim.x; i += RB_THREADS) {
        const unsigned long long x = __ldcg(&vb.part[i]);
        total += x;
        if (i < blockIdx.x) base += x;
    }
    {
        unsigned long long t1, t2;
        block_exclusive_scan_u64<RB_THREADS>(base, s_warp64, &t1);
        block_exclusive_scan_u64<RB_THREADS>(total, s_warp64, &t2);
        base = t1;
        total = t2;
    }
    if (blockIdx.x == 0 && threadIdx.x == 0) ctl->st.pool_top = total;
    if (total > alt_cap) {  // cannot happen: the host sizes the other pool (uniform exit)
        if (blockIdx.x == 0 && threadIdx.x == 0) atomicCAS(&ctl->st.err, KERR_OK, KERR_OVERFLOW);
        return 0;
    }
    // phase 3: offsets and the copy of short untouched slabs (thread per vertex);
    // long or changed slabs go to the warp-wide list
    for (uint64_t vb0 = v0; vb0 < v1; vb0 += RB_THREADS) {
        const uint64_t v = vb0 + threadIdx.x;
        const uint32_t nc = v < v1 ? vb.newcap[v] : 0u;
        uint32_t tot;
        const uint32_t ex = block_exclusive_scan_u32<RB_THREADS>(nc, s_warp, &tot);
        bool big = false;
        if (v < v1) {
            const unsigned long long no = base + ex;
            vb.newoff[v] = no;
            const Slab sl = get_slab<PK>(g, v);
            big = vb.vseg[v] != NONE || sl.len > 16;
            if (!big) {
                for (uint32_t j = 0; j < sl.len; j++) pool_copy(g, dst, no + j, src, sl.off + j);
                for (uint32_t j = sl.len; j < nc; j++) pool_clear(g, dst, no + j);
                Slab ns;
                ns.off = no;
                ns.len = sl.len;
                ns.cap = nc;
                put_slab<PK>(g, v, ns);
            }
        }
        base += tot;
        const unsigned m = __ballot_sync(0xffffffffu, big);
        if (m) {
            unsigned wb = 0;
            if (lane == 0) wb = atomicAdd(&ctl->st.n_big, (unsigned)__popc(m));
            wb = __shfl_sync(0xffffffffu, wb, 0);
            if (big) vb.big[wb + __popc(m & ((1u << lane) - 1u))] = (uint32_t)v;
        }
    }
    grid_sync(ctl);
    // phase 4: warp per long / changed slab
    const uint32_t nbig = *(volatile unsigned*)&ctl->st.n_big;
    const uint64_t warp = ((uint64_t)blockIdx.x * RB_THREADS + threadIdx.x) >> 5;
    const uint64_t nwarps = ((uint64_t)gridDim.x * RB_THREADS) >> 5;
    for (uint64_t w = warp; w < nbig; w += nwarps) {
        const uint32_t v = __ldcg(&vb.big[w]);
        const Slab sl = get_slab<PK>(g, v);
        const unsigned long long no = __ldcg(&vb.newoff[v]);
        const uint32_t len = copy_merged_warp(g, src, dst, sl, no, __ldcg(&vb.newcap[v]), kv, b, vb.vseg[v]);
        if (lane == 0) {
            Slab ns;
            ns.off = no;
            ns.len = len;
            ns.cap = __ldcg(&vb.newcap[v]);
            put_slab<PK>(g, v, ns);
        }
    }
    grid_sync(ctl);
    if (blockIdx.x == 0 && threadIdx.x == 0) ctl->st.active_pool = act ^ 1u;
    return total;
}

// The end of a batch's store pipeline, one cooperative launch:
//  * the rebuild (only if a slab would overflow; the decision is uniform: it was
//    made by the validation before this launch);
//  * with `finish`: the reset of the batch's v -> segment map, and the degree
//    refresh -- every entry of the active pool whose cached d_out (PoolEnt) no
//    longer matches d_out after this batch's restore is rewritten, a coalesced
//    stream over the pool's [0, extent) with one d_out gather per entry.
template <bool PK>
__global__ void __launch_bounds__(RB_THREADS) k_rebuild(const __grid_constant__ DevGraph g,
                                                        const uint64_t* __restrict__ kv, BatchBufs b,
                                                        VertexBufs vb, double slack, uint32_t min_cap,
                                                        uint64_t cap0, uint64_t cap1, DevCtl* ctl,
                                                        int finish) {
    const bool ok = *(volatile int*)&ctl->st.err == KERR_OK;
    unsigned act = *(volatile unsigned*)&ctl->st.active_pool;  // read before any flip
    unsigned long long ext = *(volatile unsigned long long*)&ctl->st.pool_extent;
    if (ok && *(volatile int*)&ctl->st.rebuild) {
        const unsigned long long e = rebuild_body<PK>(g, kv, b, vb, slack, min_cap, cap0, cap1, ctl);
        if (e) {
            act ^= 1u;
            ext = e;
            if (blockIdx.x == 0 && threadIdx.x == 0) ctl->st.pool_extent = e;
        }
    }
    if (!finish) return;
    const uint64_t tid = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x;
    const uint64_t nth = (uint64_t)gridDim.x * blockDim.x;
    const uint32_t nseg = *(volatile unsigned*)&ctl->st.n_vheads;
    for (uint64_t w = tid; w < nseg; w += nth) vb.vseg[kv[b.vheads[w]] >> 32] = NONE;
    if (PPR_REFRESH_FILTER || !ok || !g.pool_wide || !*(volatile unsigned*)&ctl->st.n_touched)
        return;  // nothing cached changed (or k_refresh_degrees does it)
    // stream the active pool; gather d_out for every entry (8 gathers in flight per
    // thread) and rewrite the stale ones.  (Testing a bitmap of the batch's touched
    // vertices first was slower: its gather costs as much as the hub-concentrated
    // d_out gather -- Twitter shape 19.4 vs 9.9 ms per batch.)
    PoolEnt* pool = g.pool[act];
    constexpr int RQ = 8;
    for (uint64_t p0 = tid; p0 < ext; p0 += nth * RQ) {
        PoolEnt e[RQ];
        uint32_t d[RQ];
#pragma unroll
        for (int q = 0; q < RQ; q++) {
            const uint64_t p = p0 + (uint64_t)q * nth;
            e[q] = p < ext ? __ldcs(&pool[p]) : POOL_EMPTY;
        }
#pragma unroll
        for (int q = 0; q < RQ; q++) {
            const uint32_t v = pe_v(e[q]);
            d[q] = v != 0xFFFFFFFFu ? *doutp<PK>(g, v) : 0u;  // empty slots are skipped
        }
#pragma unroll
        for (int q = 0; q < RQ; q++) {
            const uint32_t v = pe_v(e[q]);
            if (v != 0xFFFFFFFFu && pe_d(e[q]) != d[q]) pool[p0 + (uint64_t)q * nth] = pe_make(v, d[q]);
        }
    }
}

// Degree refresh of wide pool entries (PPR_REFRESH_FILTER): one CTA per SM
// holds a 2^20-bit filter of this batch's touched vertices (the only ones whose
// d_out changed; bit = v mod 2^20, so the 10^6 highest-degree relabelled ids
// are exact) in shared memory, streams the active pool and gathers d_out(v)
// only for entries whose v passes the filter -- instead of a d_out gather per
// entry.
constexpr int RF_THREADS = 1024;
constexpr uint32_t RF_BITS = 1u << 20;
template <bool PK>
__global__ void __launch_bounds__(RF_THREADS) k_refresh_degrees(const __grid_constant__ DevGraph g,
                                                                const uint32_t* __restrict__ touched,
                                                                DevCtl* ctl) {
    extern __shared__ uint32_t s_bits[];  // RF_BITS / 32 words
    if (*(volatile int*)&ctl->st.err != KERR_OK) return;
    const uint32_t nt = *(volatile unsigned*)&ctl->st.n_touched;
    if (!nt) return;
    for (uint32_t i = threadIdx.x; i < RF_BITS / 32; i += RF_THREADS) s_bits[i] = 0u;
    __syncthreads();
    for (uint32_t i = threadIdx.x; i < nt; i += RF_THREADS) {
        const uint32_t h = touched[i] & (RF_BITS - 1u);
        atomicOr(&s_bits[h >> 5], 1u << (h & 31u));
    }
    __syncthreads();
    const unsigned act = *(volatile unsigned*)&ctl->st.active_pool;
    const unsigned long long ext = *(volatile unsigned long long*)&ctl->st.pool_extent;
    PoolEnt* pool = g.pool[act];
    const uint64_t tid = (uint64_t)blockIdx.x * RF_THREADS + threadIdx.x;
    const uint64_t nth = (uint64_t)gridDim.x * RF_THREADS;
    // 16-byte loads: entry pairs [2j, 2j + 1]; RQ pairs in flight per thread
    constexpr int RQ = 8;
    const uint64_t npair = (ext + 1) / 2;
    const ulonglong2* pairs = reinterpret_cast<const ulonglong2*>(pool);
    for (uint64_t j0 = tid; j0 < npair; j0 += nth * RQ) {
        ulonglong2 e[RQ];
#pragma unroll
        for (int q = 0; q < RQ; q++) {
            const uint64_t j = j0 + (uint64_t)q * nth;
            e[q] = j < npair ? __ldcs(&pairs[j]) : make_ulonglong2(POOL_EMPTY, POOL_EMPTY);
        }
#pragma unroll
        for (int q = 0; q < RQ; q++) {
#pragma unroll
            for (int half = 0; half < 2; half++) {
                const PoolEnt x = half ? e[q].y : e[q].x;
                const uint64_t p = 2 * (j0 + (uint64_t)q * nth) + half;
                const uint32_t v = pe_v(x);
                if (v == 0xFFFFFFFFu || p >= ext) continue;
                const uint32_t h = v & (RF_BITS - 1u);
                if (!(s_bits[h >> 5] & (1u << (h & 31u)))) continue;  // d_out(v) unchanged this batch
                const uint32_t d = *doutp<PK>(g, v);
                if (pe_d(x) != d) pool[p] = pe_make(v, d);
            }
        }
    }
}

__global__ void k_seg_cleanup(const uint64_t* __restrict__ kv, BatchBufs b,
                              uint32_t* __restrict__ vseg, DevCtl* ctl) {
    const uint32_t nseg = *(volatile unsigned*)&ctl->st.n_vheads;
    for (uint64_t w = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; w < nseg;
         w += (uint64_t)gridDim.x * blockDim.x)
        vseg[kv[b.vheads[w]] >> 32] = NONE;
}

// ---------------------------------------------------------------- a2 restore

// Lemma 3 closed form for the u-segment starting at i0 and the sources
// si = s0, s0 + ds, ... (one thread per segment: s0 = 0, ds = 1; one warp per
// segment: s0 = lane, ds = 32 -- the S residuals of u are one vertex-major row,
// so the lanes' loads coalesce).  Returns false if the segment's updates all
// cancelled (nothing to restore).
template <bool PK>
__device__ __forceinline__ bool restore_segment(const DevGraph& g, const uint64_t* __restrict__ ku,
                                                uint64_t N, const BatchBufs& b, uint64_t i0,
                                                uint32_t s0, uint32_t ds, bool write_dout) {
    const double a = g.alpha;
    const uint32_t u = (uint32_t)(ku[i0] >> 32);
    int64_t S0 = 0;
    bool any = false;
    uint64_t i1 = i0;
    for (; i1 < N && (ku[i1] >> 32) == u; i1++) {
        if (is_run_head(ku, i1, i0)) {
            const int32_t net = b.rnu[i1];
            S0 += net;
            any |= net != 0;
        }
    }
    if (!any) return false;
    const int64_t dk = (int64_t)*doutp<PK>(g, u) + S0;  // post-batch d_out(u) (reading R3)
    for (uint32_t si = s0; si < g.S; si += ds) {
        double s1 = 0.0;
        for (uint64_t j = i0; j < i1; j++) {
            if (!is_run_head(ku, j, i0)) continue;
            const int32_t net = b.rnu[j];
            if (net != 0) s1 += (double)net * *Pp<PK>(g, si, (uint32_t)ku[j]);
        }
        const double S1 = (1.0 - a) * s1;
        const double one = (u == g.sources[si]) ? 1.0 : 0.0;
        const double pu = *Pp<PK>(g, si, u);
        const double r0 = *Rp<PK>(g, si, u);
        double r;
        if (dk > 0)
            r = r0 + (S1 + (double)S0 * (a * one - pu - a * r0)) / (a * (double)dk);
        else
            r = one - pu / a;  // Eq. 2 with an empty sum (reading R4)
        *Rp<PK>(g, si, u) = r;
    }
    if (ds == 32) __syncwarp();  // every lane has read d_out(u) above
    if (write_dout) *doutp<PK>(g, u) = (uint32_t)dk;
    return true;
}

// every u-segment: thread per segment (S == 1) or warp per segment (S > 1);
// `item` / `nitems` index threads or warps of the participating blocks
template <bool PK>
__device__ __forceinline__ void restore_segments(const DevGraph& g, const uint64_t* __restrict__ ku,
                                                 uint64_t N, const BatchBufs& b,
                                                 uint32_t* __restrict__ touched, DevCtl* ctl,
                                                 uint64_t item, uint64_t nitems) {
    const uint32_t nseg = *(volatile unsigned*)&ctl->st.n_uheads;
    const unsigned lane = threadIdx.x & 31u;
    if (g.S == 1) {
        for (uint64_t k = item; k < nseg; k += nitems) {
            const uint64_t i0 = b.uheads[k];
            if (restore_segment<PK>(g, ku, N, b, i0, 0, 1, true))
                touched[atomicAdd(&ctl->st.n_touched, 1u)] = (uint32_t)(ku[i0] >> 32);
        }
    } else {
        for (uint64_t k = item; k < nseg; k += nitems) {
            const uint64_t i0 = b.uheads[k];
            if (restore_segment<PK>(g, ku, N, b, i0, lane, 32, lane == 0) && lane == 0)
                touched[atomicAdd(&ctl->st.n_touched, 1u)] = (uint32_t)(ku[i0] >> 32);
        }
    }
}

// restore grid: threads (S == 1) or warps (S > 1) over the u-segments
inline unsigned restore_blocks(uint64_t N, uint32_t S, unsigned threads) {
    const uint64_t items = S == 1 ? N : N * 32;
    uint64_t blocks = (items + threads - 1) / threads;
    if (blocks < 1) blocks = 1;
    if (blocks > 148 * 32) blocks = 148 * 32;
    return (unsigned)blocks;
}

template <bool PK>
__global__ void k_restore(const __grid_constant__ DevGraph g, const uint64_t* __restrict__ ku,
                          uint64_t N, BatchBufs b, uint32_t* __restrict__ touched, DevCtl* ctl) {
    if (*(volatile int*)&ctl->st.err != KERR_OK) return;
    if (threadIdx.x == 0) atomicMin(&ctl->st.t_restore[0], globaltimer_ns());
    const uint64_t tid = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x;
    const uint64_t nth = (uint64_t)gridDim.x * blockDim.x;
    if (g.S == 1) restore_segments<PK>(g, ku, N, b, touched, ctl, tid, nth);
    else restore_segments<PK>(g, ku, N, b, touched, ctl, tid >> 5, nth >> 5);
    __syncthreads();
    if (threadIdx.x == 0) atomicMax(&ctl->st.t_restore[1], globaltimer_ns());
}

// small-batch path: the in-place apply (blocks [0, apply_blocks)) and the
// restore (the other blocks) in one launch -- both need only the validation
template <bool PK>
__global__ void k_apply_restore(const __grid_constant__ DevGraph g, const uint64_t* __restrict__ kv,
                                const uint64_t* __restrict__ ku, uint64_t N, BatchBufs b,
                                uint32_t* __restrict__ touched, DevCtl* ctl, unsigned apply_blocks) {
    if (*(volatile int*)&ctl->st.err != KERR_OK) return;
    if (blockIdx.x < apply_blocks) {
        if (!*(volatile int*)&ctl->st.rebuild)
            apply_segments<PK>(g, kv, b, ctl, ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5,
                               ((uint64_t)apply_blocks * blockDim.x) >> 5);
        return;
    }
    if (threadIdx.x == 0) atomicMin(&ctl->st.t_restore[0], globaltimer_ns());
    const uint64_t tid = (uint64_t)(blockIdx.x - apply_blocks) * blockDim.x + threadIdx.x;
    const uint64_t nth = (uint64_t)(gridDim.x - apply_blocks) * blockDim.x;
    if (g.S == 1) restore_segments<PK>(g, ku, N, b, touched, ctl, tid, nth);
    else restore_segments<PK>(g, ku, N, b, touched, ctl, tid >> 5, nth >> 5);
    __syncthreads();
    if (threadIdx.x == 0) atomicMax(&ctl->st.t_restore[1], globaltimer_ns());
}

// ---------------------------------------------------------------- build / init / export

template <bool PK>
__global__ void k_build_count(const uint32_t* __restrict__ src, const uint32_t* __restrict__ dst,
                              uint64_t m, int undirected, const __grid_constant__ DevGraph g) {
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < m;
         i += (uint64_t)gridDim.x * blockDim.x) {
        const uint32_t u = src[i], v = dst[i];
        atomicAdd(lenp<PK>(g, v), 1u);
        atomicAdd(doutp<PK>(g, u), 1u);
        if (undirected && u != v) {
            atomicAdd(lenp<PK>(g, u), 1u);
            atomicAdd(doutp<PK>(g, v), 1u);
        }
    }
}

template <bool PK>
__global__ void k_caps_from_len(const __grid_constant__ DevGraph g, uint32_t* __restrict__ newcap, double slack,
                                uint32_t min_cap) {
    for (uint64_t v = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; v < g.n;
         v += (uint64_t)gridDim.x * blockDim.x) {
        const uint32_t len = *lenp<PK>(g, (uint32_t)v);
        uint32_t extra = (uint32_t)ceil((double)len * slack);
        newcap[v] = len + (extra > min_cap ? extra : min_cap);
    }
}

template <bool PK>
__global__ void k_set_slabs(const __grid_constant__ DevGraph g, const unsigned long long* __restrict__ off,
                            const uint32_t* __restrict__ cap) {
    for (uint64_t v = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; v < g.n;
         v += (uint64_t)gridDim.x * blockDim.x) {
        Slab s;
        s.off = off[v];
        s.len = 0;
        s.cap = cap[v];
        put_slab<PK>(g, v, s);
    }
}

template <bool PK>
__global__ void k_build_fill(const uint32_t* __restrict__ src, const uint32_t* __restrict__ dst,
                             uint64_t m, int undirected, const __grid_constant__ DevGraph g) {
    PoolEnt* pool = g.pool[0];  // d_out is final here (k_build_count)
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < m;
         i += (uint64_t)gridDim.x * blockDim.x) {
        const uint32_t u = src[i], v = dst[i];
        uint32_t p = atomicAdd(lenp<PK>(g, v), 1u);
        pool_put(g, pool, get_slab<PK>(g, v).off + p, u, *doutp<PK>(g, u));
        if (undirected && u != v) {
            p = atomicAdd(lenp<PK>(g, u), 1u);
            pool_put(g, pool, get_slab<PK>(g, u).off + p, v, *doutp<PK>(g, v));
        }
    }
}

template <bool PK>
__global__ void k_init_state(const __grid_constant__ DevGraph g) {
    // P = 0 and R = 0 are set by memset; R(s) = 1 for each source (Fig. 3 a(1))
    for (uint32_t i = blockIdx.x * blockDim.x + threadIdx.x; i < g.S; i += gridDim.x * blockDim.x)
        *Rp<PK>(g, i, g.sources[i]) = 1.0;
}

template <bool PK>
__global__ void k_len_to_u32(const __grid_constant__ DevGraph g, uint32_t* __restrict__ out) {
    for (uint64_t v = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; v < g.n;
         v += (uint64_t)gridDim.x * blockDim.x)
        out[v] = *lenp<PK>(g, (uint32_t)v);
}

template <bool PK>
__global__ void k_export(const __grid_constant__ DevGraph g, int active, const unsigned long long* __restrict__ off,
                         uint64_t* __restrict__ keys, const uint32_t* __restrict__ inv) {
    const PoolEnt* pool = g.pool[active];
    for (uint64_t v = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; v < g.n;
         v += (uint64_t)gridDim.x * blockDim.x) {
        const Slab sl = get_slab<PK>(g, v);
        const uint64_t vo = inv ? inv[v] : v;  // external id
        for (uint32_t j = 0; j < sl.len; j++) {
            const uint32_t x = pool_id(g, pool, sl.off + j);
            keys[off[v] + j] = (vo << 32) | (inv ? inv[x] : x);
        }
    }
}

// ---------------------------------------------------------------- degree-ordered relabelling
// Vertices are renumbered by G0 out-degree (descending, ties by id) so that
// the heaviest receivers of pushes (a vertex is pushed to once per frontier
// out-neighbour) share residual / d_out cache lines.  perm: external ->
// internal id, inv: internal -> external.

__global__ void k_count_out(const uint32_t* __restrict__ src, const uint32_t* __restrict__ dst,
                            uint64_t m, int undirected, uint32_t* __restrict__ deg) {
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < m;
         i += (uint64_t)gridDim.x * blockDim.x) {
        atomicAdd(&deg[src[i]], 1u);
        if (undirected && src[i] != dst[i]) atomicAdd(&deg[dst[i]], 1u);
    }
}

__global__ void k_degree_keys(const uint32_t* __restrict__ deg, uint32_t n, uint64_t* __restrict__ keys,
                              uint32_t* __restrict__ vals) {
    for (uint64_t v = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; v < n;
         v += (uint64_t)gridDim.x * blockDim.x) {
        keys[v] = ((uint64_t)(0xFFFFFFFFu - deg[v]) << 32) | v;
        vals[v] = 0;
    }
}

// spread = k > 0 (1 is used): inside every full block of
// 16 L ranks (L = 16^k lines of 16 residuals) rank i goes to line i % L, slot
// i / L, so consecutive (equally hot) ranks land on different 128-byte residual
// lines -- and L2 slices -- while the block's footprint stays L lines (measured:
// Orkut-shaped relabelled push 29.8 -> 27.9 ms, LJ 3.26 -> 3.23 ms; DESIGN.md
// "Relabelling")
__global__ void k_perm_from_sorted(const uint64_t* __restrict__ keys, uint32_t n,
                                   uint32_t* __restrict__ perm, uint32_t* __restrict__ inv, int spread) {
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
         i += (uint64_t)gridDim.x * blockDim.x) {
        const uint32_t v = (uint32_t)keys[i];
        uint32_t id = (uint32_t)i;
        if (spread) {  // block of 16 * L ranks: rank i -> line i % L, slot i / L
            const uint32_t L = 16u << (4 * (spread - 1)), B = 16u * L;
            if ((id / B + 1) * (uint64_t)B <= n) {
                const uint32_t j = id % B;
                id = id - j + (j % L) * 16u + j / L;
            }
        }
        inv[id] = v;
        perm[v] = id;
    }
}

__global__ void k_map_ids(uint32_t* __restrict__ a, uint64_t m, const uint32_t* __restrict__ perm) {
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < m;
         i += (uint64_t)gridDim.x * blockDim.x)
        a[i] = perm[a[i]];
}

__global__ void k_gather_u32(const uint32_t* __restrict__ src, const uint32_t* __restrict__ perm,
                             uint32_t n, uint32_t* __restrict__ dst) {
    for (uint64_t v = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; v < n;
         v += (uint64_t)gridDim.x * blockDim.x)
        dst[v] = src[perm ? perm[v] : v];
}

// packed layout: P, R, d_out out of the records (query / export / reset)
__global__ void k_gather_rec(const __grid_constant__ DevGraph g, double* __restrict__ P, double* __restrict__ R,
                             uint32_t* __restrict__ dout, int zero_pr,
                             const uint32_t* __restrict__ perm) {
    for (uint64_t v = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; v < g.n;
         v += (uint64_t)gridDim.x * blockDim.x) {
        VRec* rc = &g.rec[perm ? perm[v] : v];
        if (P) P[v] = rc->p;
        if (R) R[v] = rc->r;
        if (dout) dout[v] = rc->dout;
        if (zero_pr) rc->p = rc->r = 0.0;
    }
}

// arrays layout, S > 1: column `sidx` of a vertex-major [n][S] array
__global__ void k_gather_col(const double* __restrict__ src, uint32_t S, uint32_t sidx, uint32_t n,
                             double* __restrict__ dst, const uint32_t* __restrict__ perm) {
    for (uint64_t v = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; v < n;
         v += (uint64_t)gridDim.x * blockDim.x)
        dst[v] = src[(uint64_t)(perm ? perm[v] : v) * S + sidx];
}

// the kernel instance for the handle's layout
#define LAUNCH_PK(k) (g.rec ? k<true> : k<false>)

inline unsigned grid_for(uint64_t n, unsigned threads, unsigned cap = 148 * 32) {
    uint64_t b = (n + threads - 1) / threads;
    if (b < 1) b = 1;
    if (b > cap) b = cap;
    return (unsigned)b;
}

}  // namespace

void launch_ctl_reset(DevCtl* ctl, cudaStream_t st, uint32_t* launches) {
    k_ctl_reset<<<1, 1, 0, st>>>(ctl);
    ++*launches;
}

void launch_batch_keys(const uint32_t* is, const uint32_t* id, uint64_t n_ins, const uint32_t* ds,
                       const uint32_t* dd, uint64_t n_del, int undirected, uint32_t n,
                       const BatchBufs& b, int slot, DevCtl* ctl, const uint32_t* perm,
                       cudaStream_t st, uint32_t* launches) {
    k_batch_keys<<<grid_for(n_ins + n_del, 256), 256, 0, st>>>(
        is, id, n_ins, ds, dd, n_del, undirected, n, b.kv[slot], b.ov[slot], b.ku[slot],
        b.ou[slot], ctl, perm);
    ++*launches;
}

void launch_heads(const uint64_t* keys, const uint32_t* ops, uint64_t N, int32_t* run_net,
                  uint32_t* heads, unsigned int* nheads, cudaStream_t st, uint32_t* launches) {
    k_heads<<<grid_for(N, 256), 256, 0, st>>>(keys, ops, N, run_net, heads, nheads);
    ++*launches;
}

void launch_store_validate(const DevGraph& g, const uint64_t* kv, uint64_t N, const BatchBufs& b,
                           const VertexBufs& vb, DevCtl* ctl, int force_rebuild, cudaStream_t st,
                           uint32_t* launches) {
    LAUNCH_PK(k_store_validate)<<<grid_for(N * 32, 256), 256, 0, st>>>(g, kv, N, b, vb.vseg, ctl,
                                                            force_rebuild);
    ++*launches;
}

void launch_store_apply(const DevGraph& g, const uint64_t* kv, uint64_t N, const BatchBufs& b,
                        DevCtl* ctl, cudaStream_t st, uint32_t* launches) {
    LAUNCH_PK(k_store_apply)<<<grid_for(N * 32, 256), 256, 0, st>>>(g, kv, b, ctl);
    ++*launches;
}

cudaError_t launch_store_rebuild(const DevGraph& g, const uint64_t* kv, uint64_t N, const BatchBufs& b,
                                 const VertexBufs& vb, const StoreParams& sp, DevCtl* ctl,
                                 cudaStream_t st, uint32_t* launches, bool finish) {
    (void)N;
    const void* fn = g.rec ? (const void*)k_rebuild<true> : (const void*)k_rebuild<false>;
    int per_sm = 0, sms = 0, dev = 0;
    cudaError_t e = cudaGetDevice(&dev);
    if (e == cudaSuccess) e = cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    if (e == cudaSuccess) e = blocks_per_sm(fn, RB_THREADS, 4, &per_sm);
    if (e != cudaSuccess) return e;
    const int grid = sms * per_sm;
    DevGraph gg = g;
    const uint64_t* kk = kv;
    BatchBufs bb = b;
    VertexBufs vv = vb;
    double slack = sp.slack;
    uint32_t min_cap = sp.min_cap;
    uint64_t cap0 = sp.cap0, cap1 = sp.cap1;
    DevCtl* c = ctl;
    int cl = finish ? 1 : 0;
    void* args[] = {&gg, &kk, &bb, &vv, &slack, &min_cap, &cap0, &cap1, &c, &cl};
    e = cudaLaunchCooperativeKernel(fn, dim3(grid), dim3(RB_THREADS), args, 0, st);
    ++*launches;
    return e;
}

void launch_refresh_degrees(const DevGraph& g, const VertexBufs& vb, DevCtl* ctl, cudaStream_t st,
                            uint32_t* launches) {
    if (!PPR_REFRESH_FILTER || !g.pool_wide) return;
    int dev = 0, sms = 0;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    LAUNCH_PK(k_refresh_degrees)<<<sms, RF_THREADS, RF_BITS / 8, st>>>(g, vb.touched, ctl);
    ++*launches;
}

cudaError_t prepare_refresh_degrees() {
    // 128 KB of dynamic shared memory (opt-in, per device: called by ppr_create on its device)
    cudaError_t e = cudaFuncSetAttribute((const void*)k_refresh_degrees<false>,
                                         cudaFuncAttributeMaxDynamicSharedMemorySize, RF_BITS / 8);
    if (e == cudaSuccess)
        e = cudaFuncSetAttribute((const void*)k_refresh_degrees<true>,
                                 cudaFuncAttributeMaxDynamicSharedMemorySize, RF_BITS / 8);
    return e;
}

void launch_seg_cleanup(const uint64_t* kv, uint64_t N, const BatchBufs& b, const VertexBufs& vb,
                        DevCtl* ctl, cudaStream_t st, uint32_t* launches) {
    k_seg_cleanup<<<grid_for(N, 256), 256, 0, st>>>(kv, b, vb.vseg, ctl);
    ++*launches;
}

void launch_restore(const DevGraph& g, const uint64_t* ku, uint64_t N, const BatchBufs& b,
                    const VertexBufs& vb, DevCtl* ctl, cudaStream_t st, uint32_t* launches) {
    LAUNCH_PK(k_restore)<<<restore_blocks(N, g.S, 128), 128, 0, st>>>(g, ku, N, b, vb.touched, ctl);
    ++*launches;
}

void launch_apply_restore(const DevGraph& g, const uint64_t* kv, const uint64_t* ku, uint64_t N,
                          const BatchBufs& b, const VertexBufs& vb, DevCtl* ctl, cudaStream_t st,
                          uint32_t* launches) {
    const unsigned ab = grid_for(N * 32, 256);
    LAUNCH_PK(k_apply_restore)<<<ab + restore_blocks(N, g.S, 256), 256, 0, st>>>(g, kv, ku, N, b,
                                                                              vb.touched, ctl, ab);
    ++*launches;
}

void launch_build_count(const uint32_t* src, const uint32_t* dst, uint64_t m, int undirected,
                        const DevGraph& g, uint32_t n, cudaStream_t st, uint32_t* launches) {
    (void)n;
    LAUNCH_PK(k_build_count)<<<grid_for(m, 256), 256, 0, st>>>(src, dst, m, undirected, g);
    ++*launches;
}

void launch_caps_from_len(const DevGraph& g, const VertexBufs& vb, double slack, uint32_t min_cap,
                          cudaStream_t st, uint32_t* launches) {
    LAUNCH_PK(k_caps_from_len)<<<grid_for(g.n, 256), 256, 0, st>>>(g, vb.newcap, slack, min_cap);
    ++*launches;
}

void launch_build_fill(const uint32_t* src, const uint32_t* dst, uint64_t m, int undirected,
                       const DevGraph& g, const VertexBufs& vb, cudaStream_t st,
                       uint32_t* launches) {
    LAUNCH_PK(k_set_slabs)<<<grid_for(g.n, 256), 256, 0, st>>>(g, vb.newoff, vb.newcap);
    LAUNCH_PK(k_build_fill)<<<grid_for(m, 256), 256, 0, st>>>(src, dst, m, undirected, g);
    *launches += 2;
}

void launch_init_state(const DevGraph& g, cudaStream_t st, uint32_t* launches) {
    LAUNCH_PK(k_init_state)<<<grid_for(g.S, 256), 256, 0, st>>>(g);
    ++*launches;
}

void launch_export(const DevGraph& g, int active, const unsigned long long* off, uint64_t* keys,
                   const uint32_t* inv, cudaStream_t st, uint32_t* launches) {
    LAUNCH_PK(k_export)<<<grid_for(g.n, 256), 256, 0, st>>>(g, active, off, keys, inv);
    ++*launches;
}

void launch_gather_rec(const DevGraph& g, double* P, double* R, uint32_t* dout, int zero_pr,
                       const uint32_t* perm, cudaStream_t st, uint32_t* launches) {
    k_gather_rec<<<grid_for(g.n, 256), 256, 0, st>>>(g, P, R, dout, zero_pr, perm);
    ++*launches;
}

void launch_gather_col(const double* src, uint32_t S, uint32_t sidx, uint32_t n, double* dst,
                       const uint32_t* perm, cudaStream_t st, uint32_t* launches) {
    k_gather_col<<<grid_for(n, 256), 256, 0, st>>>(src, S, sidx, n, dst, perm);
    ++*launches;
}

void launch_relabel(const uint32_t* src, const uint32_t* dst, uint64_t m, int undirected, uint32_t n,
                    uint32_t* deg, uint64_t* k0, uint32_t* v0, uint64_t* k1, uint32_t* v1,
                    uint32_t* hist, uint32_t* perm, uint32_t* inv, cudaStream_t st,
                    uint32_t* launches) {
    cudaMemsetAsync(deg, 0, sizeof(uint32_t) * n, st);
    k_count_out<<<grid_for(m, 256), 256, 0, st>>>(src, dst, m, undirected, deg);
    k_degree_keys<<<grid_for(n, 256), 256, 0, st>>>(deg, n, k0, v0);
    int shifts[8], np = 0, lg = 0;
    while ((1ull << lg) < n) lg++;
    for (int s = 0; s < lg; s += 8) shifts[np++] = s;
    for (int s = 32; s < 64; s += 8) shifts[np++] = s;
    const int w = radix_sort_pairs(k0, v0, k1, v1, n, shifts, np, hist, st, launches);
    const int spread = 1;  // measured best of 0..3 (round 1)
    k_perm_from_sorted<<<grid_for(n, 256), 256, 0, st>>>(w ? k1 : k0, n, perm, inv, spread);
    *launches += 3;
}

void launch_map_ids(uint32_t* a, uint64_t m, const uint32_t* perm, cudaStream_t st,
                    uint32_t* launches) {
    if (!m) return;
    k_map_ids<<<grid_for(m, 256), 256, 0, st>>>(a, m, perm);
    ++*launches;
}

void launch_gather_u32(const uint32_t* src, const uint32_t* perm, uint32_t n, uint32_t* dst,
                       cudaStream_t st, uint32_t* launches) {
    k_gather_u32<<<grid_for(n, 256), 256, 0, st>>>(src, perm, n, dst);
    ++*launches;
}

void launch_len_to_u32(const DevGraph& g, uint32_t* out, cudaStream_t st, uint32_t* launches) {
    LAUNCH_PK(k_len_to_u32)<<<grid_for(g.n, 256), 256, 0, st>>>(g, out);
    ++*launches;
}

}  // namespace ppr
