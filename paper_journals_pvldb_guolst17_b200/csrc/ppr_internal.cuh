// ppr_internal.cuh -- device-side data layout and helpers shared by the
// kernels of libppr.so (sm_100a).  Nothing here is used by oracle/.
//
// HBM layout:
//   dout   u32[n]                 d_out(v)                       (Table 1)
//   slab   SlabRec[n] (8 B each) {u32 off, u32 len} of N_in(v); cap u32[n] (store only)
//   pool   u32[pool_cap] x 2      slab storage; one active, one rebuild target
//   P, R   f64[S][n]              estimate / residual per source (Table 1)
//   F      u64[S*n] x 2           frontier entries (sidx << 32 | v), double-buffered
//   W      f64[S*n]               Alg 3 snapshot w aligned with F (Vanilla/DupDetect)
//   bitmap u32[ceil(S*n/32)]      UniqueEnqueue bits (Vanilla/Eager)
//   ctl    DevCtl                 counters, flags, stats, grid barrier
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

namespace ppr {

// Logical slab descriptor of N_in(v) (what the store code works with).
struct Slab {
    unsigned long long off;  // first pool index of N_in(v)
    uint32_t len;            // |N_in(v)| (multiset)
    uint32_t cap;            // reserved entries
};
// Stored form (array layout): the push reads only {off, len} of a pushed vertex,
// so they are one 8-byte record and the capacity (used by the store alone) is a
// separate array -- the descriptor array the push gathers from is n x 8 B (LJ
// shape: 39 MB instead of 78 MB of the 126 MB L2).  Pool offsets are u32: a
// pool holds fewer than 2^32 entries (checked at create).
struct __align__(8) SlabRec {
    uint32_t off;
    uint32_t len;
};

// Packed layout (single-source handles): every per-vertex field the hot path
// touches lives in one 32-byte record = one DRAM/L2 sector, so a pushed
// vertex (R, P, slab) and an edge target (R, d_out) each cost one sector.
struct __align__(32) VRec {
    double r;       // R_s(v)
    double p;       // P_s(v)
    uint32_t off;   // first pool index of N_in(v)
    uint32_t len;   // |N_in(v)|
    uint32_t dout;  // d_out(v)
    uint32_t cap;   // reserved slab entries
};

// error codes written by kernels into DevCtl::err (mirror ppr_status)
enum : int { KERR_OK = 0, KERR_RANGE = -2, KERR_NOENT = -3, KERR_NOCONV = -7, KERR_OVERFLOW = -8 };

// Statistics and flags the host reads back after every call (one D2H copy).
struct DevStats {
    unsigned long long pushes;
    unsigned long long pushed_edges;
    unsigned long long max_frontier;
    unsigned int iters[2];     // [0] = POS, [1] = NEG
    int err;                   // KERR_*
    int rebuild;               // 1: the store takes the rebuild path this batch
    unsigned int active_pool;  // index of the active slab pool
    unsigned int n_vheads;     // v-segments in the (v,u)-sorted batch
    unsigned int n_uheads;     // u-segments in the (u,v)-sorted batch
    unsigned int n_touched;    // distinct u restored
    unsigned long long pool_top; // scan total (rebuild / build)
    long long arc_delta;       // net change of the arc count this batch
    unsigned int n_big;        // vertices copied warp-wide in a rebuild
    unsigned int pad0;
    unsigned long long walk_edges; // in-arc walks (SHARED: one per (source group, arc))
    unsigned long long entries;    // frontier entries processed (SHARED: (vertex, group) rows that pushed)
    unsigned long long pool_extent; // slots [0, extent) of the active pool hold slabs (build / rebuild)
    // device clock (%globaltimer, ns): POS / NEG phase durations summed over the
    // push launches of a call (one, or one per source wave); restore kernel
    // first-CTA start (atomicMin) and last-CTA end (atomicMax)
    unsigned long long ns_push[2];
    unsigned long long t_restore[2];
    unsigned long long dup_enq;    // PPR_OPT_CHECK_ENQUEUE: enqueues of an already queued entry
};

__device__ __forceinline__ unsigned long long globaltimer_ns() {
    unsigned long long t;
    asm volatile("mov.u64 %0, %globaltimer;" : "=l"(t));
    return t;
}

// A counter alone on its 128-byte line: the per-round counters, the tile
// claims and the grid barrier are hammered by every CTA, so none of them
// may share a line with another.
struct __align__(128) HotU64 {
    unsigned long long v;
    unsigned long long pad[15];
};
struct __align__(128) HotU32 {
    unsigned int v;
    unsigned int pad[31];
};

struct DevCtl {
    HotU64 fcount[3];   // frontier counters, triple-buffered by round (push.cu)
    HotU64 tilectr[3];  // tile claims, triple-buffered by round
    HotU64 hyb[3];      // hybrid tail ring: head, tail, done (push.cu)
    HotU32 bar_count;   // grid barrier arrivals
    HotU32 bar_gen;     // grid barrier generation
    DevStats st;
};

// Slab-pool entries of N_in(v), two formats chosen per handle (DevGraph::pool_wide):
//  * wide (PoolEnt): the in-neighbour u AND its current out-degree,
//    (d_out(u) << 32) | u.  The push reads the divisor d(u) of Alg 3 line 19 with
//    the in-list entry itself -- one dependent random access per pushed edge
//    fewer than a separate d_out[u] gather, which matters when d_out is
//    DRAM-resident (Twitter shape: push 96 -> 69 ms per batch).  The store keeps
//    the cached degrees exact: after every batch's restore has updated d_out, the
//    last store launch streams the active pool and rewrites the entries whose
//    degree changed.  Unused slots (slab slack) hold POOL_EMPTY so that stream
//    needs no slab descriptors.
//  * narrow (u32 ids, d_out gathered per edge): when R and d_out are L2-resident
//    the gather is cheap and the refresh stream would cost more than it saves
//    (LJ shape: 3.30 vs 3.49 ms per batch).
// Vertex ids are < 2^32 - 1 (ppr_create), so u = 0xFFFFFFFF marks an empty slot.
using PoolEnt = unsigned long long;
constexpr PoolEnt POOL_EMPTY = ~0ull;
__host__ __device__ __forceinline__ uint32_t pe_v(PoolEnt e) { return (uint32_t)e; }
__host__ __device__ __forceinline__ uint32_t pe_d(PoolEnt e) { return (uint32_t)(e >> 32); }
__host__ __device__ __forceinline__ PoolEnt pe_make(uint32_t v, uint32_t d) {
    return ((PoolEnt)d << 32) | v;
}

struct DevGraph {
    uint32_t n;
    uint32_t S;
    double alpha;
    double eps;
    uint32_t* dout;
    SlabRec* slab;            // {off, len} of N_in(v)
    uint32_t* cap;            // reserved entries of N_in(v)
    PoolEnt* pool[2];         // slab pools (one active, one rebuild target); u32 entries if !pool_wide
    uint32_t pool_wide;       // 1: PoolEnt entries carry d_out; 0: u32 in-neighbour ids
    double* P;
    double* R;
    const uint32_t* sources;  // [S]
    VRec* rec;                // packed layout (S == 1): replaces dout, slab, R, P
};

// ------------------------------------------------------------------ layout accessors
// PK = packed (VRec) layout; otherwise arrays with R, P vertex-major [n][S] (the S
// residuals of a vertex share cache lines; identical to [S][n] for S = 1).

template <bool PK>
__device__ __forceinline__ double* Rp(const DevGraph& g, uint32_t sidx, uint32_t v) {
    if (PK) return &g.rec[v].r;
    return g.R + (size_t)v * g.S + sidx;  // vertex-major [n][S]
}
template <bool PK>
__device__ __forceinline__ double* Pp(const DevGraph& g, uint32_t sidx, uint32_t v) {
    if (PK) return &g.rec[v].p;
    return g.P + (size_t)v * g.S + sidx;
}
template <bool PK>
__device__ __forceinline__ uint32_t* doutp(const DevGraph& g, uint32_t v) {
    if (PK) return &g.rec[v].dout;
    return &g.dout[v];
}
template <bool PK>
__device__ __forceinline__ uint32_t* lenp(const DevGraph& g, uint32_t v) {
    if (PK) return &g.rec[v].len;
    return &g.slab[v].len;
}
template <bool PK>
__device__ __forceinline__ Slab get_slab(const DevGraph& g, uint64_t v) {
    Slab s;
    if (PK) {
        const uint4 q = __ldcg(reinterpret_cast<const uint4*>(&g.rec[v].off));
        s.off = q.x;
        s.len = q.y;
        s.cap = q.w;
    } else {
        const SlabRec r = g.slab[v];
        s.off = r.off;
        s.len = r.len;
        s.cap = g.cap[v];
    }
    return s;
}
template <bool PK>
__device__ __forceinline__ void put_slab(const DevGraph& g, uint64_t v, const Slab& s) {
    if (PK) {
        g.rec[v].off = (uint32_t)s.off;
        g.rec[v].len = s.len;
        g.rec[v].cap = s.cap;
    } else {
        SlabRec r;
        r.off = (uint32_t)s.off;
        r.len = s.len;
        g.slab[v] = r;
        g.cap[v] = s.cap;
    }
}

// ------------------------------------------------------------------ pool entries (either format)

__device__ __forceinline__ uint32_t pool_id(const DevGraph& g, const PoolEnt* pool, uint64_t i) {
    return g.pool_wide ? pe_v(pool[i]) : reinterpret_cast<const uint32_t*>(pool)[i];
}
__device__ __forceinline__ void pool_copy(const DevGraph& g, PoolEnt* dst, uint64_t j,
                                          const PoolEnt* src, uint64_t i) {
    if (g.pool_wide) dst[j] = src[i];
    else reinterpret_cast<uint32_t*>(dst)[j] = reinterpret_cast<const uint32_t*>(src)[i];
}
// d: d_out(v) for the wide format (0 = "not yet known", set by the degree refresh)
__device__ __forceinline__ void pool_put(const DevGraph& g, PoolEnt* pool, uint64_t i, uint32_t v,
                                         uint32_t d) {
    if (g.pool_wide) pool[i] = pe_make(v, d);
    else reinterpret_cast<uint32_t*>(pool)[i] = v;
}
__device__ __forceinline__ void pool_clear(const DevGraph& g, PoolEnt* pool, uint64_t i) {
    if (g.pool_wide) pool[i] = POOL_EMPTY;
    else reinterpret_cast<uint32_t*>(pool)[i] = 0xFFFFFFFFu;
}

// ------------------------------------------------------------------ helpers

__device__ __forceinline__ double ld_relaxed_f64(const double* p) {
    double v;
    asm volatile("ld.relaxed.gpu.global.f64 %0, [%1];" : "=d"(v) : "l"(p) : "memory");
    return v;
}

__device__ __forceinline__ unsigned int ld_acquire_u32(const unsigned int* p) {
    unsigned int v;
    asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
    return v;
}

__device__ __forceinline__ unsigned long long ld_acquire_u64(const unsigned long long* p) {
    unsigned long long v;
    asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}

__device__ __forceinline__ void st_release_u32(unsigned int* p, unsigned int v) {
    asm volatile("st.release.gpu.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}

// Sense-free generation barrier over all CTAs of a cooperative launch.
#ifndef PPR_BAR_SLEEP
#define PPR_BAR_SLEEP 32
#endif
__device__ __forceinline__ void grid_sync(DevCtl* ctl) {
    __syncthreads();
    if (threadIdx.x == 0) {
        unsigned int gen = ld_acquire_u32(&ctl->bar_gen.v);
        __threadfence();
        unsigned int arrived = atomicAdd(&ctl->bar_count.v, 1u) + 1u;
        if (arrived == gridDim.x) {
            ctl->bar_count.v = 0;
            __threadfence();
            st_release_u32(&ctl->bar_gen.v, gen + 1u);
        } else {
            while (ld_acquire_u32(&ctl->bar_gen.v) == gen)
                if (PPR_BAR_SLEEP) __nanosleep(PPR_BAR_SLEEP);
        }
        __threadfence();
    }
    __syncthreads();
}

__device__ __forceinline__ unsigned lane_id() { return threadIdx.x & 31u; }

// ------------------------------------------------------------------ L2 cache policies
// The push is bound by random fp64 atomics: ~120 G/s when the residual array
// is L2-resident vs ~43 G/s once it spills to DRAM (tools/atomic_bench.cu on
// B200).  R and d_out (the per-edge random targets) are therefore accessed
// with an evict_last policy and the streamed data (slab pool, descriptors,
// P, frontiers) with evict_first.
__device__ __forceinline__ unsigned long long l2_keep() {
    unsigned long long p;
#if defined(PPR_KEEP_NORMAL)  // experiment builds only
    asm("createpolicy.fractional.L2::evict_normal.b64 %0, 1.0;" : "=l"(p));
#elif defined(PPR_KEEP_HALF)
    asm("createpolicy.fractional.L2::evict_last.L2::evict_unchanged.b64 %0, 0.5;" : "=l"(p));
#else
    asm("createpolicy.fractional.L2::evict_last.b64 %0, 1.0;" : "=l"(p));
#endif
    return p;
}
__device__ __forceinline__ unsigned long long l2_stream() {
    unsigned long long p;
    asm("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(p));
    return p;
}
// policies of the pool (per-edge in-list reads) and slab-descriptor reads (per
// pushed vertex): 0 = evict_first (streamed), 1 = evict_normal, 2 = evict_last
#ifndef PPR_POOL_POL
#define PPR_POOL_POL 0
#endif
// (-1, the default for the slab reads: evict_normal when the push runs with the
// persisting L2 window, i.e. the hot set is L2-resident -- the 8-byte descriptors
// then stay in L2 between rounds, LJ push -1.6%; evict_first otherwise, Twitter)
#ifndef PPR_SLAB_POL
#define PPR_SLAB_POL -1
#endif
template <int K>
__device__ __forceinline__ unsigned long long l2_pol() {
    unsigned long long p;
    if (K == 2) asm("createpolicy.fractional.L2::evict_last.b64 %0, 1.0;" : "=l"(p));
    else if (K == 1) asm("createpolicy.fractional.L2::evict_normal.b64 %0, 1.0;" : "=l"(p));
    else asm("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(p));
    return p;
}
__device__ __forceinline__ double atom_add_pol(double* a, double v, unsigned long long pol) {
    double r;
    asm volatile("atom.global.add.L2::cache_hint.f64 %0, [%1], %2, %3;"
                 : "=d"(r) : "l"(a), "d"(v), "l"(pol) : "memory");
    return r;
}
__device__ __forceinline__ double atom_exch_f64_pol(double* a, double v, unsigned long long pol) {
    unsigned long long r;
    asm volatile("atom.global.exch.L2::cache_hint.b64 %0, [%1], %2, %3;"
                 : "=l"(r) : "l"(a), "l"(__double_as_longlong(v)), "l"(pol) : "memory");
    return __longlong_as_double(r);
}
__device__ __forceinline__ void red_add_pol(double* a, double v, unsigned long long pol) {
    asm volatile("red.global.add.L2::cache_hint.f64 [%0], %1, %2;" ::"l"(a), "d"(v), "l"(pol)
                 : "memory");
}
__device__ __forceinline__ uint32_t ld_u32_pol(const uint32_t* a, unsigned long long pol) {
    uint32_t r;
    asm volatile("ld.global.nc.L2::cache_hint.u32 %0, [%1], %2;" : "=r"(r) : "l"(a), "l"(pol));
    return r;
}
__device__ __forceinline__ uint32_t ld_u32_nc_pol(const uint32_t* a, unsigned long long pol) {
    uint32_t r;
    asm volatile("ld.global.nc.L2::cache_hint.u32 %0, [%1], %2;" : "=r"(r) : "l"(a), "l"(pol));
    return r;
}
__device__ __forceinline__ PoolEnt ld_pool_ent(const PoolEnt* a, unsigned long long pol) {
    PoolEnt r;
    asm volatile("ld.global.nc.L2::cache_hint.u64 %0, [%1], %2;" : "=l"(r) : "l"(a), "l"(pol));
    return r;
}
__device__ __forceinline__ uint2 ld_slab_pol(const SlabRec* a, unsigned long long pol) {
    uint2 r;
    asm volatile("ld.global.nc.L2::cache_hint.v2.u32 {%0, %1}, [%2], %3;"
                 : "=r"(r.x), "=r"(r.y) : "l"(a), "l"(pol));
    return r;
}
__device__ __forceinline__ ulonglong2 ld_u64x2_pol(const void* a, unsigned long long pol) {
    ulonglong2 r;
    asm volatile("ld.global.nc.L2::cache_hint.v2.u64 {%0, %1}, [%2], %3;"
                 : "=l"(r.x), "=l"(r.y) : "l"(a), "l"(pol));
    return r;
}

// pushCond of Alg 3 lines 8-10: POS r > eps, NEG r < -eps
template <bool POS>
__device__ __forceinline__ bool push_cond(double r, double eps) {
    return POS ? (r > eps) : (r < -eps);
}

// PushCondLocal of Alg 4 lines 1-5: the add crossed the threshold
template <bool POS>
__device__ __forceinline__ bool crossed(double pre, double cur, double eps) {
    return !push_cond<POS>(pre, eps) && push_cond<POS>(cur, eps);
}

}  // namespace ppr
