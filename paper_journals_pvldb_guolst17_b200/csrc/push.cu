// push.cu -- persistent two-phase frontier push (steps a3-a6 of the hot path).
//
// One cooperative launch runs every round of both phases (POS: r > eps, then
// NEG: r < -eps; Alg 3 lines 1-7) with a grid barrier between
// rounds, so there is no host round-trip per round (north_star "persistent
// ... iteration loop").  Frontier entries are (source index << 32 | vertex),
// so all sources of a multi-source handle advance in the same rounds.
//
// Round structure per mode (Table 3):
//   OPT       Alg 4 with the self-update fused into the same
//             pass: r_u is read ONCE with a relaxed load (eager propagation,
//             P:1102-1112), every v in N_in(u) gets
//             atomicAdd(R(v), (1-a) r_u / d(v)) and is enqueued iff this add
//             crossed the threshold (local duplicate detection, Alg 4 lines
//             14-17); then R(u) -= r_u atomically and u is
//             re-enqueued iff the value that subtraction produced still meets
//             pushCond (lines 21-23).  Exactly-once enqueue:
//             DESIGN.md K-PUSH.
//   EAGER     Alg 4 order (propagate, grid barrier, self-update) with
//             UniqueEnqueue through a bitmap instead of the crossing test.
//   DUPDETECT Alg 3 order (snapshot/self-update, grid barrier, propagate)
//             with the crossing test.
//   VANILLA   Alg 3 as printed: snapshot, grid barrier,
//             propagate, UniqueEnqueue through a bitmap.
// OPT's default schedule runs each phase's rounds on the asynchronous ring
// worklist from the seed round on (hybrid_tail with PushArgs::hyb_all; any push
// order is valid, Lemma 1), with lazy done-accounting (async_loop, RING_LAZY);
// frontier rounds with the ring only for the post-peak tail on request.
//
// Work distribution (north_star "degree-binned scheduling"): a CTA takes a
// tile of T <= 512 frontier entries (T shrinks with the frontier so small
// rounds still spread over all SMs; the first tile of every CTA is static,
// later ones are claimed with one atomic per CTA), scans the entries'
// in-degrees in shared memory, and its warps then walk the tile's edge range
// in blocks of U x 32 edges (U independent load/atomic chains per lane for
// memory-level parallelism), each edge finding its owner entry by binary
// search in the shared prefix array.  In-lists of any size -- thread-, warp-
// or CTA-sized -- are thereby balanced across all lanes of the CTA, slab
// reads are coalesced, and no CTA barrier is needed inside the edge walk.
// Enqueues go into a per-warp shared-memory queue slice (ballot + popc); a
// full slice is flushed by its warp with one global atomic, and the CTA
// flushes all slices with one atomic at the end of a round.
#include "block_scan.cuh"
#include "primitives.cuh"
#include "push.cuh"

namespace ppr {

namespace {

// vertex layout / pool format of a push instantiation (template parameter LAY):
// arrays with u32 in-list entries, packed VRec records, arrays with PoolEnt entries
// that carry d_out (ppr_internal.cuh) -- compile-time, so the hot loop of each
// format has no branch and no registers for the other
constexpr int LAY_ARRAYS = 0, LAY_PACKED = 1, LAY_WIDE = 2;

constexpr int PT = PUSH_THREADS;
constexpr int NW = PT / 32;     // warps per CTA
#ifndef PPR_PUSH_U
#define PPR_PUSH_U 2
#endif
// push_chk.cu compiles the Opt push with the exactly-once enqueue check
#ifndef PPR_CHECK_ENQ
#define PPR_CHECK_ENQ 0
#endif
#ifndef PPR_RING_LAZY
#define PPR_RING_LAZY 1
#endif
#ifndef PPR_RING_FLUSH_EVERY
#define PPR_RING_FLUSH_EVERY 16
#endif
#ifndef PPR_RING_LOW
#define PPR_RING_LOW 256
#endif
// RING_PRECLAIM + RING_TCACHE (default on): the next chunk is claimed a tile ahead
// and served from a cached tail value, so the claim barrier no longer waits for
// memory round trips (they were ~22% of the LJ push's warp-state samples:
// profiles/round2_s3_final/push_lj_top_stall_sass.txt; push 2.85 -> 2.79 ms)
#ifndef PPR_RING_TCACHE
#define PPR_RING_TCACHE 1
#endif
#ifndef PPR_RING_PRECLAIM
#define PPR_RING_PRECLAIM 1
#endif
#ifndef PPR_RING_SPLIT
#define PPR_RING_SPLIT 1
#endif
#ifndef PPR_RING_MIN_TILE
#define PPR_RING_MIN_TILE 32
#endif
constexpr unsigned long long RING_SPLIT = PPR_RING_SPLIT;        // a claim takes 1/(SPLIT * grid) of the queue
constexpr unsigned long long RING_MIN_TILE = PPR_RING_MIN_TILE;  // ... but at least this many entries
constexpr int RING_FLUSH_EVERY = PPR_RING_FLUSH_EVERY;  // RING_LAZY: tiles between CTA-wide flushes
constexpr unsigned long long RING_LOW = PPR_RING_LOW;   // ... or flush at once when fewer than this
                                                        // many entries per CTA are queued
#ifndef PPR_PUSH_TMAX
#define PPR_PUSH_TMAX PT
#endif
#ifndef PPR_PUSH_PREF
#define PPR_PUSH_PREF 0
#endif
// PIPE (software-pipelined edge walk, walk_edges): on for the 2-chain build;
// the 3-chain build of the dense graphs keeps the plain walk (Twitter shape, wide
// entries, ring schedule: push 84.4 ms plain vs 89.2 ms pipelined)
#ifndef PPR_PUSH_PIPE
#define PPR_PUSH_PIPE (PPR_PUSH_U == 2)
#endif
#ifndef PPR_PUSH_OPT_ONLY
#define PPR_PUSH_OPT_ONLY 0
#endif
// per-CTA time split of the trace (PPR_TRACE): compiled in only on request,
// its counters would otherwise cost registers in every thread
#ifndef PPR_PUSH_TIMESPLIT
#define PPR_PUSH_TIMESPLIT 0
#endif
constexpr bool kTimeSplit = PPR_PUSH_TIMESPLIT;
constexpr int U = PPR_PUSH_U;   // edges per lane per step
#ifndef PPR_PUSH_QW
#define PPR_PUSH_QW 256
#endif
constexpr int QW = PPR_PUSH_QW; // per-warp queue slice (entries)
enum { M_OPT = 0, M_EAGER = 1, M_DUP = 2, M_VAN = 3, M_ASYNC = 4, M_SCAN = 5 };
// how a warp tile gets r and decides enqueues
enum { K_OPT = 0, K_EAGER = 1, K_DUP = 2, K_VAN = 3, K_SCAN = 4 };
// K_SCAN (mode EAGER_SCAN): eager read as in Opt, but every residual change is a
// fire-and-forget reduction that also marks the touched vertex in a bitmap;
// the next frontier is decided after a grid barrier by scanning the bitmap.

struct TileArrays {
    uint32_t scan[PT + 1];                // exclusive in-degree prefix of the tile
    uint32_t sid[PT];                     // source index of each entry
    unsigned long long off[PT];           // slab offset of each entry
    double w[PT];                         // (1-a) * r of each entry
};
// PPR_PUSH_LEAN (default 1): two tile buffers alternate between consecutive
// tiles of a round and the next tile is claimed as a tile starts, so a tile
// costs two CTA barriers (warp totals, prefix) instead of six; warps that
// finish walking tile t go on to tile t+1's entry loads and exchange while
// the last warps of tile t are still walking (the barrier after the warp
// totals of t+1 is the first point that waits for them).
#ifndef PPR_PUSH_LEAN
#define PPR_PUSH_LEAN 1
#endif
constexpr int NBUF = PPR_PUSH_LEAN ? 2 : 1;
struct Smem {
    TileArrays tb[NBUF];                  // the CTA's current tile (LEAN: alternating buffers)
    uint32_t wtot[NBUF][NW];              // LEAN: per-warp in-degree totals of a tile
    unsigned long long nxt[NBUF];         // LEAN: the tile claimed while this one runs
    unsigned int chunkb[NBUF];            // LEAN: next 32-edge chunk of each buffer
    unsigned long long q[NW][QW];         // per-warp enqueue slices
    unsigned int wq[NW];                  // slice fill at the end-of-round flush
    unsigned long long gbase;
    unsigned long long next;              // next claimed tile
    unsigned long long cround;            // this round's frontier size
    unsigned int chunk;                   // next 32-edge chunk of the tile (dynamic claims)
    uint32_t warp_tmp[NW + 1];            // block-scan scratch
};


struct Ctx {
    const PoolEnt* pool;
    unsigned long long* Fout;
    unsigned long long* cnt_out;
    unsigned long long* trace_edges;  // this round's edge counter (trace mode) or null
    unsigned long long ring_cap;      // async mode: Fout is a ring of this many slots (0: linear)
    uint32_t qn;                      // warp-uniform fill of this warp's slice
    unsigned long long pushes;        // per-thread counters
    unsigned long long edges;
    unsigned long long t_work, t_flush, t_bar;  // trace mode: ns per CTA in tiles / flush / barrier
    unsigned long long t_pro, t_claim, t_mark, t_mark2;  // tile prologue, claims
};

__device__ __forceinline__ unsigned lane() { return threadIdx.x & 31u; }
__device__ __forceinline__ unsigned warp() { return threadIdx.x >> 5; }

constexpr unsigned long long EMPTY = ~0ull;  // free ring slot (async mode)

// writes entry e at queue position pos: a linear frontier (rounds), or a
// ring slot (async) that must first have been freed by its consumer
__device__ __forceinline__ void put_entry(Ctx& c, unsigned long long pos, unsigned long long e) {
    if (c.ring_cap) {
        pos %= c.ring_cap;
        while (*(volatile unsigned long long*)&c.Fout[pos] != EMPTY) __nanosleep(64);
    }
    __stcg(&c.Fout[pos], e);
}

__device__ __forceinline__ void warp_flush(Smem& s, Ctx& c) {
    if (c.qn == 0) return;  // warp-uniform
    unsigned long long base = 0;
    if (lane() == 0) base = atomicAdd(c.cnt_out, (unsigned long long)c.qn);
    base = __shfl_sync(0xffffffffu, base, 0);
    const unsigned w = warp();
    for (uint32_t i = lane(); i < c.qn; i += 32) put_entry(c, base + i, s.q[w][i]);
    __syncwarp();
    c.qn = 0;
}

// warp-wide enqueue; caller guarantees c.qn + 32 <= QW
__device__ __forceinline__ void warp_enqueue(Smem& s, Ctx& c, const PushArgs& a, bool flag,
                                             unsigned long long e) {
    // CHECK_ENQUEUE (push_chk.cu build, Opt only): an entry must not be enqueued
    // while it is queued; the UniqueEnqueue bitmap serves as the in-queue flags
    if (PPR_CHECK_ENQ && flag) {
        const unsigned long long bit = (e >> 32) * a.g.n + (uint32_t)e;
        const uint32_t m = 1u << (bit & 31u);
        if (atomicOr(&a.bitmap[bit >> 5], m) & m) atomicAdd(&a.ctl->st.dup_enq, 1ull);
    }
    const unsigned b = __ballot_sync(0xffffffffu, flag);
    if (flag) s.q[warp()][c.qn + __popc(b & ((1u << lane()) - 1u))] = e;
    c.qn += __popc(b);
}

__device__ __forceinline__ void ensure_room(Smem& s, Ctx& c, uint32_t need) {
    if (c.qn + need > QW) {
        __syncwarp();
        warp_flush(s, c);
    }
}

// end of a round: all slices of the CTA go out with one global atomic
__device__ __forceinline__ void block_flush(Smem& s, Ctx& c) {
    const unsigned w = warp();
    __syncwarp();
    if (lane() == 0) s.wq[w] = c.qn;
    __syncthreads();
    if (threadIdx.x == 0) {
        unsigned long long tot = 0;
        for (int i = 0; i < NW; i++) {
            unsigned x = s.wq[i];
            s.wq[i] = (unsigned)tot;
            tot += x;
        }
        s.gbase = tot ? atomicAdd(c.cnt_out, tot) : 0ull;
    }
    __syncthreads();
    const unsigned long long base = s.gbase + s.wq[w];
    for (uint32_t i = lane(); i < c.qn; i += 32) put_entry(c, base + i, s.q[w][i]);
    c.qn = 0;
    __syncthreads();
}

__device__ __forceinline__ bool test_and_set(uint32_t* bitmap, unsigned long long bit) {
    const uint32_t mask = 1u << (bit & 31u);
    const uint32_t old = atomicOr(&bitmap[bit >> 5], mask);
    return (old & mask) == 0;
}

__device__ __forceinline__ void mark_bit(uint32_t* bitmap, unsigned long long bit) {
    // Test before set: hub vertices are pushed to many times per round, and an
    // unconditional RED.OR flood on their few words serialises at the L2 slice.
    // The test load may be stale (L1, invalidated at every grid barrier); a
    // stale 0 only costs a redundant RED.OR.
    const uint32_t m = 1u << (bit & 31u);
    if (!(bitmap[bit >> 5] & m)) atomicOr(&bitmap[bit >> 5], m);  // result unused: RED.OR
}

__device__ __forceinline__ void clear_bit(uint32_t* bitmap, unsigned long long bit) {
    atomicAnd(&bitmap[bit >> 5], ~(1u << (bit & 31u)));
}

// largest i with scan[i] <= e, i in [0, T): scan[T..] hold 0xFFFFFFFF
__device__ __forceinline__ int owner_of(const uint32_t* scan, uint32_t e, int top) {
    int lo = 0;
    for (int step = top; step > 0; step >>= 1)
        if (scan[lo + step] <= e) lo += step;
    return lo;
}

// ---------------------------------------------------------------- CTA tile

template <bool POS, int KIND, int LAY>
__device__ __forceinline__ void tile_body(Smem& s, Ctx& c, const PushArgs& a, bool valid,
                                          unsigned long long ent, uint64_t idx, uint32_t T,
                                          int top, int buf = 0, unsigned long long nxt = 0,
                                          unsigned long long* pf = nullptr,
                                          const unsigned long long* Fin = nullptr, uint64_t C = 0);

// Processes the T entries Fin[base_idx .. base_idx+T) (thread i = entry i):
// neighbour propagation of every pushed entry and, for K_OPT, the fused
// self-update.  Must be called by all threads of the CTA.
template <bool POS, int KIND, int LAY>
__device__ __forceinline__ void cta_tile(Smem& s, Ctx& c, const PushArgs& a,
                                         const unsigned long long* Fin, uint64_t C,
                                         uint64_t base_idx, uint32_t T, int top, int buf = 0,
                                         unsigned long long nxt = 0) {
    const uint64_t idx = base_idx + threadIdx.x;
    const bool valid = threadIdx.x < T && idx < C;
    const unsigned long long ent = valid ? __ldcg(&Fin[idx]) : 0ull;
    tile_body<POS, KIND, LAY>(s, c, a, valid, ent, idx, T, top, buf, nxt);
}

// in-list entry i of the active pool: v, and d_out(v) for the wide format
template <int LAY>
__device__ __forceinline__ void load_entry(const PoolEnt* pool, uint64_t i, unsigned long long pol,
                                           uint32_t& v, uint32_t& d) {
    if constexpr (LAY == LAY_WIDE) {
        const PoolEnt pe = ld_pool_ent(&pool[i], pol);
        v = pe_v(pe);
        d = pe_d(pe);
    } else {
        v = ld_u32_nc_pol(reinterpret_cast<const uint32_t*>(pool) + i, pol);
    }
}

// Walks the E edges of one prepared tile (scan/off/w/sid, the entries' in-lists
// concatenated): warps claim U consecutive 32-edge chunks at a time from
// *chunkp, lane k of a chunk takes edge k, finds its owner entry by binary
// search in the prefix, and runs the chain pool entry -> d_out(v) ->
// atomicAdd(R(v), (1-a) r_u / d(v)) (Alg 3 lines 17-20 / Alg 4 lines 11-17).
// All U atomics of a step are issued before any result is consumed.
template <bool POS, int KIND, int LAY>
__device__ __forceinline__ void walk_edges(Smem& s, Ctx& c, const PushArgs& a, const TileArrays& t,
                                           uint32_t E, int top, unsigned int* chunkp) {
    const unsigned L = lane(), w = warp();
    const double eps = a.g.eps;
    const uint32_t n = a.g.n;
    const unsigned long long pol_keep = l2_keep(), pol_stream = l2_pol<PPR_POOL_POL>();
    if constexpr (KIND == K_SCAN) {  // fire-and-forget edge walk: no enqueue decisions here
        for (uint32_t cb = w; cb * 32 < E; cb += NW * U) {
            uint32_t v[U], d[U];
            int j[U];
#pragma unroll
            for (int k = 0; k < U; k++) {
                const uint32_t e = (cb + NW * k) * 32 + L;
                j[k] = -1;
                v[k] = 0;
                d[k] = 1;
                if (e < E) {
                    j[k] = owner_of(t.scan, e, top);
                    load_entry<LAY>(c.pool, t.off[j[k]] + (e - t.scan[j[k]]), pol_stream, v[k], d[k]);
                }
            }
            if constexpr (LAY != LAY_WIDE) {
#pragma unroll
                for (int k = 0; k < U; k++)
                    if (j[k] >= 0) d[k] = (LAY == LAY_PACKED) ? __ldcg(&a.g.rec[v[k]].dout) : ld_u32_nc_pol(&a.g.dout[v[k]], pol_keep);
            }
#pragma unroll
            for (int k = 0; k < U; k++) {
                if (j[k] >= 0) {
                    const uint32_t sj = t.sid[j[k]];
                    red_add_pol(Rp<(LAY == LAY_PACKED)>(a.g, sj, v[k]), __ddiv_rn(t.w[j[k]], (double)d[k]), pol_keep);
                    mark_bit(a.bitmap, (size_t)v[k] * a.g.S + sj);
                }
            }
        }
    } else if constexpr (PPR_PUSH_PIPE) {
    // software-pipelined walk: the next claim's pool entries are loaded while
    // this claim's atomics are in flight, so a warp step costs about one
    // atomic round trip instead of pool load + d_out gather + atomic
    uint32_t cb = 0;
    if (L == 0) cb = atomicAdd(chunkp, (unsigned)U);
    cb = __shfl_sync(0xffffffffu, cb, 0);
    uint32_t v[U], dw[U];
    int j[U];
#pragma unroll
    for (int k = 0; k < U; k++) {
        const uint32_t e = (cb + k) * 32 + L;
        j[k] = -1;
        v[k] = 0;
        dw[k] = 1;
        if (e < E) {
            j[k] = owner_of(t.scan, e, top);
            load_entry<LAY>(c.pool, t.off[j[k]] + (e - t.scan[j[k]]), pol_stream, v[k], dw[k]);
        }
    }
    while (cb * 32 < E) {
        ensure_room(s, c, 32 * U);
        uint32_t d[U];
#pragma unroll
        for (int k = 0; k < U; k++)
            d[k] = (LAY == LAY_WIDE || j[k] < 0) ? dw[k]
                   : ((LAY == LAY_PACKED) ? __ldcg(&a.g.rec[v[k]].dout) : ld_u32_nc_pol(&a.g.dout[v[k]], pol_keep));
        double incr[U], pre[U];
        unsigned long long ev[U];
#pragma unroll
        for (int k = 0; k < U; k++) {
            if (j[k] >= 0) {
                const uint32_t sj = t.sid[j[k]];
                incr[k] = __ddiv_rn(t.w[j[k]], (double)d[k]);
                pre[k] = atom_add_pol(Rp<(LAY == LAY_PACKED)>(a.g, sj, v[k]), incr[k], pol_keep);
                ev[k] = ((unsigned long long)sj << 32) | v[k];
            }
        }
        bool act[U];
#pragma unroll
        for (int k = 0; k < U; k++) act[k] = j[k] >= 0;
        // next claim: entries in flight with the atomics above
        if (L == 0) cb = atomicAdd(chunkp, (unsigned)U);
        cb = __shfl_sync(0xffffffffu, cb, 0);
#pragma unroll
        for (int k = 0; k < U; k++) {
            const uint32_t e = (cb + k) * 32 + L;
            j[k] = -1;
            if (e < E) {
                j[k] = owner_of(t.scan, e, top);
                load_entry<LAY>(c.pool, t.off[j[k]] + (e - t.scan[j[k]]), pol_stream, v[k], dw[k]);
            }
        }
#pragma unroll
        for (int k = 0; k < U; k++) {
            bool enq = false;
            if (act[k]) {
                const double cur = __dadd_rn(pre[k], incr[k]);  // == the stored value (no FMA)
                if (KIND == K_OPT || KIND == K_DUP)
                    enq = crossed<POS>(pre[k], cur, eps);   // Alg 4 line 16
                else
                    enq = push_cond<POS>(cur, eps) &&
                          test_and_set(a.bitmap, (size_t)(ev[k] >> 32) * n + (uint32_t)ev[k]);  // UniqueEnqueue
            }
            warp_enqueue(s, c, a, enq, ev[k]);
        }
    }
    } else {
    // warps claim U consecutive 32-edge chunks at a time from a shared counter,
    // so a warp whose atomics return late does not hold up the others
    while (true) {
        uint32_t cb = 0;
        if (L == 0) cb = atomicAdd(chunkp, (unsigned)U);
        cb = __shfl_sync(0xffffffffu, cb, 0);
        if (cb * 32 >= E) break;
        ensure_room(s, c, 32 * U);
        uint32_t v[U], d[U];
        int j[U];
#pragma unroll
        for (int k = 0; k < U; k++) {
            const uint32_t e = (cb + k) * 32 + L;
            j[k] = -1;
            v[k] = 0;
            d[k] = 1;
            if (e < E) {
                j[k] = owner_of(t.scan, e, top);
                // wide pool: one 8-byte load gives v and d_out(v) (ppr_internal.cuh PoolEnt)
                load_entry<LAY>(c.pool, t.off[j[k]] + (e - t.scan[j[k]]), pol_stream, v[k], d[k]);
            }
        }
        if constexpr (LAY != LAY_WIDE) {  // narrow pool: gather d_out(v), all U loads in flight
#pragma unroll
            for (int k = 0; k < U; k++)
                if (j[k] >= 0) d[k] = (LAY == LAY_PACKED) ? __ldcg(&a.g.rec[v[k]].dout) : ld_u32_nc_pol(&a.g.dout[v[k]], pol_keep);
        }
        double incr[U], pre[U];
        uint32_t sj[U];
#pragma unroll
        for (int k = 0; k < U; k++) {
            if (j[k] >= 0) {
                sj[k] = t.sid[j[k]];
                incr[k] = __ddiv_rn(t.w[j[k]], (double)d[k]);
                pre[k] = atom_add_pol(Rp<(LAY == LAY_PACKED)>(a.g, sj[k], v[k]), incr[k], pol_keep);
            }
        }
#pragma unroll
        for (int k = 0; k < U; k++) {
            bool enq = false;
            unsigned long long ev = 0;
            if (j[k] >= 0) {
                const double cur = __dadd_rn(pre[k], incr[k]);  // == the stored value (no FMA)
                ev = ((unsigned long long)sj[k] << 32) | v[k];
                if (KIND == K_OPT || KIND == K_DUP)
                    enq = crossed<POS>(pre[k], cur, eps);   // Alg 4 line 16
                else
                    enq = push_cond<POS>(cur, eps) &&
                          test_and_set(a.bitmap, (size_t)sj[k] * n + v[k]);  // UniqueEnqueue
            }
            warp_enqueue(s, c, a, enq, ev);
        }
    }
    }  // not K_SCAN
}

// The tile's work once thread i holds entry i (valid, ent; idx indexes W):
// the entry's residual read / self-update, the CTA-wide prefix of the
// pushed entries' in-degrees, then the edge walk by all warps.
template <bool POS, int KIND, int LAY>
__device__ __forceinline__ void tile_body(Smem& s, Ctx& c, const PushArgs& a, bool valid,
                                          unsigned long long ent, uint64_t idx, uint32_t T,
                                          int top, int buf, unsigned long long nxt,
                                          unsigned long long* pf, const unsigned long long* Fin,
                                          uint64_t C) {
    const double eps = a.g.eps, alpha = a.g.alpha;
    const uint32_t sidx = (uint32_t)(ent >> 32), u = (uint32_t)ent;
    double* ru = Rp<(LAY == LAY_PACKED)>(a.g, sidx, u);
    double r = 0.0;
    bool push = false;
    // the slab descriptor depends only on u: issued before (and overlapping)
    // the residual read below, used only if the entry pushes
    uint32_t len = 0;
    unsigned long long off = 0;
    if (valid) {
        if ((LAY == LAY_PACKED)) {  // {off, len} of the vertex record (same sector as R(u), P(u))
            const uint2 q = __ldcg(reinterpret_cast<const uint2*>(&a.g.rec[u].off));
            off = q.x;
            len = q.y;
        } else {
            unsigned long long spol;
            if constexpr (PPR_SLAB_POL >= 0) spol = l2_pol<PPR_SLAB_POL>();
            else spol = a.l2_bytes ? l2_pol<1>() : l2_pol<0>();
            const uint2 sl = ld_slab_pol(&a.g.slab[u], spol);
            off = sl.x;               // SlabRec::off
            len = sl.y;               // SlabRec::len
        }
    }
    if (KIND == K_OPT) {
        // Alg 4 lines 10 and 20-21 as one atomic: r_u = R(u), R(u) = 0.  Adds that
        // reach u before the exchange are absorbed into r_u; adds
        // after it start from 0, so u's next crossing re-enqueues it exactly once
        // (DESIGN.md K-PUSH).
        if (PPR_CHECK_ENQ && valid) {  // CHECK_ENQUEUE: dequeued before the exchange can re-enqueue it
            const unsigned long long bit = (unsigned long long)sidx * a.g.n + u;
            atomicAnd(&a.bitmap[bit >> 5], ~(1u << (bit & 31u)));
            __threadfence();
        }
        r = valid ? atom_exch_f64_pol(ru, 0.0, l2_keep()) : 0.0;
        push = valid && r != 0.0;
        if (push) red_add_pol(Pp<(LAY == LAY_PACKED)>(a.g, sidx, u), __dmul_rn(alpha, r), l2_stream());
    } else if (KIND == K_EAGER || KIND == K_SCAN) {
        r = valid ? ld_relaxed_f64(ru) : 0.0;  // Alg 4 line 10: the current R(u)
        push = valid && push_cond<POS>(r, eps);
        if (KIND == K_EAGER && valid) __stcg(&a.W[idx], push ? r : 0.0);
    } else {
        r = valid ? __ldcg(&a.W[idx]) : 0.0;   // Alg 3: the snapshot S
        push = valid;
    }
    if (KIND == K_SCAN && push) {  // self-update: no result needed; u is re-tested at the scan
        red_add_pol(ru, -r, l2_keep());
        red_add_pol(Pp<(LAY == LAY_PACKED)>(a.g, sidx, u), __dmul_rn(alpha, r), l2_stream());
        mark_bit(a.bitmap, (size_t)u * a.g.S + sidx);
    }
    if (!push) len = 0;
    if (push && KIND != K_VAN && KIND != K_DUP && KIND != K_EAGER) c.pushes++;
    uint32_t E;
    TileArrays& t = s.tb[buf];
    unsigned int* chunkp = &s.chunk;
    if constexpr (PPR_PUSH_LEAN) {
        // two barriers: warp-inclusive scans + per-warp totals, then every warp
        // scans the NW totals itself and writes its part of the prefix
        const unsigned L = lane(), wi = warp();
        uint32_t inc = len;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            const uint32_t y = __shfl_up_sync(0xffffffffu, inc, o);
            if (L >= (unsigned)o) inc += y;
        }
        if (L == 31) s.wtot[buf][wi] = inc;
        t.off[threadIdx.x] = off;
        t.w[threadIdx.x] = __dmul_rn(1.0 - alpha, r);
        t.sid[threadIdx.x] = sidx;
        if (threadIdx.x == 0) {
            t.scan[PT] = 0xFFFFFFFFu;
            s.chunkb[buf] = 0;
            s.nxt[buf] = nxt;
        }
        __syncthreads();
        if (pf) {  // PREF: the next tile's entry of this thread, in flight during the walk
            const uint64_t j = s.nxt[buf] * T + threadIdx.x;
            *pf = (threadIdx.x < T && j < C) ? __ldcg(&Fin[j]) : 0ull;
        }
        const uint32_t wt = L < (unsigned)NW ? s.wtot[buf][L] : 0u;
        uint32_t wsc = wt;
#pragma unroll
        for (int o = 1; o < NW; o <<= 1) {
            const uint32_t y = __shfl_up_sync(0xffffffffu, wsc, o);
            if (L >= (unsigned)o) wsc += y;
        }
        const uint32_t wbase = __shfl_sync(0xffffffffu, wsc - wt, wi);
        E = __shfl_sync(0xffffffffu, wsc, NW - 1);
        t.scan[threadIdx.x] = threadIdx.x < T ? wbase + inc - len : 0xFFFFFFFFu;
        chunkp = &s.chunkb[buf];
    } else {
        const uint32_t ex = block_exclusive_scan_u32<PT>(len, s.warp_tmp, &E);
        t.scan[threadIdx.x] = threadIdx.x < T ? ex : 0xFFFFFFFFu;
        if (threadIdx.x == 0) {
            t.scan[PT] = 0xFFFFFFFFu;
            s.chunk = 0;
        }
        t.off[threadIdx.x] = off;
        t.w[threadIdx.x] = __dmul_rn(1.0 - alpha, r);
        t.sid[threadIdx.x] = sidx;
    }
    __syncthreads();
    if (kTimeSplit && a.trace && threadIdx.x == 0) c.t_pro += globaltimer_ns() - c.t_mark;
    if (threadIdx.x == 0) {
        c.edges += E;
        if (c.trace_edges && E) atomicAdd(c.trace_edges, (unsigned long long)E);
    }
    walk_edges<POS, KIND, LAY>(s, c, a, t, E, top, chunkp);
}

// Every CTA takes tiles of T entries: its first tile statically, the rest by
// one atomic claim each, until C is covered.
template <bool POS, int KIND, int LAY>
__device__ __forceinline__ void propagate_all(Smem& s, Ctx& c, const PushArgs& a, const unsigned long long* Fin,
                              uint64_t C, unsigned long long* tc) {
    uint64_t per = (C + gridDim.x - 1) / gridDim.x;
    uint32_t T = (uint32_t)((per + 31) / 32 * 32);
    if (T > PPR_PUSH_TMAX) T = PPR_PUSH_TMAX;
    if (T < 32) T = 32;
    int top = 1;
    while (top * 2 < (int)T) top <<= 1;
    const uint64_t ntiles = (C + T - 1) / T;
    uint64_t t = blockIdx.x;
    if constexpr (PPR_PUSH_LEAN) {
        // the claim of the next tile is issued as a tile starts and published
        // with the tile's first barrier; buffers alternate (see Smem)
        const bool claims = ntiles > gridDim.x;
        int buf = 0;
        unsigned long long pent = 0;
        bool have = false;
        while (t < ntiles) {
            unsigned long long nxt = ~0ull;
            if (claims && threadIdx.x == 0) nxt = atomicAdd(tc, 1ull) + gridDim.x;
            const uint64_t idx = t * T + threadIdx.x;
            const bool valid = threadIdx.x < T && idx < C;
            const unsigned long long ent = have ? pent : (valid ? __ldcg(&Fin[idx]) : 0ull);
            tile_body<POS, KIND, LAY>(s, c, a, valid, ent, idx, T, top, buf, nxt,
                                      (PPR_PUSH_PREF && claims) ? &pent : nullptr, Fin, C);
            have = PPR_PUSH_PREF && claims;
            t = claims ? s.nxt[buf] : ntiles;
            buf ^= 1;
        }
        __syncthreads();  // every warp is done with both buffers before the round's flush
    } else {
    while (t < ntiles) {
        if (kTimeSplit && a.trace && threadIdx.x == 0) c.t_mark = globaltimer_ns();
        cta_tile<POS, KIND, LAY>(s, c, a, Fin, C, t * T, T, top);
        if (kTimeSplit && a.trace && threadIdx.x == 0) c.t_mark2 = globaltimer_ns();
        if (ntiles <= gridDim.x) break;  // every tile was assigned statically
        if (threadIdx.x == 0) s.next = atomicAdd(tc, 1ull) + gridDim.x;
        __syncthreads();
        t = s.next;
        __syncthreads();
        if (kTimeSplit && a.trace && threadIdx.x == 0) c.t_claim += globaltimer_ns() - c.t_mark2;
    }
    }
}


// ---------------------------------------------------------------- Alg 3 / Eager sessions

// self-update session of Alg 3 (lines 13-16): w = R(u), P(u) += a w, R(u) = 0
template <int LAY>
__device__ __forceinline__ void session_snapshot(Ctx& c, const PushArgs& a, const unsigned long long* Fin,
                                 uint64_t C, bool bitmap) {
    const double alpha = a.g.alpha;
    for (uint64_t idx = (uint64_t)blockIdx.x * PT + threadIdx.x; idx < C;
         idx += (uint64_t)gridDim.x * PT) {
        const unsigned long long ent = __ldcg(&Fin[idx]);
        const size_t i = (size_t)(ent >> 32) * a.g.n + (uint32_t)ent;
        double* rp = Rp<(LAY == LAY_PACKED)>(a.g, (uint32_t)(ent >> 32), (uint32_t)ent);
        double* pp = Pp<(LAY == LAY_PACKED)>(a.g, (uint32_t)(ent >> 32), (uint32_t)ent);
        const double w = __ldcg(rp);
        __stcg(pp, __dadd_rn(__ldcg(pp), __dmul_rn(alpha, w)));
        __stcg(rp, 0.0);
        __stcg(&a.W[idx], w);
        if (bitmap) clear_bit(a.bitmap, i);
        c.pushes++;
    }
}

// Eager: self-update with the r_u recorded during propagation (Alg 4 lines 19-23)
template <bool POS, int LAY>
__device__ __forceinline__ void session_eager_self(Smem& s, Ctx& c, const PushArgs& a,
                                   const unsigned long long* Fin, uint64_t C) {
    const double eps = a.g.eps, alpha = a.g.alpha;
    const uint64_t stride = (uint64_t)gridDim.x * PT;
    for (uint64_t b = (uint64_t)blockIdx.x * PT + warp() * 32; b < C; b += stride) {
        const uint64_t idx = b + lane();
        bool enq = false;
        unsigned long long ent = 0;
        if (idx < C) {
            ent = __ldcg(&Fin[idx]);
            const double r = __ldcg(&a.W[idx]);
            if (r != 0.0) {
                const size_t i = (size_t)(ent >> 32) * a.g.n + (uint32_t)ent;
                const double old = atomicAdd(Rp<(LAY == LAY_PACKED)>(a.g, (uint32_t)(ent >> 32), (uint32_t)ent), -r);
                const double cur = __dadd_rn(old, -r);
                atomicAdd(Pp<(LAY == LAY_PACKED)>(a.g, (uint32_t)(ent >> 32), (uint32_t)ent), __dmul_rn(alpha, r));
                c.pushes++;
                enq = push_cond<POS>(cur, eps) && test_and_set(a.bitmap, i);
            }
        }
        ensure_room(s, c, 32);
        warp_enqueue(s, c, a, enq, ent);
    }
}

__device__ __forceinline__ void clear_frontier_bits(Ctx& c, const PushArgs& a, const unsigned long long* Fin,
                                    uint64_t C) {
    for (uint64_t idx = (uint64_t)blockIdx.x * PT + threadIdx.x; idx < C;
         idx += (uint64_t)gridDim.x * PT) {
        const unsigned long long ent = __ldcg(&Fin[idx]);
        clear_bit(a.bitmap, (ent >> 32) * a.g.n + (uint32_t)ent);
    }
}

// ---------------------------------------------------------------- bitmap-scan frontier
//
// After the round's reductions are complete (grid barrier), every marked
// (vertex, source) bit is tested once: it joins the next frontier iff its
// residual meets pushCond.  Words are scanned warp-wide (lane = word), the
// hits are compacted with ballot/popc into the warp's queue slice, and the
// words are cleared.  Every vertex whose residual changed this round was
// marked, and every other residual is unchanged and fails pushCond, so the
// emitted frontier is exactly {(s,v) : pushCond(R_s(v))} (Alg 3 line 1,
// restricted to the vertices the round touched) and is sorted by vertex
// within each warp's word range.
template <bool POS, int LAY>
__device__ __forceinline__ void scan_bitmap(Smem& s, Ctx& c, const PushArgs& a) {
    const double eps = a.g.eps;
    const uint64_t nbits = (uint64_t)a.g.S * a.g.n;
    const uint64_t nwords = (nbits + 31) / 32;
    const uint64_t gw = (uint64_t)blockIdx.x * NW + warp(), nw = (uint64_t)gridDim.x * NW;
    for (uint64_t w0 = gw * 32; w0 < nwords; w0 += nw * 32) {
        const uint64_t wi = w0 + lane();
        uint32_t word = wi < nwords ? __ldcg(&a.bitmap[wi]) : 0u;
        if (word) __stcg(&a.bitmap[wi], 0u);
        // lanes drain their words bit by bit; the warp advances while any lane has bits
        while (__any_sync(0xffffffffu, word != 0)) {
            bool enq = false;
            unsigned long long ent = 0;
            if (word) {
                const int b = __ffs(word) - 1;
                word &= word - 1;
                const uint64_t bit = wi * 32 + b;
                const uint32_t v = (uint32_t)(bit / a.g.S), sidx = (uint32_t)(bit % a.g.S);
                enq = push_cond<POS>(__ldcg(Rp<(LAY == LAY_PACKED)>(a.g, sidx, v)), eps);
                ent = ((unsigned long long)sidx << 32) | v;
            }
            ensure_room(s, c, 32);
            warp_enqueue(s, c, a, enq, ent);
        }
    }
}

// ---------------------------------------------------------------- seeding

template <bool POS, int LAY>
__device__ __forceinline__ void seed_phase(Smem& s, Ctx& c, const PushArgs& a) {
    const double eps = a.g.eps;
    const uint64_t stride = (uint64_t)gridDim.x * PT;
    uint64_t total;
    const uint64_t nv = a.seed_v ? (uint64_t)(*a.n_seed_v_dev) : 0;
    if (a.seed_all)
        total = (uint64_t)a.g.S * a.g.n;
    else if (a.seed_v)
        total = nv * a.g.S;
    else
        total = a.n_seed_e;
    for (uint64_t b = (uint64_t)blockIdx.x * PT + warp() * 32; b < total; b += stride) {
        const uint64_t k = b + lane();
        bool enq = false;
        unsigned long long ent = 0;
        if (k < total) {
            uint32_t sidx, v;
            if (a.seed_all) {
                sidx = (uint32_t)(k / a.g.n);
                v = (uint32_t)(k % a.g.n);
            } else if (a.seed_v) {
                sidx = (uint32_t)(k / nv);
                v = a.seed_v[k % nv];
            } else {
                ent = a.seed_e[k];
                sidx = (uint32_t)(ent >> 32);
                v = (uint32_t)ent;
            }
            ent = ((unsigned long long)sidx << 32) | v;
            enq = push_cond<POS>(__ldcg(Rp<(LAY == LAY_PACKED)>(a.g, sidx, v)), eps);
        }
        ensure_room(s, c, 32);
        warp_enqueue(s, c, a, enq, ent);
    }
}

// ---------------------------------------------------------------- hybrid tail
//
// Opt mode, PushArgs::hyb_thresh > 0: once a phase's frontier has shrunk to
// at most hyb_thresh entries, its remaining rounds are latency-bound (a few
// microseconds of dependent loads and atomics plus a grid barrier per round,
// for a few thousand pushes), so the rest of the phase runs on the
// asynchronous ring schedule instead (the same operations without round
// barriers; any push order is valid, Lemma 1; DESIGN.md K-ASYNC).
template <bool POS, int LAY>
__device__ __forceinline__ void async_loop(Smem& s, Ctx& c, const PushArgs& a, unsigned long long* head,
                                           unsigned long long* tail, unsigned long long* done);

template <bool POS, int LAY>
__device__ __forceinline__ void hybrid_tail(Smem& s, Ctx& c, const PushArgs& a,
                                            const unsigned long long* Fin, uint64_t C) {
    DevCtl* ctl = a.ctl;
    unsigned long long* head = &ctl->hyb[0].v;
    unsigned long long* tail = &ctl->hyb[1].v;
    unsigned long long* done = &ctl->hyb[2].v;
    for (uint64_t i = (uint64_t)blockIdx.x * PT + threadIdx.x; i < C; i += (uint64_t)gridDim.x * PT)
        __stcg(&a.ring[i], __ldcg(&Fin[i]));  // ring slots are EMPTY between uses
    if (blockIdx.x == 0 && threadIdx.x == 0) *tail = C;
    grid_sync(ctl);
    c.Fout = a.ring;
    c.cnt_out = tail;
    c.ring_cap = a.ring_cap;
    async_loop<POS, LAY>(s, c, a, head, tail, done);
    c.ring_cap = 0;
    grid_sync(ctl);
    if (blockIdx.x == 0 && threadIdx.x == 0) *head = *tail = *done = 0;
}

// ---------------------------------------------------------------- phase driver

template <int MODE, bool POS, int LAY>
__device__ __forceinline__ void run_phase(Smem& s, Ctx& c, const PushArgs& a, unsigned& it) {
    DevCtl* ctl = a.ctl;
    const int ph = POS ? 0 : 1;
    // seed into F[it%2] / fcount[it%3]; both that and the next counter are 0 here
    c.Fout = a.F[it & 1];
    c.cnt_out = &ctl->fcount[it % 3].v;
    seed_phase<POS, LAY>(s, c, a);
    block_flush(s, c);
    grid_sync(ctl);
    uint32_t pit = 0;
    uint64_t C = 0, Cprev = ~0ull;
    while (true) {
        // one load per CTA (grid_sync ended with __syncthreads)
        if (threadIdx.x == 0) s.cround = *(volatile unsigned long long*)&ctl->fcount[it % 3].v;
        __syncthreads();
        C = s.cround;
        c.trace_edges = (a.trace && it < a.trace_cap) ? &a.trace[4ull * it + 2] : nullptr;
        if (blockIdx.x == 0 && threadIdx.x == 0) {
            if (c.trace_edges) {
                a.trace[4ull * it] = C | ((unsigned long long)ph << 63);
                a.trace[4ull * it + 1] = globaltimer_ns();
            }
            ctl->fcount[(it + 2) % 3].v = 0;
            ctl->tilectr[(it + 2) % 3].v = 0;
            if (C > 0 && !(a.max_iters && pit >= a.max_iters)) {
                ctl->st.iters[ph]++;
                atomicMax(&ctl->st.max_frontier, (unsigned long long)C);
            }
            if (C > 0 && pit >= a.iter_cap) atomicCAS(&ctl->st.err, KERR_OK, KERR_NOCONV);
        }
        if (C == 0 || (a.max_iters && pit >= a.max_iters) || pit >= a.iter_cap) break;
        const unsigned long long* Fin = a.F[it & 1];
        // the ring takes over: for the whole phase on dense graphs (hyb_all), else
        // once the frontier is past its peak and at most hyb_thresh entries
        if (MODE == M_OPT && a.ring && !a.max_iters &&
            (a.hyb_all || (pit > 0 && C <= a.hyb_thresh && C <= Cprev))) {
            hybrid_tail<POS, LAY>(s, c, a, Fin, C);  // the phase ends on the ring
            it++;
            C = 0;
            break;
        }
        c.Fout = a.F[(it + 1) & 1];
        c.cnt_out = &ctl->fcount[(it + 1) % 3].v;
        unsigned long long* tc = &ctl->tilectr[it % 3].v;
        const unsigned long long t0 = (kTimeSplit && a.trace) ? globaltimer_ns() : 0;
        if (MODE == M_OPT) {
            propagate_all<POS, K_OPT, LAY>(s, c, a, Fin, C, tc);
        } else if (MODE == M_SCAN) {
            propagate_all<POS, K_SCAN, LAY>(s, c, a, Fin, C, tc);
            grid_sync(ctl);  // every reduction of the round has landed
            scan_bitmap<POS, LAY>(s, c, a);
        } else if (MODE == M_VAN || MODE == M_DUP) {
            session_snapshot<LAY>(c, a, Fin, C, MODE == M_VAN);
            grid_sync(ctl);
            if (MODE == M_VAN)
                propagate_all<POS, K_VAN, LAY>(s, c, a, Fin, C, tc);
            else
                propagate_all<POS, K_DUP, LAY>(s, c, a, Fin, C, tc);
        } else {  // M_EAGER
            clear_frontier_bits(c, a, Fin, C);
            grid_sync(ctl);
            propagate_all<POS, K_EAGER, LAY>(s, c, a, Fin, C, tc);
            grid_sync(ctl);
            session_eager_self<POS, LAY>(s, c, a, Fin, C);
        }
        const unsigned long long t1 = (kTimeSplit && a.trace) ? globaltimer_ns() : 0;
        block_flush(s, c);
        const unsigned long long t2 = (kTimeSplit && a.trace) ? globaltimer_ns() : 0;
        grid_sync(ctl);
        if (kTimeSplit && a.trace) {
            const unsigned long long t3 = globaltimer_ns();
            c.t_work += t1 - t0;
            c.t_flush += t2 - t1;
            c.t_bar += t3 - t2;
        }
        it++;
        pit++;
        Cprev = C;
    }
    // a frontier left by max_iters keeps its UniqueEnqueue bits: drop them
    if ((MODE == M_VAN || MODE == M_EAGER) && C > 0) clear_frontier_bits(c, a, a.F[it & 1], C);
    // leave the counters of the next phase's seed round at zero
    grid_sync(ctl);
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        ctl->fcount[0].v = ctl->fcount[1].v = ctl->fcount[2].v = 0;
        ctl->tilectr[0].v = ctl->tilectr[1].v = ctl->tilectr[2].v = 0;
    }
    grid_sync(ctl);
}

template <int MODE, int LAY>
__global__ void __launch_bounds__(PT, PUSH_MIN_BLOCKS) k_push(const __grid_constant__ PushArgs a) {
    __shared__ Smem s;
    Ctx c;
    c.trace_edges = nullptr;
    c.ring_cap = 0;
    c.qn = 0;
    c.pushes = 0;
    c.edges = 0;
    c.t_work = c.t_flush = c.t_bar = 0;
    c.t_pro = c.t_claim = c.t_mark = c.t_mark2 = 0;
    if (*(volatile int*)&a.ctl->st.err != KERR_OK) return;  // earlier stage failed: uniform exit
    c.pool = *(volatile unsigned*)&a.ctl->st.active_pool ? a.g.pool[1] : a.g.pool[0];
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        for (int i = 0; i < 3; i++) a.ctl->fcount[i].v = a.ctl->tilectr[i].v = 0;
    }
    grid_sync(a.ctl);
    const bool stamp = blockIdx.x == 0 && threadIdx.x == 0;
    const unsigned long long t0 = stamp ? globaltimer_ns() : 0;
    unsigned it = 0;
    if (a.phases & 1) run_phase<MODE, true, LAY>(s, c, a, it);
    const unsigned long long t1 = stamp ? globaltimer_ns() : 0;  // run_phase ends with a grid barrier
    if (a.phases & 2) run_phase<MODE, false, LAY>(s, c, a, it);
    if (stamp) {  // phase durations, summed over launches (source waves)
        atomicAdd(&a.ctl->st.ns_push[0], t1 - t0);
        atomicAdd(&a.ctl->st.ns_push[1], globaltimer_ns() - t1);
    }
    if (a.trace && blockIdx.x == 0 && threadIdx.x == 0 && it < a.trace_cap) {
        a.trace[4ull * it] = ~0ull;  // end marker
        a.trace[4ull * it + 1] = globaltimer_ns();
    }
    if (kTimeSplit && a.trace && threadIdx.x == 0) {  // per-CTA time split, summed over CTAs
        atomicAdd(&a.trace[4ull * a.trace_cap + 0], c.t_work);
        atomicAdd(&a.trace[4ull * a.trace_cap + 1], c.t_flush);
        atomicAdd(&a.trace[4ull * a.trace_cap + 2], c.t_bar);
        atomicAdd(&a.trace[4ull * a.trace_cap + 3], 1ull);
        atomicAdd(&a.trace[4ull * a.trace_cap + 4], c.t_pro);
        atomicAdd(&a.trace[4ull * a.trace_cap + 5], c.t_claim);
    }
    // statistics
    __shared__ unsigned long long s_red[2];
    if (threadIdx.x == 0) s_red[0] = s_red[1] = 0;
    __syncthreads();
    if (c.pushes) atomicAdd(&s_red[0], c.pushes);
    if (c.edges) atomicAdd(&s_red[1], c.edges);
    __syncthreads();
    if (threadIdx.x == 0) {
        if (s_red[0]) atomicAdd(&a.ctl->st.pushes, s_red[0]);
        if (s_red[1]) atomicAdd(&a.ctl->st.pushed_edges, s_red[1]);
    }
}

// cooperative launch carrying the L2 access-policy window as a launch attribute
inline cudaError_t coop_launch(const void* fn, int grid, const PushArgs& a, cudaStream_t st) {
    PushArgs copy = a;
    void* args[] = {&copy};
    cudaLaunchConfig_t cfg{};
    cfg.gridDim = dim3(grid);
    cfg.blockDim = dim3(PT);
    cfg.stream = st;
    cudaLaunchAttribute at[2];
    int na = 0;
    at[na].id = cudaLaunchAttributeCooperative;
    at[na].val.cooperative = 1;
    na++;
    if (a.l2_bytes) {
        at[na].id = cudaLaunchAttributeAccessPolicyWindow;
        at[na].val.accessPolicyWindow.base_ptr = a.l2_base;
        at[na].val.accessPolicyWindow.num_bytes = a.l2_bytes;
        at[na].val.accessPolicyWindow.hitRatio = a.l2_hit;
        at[na].val.accessPolicyWindow.hitProp = cudaAccessPropertyPersisting;
        at[na].val.accessPolicyWindow.missProp = cudaAccessPropertyStreaming;
        na++;
    }
    cfg.attrs = at;
    cfg.numAttrs = na;
    return cudaLaunchKernelExC(&cfg, fn, args);
}

// ---------------------------------------------------------------- asynchronous schedule
//
// PPR_MODE_ASYNC: the same Alg 4 operations on every frontier vertex (eager
// r_u read, crossing-test enqueue, fused self-update), but without rounds.
// The frontier is one ring queue per phase: producers reserve slots with
// atomicAdd(tail) (per warp slice / per tile flush), CTAs claim chunks with
// atomicAdd(head) and process each chunk as a tile as soon as its slots are
// filled, consumers free slots after reading them.  Lemma 1
// allows any push order; within a phase residuals stay monotone, so each
// vertex is still enqueued exactly once per crossing and is in the queue at
// most once at a time (capacity S*n suffices; the ring has 2*S*n slots).
// Termination: `done` counts processed entries and `tail` enqueued ones; an
// entry's children are added to tail before the entry is added to done, so
// reading done == tail (done first) means no entry is queued or in progress.

// The ring loop: CTAs claim chunks of queued entries and process each chunk
// as a tile until done == tail.  Entry: the ring holds the seeds, tail = their
// count, head = done = 0, c.Fout/c.cnt_out/c.ring_cap point at the ring.
template <bool POS, int LAY>
__device__ __forceinline__ void async_loop(Smem& s, Ctx& c, const PushArgs& a, unsigned long long* head,
                                           unsigned long long* tail, unsigned long long* done) {
    __shared__ unsigned long long s_h, s_k;
    __shared__ int s_flag, s_flushnow;
    unsigned long long debt_lo = 0, debt_hi = 0;  // thread 0: claimed, not yet served
    // RING_LAZY: thread 0's processed entries whose children may still sit in the
    // warps' queue slices -- added to `done` only after a CTA-wide flush, which
    // happens every RING_FLUSH_EVERY tiles, when the ring runs low, and before the
    // CTA idles (so done == tail still implies that nothing is queued or pending)
    unsigned long long pend = 0;
    int since = 0;
    unsigned long long t_seen = 0;  // thread 0: the last tail value read
    while (true) {
        if (threadIdx.x == 0) {
            unsigned long long h0 = 0, k0 = 0;
            int flag = 0, spins = 0, flushnow = 0;
            while (true) {
                // RING_TCACHE: a claimed range below a tail value read earlier (tail only
                // grows) is served without another read, so the claim barrier waits for
                // no memory round trip when the claim was issued a tile ahead
                unsigned long long t;
                if (PPR_RING_TCACHE && debt_lo < debt_hi && debt_lo < t_seen) {
                    t = t_seen;
                } else {
                    t = *(volatile unsigned long long*)tail;
                    t_seen = t;
                }
                if (debt_lo < debt_hi) {
                    if (t > debt_lo) {
                        h0 = debt_lo;
                        k0 = (t < debt_hi ? t : debt_hi) - debt_lo;
                        debt_lo += k0;
                        if (PPR_RING_LAZY)
                            flushnow = ++since >= RING_FLUSH_EVERY || t - debt_lo < RING_LOW * gridDim.x;
                        // RING_PRECLAIM: claim the next chunk now, while the queue is long; the
                        // atomic's result is only needed at the next claim, after this tile
                        if (PPR_RING_PRECLAIM && debt_lo == debt_hi) {
                            const unsigned long long hh = debt_hi;  // <= head: no extra read
                            if (t > hh && t - hh >= RING_LOW * gridDim.x) {
                                unsigned long long want = (t - hh + RING_SPLIT * gridDim.x - 1) / (RING_SPLIT * gridDim.x);
                                want = want < RING_MIN_TILE ? RING_MIN_TILE : (want > PT ? PT : want);
                                debt_lo = atomicAdd(head, want);
                                debt_hi = debt_lo + want;
                            }
                        }
                        break;
                    }
                } else {
                    const unsigned long long h = *(volatile unsigned long long*)head;
                    if (t > h) {
                        unsigned long long want = (t - h + RING_SPLIT * gridDim.x - 1) / (RING_SPLIT * gridDim.x);
                        want = want < RING_MIN_TILE ? RING_MIN_TILE : (want > PT ? PT : want);
                        debt_lo = atomicAdd(head, want);
                        debt_hi = debt_lo + want;
                        continue;
                    }
                }
                if (PPR_RING_LAZY && pend) {  // no work in sight: publish the pending entries first
                    flag = 2;
                    break;
                }
                // acquire: a `done` that counts an entry makes that entry's
                // children (added to `tail` before it, released below) visible
                const unsigned long long d = ld_acquire_u64(done);
                const unsigned long long t2 = ld_acquire_u64(tail);
                if (d == t2) {
                    flag = 1;
                    break;
                }
                __nanosleep(spins < 16 ? 64 : 512);
                spins++;
            }
            s_h = h0;
            s_k = k0;
            s_flag = flag;
            s_flushnow = flushnow;
        }
        __syncthreads();
        const int fl = s_flag, flushnow = s_flushnow;  // read before thread 0 can rewrite them
        if (fl == 1) break;
        if (PPR_RING_LAZY && fl == 2) {
            block_flush(s, c);  // the pending entries' children reach `tail` ...
            if (threadIdx.x == 0) {  // ... before the entries count as done
                __threadfence();
                atomicAdd(done, pend);
                pend = 0;
                since = 0;
            }
            continue;
        }
        const unsigned long long h = s_h;
        const uint32_t k = (uint32_t)s_k;
        // thread i takes slot h + i: wait for its producer, read, free the slot
        const bool valid = threadIdx.x < k;
        unsigned long long ent = 0;
        if (valid) {
            const unsigned long long pos = (h + threadIdx.x) % a.ring_cap;
            volatile unsigned long long* slot = (volatile unsigned long long*)&a.ring[pos];
            while ((ent = *slot) == EMPTY) __nanosleep(32);
            *slot = EMPTY;
        }
        int top = 1;
        while (top * 2 < (int)k) top <<= 1;
        tile_body<POS, K_OPT, LAY>(s, c, a, valid, ent, 0, k, top);
        if (PPR_RING_LAZY) {
            if (threadIdx.x == 0) pend += k;
            if (!flushnow) continue;  // the next claim's barrier separates the tiles
        }
        block_flush(s, c);  // this tile's children reach `tail` ...
        if (threadIdx.x == 0) {  // ... before it counts as done (release: tail and the slots first)
            __threadfence();
            atomicAdd(done, PPR_RING_LAZY ? pend : (unsigned long long)k);
            pend = 0;
            since = 0;
        }
    }
}

template <bool POS, int LAY>
__device__ __forceinline__ void async_phase(Smem& s, Ctx& c, const PushArgs& a) {
    DevCtl* ctl = a.ctl;
    unsigned long long* head = &ctl->tilectr[0].v;
    unsigned long long* tail = &ctl->fcount[0].v;
    unsigned long long* done = &ctl->fcount[1].v;
    c.Fout = a.ring;
    c.cnt_out = tail;
    c.ring_cap = a.ring_cap;
    seed_phase<POS, LAY>(s, c, a);
    block_flush(s, c);
    grid_sync(ctl);
    async_loop<POS, LAY>(s, c, a, head, tail, done);
    grid_sync(ctl);
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        *head = 0;
        *tail = 0;
        *done = 0;
    }
    grid_sync(ctl);
}

template <int LAY>
__global__ void __launch_bounds__(PT, PUSH_MIN_BLOCKS) k_push_async(const __grid_constant__ PushArgs a) {
    __shared__ Smem s;
    Ctx c;
    c.trace_edges = nullptr;
    c.ring_cap = 0;
    c.qn = 0;
    c.pushes = 0;
    c.edges = 0;
    c.t_work = c.t_flush = c.t_bar = 0;
    c.t_pro = c.t_claim = c.t_mark = c.t_mark2 = 0;
    if (*(volatile int*)&a.ctl->st.err != KERR_OK) return;  // earlier stage failed: uniform exit
    c.pool = *(volatile unsigned*)&a.ctl->st.active_pool ? a.g.pool[1] : a.g.pool[0];
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        for (int i = 0; i < 3; i++) a.ctl->fcount[i].v = a.ctl->tilectr[i].v = 0;
    }
    grid_sync(a.ctl);
    const bool stamp = blockIdx.x == 0 && threadIdx.x == 0;
    const unsigned long long t0 = stamp ? globaltimer_ns() : 0;
    if (a.phases & 1) async_phase<true, LAY>(s, c, a);
    const unsigned long long t1 = stamp ? globaltimer_ns() : 0;  // async_phase ends with a grid barrier
    if (a.phases & 2) async_phase<false, LAY>(s, c, a);
    if (stamp) {  // phase durations, summed over launches (source waves)
        atomicAdd(&a.ctl->st.ns_push[0], t1 - t0);
        atomicAdd(&a.ctl->st.ns_push[1], globaltimer_ns() - t1);
    }
    __shared__ unsigned long long s_red[2];
    if (threadIdx.x == 0) s_red[0] = s_red[1] = 0;
    __syncthreads();
    if (c.pushes) atomicAdd(&s_red[0], c.pushes);
    if (c.edges) atomicAdd(&s_red[1], c.edges);
    __syncthreads();
    if (threadIdx.x == 0) {
        if (s_red[0]) atomicAdd(&a.ctl->st.pushes, s_red[0]);
        if (s_red[1]) atomicAdd(&a.ctl->st.pushed_edges, s_red[1]);
    }
}

template <int LAY>
cudaError_t launch_async(const PushArgs& a, int num_sms, cudaStream_t st) {
    int bps = 0;
    const cudaError_t e = blocks_per_sm((const void*)k_push_async<LAY>, PT, PUSH_MIN_BLOCKS, &bps);
    if (e != cudaSuccess) return e;
    return coop_launch((const void*)k_push_async<LAY>, num_sms * bps, a, st);
}

template <int MODE, int LAY>
cudaError_t launch_mode(const PushArgs& a, int num_sms, cudaStream_t st) {
    int bps = 0;
    const cudaError_t e = blocks_per_sm((const void*)k_push<MODE, LAY>, PT, PUSH_MIN_BLOCKS, &bps);
    if (e != cudaSuccess) return e;
    return coop_launch((const void*)k_push<MODE, LAY>, num_sms * bps, a, st);
}

template <int LAY>
cudaError_t launch_layout(int mode, const PushArgs& a, int num_sms, cudaStream_t st) {
#if PPR_PUSH_OPT_ONLY
    return mode == M_OPT ? launch_mode<M_OPT, LAY>(a, num_sms, st) : cudaErrorInvalidValue;
#endif
    switch (mode) {
        case M_OPT: return launch_mode<M_OPT, LAY>(a, num_sms, st);
        case M_EAGER: return launch_mode<M_EAGER, LAY>(a, num_sms, st);
        case M_DUP: return launch_mode<M_DUP, LAY>(a, num_sms, st);
        case M_VAN: return launch_mode<M_VAN, LAY>(a, num_sms, st);
        case M_ASYNC: return launch_async<LAY>(a, num_sms, st);
        case M_SCAN: return launch_mode<M_SCAN, LAY>(a, num_sms, st);
        default: return cudaErrorInvalidValue;
    }
}

}  // namespace

// push_u3.cu compiles this file a second time with 3 edge chains per lane
// (PPR_PUSH_U=3), Opt only, as launch_push_u3 (dense graphs, ppr_api.cu)
#ifndef PPR_PUSH_ENTRY
#define PPR_PUSH_ENTRY launch_push
#endif
cudaError_t PPR_PUSH_ENTRY(int mode, const PushArgs& a, int num_sms, cudaStream_t st) {
    if (mode == 6 /* PPR_MODE_SHARED */) return a.g.rec ? cudaErrorInvalidValue : launch_push_ms(a, num_sms, st);
    if (a.g.rec) return launch_layout<LAY_PACKED>(mode, a, num_sms, st);
    return a.g.pool_wide ? launch_layout<LAY_WIDE>(mode, a, num_sms, st)
                         : launch_layout<LAY_ARRAYS>(mode, a, num_sms, st);
}

}  // namespace ppr
