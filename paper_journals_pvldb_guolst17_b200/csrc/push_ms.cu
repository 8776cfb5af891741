// push_ms.cu -- shared-adjacency multi-source push (PPR_MODE_SHARED; SURVEY
// 8(f) NEXT-3, steps a3-a6 of the hot path for S > 1 sources).
//
// The S sources of a handle are independent unit-vector problems
// over one graph, so their pushes walk the same in-lists.  This kernel makes
// a frontier entry a (group, vertex) pair, where a group is 32 consecutive
// source columns of the vertex-major [n][S] residual array, and gives every
// lane of a warp one source of the group:
//   * Alg 4 line 10 (eager read): lane l reads R_{32g+l}(u) with
//     a relaxed load -- one coalesced 256-byte row read per entry -- and the
//     lanes whose residual meets pushCond form the entry's push mask.
//   * Alg 4 lines 20-21 (self-update): P(u) += a r, R(u) -= r for the masked
//     lanes, as fire-and-forget reductions (coalesced).
//   * Alg 4 lines 11-13 (propagation): N_in(u) is read ONCE for the whole
//     group; for every v the masked lanes add (1-a) r_l / d(v) to
//     R_{32g+l}(v): one warp-wide reduction onto one contiguous row segment
//     instead of up to 32 random single-word atomics.
//   * Frontier generation (north_star "bitmap dedup plus warp-ballot/scan
//     compaction"): every changed (v, g) is marked in a bitmap; after a grid
//     barrier the bitmap is compacted into the next frontier.  Whether an
//     entry pushes any lane is decided when it is processed (the row read
//     above), so the scan is pure bit compaction.
// Termination and correctness follow DESIGN.md K-SCAN: every residual change
// marks its (v, g), the next round re-reads every marked row after the
// barrier, so a round that finds no lane meeting pushCond changes nothing
// and the phase ends with -eps <= R <= eps everywhere.  Each entry is in a
// frontier at most once per round (the bitmap deduplicates), so no residual
// mass is pushed twice.  Seeding: the touched vertices (every group), the
// sources (create) or every (v, g) (ppr_push) are marked and compacted.
//
// The increment is ((1-a) r) * (1/d(v)): the reciprocal is computed once per
// edge and shared by the 32 lanes (reading R-RCP; the oracle
// divides, the two differ by at most one rounding per increment, far inside
// the invariant tolerance R18).
#include "block_scan.cuh"
#include "primitives.cuh"
#include "push.cuh"

namespace ppr {

namespace {

constexpr int PT = PUSH_THREADS;
constexpr int NW = PT / 32;
#ifndef PPR_MS_MT
#define PPR_MS_MT 64
#endif
#ifndef PPR_MS_CLAIM_AHEAD
#define PPR_MS_CLAIM_AHEAD 1
#endif
#ifndef PPR_MS_WSCAN
#define PPR_MS_WSCAN 1
#endif
constexpr int MT = PPR_MS_MT;  // frontier entries per CTA tile (a multiple of 32)
static_assert(MT % 32 == 0, "MT");
#ifndef PPR_MS_DIV
#define PPR_MS_DIV 0
#endif
#ifndef PPR_MS_QW
#define PPR_MS_QW 256
#endif
constexpr int QW = PPR_MS_QW;  // per-warp queue slice (entries)

struct MsSmem {
    double w[MT][32];                 // (1-a) r of every lane of every entry (0: lane idle)
    unsigned long long off[MT];       // slab offset of each entry
    uint32_t scan[2 * MT];            // exclusive prefix of the entries' walk lengths
    uint32_t grp[MT];                 // source group of each entry
    uint32_t len[MT];                 // walk length (in-degree, or 0 if no lane pushes)
    unsigned long long q[NW][QW];     // per-warp enqueue slices
    unsigned int wq[NW];
    unsigned long long gbase;
    unsigned long long next;
    unsigned long long cround;
    unsigned int chunk;
    uint32_t E;
#if PPR_MS_WSCAN
    uint32_t wscan[NW][2 * MT];       // every warp's own copy of the prefix (no scan barrier)
    unsigned int chunk2[2];           // chunk counters of even / odd tiles
#endif
};

struct MsCtx {
    const PoolEnt* pool;
    unsigned long long* Fout;
    unsigned long long* cnt_out;
    uint32_t qn;
    unsigned long long pushes;     // (source, vertex) self-updates
    unsigned long long edges;      // (source, arc) propagations
    unsigned long long walks;      // (group, arc) walks
    unsigned long long entries;    // (vertex, group) entries with at least one pushing lane
    uint32_t tiles;                // tiles processed by this CTA (chunk-counter parity)
};

__device__ __forceinline__ unsigned lane() { return threadIdx.x & 31u; }
__device__ __forceinline__ unsigned warp() { return threadIdx.x >> 5; }

__device__ __forceinline__ void warp_flush(MsSmem& s, MsCtx& c) {
    if (c.qn == 0) return;  // warp-uniform
    unsigned long long base = 0;
    if (lane() == 0) base = atomicAdd(c.cnt_out, (unsigned long long)c.qn);
    base = __shfl_sync(0xffffffffu, base, 0);
    for (uint32_t i = lane(); i < c.qn; i += 32) __stcg(&c.Fout[base + i], s.q[warp()][i]);
    __syncwarp();
    c.qn = 0;
}

__device__ __forceinline__ void warp_enqueue(MsSmem& s, MsCtx& c, bool flag, unsigned long long e) {
    if (c.qn + 32 > QW) {
        __syncwarp();
        warp_flush(s, c);
    }
    const unsigned b = __ballot_sync(0xffffffffu, flag);
    if (flag) s.q[warp()][c.qn + __popc(b & ((1u << lane()) - 1u))] = e;
    c.qn += __popc(b);
}

__device__ __forceinline__ void block_flush(MsSmem& s, MsCtx& c) {
    const unsigned w = warp();
    __syncwarp();
    if (lane() == 0) s.wq[w] = c.qn;
    __syncthreads();
    if (threadIdx.x == 0) {
        unsigned long long tot = 0;
        for (int i = 0; i < NW; i++) {
            const unsigned x = s.wq[i];
            s.wq[i] = (unsigned)tot;
            tot += x;
        }
        s.gbase = tot ? atomicAdd(c.cnt_out, tot) : 0ull;
    }
    __syncthreads();
    const unsigned long long base = s.gbase + s.wq[w];
    for (uint32_t i = lane(); i < c.qn; i += 32) __stcg(&c.Fout[base + i], s.q[w][i]);
    c.qn = 0;
    __syncthreads();
}

// Marks (v, g).  The test reads the word at L2 (never a stale L1 copy: the
// scan clears words between rounds), so a set bit is only skipped when it is
// really set.
__device__ __forceinline__ void mark(uint32_t* bitmap, unsigned long long bit) {
    const uint32_t m = 1u << (bit & 31u);
    uint32_t* p = &bitmap[bit >> 5];
    if (!(__ldcg(p) & m)) atomicOr(p, m);
}

// largest i with scan[i] <= e (scan[T..] hold 0xFFFFFFFF)
__device__ __forceinline__ int owner_of(const uint32_t* scan, uint32_t e, int top) {
    int lo = 0;
    for (int step = top; step > 0; step >>= 1)
        if (scan[lo + step] <= e) lo += step;
    return lo;
}

// ---------------------------------------------------------------- one tile

template <bool POS, bool WIDE>
__device__ __forceinline__ void ms_tile(MsSmem& s, MsCtx& c, const PushArgs& a, uint32_t SG,
                                        const unsigned long long* Fin, uint64_t C, uint64_t base,
                                        uint32_t T, int top) {
    const unsigned L = lane(), w = warp();
    const uint32_t S = a.g.S;
    const double eps = a.g.eps, alpha = a.g.alpha;
    const unsigned long long pol_keep = l2_keep(), pol_stream = l2_stream();
    // Phase A: one warp per entry -- eager row read, push mask, self-update.
    // A warp's entries are j = w + NW*i, i < PA (at most MT/NW): lane i loads
    // entry i and its slab descriptor, then the warp issues all PA row reads
    // before consuming any, so the entries' dependent loads overlap instead of
    // running one chain per entry.
    constexpr int PA = MT / NW;
    static_assert(PA <= 32, "one lane per entry of the warp");
    unsigned long long myent = 0;
    uint2 mysl = make_uint2(0, 0);
    {
        const uint32_t j = w + NW * L;
        if (L < (unsigned)PA && j < T && base + j < C) {
            myent = __ldcg(&Fin[base + j]);
            mysl = ld_slab_pol(&a.g.slab[(uint32_t)myent], pol_stream);  // SlabRec {off, len}
        }
    }
    unsigned mymask = 0;
    constexpr int PB = 4;  // row reads in flight per batch (registers)
#pragma unroll
    for (int i0 = 0; i0 < PA; i0 += PB) {
        if (w + NW * i0 >= T) break;  // warp-uniform
        double r[PB];
#pragma unroll
        for (int q = 0; q < PB; q++) {
            const int i = i0 + q;
            const unsigned long long ent = __shfl_sync(0xffffffffu, myent, i);
            const uint32_t j = w + NW * i;
            const uint32_t sidx = (uint32_t)(ent >> 32) * 32 + L;
            const bool lok = j < T && base + j < C && sidx < S;
            r[q] = lok ? ld_relaxed_f64(a.g.R + (size_t)(uint32_t)ent * S + sidx) : 0.0;
        }
#pragma unroll
        for (int q = 0; q < PB; q++) {
            const int i = i0 + q;
            const uint32_t j = w + NW * i;
            if (j >= T) break;  // warp-uniform
            const unsigned long long ent = __shfl_sync(0xffffffffu, myent, i);
            const uint32_t g = (uint32_t)(ent >> 32), u = (uint32_t)ent;
            const uint32_t sidx = g * 32 + L;
            const bool p = base + j < C && sidx < S && push_cond<POS>(r[q], eps);
            const unsigned mask = __ballot_sync(0xffffffffu, p);
            if (p) {
                red_add_pol(a.g.R + (size_t)u * S + sidx, -r[q], pol_keep);
                red_add_pol(a.g.P + (size_t)u * S + sidx, __dmul_rn(alpha, r[q]), pol_stream);
            }
            s.w[j][L] = p ? __dmul_rn(1.0 - alpha, r[q]) : 0.0;
            if (L == (unsigned)i) mymask = mask;
            if (L == 0 && mask) {  // u's row changed (one mark per entry: no test needed)
                const unsigned long long bit = (unsigned long long)u * SG + g;
                atomicOr(&a.bitmap[bit >> 5], 1u << (bit & 31u));
            }
        }
    }
    if (L < (unsigned)PA && w + NW * L < T) {  // lane i publishes entry i
        const uint32_t j = w + NW * L;
        const uint32_t len = mymask ? mysl.y : 0u;
        s.len[j] = len;
        s.off[j] = mysl.x;
        s.grp[j] = (uint32_t)(myent >> 32);
        if (mymask) {
            const unsigned k = __popc(mymask);
            c.pushes += k;
            c.edges += (unsigned long long)k * len;
            c.walks += len;
            c.entries++;
        }
    }
    __syncthreads();
    // exclusive scan of the T walk lengths (MT/32 consecutive entries per lane);
    // with PPR_MS_WSCAN every warp computes it into its own copy, so the walk
    // starts without a second CTA barrier (the chunk counter of this tile's
    // parity was reset during the previous tile)
#if PPR_MS_WSCAN
    uint32_t Ew = 0;  // the tile's walk length, from every warp's own scan
    const uint32_t par = c.tiles & 1u;
    uint32_t* scan = s.wscan[w];
    if (true) {
#else
    uint32_t* scan = s.scan;
    if (w == 0) {
#endif
        constexpr int EPL = MT / 32;
        uint32_t x[EPL];
        uint32_t sum = 0;
#pragma unroll
        for (int q = 0; q < EPL; q++) {
            x[q] = EPL * L + q < T ? s.len[EPL * L + q] : 0u;
            sum += x[q];
        }
        uint32_t inc = sum;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            const uint32_t y = __shfl_up_sync(0xffffffffu, inc, o);
            if (L >= (unsigned)o) inc += y;
        }
        uint32_t ex = inc - sum;
#pragma unroll
        for (int q = 0; q < EPL; q++) {
            scan[EPL * L + q] = EPL * L + q < T ? ex : 0xFFFFFFFFu;
            scan[EPL * L + q + MT] = 0xFFFFFFFFu;
            ex += x[q];
        }
#if PPR_MS_WSCAN
        Ew = __shfl_sync(0xffffffffu, inc, 31);
#else
        if (L == 31) {
            s.E = inc;
            s.chunk = 0;
        }
#endif
    }
#if PPR_MS_WSCAN
    __syncwarp();
    const uint32_t E = Ew;
    if (threadIdx.x == 0) s.chunk2[par ^ 1u] = 0;  // the next tile's counter (its last user finished)
    unsigned int* chunkp = &s.chunk2[par];
#else
    __syncthreads();
    const uint32_t E = s.E;
    unsigned int* chunkp = &s.chunk;
#endif
    // Phase B: warps claim 32-arc chunks of the tile's walk; lane k loads arc k
    // (v, d(v), 1/d(v)) and marks (v, g), then the warp applies the 32 arcs one
    // by one, every lane adding its source's increment to the shared row
    while (true) {
        uint32_t cb = 0;
        if (L == 0) cb = atomicAdd(chunkp, 1u);
        cb = __shfl_sync(0xffffffffu, cb, 0);
        if (cb * 32 >= E) break;
        const uint32_t e = cb * 32 + L;
        const bool ok = e < E;
        int j = 0;
        uint32_t v = 0, d = 1;
        if (ok) {
            j = owner_of(scan, e, top);
            const uint64_t i = s.off[j] + (e - scan[j]);
            if constexpr (WIDE) {  // d_out(v) travels with the in-list entry
                const PoolEnt pe = ld_pool_ent(&c.pool[i], pol_stream);
                v = pe_v(pe);
                d = pe_d(pe);
            } else {
                v = ld_u32_nc_pol(reinterpret_cast<const uint32_t*>(c.pool) + i, pol_stream);
                d = ld_u32_nc_pol(&a.g.dout[v], pol_keep);
            }
            mark(a.bitmap, (unsigned long long)v * SG + s.grp[j]);
        }
#if PPR_MS_DIV  // experiment: every lane divides (as the oracle), no shared reciprocal
        const double rd = (double)d;
#else
        const double rd = __drcp_rn((double)d);
#endif
        const uint32_t nk = E - cb * 32 < 32 ? E - cb * 32 : 32;
        for (uint32_t k = 0; k < nk; k++) {
            const uint32_t vk = __shfl_sync(0xffffffffu, v, k);
            const int jk = __shfl_sync(0xffffffffu, j, k);
            const double rk = __shfl_sync(0xffffffffu, rd, k);
            const double wl = s.w[jk][L];
            if (wl != 0.0)
#if PPR_MS_DIV
                red_add_pol(a.g.R + (size_t)vk * S + s.grp[jk] * 32 + L, __ddiv_rn(wl, rk), pol_keep);
#else
                red_add_pol(a.g.R + (size_t)vk * S + s.grp[jk] * 32 + L, __dmul_rn(wl, rk), pol_keep);
#endif
        }
    }
    __syncthreads();  // smem of this tile is reused by the next
    c.tiles++;
}

// every CTA takes tiles of T entries (first statically, the rest by claims)
template <bool POS, bool WIDE>
__device__ __forceinline__ void ms_round(MsSmem& s, MsCtx& c, const PushArgs& a, uint32_t SG,
                                         const unsigned long long* Fin, uint64_t C,
                                         unsigned long long* tc) {
    const uint64_t per = (C + gridDim.x - 1) / gridDim.x;
    uint32_t T = (uint32_t)((per + NW - 1) / NW * NW);
    if (T > MT) T = MT;
    if (T < NW) T = NW;
    int top = 1;
    while (top * 2 < (int)T) top <<= 1;
    const uint64_t ntiles = (C + T - 1) / T;
    const bool dyn = ntiles > gridDim.x;
    uint64_t t = blockIdx.x;
    while (t < ntiles) {
        // the next tile is claimed as this one starts, so the claim's latency
        // overlaps the tile (thread 0 first needs the result after it)
        unsigned long long claim = 0;
        if (PPR_MS_CLAIM_AHEAD && dyn && threadIdx.x == 0) claim = atomicAdd(tc, 1ull);
        ms_tile<POS, WIDE>(s, c, a, SG, Fin, C, t * T, T, top);  // ends with a CTA barrier
        if (!dyn) break;
        if (!PPR_MS_CLAIM_AHEAD && threadIdx.x == 0) claim = atomicAdd(tc, 1ull);
        if (threadIdx.x == 0) s.next = claim + gridDim.x;
        __syncthreads();
        t = s.next;  // rewritten only after the next tile's first barrier
    }
}

// compacts the marked (v, g) bits into the frontier (bit = v * SG + g) and
// clears them; emitted entries are sorted by vertex within a warp's words
__device__ __forceinline__ void ms_scan(MsSmem& s, MsCtx& c, const PushArgs& a, uint32_t SG) {
    const uint64_t nwords = ((uint64_t)SG * a.g.n + 31) / 32;
    const uint64_t gw = (uint64_t)blockIdx.x * NW + warp(), nw = (uint64_t)gridDim.x * NW;
    for (uint64_t w0 = gw * 32; w0 < nwords; w0 += nw * 32) {
        const uint64_t wi = w0 + lane();
        uint32_t word = wi < nwords ? __ldcg(&a.bitmap[wi]) : 0u;
        if (word) __stcg(&a.bitmap[wi], 0u);
        while (__any_sync(0xffffffffu, word != 0)) {
            bool enq = false;
            unsigned long long ent = 0;
            if (word) {
                const int b = __ffs(word) - 1;
                word &= word - 1;
                const uint64_t bit = wi * 32 + b;
                ent = ((bit % SG) << 32) | (bit / SG);
                enq = true;
            }
            warp_enqueue(s, c, enq, ent);
        }
    }
}

// marks the phase's seeds: every (seed vertex, group) of the launch's group
// range [g0, g1) (all groups, or one wave of them)
__device__ __forceinline__ void ms_seed(const PushArgs& a, uint32_t SG) {
    const uint64_t stride = (uint64_t)gridDim.x * PT;
    const uint64_t t0 = (uint64_t)blockIdx.x * PT + threadIdx.x;
    const uint32_t g0 = a.g_hi ? a.g_lo : 0u, g1 = a.g_hi ? a.g_hi : SG, G = g1 - g0;
    if (a.seed_all) {
        if (G == SG) {
            const uint64_t nbits = (uint64_t)SG * a.g.n, nwords = (nbits + 31) / 32;
            for (uint64_t wi = t0; wi < nwords; wi += stride) {
                const uint64_t rem = nbits - wi * 32;
                a.bitmap[wi] = rem >= 32 ? 0xFFFFFFFFu : ((1u << rem) - 1u);
            }
        } else {
            for (uint64_t k = t0; k < (uint64_t)a.g.n * G; k += stride)
                mark(a.bitmap, (k / G) * SG + g0 + k % G);
        }
    } else if (a.seed_v) {
        const uint64_t nv = *a.n_seed_v_dev;
        for (uint64_t k = t0; k < nv * G; k += stride)
            mark(a.bitmap, (unsigned long long)a.seed_v[k / G] * SG + g0 + (k % G));
    } else {
        for (uint64_t k = t0; k < a.n_seed_e; k += stride) {
            const unsigned long long ent = a.seed_e[k];
            const uint32_t g = (uint32_t)(ent >> 32) / 32;
            if (g >= g0 && g < g1) mark(a.bitmap, (unsigned long long)(uint32_t)ent * SG + g);
        }
    }
}

template <bool POS, bool WIDE>
__device__ __forceinline__ void ms_phase(MsSmem& s, MsCtx& c, const PushArgs& a, uint32_t SG,
                                         unsigned& it) {
    DevCtl* ctl = a.ctl;
    const int ph = POS ? 0 : 1;
    ms_seed(a, SG);
    grid_sync(ctl);
    c.Fout = a.F[it & 1];
    c.cnt_out = &ctl->fcount[it % 3].v;
    ms_scan(s, c, a, SG);
    block_flush(s, c);
    grid_sync(ctl);
    uint32_t pit = 0;
    while (true) {
        if (threadIdx.x == 0) s.cround = *(volatile unsigned long long*)&ctl->fcount[it % 3].v;
        __syncthreads();
        const uint64_t C = s.cround;
        if (blockIdx.x == 0 && threadIdx.x == 0) {
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
        c.Fout = a.F[(it + 1) & 1];
        c.cnt_out = &ctl->fcount[(it + 1) % 3].v;
        ms_round<POS, WIDE>(s, c, a, SG, Fin, C, &ctl->tilectr[it % 3].v);
        grid_sync(ctl);  // every reduction and mark of the round has landed
        ms_scan(s, c, a, SG);
        block_flush(s, c);
        grid_sync(ctl);
        it++;
        pit++;
    }
    grid_sync(ctl);
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        ctl->fcount[0].v = ctl->fcount[1].v = ctl->fcount[2].v = 0;
        ctl->tilectr[0].v = ctl->tilectr[1].v = ctl->tilectr[2].v = 0;
    }
    grid_sync(ctl);
}

template <bool WIDE>  // PoolEnt in-list entries carrying d_out (ppr_internal.cuh), else u32 ids
__global__ void __launch_bounds__(PT, PUSH_MIN_BLOCKS) k_push_ms(const __grid_constant__ PushArgs a) {
    __shared__ MsSmem s;
    MsCtx c;
    c.qn = 0;
    c.pushes = c.edges = c.walks = c.entries = 0;
    c.tiles = 0;
#if PPR_MS_WSCAN
    if (threadIdx.x == 0) s.chunk2[0] = s.chunk2[1] = 0;  // ordered by the grid barrier below
#endif
    if (*(volatile int*)&a.ctl->st.err != KERR_OK) return;  // earlier stage failed: uniform exit
    c.pool = *(volatile unsigned*)&a.ctl->st.active_pool ? a.g.pool[1] : a.g.pool[0];
    const uint32_t SG = (a.g.S + 31) / 32;
    if (blockIdx.x == 0 && threadIdx.x == 0)
        for (int i = 0; i < 3; i++) a.ctl->fcount[i].v = a.ctl->tilectr[i].v = 0;
    grid_sync(a.ctl);
    const bool stamp = blockIdx.x == 0 && threadIdx.x == 0;
    const unsigned long long t0 = stamp ? globaltimer_ns() : 0;
    unsigned it = 0;
    if (a.phases & 1) ms_phase<true, WIDE>(s, c, a, SG, it);
    const unsigned long long t1 = stamp ? globaltimer_ns() : 0;  // ms_phase ends with a grid barrier
    if (a.phases & 2) ms_phase<false, WIDE>(s, c, a, SG, it);
    if (stamp) {  // phase durations, summed over launches (source waves)
        atomicAdd(&a.ctl->st.ns_push[0], t1 - t0);
        atomicAdd(&a.ctl->st.ns_push[1], globaltimer_ns() - t1);
    }
    __shared__ unsigned long long s_red[4];
    if (threadIdx.x < 4) s_red[threadIdx.x] = 0;
    __syncthreads();
    if (c.pushes) atomicAdd(&s_red[0], c.pushes);
    if (c.edges) atomicAdd(&s_red[1], c.edges);
    if (c.walks) atomicAdd(&s_red[2], c.walks);
    if (c.entries) atomicAdd(&s_red[3], c.entries);
    __syncthreads();
    if (threadIdx.x == 0) {
        if (s_red[0]) atomicAdd(&a.ctl->st.pushes, s_red[0]);
        if (s_red[1]) atomicAdd(&a.ctl->st.pushed_edges, s_red[1]);
        if (s_red[2]) atomicAdd(&a.ctl->st.walk_edges, s_red[2]);
        if (s_red[3]) atomicAdd(&a.ctl->st.entries, s_red[3]);
    }
}

}  // namespace

cudaError_t launch_push_ms(const PushArgs& a, int num_sms, cudaStream_t st) {
    int bps = 0;
    const void* fn = a.g.pool_wide ? (const void*)k_push_ms<true> : (const void*)k_push_ms<false>;
    const cudaError_t e = blocks_per_sm(fn, PT, PUSH_MIN_BLOCKS, &bps);
    if (e != cudaSuccess) return e;
    PushArgs copy = a;
    void* args[] = {&copy};
    cudaLaunchConfig_t cfg{};
    cfg.gridDim = dim3(num_sms * bps);
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

}  // namespace ppr
