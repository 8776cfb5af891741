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
//             pass: per frontier tile, r_u is read ONCE with a relaxed load
//             (eager propagation), every v in N_in(u) gets
//             atomicAdd(R(v), (1-a) r_u / d(v)) and is enqueued iff this add
//             crossed the threshold (local duplicate detection, Alg 4 lines
//             14-17); then R(u) -= r_u atomically and u is
//             re-enqueued iff the value that subtraction produced still meets
//             pushCond (lines 21-23).  Exactly-once enqueue
//             argument: DESIGN.md K-PUSH.
//   EAGER     Alg 4 order (propagate, barrier, self-update) with UniqueEnqueue
//             through a bitmap instead of the crossing test.
//   DUPDETECT Alg 3 order (snapshot/self-update, barrier, propagate) with the
//             crossing test.
//   VANILLA   Alg 3 as printed: snapshot, barrier, propagate,
//             UniqueEnqueue through a bitmap.
//
// Work distribution (north_star "degree-binned scheduling"): a CTA takes a
// tile of PUSH_THREADS frontier entries, scans their in-degrees in shared
// memory and then walks the tile's edges PUSH_THREADS at a time, each thread
// binary-searching its owner entry -- thread-, warp- and CTA-sized in-lists
// are balanced inside the tile and slab reads are coalesced.  Tiles are
// claimed dynamically with an atomic counter.
// Enqueues go through a per-CTA shared-memory queue flushed with one global
// atomic per flush (warp ballot + __syncthreads_count aggregation).
#include "block_scan.cuh"
#include "push.cuh"

namespace ppr {

namespace {

constexpr int PT = PUSH_THREADS;
constexpr int QCAP = PUSH_QCAP;
constexpr int NWARP = PT / 32;
enum { M_OPT = 0, M_EAGER = 1, M_DUP = 2, M_VAN = 3 };

struct Smem {
    unsigned long long q[QCAP];       // enqueue buffer
    unsigned long long off[PT];       // slab offset of each tile entry
    double w[PT];                     // (1-a) * r of each tile entry
    uint32_t scan[PT];                // exclusive prefix of in-degrees
    uint32_t sidx[PT];                // source index of each tile entry
    uint32_t warp[NWARP + 1];         // block-scan scratch
    unsigned int qn;                  // entries in q
    unsigned long long gbase;         // flush base
    unsigned long long tile;          // claimed tile
};

struct Ctx {
    DevGraph g;
    DevCtl* ctl;
    const uint32_t* pool;
    unsigned long long* Fout;
    unsigned long long* cnt_out;
    uint32_t qn;                // block-uniform queue fill
    unsigned long long pushes;  // per-thread counters
    unsigned long long edges;
};

__device__ __forceinline__ void flush(Smem& s, Ctx& c) {
    if (c.qn == 0) return;  // block-uniform
    if (threadIdx.x == 0) s.gbase = atomicAdd(c.cnt_out, (unsigned long long)c.qn);
    __syncthreads();
    const unsigned long long gb = s.gbase;
    for (uint32_t i = threadIdx.x; i < c.qn; i += PT) c.Fout[gb + i] = s.q[i];
    __syncthreads();
    if (threadIdx.x == 0) s.qn = 0;
    __syncthreads();
    c.qn = 0;
}

// Block-wide enqueue of `e` where flag is set.  Must be called by all threads.
__device__ __forceinline__ void enqueue(Smem& s, Ctx& c, bool flag, unsigned long long e) {
    const unsigned lane = threadIdx.x & 31u;
    const unsigned b = __ballot_sync(0xffffffffu, flag);
    if (b) {
        unsigned base = 0;
        if (lane == 0) base = atomicAdd(&s.qn, (unsigned)__popc(b));
        base = __shfl_sync(0xffffffffu, base, 0);
        if (flag) s.q[base + __popc(b & ((1u << lane) - 1u))] = e;
    }
    c.qn += (uint32_t)__syncthreads_count(flag);
    if (c.qn > QCAP - PT) flush(s, c);
}

__device__ __forceinline__ int owner_of(const Smem& s, uint32_t e) {
    int lo = 0, hi = PT;
    while (hi - lo > 1) {
        int mid = (lo + hi) >> 1;
        if (s.scan[mid] <= e) lo = mid; else hi = mid;
    }
    return lo;
}

__device__ __forceinline__ bool claim_tile(Smem& s, unsigned long long* tc, uint32_t ntiles,
                                           unsigned long long& t) {
    if (threadIdx.x == 0) s.tile = atomicAdd(tc, 1ull);
    __syncthreads();
    t = s.tile;
    return t < ntiles;
}

// Loads a tile's entries: the slab of u, the weight (1-a)*r and the
// in-degree prefix.  Returns the tile's edge count E (block-uniform).
__device__ __forceinline__ uint32_t load_tile(Smem& s, Ctx& c, bool push, uint32_t sidx,
                                              uint32_t u, double r) {
    uint32_t len = 0;
    unsigned long long off = 0;
    if (push) {
        const ulonglong2 sl = __ldg(reinterpret_cast<const ulonglong2*>(&c.g.slab[u]));
        off = sl.x;                   // Slab::off
        len = (uint32_t)sl.y;         // Slab::len (low word of {len, cap})
    }
    s.off[threadIdx.x] = off;
    s.w[threadIdx.x] = __dmul_rn(1.0 - c.g.alpha, r);
    s.sidx[threadIdx.x] = sidx;
    uint32_t E;
    s.scan[threadIdx.x] = block_exclusive_scan_u32<PT>(len, s.warp, &E);
    __syncthreads();
    if (threadIdx.x == 0) c.edges += E;
    return E;
}

// One neighbour propagation: R(v) += (1-a) w / d(v) (Alg 3 line 21, Alg 4
// lines 13-15).  Returns pre and sets cur = pre + inc exactly as stored.
__device__ __forceinline__ double propagate_edge(const Smem& s, Ctx& c, uint32_t e,
                                                 unsigned long long& ev, double& cur) {
    const int j = owner_of(s, e);
    const uint32_t v = __ldg(&c.pool[s.off[j] + (e - s.scan[j])]);
    const uint32_t d = __ldg(&c.g.dout[v]);
    const double inc = __ddiv_rn(s.w[j], (double)d);
    const uint32_t sj = s.sidx[j];
    double* rp = c.g.R + (size_t)sj * c.g.n + v;
    const double pre = atomicAdd(rp, inc);
    cur = __dadd_rn(pre, inc);  // bit-identical to the stored value (no FMA)
    ev = ((unsigned long long)sj << 32) | v;
    return pre;
}

__device__ __forceinline__ bool test_and_set(uint32_t* bitmap, unsigned long long bit) {
    const uint32_t mask = 1u << (bit & 31u);
    const uint32_t old = atomicOr(&bitmap[bit >> 5], mask);
    return (old & mask) == 0;
}

__device__ __forceinline__ void clear_bit(uint32_t* bitmap, unsigned long long bit) {
    atomicAnd(&bitmap[bit >> 5], ~(1u << (bit & 31u)));
}

// ---------------------------------------------------------------- OPT round

template <bool POS>
__device__ void round_opt(Smem& s, Ctx& c, const PushArgs& a, const unsigned long long* Fin,
                          uint64_t C, unsigned long long* tc) {
    const uint32_t ntiles = (uint32_t)((C + PT - 1) / PT);
    const double eps = c.g.eps, alpha = c.g.alpha;
    unsigned long long t;
    while (claim_tile(s, tc, ntiles, t)) {
        const uint64_t idx = t * PT + threadIdx.x;
        const bool valid = idx < C;
        const unsigned long long ent = valid ? __ldcg(&Fin[idx]) : 0ull;
        const uint32_t sidx = (uint32_t)(ent >> 32), u = (uint32_t)ent;
        double* ru = c.g.R + (size_t)sidx * c.g.n + u;
        const double r = valid ? ld_relaxed_f64(ru) : 0.0;  // Alg 4 line 10
        const bool push = valid && push_cond<POS>(r, eps);
        const uint32_t E = load_tile(s, c, push, sidx, u, r);
        for (uint32_t e0 = 0; e0 < E; e0 += PT) {
            const uint32_t e = e0 + threadIdx.x;
            bool cross = false;
            unsigned long long ev = 0;
            if (e < E) {
                double cur;
                const double pre = propagate_edge(s, c, e, ev, cur);
                cross = crossed<POS>(pre, cur, eps);  // Alg 4 line 16
            }
            enqueue(s, c, cross, ev);
        }
        bool re = false;
        if (push) {  // Alg 4 lines 20-23, fused: atomic subtract, re-enqueue on its result
            const double old = atomicAdd(ru, -r);
            const double cur = __dadd_rn(old, -r);
            double* pu = c.g.P + (size_t)sidx * c.g.n + u;
            __stcg(pu, __dadd_rn(__ldcg(pu), __dmul_rn(alpha, r)));
            re = push_cond<POS>(cur, eps);
            c.pushes++;
        }
        enqueue(s, c, re, ent);
    }
}

// ---------------------------------------------------------------- Alg 3 rounds

// self-update session (Alg 3 lines 13-16): w = R(u), P(u) += a w, R(u) = 0.
__device__ void session_snapshot(Ctx& c, const PushArgs& a, const unsigned long long* Fin,
                                 uint64_t C, bool bitmap) {
    const double alpha = c.g.alpha;
    for (uint64_t idx = (uint64_t)blockIdx.x * PT + threadIdx.x; idx < C;
         idx += (uint64_t)gridDim.x * PT) {
        const unsigned long long ent = __ldcg(&Fin[idx]);
        const size_t i = (size_t)(ent >> 32) * c.g.n + (uint32_t)ent;
        const double w = __ldcg(&c.g.R[i]);
        __stcg(&c.g.P[i], __dadd_rn(__ldcg(&c.g.P[i]), __dmul_rn(alpha, w)));
        __stcg(&c.g.R[i], 0.0);
        __stcg(&a.W[idx], w);
        if (bitmap) clear_bit(a.bitmap, i);
        c.pushes++;
    }
}

// neighbour-propagation session of Alg 3 (lines 19-23) using the snapshot W.
template <bool POS, bool UNIQUE>
__device__ void session_propagate(Smem& s, Ctx& c, const PushArgs& a,
                                  const unsigned long long* Fin, uint64_t C,
                                  unsigned long long* tc) {
    const uint32_t ntiles = (uint32_t)((C + PT - 1) / PT);
    const double eps = c.g.eps;
    unsigned long long t;
    while (claim_tile(s, tc, ntiles, t)) {
        const uint64_t idx = t * PT + threadIdx.x;
        const bool valid = idx < C;
        const unsigned long long ent = valid ? __ldcg(&Fin[idx]) : 0ull;
        const double w = valid ? __ldcg(&a.W[idx]) : 0.0;
        const uint32_t E = load_tile(s, c, valid, (uint32_t)(ent >> 32), (uint32_t)ent, w);
        for (uint32_t e0 = 0; e0 < E; e0 += PT) {
            const uint32_t e = e0 + threadIdx.x;
            bool enq = false;
            unsigned long long ev = 0;
            if (e < E) {
                double cur;
                const double pre = propagate_edge(s, c, e, ev, cur);
                if (UNIQUE) {  // UniqueEnqueue if pushCond(R(v)) (line 22-23)
                    enq = push_cond<POS>(cur, eps) &&
                          test_and_set(a.bitmap, (ev >> 32) * c.g.n + (uint32_t)ev);
                } else {       // local duplicate detection
                    enq = crossed<POS>(pre, cur, eps);
                }
            }
            enqueue(s, c, enq, ev);
        }
    }
}

// Eager (Alg 4 order) with UniqueEnqueue: propagate with the current r_u ...
template <bool POS>
__device__ void session_eager_propagate(Smem& s, Ctx& c, const PushArgs& a,
                                        const unsigned long long* Fin, uint64_t C,
                                        unsigned long long* tc) {
    const uint32_t ntiles = (uint32_t)((C + PT - 1) / PT);
    const double eps = c.g.eps;
    unsigned long long t;
    while (claim_tile(s, tc, ntiles, t)) {
        const uint64_t idx = t * PT + threadIdx.x;
        const bool valid = idx < C;
        const unsigned long long ent = valid ? __ldcg(&Fin[idx]) : 0ull;
        const uint32_t sidx = (uint32_t)(ent >> 32), u = (uint32_t)ent;
        const double r = valid ? ld_relaxed_f64(c.g.R + (size_t)sidx * c.g.n + u) : 0.0;
        const bool push = valid && push_cond<POS>(r, eps);
        if (valid) __stcg(&a.W[idx], push ? r : 0.0);
        const uint32_t E = load_tile(s, c, push, sidx, u, r);
        for (uint32_t e0 = 0; e0 < E; e0 += PT) {
            const uint32_t e = e0 + threadIdx.x;
            bool enq = false;
            unsigned long long ev = 0;
            if (e < E) {
                double cur;
                propagate_edge(s, c, e, ev, cur);
                enq = push_cond<POS>(cur, eps) &&
                      test_and_set(a.bitmap, (ev >> 32) * c.g.n + (uint32_t)ev);
            }
            enqueue(s, c, enq, ev);
        }
    }
}

// ... then self-update with the same r_u (Alg 4 lines 19-23).
template <bool POS>
__device__ void session_eager_self(Smem& s, Ctx& c, const PushArgs& a,
                                   const unsigned long long* Fin, uint64_t C) {
    const double eps = c.g.eps, alpha = c.g.alpha;
    const uint64_t stride = (uint64_t)gridDim.x * PT;
    for (uint64_t b = (uint64_t)blockIdx.x * PT; b < C; b += stride) {
        const uint64_t idx = b + threadIdx.x;
        bool enq = false;
        unsigned long long ent = 0;
        if (idx < C) {
            ent = __ldcg(&Fin[idx]);
            const double r = __ldcg(&a.W[idx]);
            if (r != 0.0) {
                const size_t i = (size_t)(ent >> 32) * c.g.n + (uint32_t)ent;
                const double old = atomicAdd(&c.g.R[i], -r);
                const double cur = __dadd_rn(old, -r);
                __stcg(&c.g.P[i], __dadd_rn(__ldcg(&c.g.P[i]), __dmul_rn(alpha, r)));
                c.pushes++;
                enq = push_cond<POS>(cur, eps) && test_and_set(a.bitmap, i);
            }
        }
        enqueue(s, c, enq, ent);
    }
}

__device__ void clear_frontier_bits(Ctx& c, const PushArgs& a, const unsigned long long* Fin,
                                    uint64_t C) {
    for (uint64_t idx = (uint64_t)blockIdx.x * PT + threadIdx.x; idx < C;
         idx += (uint64_t)gridDim.x * PT) {
        const unsigned long long ent = __ldcg(&Fin[idx]);
        clear_bit(a.bitmap, (ent >> 32) * c.g.n + (uint32_t)ent);
    }
}

// ---------------------------------------------------------------- seeding

template <bool POS>
__device__ void seed_phase(Smem& s, Ctx& c, const PushArgs& a) {
    const double eps = c.g.eps;
    const uint64_t stride = (uint64_t)gridDim.x * PT;
    uint64_t total;
    if (a.seed_all)
        total = (uint64_t)c.g.S * c.g.n;
    else if (a.seed_v)
        total = (uint64_t)(*a.n_seed_v_dev) * c.g.S;
    else
        total = a.n_seed_e;
    const uint64_t nv = a.seed_v ? (uint64_t)(*a.n_seed_v_dev) : 0;
    for (uint64_t b = (uint64_t)blockIdx.x * PT; b < total; b += stride) {
        const uint64_t k = b + threadIdx.x;
        bool enq = false;
        unsigned long long ent = 0;
        if (k < total) {
            uint32_t sidx, v;
            if (a.seed_all) {
                sidx = (uint32_t)(k / c.g.n);
                v = (uint32_t)(k % c.g.n);
            } else if (a.seed_v) {
                sidx = (uint32_t)(k / nv);
                v = a.seed_v[k % nv];
            } else {
                ent = a.seed_e[k];
                sidx = (uint32_t)(ent >> 32);
                v = (uint32_t)ent;
            }
            ent = ((unsigned long long)sidx << 32) | v;
            enq = push_cond<POS>(__ldcg(&c.g.R[(size_t)sidx * c.g.n + v]), eps);
        }
        enqueue(s, c, enq, ent);
    }
}

// ---------------------------------------------------------------- phase driver

template <int MODE, bool POS>
__device__ void run_phase(Smem& s, Ctx& c, const PushArgs& a, unsigned& it) {
    DevCtl* ctl = c.ctl;
    const int ph = POS ? 0 : 1;
    // seed into F[it%2] / fcount[it%3]; both that and the next counter are 0 here
    c.Fout = a.F[it & 1];
    c.cnt_out = &ctl->fcount[it % 3];
    seed_phase<POS>(s, c, a);
    flush(s, c);
    grid_sync(ctl);
    uint32_t pit = 0;
    uint64_t C = 0;
    while (true) {
        C = *(volatile unsigned long long*)&ctl->fcount[it % 3];
        if (blockIdx.x == 0 && threadIdx.x == 0) {
            ctl->fcount[(it + 2) % 3] = 0;
            ctl->tilectr[(it + 2) % 3] = 0;
            if (C > 0 && !(a.max_iters && pit >= a.max_iters)) {
                ctl->iters[ph]++;
                atomicMax(&ctl->max_frontier, (unsigned long long)C);
            }
            if (C > 0 && pit >= a.iter_cap) atomicCAS(&ctl->err, KERR_OK, KERR_NOCONV);
        }
        if (C == 0 || (a.max_iters && pit >= a.max_iters) || pit >= a.iter_cap) break;
        const unsigned long long* Fin = a.F[it & 1];
        c.Fout = a.F[(it + 1) & 1];
        c.cnt_out = &ctl->fcount[(it + 1) % 3];
        unsigned long long* tc = &ctl->tilectr[it % 3];
        if (MODE == M_OPT) {
            round_opt<POS>(s, c, a, Fin, C, tc);
        } else if (MODE == M_VAN || MODE == M_DUP) {
            session_snapshot(c, a, Fin, C, MODE == M_VAN);
            grid_sync(ctl);
            session_propagate<POS, MODE == M_VAN>(s, c, a, Fin, C, tc);
        } else {  // M_EAGER
            clear_frontier_bits(c, a, Fin, C);
            grid_sync(ctl);
            session_eager_propagate<POS>(s, c, a, Fin, C, tc);
            grid_sync(ctl);
            session_eager_self<POS>(s, c, a, Fin, C);
        }
        flush(s, c);
        grid_sync(ctl);
        it++;
        pit++;
    }
    // a frontier left by max_iters keeps its UniqueEnqueue bits: drop them
    if ((MODE == M_VAN || MODE == M_EAGER) && C > 0) clear_frontier_bits(c, a, a.F[it & 1], C);
    // leave the counters of the next phase's seed round at zero
    grid_sync(ctl);
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        ctl->fcount[it % 3] = 0;
        ctl->fcount[(it + 1) % 3] = 0;
        ctl->fcount[(it + 2) % 3] = 0;
        ctl->tilectr[0] = ctl->tilectr[1] = ctl->tilectr[2] = 0;
    }
    grid_sync(ctl);
}

template <int MODE>
__global__ void __launch_bounds__(PT, 2) k_push(PushArgs a) {
    __shared__ Smem s;
    Ctx c;
    c.g = a.g;
    c.ctl = a.ctl;
    c.qn = 0;
    c.pushes = 0;
    c.edges = 0;
    if (threadIdx.x == 0) s.qn = 0;
    if (*(volatile int*)&a.ctl->err != KERR_OK) return;  // earlier stage failed: uniform exit
    c.pool = a.g.pool[*(volatile unsigned*)&a.ctl->active_pool];
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        for (int i = 0; i < 3; i++) a.ctl->fcount[i] = a.ctl->tilectr[i] = 0;
    }
    grid_sync(a.ctl);
    unsigned it = 0;
    if (a.phases & 1) run_phase<MODE, true>(s, c, a, it);
    if (a.phases & 2) run_phase<MODE, false>(s, c, a, it);
    // statistics
    __shared__ unsigned long long s_red[2];
    if (threadIdx.x == 0) s_red[0] = s_red[1] = 0;
    __syncthreads();
    if (c.pushes) atomicAdd(&s_red[0], c.pushes);
    if (c.edges) atomicAdd(&s_red[1], c.edges);
    __syncthreads();
    if (threadIdx.x == 0) {
        if (s_red[0]) atomicAdd(&a.ctl->pushes, s_red[0]);
        if (s_red[1]) atomicAdd(&a.ctl->pushed_edges, s_red[1]);
    }
}

template <int MODE>
cudaError_t launch_mode(const PushArgs& a, int num_sms, cudaStream_t st) {
    static int blocks_per_sm = 0;
    if (blocks_per_sm == 0) {
        cudaError_t e =
            cudaOccupancyMaxActiveBlocksPerMultiprocessor(&blocks_per_sm, k_push<MODE>, PT, 0);
        if (e != cudaSuccess) return e;
        if (blocks_per_sm < 1) return cudaErrorInvalidConfiguration;
        if (blocks_per_sm > 2) blocks_per_sm = 2;
    }
    dim3 grid(num_sms * blocks_per_sm), block(PT);
    PushArgs copy = a;
    void* args[] = {&copy};
    return cudaLaunchCooperativeKernel((const void*)k_push<MODE>, grid, block, args, 0, st);
}

}  // namespace

cudaError_t launch_push(int mode, const PushArgs& a, int num_sms, cudaStream_t st) {
    switch (mode) {
        case M_OPT: return launch_mode<M_OPT>(a, num_sms, st);
        case M_EAGER: return launch_mode<M_EAGER>(a, num_sms, st);
        case M_DUP: return launch_mode<M_DUP>(a, num_sms, st);
        case M_VAN: return launch_mode<M_VAN>(a, num_sms, st);
        default: return cudaErrorInvalidValue;
    }
}

}  // namespace ppr
