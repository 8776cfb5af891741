// push_sortagg.cu -- PPR_MODE_SORTAGG: Alg 3 rounds with sort-and-aggregate
// neighbour propagation instead of atomics.
//
// PAPER.md P:433-442 names the alternative to Line 21's atomics: "run a
// parallel sort on the key-value pairs consisting of the neighbor vertex ids
// and the corresponding residuals ... a parallel reduce operation to
// aggregate the residuals with the same keys and then transfer the residuals
// to the designated vertices" (rejected there for Maxwell, fn 2).
//
// One round of a phase (Alg 3 lines 9-23), host-driven:
//   self     for every frontier entry u (sorted by key):  w_u = R(u),
//            P(u) += a w_u, R(u) = 0                          (lines 13-16)
//   scan     offsets of the pairs of each entry (|N_in(u)|)
//   gen      pair (key(v, s), (1-a) w_u / d(v)) for every v in N_in(u)
//   sort     stable LSD radix sort of the pairs by key only: pairs of one key
//            stay in generation order, i.e. ascending u
//   reduce   per key, sequentially from R(v): R(v) = (..(R(v) + i_1) + i_2 ..)
//            -- the order in which a sequential Alg 3 loop over the sorted
//            frontier applies them (lines 19-21); pushCond decides FQ'
//   compact  FQ' = keys whose new residual meets pushCond, in key order
// No atomics, no data races: the result is bit-reproducible run to run and
// bit-identical to the oracle's Alg 3 emulation (ascending vertex order)
// whenever the internal ids are the caller's (no relabelling).
// Keys are v * S + sidx, so each source's frontier is in ascending v.
#include <algorithm>
#include <vector>

#include "primitives.cuh"
#include "push.cuh"

namespace ppr {

struct SortAgg {
    uint64_t cap = 0;        // pairs
    uint64_t* k[2] = {nullptr, nullptr};
    uint32_t* v[2] = {nullptr, nullptr};
    double* inc = nullptr;
    uint32_t* flag = nullptr;
    unsigned long long* pos = nullptr;
    uint32_t* hist = nullptr;
    unsigned long long* part = nullptr;
    uint64_t fcap = 0;       // frontier entries (S * n)
    uint32_t* len = nullptr;
    unsigned long long* off = nullptr;
    double* w = nullptr;
    unsigned long long* cnt = nullptr;  // device counters [0]: seed count, [1]: scan total
    unsigned long long* h_cnt = nullptr;  // pinned
    uint64_t bytes = 0;
};

namespace {

constexpr int SA_T = 256;

inline unsigned grid_for(uint64_t n, int per_block) {
    uint64_t g = (n + per_block - 1) / per_block;
    if (g < 1) g = 1;
    if (g > (1u << 20)) g = 1u << 20;
    return (unsigned)g;
}

template <bool POS>
__global__ void __launch_bounds__(SA_T) k_sa_seed(const PushArgs a, uint64_t nv, uint64_t* keys,
                                                  unsigned long long* cnt) {
    const uint64_t S = a.g.S, n = a.g.n;
    uint64_t total = a.seed_all ? S * n : (a.seed_v ? nv * S : a.n_seed_e);
    for (uint64_t k = (uint64_t)blockIdx.x * SA_T + threadIdx.x; k < total;
         k += (uint64_t)gridDim.x * SA_T) {
        uint32_t sidx, v;
        if (a.seed_all) {
            sidx = (uint32_t)(k / n);
            v = (uint32_t)(k % n);
        } else if (a.seed_v) {
            sidx = (uint32_t)(k / nv);
            v = a.seed_v[k % nv];
        } else {
            sidx = (uint32_t)(a.seed_e[k] >> 32);
            v = (uint32_t)a.seed_e[k];
        }
        if (push_cond<POS>(*Rp<false>(a.g, sidx, v), a.g.eps))
            keys[atomicAdd(cnt, 1ull)] = (uint64_t)v * S + sidx;
    }
}

// lines 13-16: w = R(u); P(u) += a w; R(u) = 0; and |N_in(u)|
__global__ void __launch_bounds__(SA_T) k_sa_self(const PushArgs a, const unsigned long long* F,
                                                  uint64_t C, double* W, uint32_t* len) {
    const uint64_t S = a.g.S;
    for (uint64_t i = (uint64_t)blockIdx.x * SA_T + threadIdx.x; i < C;
         i += (uint64_t)gridDim.x * SA_T) {
        const uint64_t key = F[i];
        const uint32_t u = (uint32_t)(key / S), sidx = (uint32_t)(key % S);
        double* rp = Rp<false>(a.g, sidx, u);
        double* pp = Pp<false>(a.g, sidx, u);
        const double w = *rp;
        *pp = __dadd_rn(*pp, __dmul_rn(a.g.alpha, w));
        *rp = 0.0;
        W[i] = w;
        len[i] = a.g.slab[u].len;
    }
}

// one warp per frontier entry: its pairs at off[i] .. off[i] + |N_in(u)|
__global__ void __launch_bounds__(SA_T) k_sa_gen(const PushArgs a, const PoolEnt* pool,
                                                 const unsigned long long* F, uint64_t C,
                                                 const unsigned long long* off, const double* W,
                                                 uint64_t* keys, uint32_t* vals, double* inc) {
    const uint64_t S = a.g.S;
    const unsigned lane = threadIdx.x & 31u;
    const double c1 = 1.0 - a.g.alpha;
    for (uint64_t i = ((uint64_t)blockIdx.x * SA_T + threadIdx.x) / 32; i < C;
         i += (uint64_t)gridDim.x * (SA_T / 32)) {
        const uint64_t key = F[i];
        const uint32_t u = (uint32_t)(key / S), sidx = (uint32_t)(key % S);
        const Slab sl = get_slab<false>(a.g, u);
        const double cw = __dmul_rn(c1, W[i]);  // (1 - a) * w_u, as the oracle's loop
        const unsigned long long o = off[i];
        for (uint32_t j = lane; j < sl.len; j += 32) {
            const uint32_t x = pool_id(a.g, pool, sl.off + j);
            const uint32_t dx = a.g.pool_wide ? pe_d(pool[sl.off + j]) : a.g.dout[x];
            const uint64_t p = o + j;
            keys[p] = (uint64_t)x * S + sidx;
            vals[p] = (uint32_t)p;
            inc[p] = __ddiv_rn(cw, (double)dx);
        }
    }
}

// lines 19-23 per key, in pair order: the run head applies the run to R(v)
template <bool POS>
__global__ void __launch_bounds__(SA_T) k_sa_reduce(const PushArgs a, const uint64_t* keys,
                                                    const uint32_t* vals, const double* inc,
                                                    uint64_t E, uint32_t* flag) {
    const uint64_t S = a.g.S;
    for (uint64_t i = (uint64_t)blockIdx.x * SA_T + threadIdx.x; i < E;
         i += (uint64_t)gridDim.x * SA_T) {
        const uint64_t key = keys[i];
        uint32_t f = 0;
        if (i == 0 || keys[i - 1] != key) {
            double* rp = Rp<false>(a.g, (uint32_t)(key % S), (uint32_t)(key / S));
            double r = *rp;
            for (uint64_t j = i; j < E && keys[j] == key; j++) r = __dadd_rn(r, inc[vals[j]]);
            *rp = r;
            f = push_cond<POS>(r, a.g.eps) ? 1u : 0u;
        }
        flag[i] = f;
    }
}

__global__ void __launch_bounds__(SA_T) k_sa_compact(const uint64_t* keys, const uint32_t* flag,
                                                     const unsigned long long* pos, uint64_t E,
                                                     unsigned long long* Fn) {
    for (uint64_t i = (uint64_t)blockIdx.x * SA_T + threadIdx.x; i < E;
         i += (uint64_t)gridDim.x * SA_T)
        if (flag[i]) Fn[pos[i]] = keys[i];
}

template <typename T>
cudaError_t sa_alloc(SortAgg* s, T** p, uint64_t count) {
    cudaError_t e = cudaMalloc((void**)p, sizeof(T) * (count ? count : 1));
    if (e == cudaSuccess) s->bytes += sizeof(T) * (count ? count : 1);
    return e;
}
template <typename T>
void sa_free(SortAgg* s, T*& p, uint64_t count) {
    if (p) {
        cudaFree(p);
        s->bytes -= sizeof(T) * (count ? count : 1);
    }
    p = nullptr;
}

void free_pairs(SortAgg* s) {
    for (int i = 0; i < 2; i++) {
        sa_free(s, s->k[i], s->cap);
        sa_free(s, s->v[i], s->cap);
    }
    sa_free(s, s->inc, s->cap);
    sa_free(s, s->flag, s->cap);
    sa_free(s, s->pos, s->cap);
    sa_free(s, s->hist, rs_hist_entries(s->cap));
    sa_free(s, s->part, scan_parts(s->cap) + 1);
    s->cap = 0;
}

cudaError_t ensure_pairs(SortAgg* s, uint64_t need) {
    if (need <= s->cap) return cudaSuccess;
    free_pairs(s);
    uint64_t cap = std::max<uint64_t>(need + need / 4, 1u << 16);
    cudaError_t e = cudaSuccess;
    for (int i = 0; i < 2 && e == cudaSuccess; i++) {
        e = sa_alloc(s, &s->k[i], cap);
        if (e == cudaSuccess) e = sa_alloc(s, &s->v[i], cap);
    }
    if (e == cudaSuccess) e = sa_alloc(s, &s->inc, cap);
    if (e == cudaSuccess) e = sa_alloc(s, &s->flag, cap);
    if (e == cudaSuccess) e = sa_alloc(s, &s->pos, cap);
    if (e == cudaSuccess) e = sa_alloc(s, &s->hist, rs_hist_entries(cap));
    if (e == cudaSuccess) e = sa_alloc(s, &s->part, scan_parts(cap) + 1);
    s->cap = cap;
    if (e != cudaSuccess) free_pairs(s);
    return e;
}

cudaError_t ensure_frontier(SortAgg* s, uint64_t Sn) {
    if (s->fcap >= Sn) return cudaSuccess;
    sa_free(s, s->len, s->fcap);
    sa_free(s, s->off, s->fcap);
    sa_free(s, s->w, s->fcap);
    cudaError_t e = sa_alloc(s, &s->len, Sn);
    if (e == cudaSuccess) e = sa_alloc(s, &s->off, Sn);
    if (e == cudaSuccess) e = sa_alloc(s, &s->w, Sn);
    if (e == cudaSuccess && !s->cnt) e = sa_alloc(s, &s->cnt, 4);
    if (e == cudaSuccess && !s->h_cnt) e = cudaMallocHost(&s->h_cnt, 4 * sizeof(unsigned long long));
    s->fcap = e == cudaSuccess ? Sn : 0;
    return e;
}

int ceil_log2_u64(uint64_t x) {
    int b = 0;
    while ((1ull << b) < x) b++;
    return b;
}

// device counter -> host (synchronises the stream)
cudaError_t read_cnt(SortAgg* s, const unsigned long long* d, cudaStream_t st, uint64_t* out) {
    cudaError_t e = cudaMemcpyAsync(s->h_cnt, d, sizeof(unsigned long long), cudaMemcpyDeviceToHost, st);
    if (e == cudaSuccess) e = cudaStreamSynchronize(st);
    *out = s->h_cnt[0];
    return e;
}

template <bool POS>
cudaError_t sa_phase(SortAgg* s, const PushArgs& a, uint64_t nv, cudaStream_t st,
                     SortAggStats* out, uint32_t* launches) {
    const uint64_t Sn = (uint64_t)a.g.S * a.g.n;
    const PoolEnt* pool = a.g.pool[out->active_pool];
    int shifts[8];
    const int bits = ceil_log2_u64(Sn);
    int np = 0;
    for (int sh = 0; sh < bits && np < 8; sh += 8) shifts[np++] = sh;
    // seed: FQ = {seeds meeting pushCond} (Alg 3 line 1 / 4), sorted by key
    const uint64_t total = a.seed_all ? Sn : (a.seed_v ? nv * a.g.S : a.n_seed_e);
    cudaError_t e = ensure_pairs(s, std::max<uint64_t>(total, 1));
    if (e != cudaSuccess) return e;
    cudaMemsetAsync(s->cnt, 0, sizeof(unsigned long long), st);
    if (total) {
        k_sa_seed<POS><<<grid_for(total, SA_T), SA_T, 0, st>>>(a, nv, s->k[0], s->cnt);
        ++*launches;
    }
    uint64_t C = 0;
    if ((e = read_cnt(s, s->cnt, st, &C)) != cudaSuccess) return e;
    if (C == 0) return cudaGetLastError();
    const int ws = radix_sort_pairs(s->k[0], s->v[0], s->k[1], s->v[1], C, shifts, np, s->hist, st,
                                    launches);
    cudaMemcpyAsync(a.F[0], s->k[ws], sizeof(uint64_t) * C, cudaMemcpyDeviceToDevice, st);
    int cur = 0;
    uint32_t pit = 0;
    const int ph = POS ? 0 : 1;
    while (C > 0) {
        if (a.max_iters && pit >= a.max_iters) break;
        if (pit >= a.iter_cap) {
            out->noconv = 1;
            break;
        }
        out->iters[ph]++;
        out->pushes += C;
        out->max_frontier = std::max<uint64_t>(out->max_frontier, C);
        const unsigned long long* F = a.F[cur];
        k_sa_self<<<grid_for(C, SA_T), SA_T, 0, st>>>(a, F, C, s->w, s->len);
        exclusive_scan_u32(s->len, s->off, C, s->part, s->cnt + 1, st, launches);
        ++*launches;
        uint64_t E = 0;
        if ((e = read_cnt(s, s->cnt + 1, st, &E)) != cudaSuccess) return e;
        out->edges += E;
        if (E >= (1ull << 32)) return cudaErrorInvalidValue;  // u32 pair positions
        if ((e = ensure_pairs(s, E)) != cudaSuccess) return e;
        if (E == 0) {
            C = 0;
            break;
        }
        k_sa_gen<<<grid_for(C, SA_T / 32), SA_T, 0, st>>>(a, pool, F, C, s->off, s->w, s->k[0],
                                                           s->v[0], s->inc);
        ++*launches;
        const int w = radix_sort_pairs(s->k[0], s->v[0], s->k[1], s->v[1], E, shifts, np, s->hist,
                                       st, launches);
        k_sa_reduce<POS><<<grid_for(E, SA_T), SA_T, 0, st>>>(a, s->k[w], s->v[w], s->inc, E,
                                                             s->flag);
        exclusive_scan_u32(s->flag, s->pos, E, s->part, s->cnt + 1, st, launches);
        k_sa_compact<<<grid_for(E, SA_T), SA_T, 0, st>>>(s->k[w], s->flag, s->pos, E,
                                                         a.F[cur ^ 1]);
        *launches += 2;
        if ((e = read_cnt(s, s->cnt + 1, st, &C)) != cudaSuccess) return e;
        cur ^= 1;
        pit++;
    }
    return cudaGetLastError();
}

}  // namespace

cudaError_t sortagg_push(SortAgg** ps, const PushArgs& a, uint64_t n_seed_v, cudaStream_t st,
                         SortAggStats* out, uint32_t* launches) {
    if (a.g.rec) return cudaErrorInvalidValue;  // arrays layout only
    if (!*ps) *ps = new SortAgg();
    SortAgg* s = *ps;
    cudaError_t e = ensure_frontier(s, (uint64_t)a.g.S * a.g.n);
    if (e != cudaSuccess) return e;
    if (a.phases & 1) e = sa_phase<true>(s, a, n_seed_v, st, out, launches);
    if (e == cudaSuccess && !out->noconv && (a.phases & 2))
        e = sa_phase<false>(s, a, n_seed_v, st, out, launches);
    return e;
}

uint64_t sortagg_bytes(const SortAgg* s) { return s ? s->bytes : 0; }

void sortagg_free(SortAgg* s) {
    if (!s) return;
    free_pairs(s);
    sa_free(s, s->len, s->fcap);
    sa_free(s, s->off, s->fcap);
    sa_free(s, s->w, s->fcap);
    sa_free(s, s->cnt, 4);
    if (s->h_cnt) cudaFreeHost(s->h_cnt);
    delete s;
}

}  // namespace ppr
