// ppr_api.cu -- the C ABI of libppr.so (include/ppr.h) and the host
// orchestrator of one batch:
//
//   a0 staging      H2D copy of the batch (PPR_MEM_HOST) or device pointers as given
//   keys            k_batch_keys: (v,u) and (u,v) keys + id range check
//   sort x2         in-house LSD radix sort (primitives.cu)
//   heads           run nets + segment heads of both orders
//   a1 store        validate (deletion claims) -> in-place apply | rebuild
//   a2 restore      Lemma 3 closed form per touched u, d_out update
//   a3-a6 push      one cooperative persistent kernel: POS then NEG (push.cu)
//   stats           one D2H copy of the device control block
//
// Every kernel checks the device error flag first, so a batch that fails
// validation (ERANGE / ENOENT) mutates nothing and costs no host round-trip
// until the final stats copy.
#include <cuda_runtime.h>

#include <algorithm>
#include <cmath>
#include <cstdarg>
#include <cstddef>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <map>
#include <mutex>
#include <new>
#include <string>
#include <vector>

#include "../../include/ppr.h"
#include "ppr_internal.cuh"
#include "primitives.cuh"
#include "push.cuh"
#include "store.cuh"

using namespace ppr;

// shape of a captured batch graph: replay only while all of it matches
struct GraphKey {
    uint64_t n_ins = 0, n_del = 0;
    bool push = false;
    int mode = -1;
    uint32_t max_iters = 0;
    bool timing = false, force_rebuild = false;
    uint64_t epoch = 0, cap0 = 0, cap1 = 0;
    const void* pool0 = nullptr;
    const void* pool1 = nullptr;
    bool operator==(const GraphKey& o) const {
        return n_ins == o.n_ins && n_del == o.n_del && push == o.push && mode == o.mode &&
               max_iters == o.max_iters && timing == o.timing && force_rebuild == o.force_rebuild &&
               epoch == o.epoch && cap0 == o.cap0 && cap1 == o.cap1 && pool0 == o.pool0 &&
               pool1 == o.pool1;
    }
};

struct ppr_ctx {
    int device = 0;
    cudaStream_t st = nullptr;
    bool own_stream = false;
    int num_sms = 0;
    uint32_t n = 0, S = 0;
    double alpha = 0, eps = 0;
    int undirected = 0;
    int mode = PPR_MODE_OPT;
    bool push_enabled = true;
    uint32_t max_iters = 0;
    bool timing = true;
    bool force_rebuild = false;
    double slack = 0.25;
    uint32_t min_cap = 4;
    uint64_t m = 0;          // arcs in the store
    unsigned active = 0;     // host mirror of DevCtl::active_pool
    uint64_t pool_cap[2] = {0, 0};
    // device state
    VRec* d_rec = nullptr;       // packed layout (S == 1, pools < 2^32 entries)
    double* d_hot = nullptr;     // arrays layout: R [S][n] followed by d_out [n] (one allocation,
    uint64_t hot_bytes = 0;      //   the L2 access-policy window / persisting set-aside)
    bool l2_window = false;
    size_t l2_win_bytes = 0;
    float l2_hit = 0.f;
    uint32_t* d_dout = nullptr;  // structure-of-arrays layout (S > 1)
    SlabRec* d_slab = nullptr;   // {off, len} of N_in(v) (ppr_internal.cuh)
    uint32_t* d_cap = nullptr;   // slab capacities
    PoolEnt* d_pool[2] = {nullptr, nullptr};  // slab pools (entries: PoolEnt if pool_wide, else u32)
    bool pool_wide = false;                   // ppr_opts.pool_degrees (ppr_internal.cuh PoolEnt)
    double* d_P = nullptr;
    double* d_R = nullptr;
    uint32_t* d_sources = nullptr;  // internal ids
    uint32_t* d_perm = nullptr;     // external -> internal vertex id (degree order), or null
    uint32_t* d_inv = nullptr;      // internal -> external
    unsigned long long* d_F[2] = {nullptr, nullptr};
    double* d_W = nullptr;
    uint32_t* d_bitmap = nullptr;
    DevCtl* d_ctl = nullptr;
    DevStats* h_ctl = nullptr;  // pinned copy of DevCtl::st
    VertexBufs vb{};
    // batch scratch
    uint64_t bcap = 0;  // sort entries
    uint64_t ucap = 0;  // input updates per kind
    BatchBufs bb{};
    uint32_t* d_in[4] = {nullptr, nullptr, nullptr, nullptr};
    int shifts[8] = {0};
    int npasses = 0;
    cudaEvent_t ev[5] = {nullptr, nullptr, nullptr, nullptr, nullptr};
    cudaStream_t st2 = nullptr;  // restore branch of a batch (fork/join with st)
    cudaEvent_t ev_fork = nullptr, ev_valid = nullptr, ev_join = nullptr;
    std::string err;
    bool poisoned = false;
    uint64_t dev_bytes = 0;
    std::vector<void*> allocs;
    bool graphs = true;                     // replay each batch shape as a CUDA graph (PPR_GRAPHS=0: off)
    cudaGraphExec_t gexec = nullptr;
    GraphKey gkey{};
    uint32_t glaunches = 0;
    uint64_t buf_epoch = 0;                 // bumped whenever batch / pool buffers are reallocated
    unsigned long long* d_ring = nullptr;   // PPR_MODE_ASYNC ring queue (2*S*n slots, EMPTY)
    unsigned long long ring_cap = 0;
    uint64_t hyb_thresh = 0;                // Opt: frontier size at which a phase finishes on the ring
    int ring_all = -1;                      // Opt: whole phases on the ring (-1: iff >= 8 arcs per vertex)
    int edge_chains = 0;                    // Opt: edge chains per lane (0: 3 iff ring_all, else 2)
    uint32_t wave = 0;                      // SHARED: sources per push launch (multiple of 32; 0: all)
    bool check_enq = false;                 // PPR_OPT_CHECK_ENQUEUE (Opt debug)
    unsigned long long* d_trace = nullptr;  // PPR_TRACE=1: per-round trace of the push
    uint32_t trace_cap = 0;
    SortAgg* sa = nullptr;                  // PPR_MODE_SORTAGG scratch (grown on demand)
};

namespace {

bool dbg_on() {  // PPR_DEBUG=1: report launch errors / L2 setup on stderr (diagnostics only)
    static const bool on = getenv("PPR_DEBUG") && atoi(getenv("PPR_DEBUG")) > 0;
    return on;
}

// Persisting-L2 set-aside per device, reference-counted over the handles that
// use an access-policy window: the first raises cudaLimitPersistingL2CacheSize
// (remembering the previous value), the last restores it.  Persisting lines
// of other handles are never reset here.
struct L2Share {
    int refs = 0;
    size_t prev = 0, cur = 0;
};
std::mutex g_l2_mu;
std::map<int, L2Share> g_l2;

bool l2_acquire(int device, size_t bytes) {
    std::lock_guard<std::mutex> lk(g_l2_mu);
    L2Share& s = g_l2[device];
    size_t cur = 0;
    if (cudaDeviceGetLimit(&cur, cudaLimitPersistingL2CacheSize) != cudaSuccess) {
        cudaGetLastError();
        return false;
    }
    if (s.refs == 0) s.prev = cur;
    if (cur < bytes && cudaDeviceSetLimit(cudaLimitPersistingL2CacheSize, bytes) != cudaSuccess) {
        cudaGetLastError();
        return false;
    }
    s.cur = std::max(cur, bytes);
    s.refs++;
    return true;
}

void l2_release(int device) {
    std::lock_guard<std::mutex> lk(g_l2_mu);
    auto it = g_l2.find(device);
    if (it == g_l2.end() || it->second.refs == 0) return;
    if (--it->second.refs == 0) {
        int cur_dev = 0;
        cudaGetDevice(&cur_dev);
        cudaSetDevice(device);
        cudaDeviceSetLimit(cudaLimitPersistingL2CacheSize, it->second.prev);
        cudaSetDevice(cur_dev);
        cudaGetLastError();
        g_l2.erase(it);
    }
}

void set_err(ppr_ctx* h, const char* fmt, ...) {
    char buf[512];
    va_list ap;
    va_start(ap, fmt);
    vsnprintf(buf, sizeof buf, fmt, ap);
    va_end(ap);
    h->err = buf;
}

ppr_status cuda_fail(ppr_ctx* h, cudaError_t e, const char* where) {
    set_err(h, "%s: %s", where, cudaGetErrorString(e));
    h->poisoned = true;
    return PPR_ECUDA;
}

template <typename T>
cudaError_t dalloc(ppr_ctx* h, T** p, uint64_t count) {
    void* q = nullptr;
    size_t bytes = (size_t)std::max<uint64_t>(count, 1) * sizeof(T);
    cudaError_t e = cudaMalloc(&q, bytes);
    if (e != cudaSuccess) {
        cudaGetLastError();
        *p = nullptr;
        return e;
    }
    h->dev_bytes += bytes;
    *p = (T*)q;
    return cudaSuccess;
}

template <typename T>
void dfree(ppr_ctx* h, T*& p, uint64_t count) {
    if (p) {
        cudaFree(p);
        h->dev_bytes -= (size_t)std::max<uint64_t>(count, 1) * sizeof(T);
    }
    p = nullptr;
}

// PoolEnt-sized words backing a pool of `cap` entries (4 or 8 bytes each)
// slab offsets are u32 (SlabRec), so a pool holds at most this many entries
constexpr uint64_t kPoolMaxEntries = 0xFFFFFFFFull - 64;

uint64_t pool_words(const ppr_ctx* h, uint64_t cap) { return h->pool_wide ? cap : (cap + 1) / 2; }

DevGraph graph_of(const ppr_ctx* h) {
    DevGraph g;
    g.n = h->n;
    g.S = h->S;
    g.alpha = h->alpha;
    g.eps = h->eps;
    g.dout = h->d_dout;
    g.slab = h->d_slab;
    g.cap = h->d_cap;
    g.pool[0] = h->d_pool[0];
    g.pool[1] = h->d_pool[1];
    g.pool_wide = h->pool_wide ? 1u : 0u;
    g.P = h->d_P;
    g.R = h->d_R;
    g.sources = h->d_sources;
    g.rec = h->d_rec;
    return g;
}

int ceil_log2(uint64_t x) {
    int b = 0;
    while ((1ull << b) < x) b++;
    return b < 1 ? 1 : b;
}

void free_batch(ppr_ctx* h) {
    BatchBufs& b = h->bb;
    for (int i = 0; i < 2; i++) {
        dfree(h, b.kv[i], h->bcap);
        dfree(h, b.ku[i], h->bcap);
        dfree(h, b.ov[i], h->bcap);
        dfree(h, b.ou[i], h->bcap);
    }
    dfree(h, b.hist, rs_hist_entries(h->bcap));
    dfree(h, b.hist2, rs_hist_entries(h->bcap));
    dfree(h, b.rnv, h->bcap);
    dfree(h, b.rnu, h->bcap);
    dfree(h, b.vheads, h->bcap);
    dfree(h, b.uheads, h->bcap);
    dfree(h, b.claim, h->bcap);
    dfree(h, b.delpos, h->bcap);
    dfree(h, b.seg_end, h->bcap);
    dfree(h, b.seg_D, h->bcap);
    dfree(h, b.seg_I, h->bcap);
    dfree(h, h->d_in[0], 4 * h->ucap);
    h->bcap = h->ucap = 0;
}

ppr_status ensure_batch(ppr_ctx* h, uint64_t nupd, uint64_t N) {
    if (N <= h->bcap && nupd <= h->ucap) return PPR_OK;
    cudaError_t e = cudaStreamSynchronize(h->st);
    if (e != cudaSuccess) return cuda_fail(h, e, "ensure_batch sync");
    free_batch(h);
    h->buf_epoch++;
    uint64_t cap = std::max<uint64_t>(N + N / 4, 1024);
    uint64_t ucap = std::max<uint64_t>(nupd + nupd / 4, 1024);
    BatchBufs& b = h->bb;
    bool ok = true;
    for (int i = 0; i < 2; i++) {
        ok = ok && dalloc(h, &b.kv[i], cap) == cudaSuccess && dalloc(h, &b.ku[i], cap) == cudaSuccess &&
             dalloc(h, &b.ov[i], cap) == cudaSuccess && dalloc(h, &b.ou[i], cap) == cudaSuccess;
    }
    ok = ok && dalloc(h, &b.hist, rs_hist_entries(cap)) == cudaSuccess &&
         dalloc(h, &b.hist2, rs_hist_entries(cap)) == cudaSuccess;
    ok = ok && dalloc(h, &b.rnv, cap) == cudaSuccess && dalloc(h, &b.rnu, cap) == cudaSuccess;
    ok = ok && dalloc(h, &b.vheads, cap) == cudaSuccess && dalloc(h, &b.uheads, cap) == cudaSuccess;
    ok = ok && dalloc(h, &b.claim, cap) == cudaSuccess && dalloc(h, &b.delpos, cap) == cudaSuccess;
    ok = ok && dalloc(h, &b.seg_end, cap) == cudaSuccess && dalloc(h, &b.seg_D, cap) == cudaSuccess &&
         dalloc(h, &b.seg_I, cap) == cudaSuccess;
    // staging: one block [ins_src | ins_dst | del_src | del_dst] at offsets set by the batch's
    // counts, so a batch packed the same way on the host arrives with one copy
    ok = ok && dalloc(h, &h->d_in[0], 4 * ucap) == cudaSuccess;
    h->bcap = cap;
    h->ucap = ucap;
    if (!ok) {
        free_batch(h);
        set_err(h, "out of device memory for a batch of %llu arcs", (unsigned long long)N);
        return PPR_ENOMEM;
    }
    return PPR_OK;
}

// the inactive pool must hold a rebuild of (m + new arcs) entries
ppr_status ensure_alt_pool(ppr_ctx* h, uint64_t new_arcs) {
    const unsigned alt = h->active ^ 1u;
    const double need_d =
        std::ceil((1.0 + h->slack) * (double)(h->m + new_arcs)) + (double)(h->min_cap + 1) * h->n + 1024;
    const uint64_t need = (uint64_t)need_d;
    if (h->pool_cap[alt] >= need) return PPR_OK;
    if (need > kPoolMaxEntries) {
        set_err(h, "a slab pool of %llu entries exceeds the 2^32 - 1 entries u32 slab offsets address",
                (unsigned long long)need);
        return PPR_ENOMEM;
    }
    cudaError_t e = cudaStreamSynchronize(h->st);
    if (e != cudaSuccess) return cuda_fail(h, e, "ensure_alt_pool sync");
    dfree(h, h->d_pool[alt], pool_words(h, h->pool_cap[alt]));
    h->pool_cap[alt] = 0;
    h->buf_epoch++;
    uint64_t cap = std::min<uint64_t>(need + need / 4, kPoolMaxEntries);
    if (dalloc(h, &h->d_pool[alt], pool_words(h, cap)) != cudaSuccess) {
        set_err(h, "out of device memory for the rebuild pool (%llu entries)",
                (unsigned long long)cap);
        return PPR_ENOMEM;
    }
    cudaMemsetAsync(h->d_pool[alt], 0xFF, sizeof(PoolEnt) * pool_words(h, cap), h->st);  // empty slots
    h->pool_cap[alt] = cap;
    return PPR_OK;
}

void fill_stats(ppr_ctx* h, ppr_batch_stats* s, uint32_t launches, bool timed,
                uint64_t h2d = 0) {
    if (!s) return;
    memset(s, 0, sizeof *s);
    s->h2d_bytes = h2d;
    s->d2h_bytes = sizeof(DevStats);
    const DevStats& c = *h->h_ctl;
    s->iters_pos = c.iters[0];
    s->iters_neg = c.iters[1];
    s->pushes = c.pushes;
    s->pushed_edges = c.pushed_edges;
    s->walk_edges = h->mode == PPR_MODE_SHARED ? c.walk_edges : c.pushed_edges;
    s->entries = h->mode == PPR_MODE_SHARED ? c.entries : c.pushes;
    s->dup_enqueues = c.dup_enq;
    s->max_frontier = c.max_frontier;
    s->touched = (uint64_t)c.n_touched * h->S;
    s->num_arcs = h->m;
    s->rebuilt = (c.rebuild && c.err == KERR_OK) ? 1u : 0u;
    s->kernel_launches = launches;
    if (timed) {
        float ms = 0;
        cudaEventElapsedTime(&ms, h->ev[0], h->ev[4]);
        s->ms_total = ms;
        cudaEventElapsedTime(&ms, h->ev[0], h->ev[1]);
        s->ms_store = ms;
        cudaEventElapsedTime(&ms, h->ev[2], h->ev[3]);
        s->ms_push = ms;
    }
    // device-clock phase times (DevStats stamps; 0 where the stage did not run)
    if (c.t_restore[1] > c.t_restore[0]) s->ms_restore = (float)((c.t_restore[1] - c.t_restore[0]) * 1e-6);
    s->ms_push_pos = (float)(c.ns_push[0] * 1e-6);
    s->ms_push_neg = (float)(c.ns_push[1] * 1e-6);
}

PushArgs push_args(ppr_ctx* h) {
    PushArgs a{};
    a.g = graph_of(h);
    a.ctl = h->d_ctl;
    a.F[0] = h->d_F[0];
    a.F[1] = h->d_F[1];
    a.W = h->d_W;
    a.bitmap = h->d_bitmap;
    a.phases = 3;
    a.max_iters = h->max_iters;
    a.iter_cap = 1000000;
    a.l2_base = h->d_hot;
    a.l2_bytes = h->l2_win_bytes;
    a.l2_hit = h->l2_hit;
    if (h->d_trace) {
        cudaMemsetAsync(h->d_trace, 0, sizeof(unsigned long long) * (4 * h->trace_cap + 8), h->st);
        a.trace = h->d_trace;
        a.trace_cap = h->trace_cap;
    }
    return a;
}

// PPR_TRACE=1: print the per-round frontier sizes, times and edges of the last push
void dump_trace(ppr_ctx* h, const char* what) {
    if (!h->d_trace) return;
    std::vector<unsigned long long> t(4ull * h->trace_cap + 8);
    cudaMemcpy(t.data(), h->d_trace, sizeof(unsigned long long) * t.size(), cudaMemcpyDeviceToHost);
    fprintf(stderr, "PPR_TRACE %s:", what);
    for (uint32_t i = 0; i + 1 < h->trace_cap; i++) {
        if (t[4 * i] == ~0ull || t[4 * i + 1] == 0) break;
        unsigned long long t1 = t[4 * (i + 1) + 1];
        fprintf(stderr, " [%c%llu %llu %.1fus]", (t[4 * i] >> 63) ? 'N' : 'P',
                t[4 * i] & ~(1ull << 63), t[4 * i + 2], t1 ? (t1 - t[4 * i + 1]) / 1e3 : -1.0);
    }
    const unsigned long long* x = &t[4ull * h->trace_cap];
    if (x[3])
        fprintf(stderr, "\nPPR_TRACE split per CTA (us): tiles %.1f [prologue %.1f claim %.1f] flush %.1f barrier %.1f (%llu CTAs)",
                x[0] / 1e3 / x[3], x[4] / 1e3 / x[3], x[5] / 1e3 / x[3], x[1] / 1e3 / x[3],
                x[2] / 1e3 / x[3], x[3]);
    fprintf(stderr, "\n");
}

ppr_status status_of_kerr(ppr_ctx* h, int kerr) {
    switch (kerr) {
        case KERR_OK: return PPR_OK;
        case KERR_RANGE: set_err(h, "vertex id >= n"); return PPR_ERANGE;
        case KERR_NOENT: set_err(h, "deletion of an absent arc"); return PPR_ENOENT;
        case KERR_NOCONV:
            set_err(h, "push exceeded the iteration cap");
            h->poisoned = true;
            return PPR_ENOCONV;
        default:
            set_err(h, "internal store overflow (%d)", kerr);
            h->poisoned = true;
            return PPR_ECUDA;
    }
}

// synchronise, copy the control block, map errors
ppr_status finish(ppr_ctx* h, const char* where) {
    cudaError_t e = cudaMemcpyAsync(h->h_ctl, &h->d_ctl->st, sizeof(DevStats), cudaMemcpyDeviceToHost, h->st);
    if (e != cudaSuccess) return cuda_fail(h, e, where);
    e = cudaStreamSynchronize(h->st);
    if (e != cudaSuccess) return cuda_fail(h, e, (std::string(where) + " (stream)").c_str());
    e = cudaGetLastError();
    if (e != cudaSuccess) return cuda_fail(h, e, (std::string(where) + " (last error)").c_str());
    return status_of_kerr(h, h->h_ctl->err);
}

void record(ppr_ctx* h, int i) {
    if (h->timing) {
        cudaError_t e = cudaEventRecord(h->ev[i], h->st);
        if (e != cudaSuccess && dbg_on())
            fprintf(stderr, "PPR_DEBUG: event record %d: %s\n", i, cudaGetErrorString(e));
    }
}

void destroy_all(ppr_ctx* h) {
    if (h->st) cudaStreamSynchronize(h->st);
    if (h->gexec) cudaGraphExecDestroy(h->gexec), h->gexec = nullptr;
    free_batch(h);
    dfree(h, h->d_rec, h->n);
    if (h->l2_window) {
        l2_release(h->device);
        h->l2_window = false;
    }
    if (h->d_hot) {
        dfree(h, h->d_hot, (uint64_t)h->S * h->n + (h->n + 1) / 2 + 32);
        h->d_R = nullptr;
        h->d_dout = nullptr;
    }
    dfree(h, h->d_dout, h->n);
    dfree(h, h->d_slab, h->n);
    dfree(h, h->d_cap, h->n);
    dfree(h, h->d_pool[0], pool_words(h, h->pool_cap[0]));
    dfree(h, h->d_pool[1], pool_words(h, h->pool_cap[1]));
    dfree(h, h->d_P, (uint64_t)h->S * h->n);
    dfree(h, h->d_R, (uint64_t)h->S * h->n);
    dfree(h, h->d_sources, h->S);
    dfree(h, h->d_perm, h->n);
    dfree(h, h->d_inv, h->n);
    dfree(h, h->d_F[0], (uint64_t)h->S * h->n);
    dfree(h, h->d_F[1], (uint64_t)h->S * h->n);
    dfree(h, h->d_W, (uint64_t)h->S * h->n);
    dfree(h, h->d_bitmap, ((uint64_t)h->S * h->n + 31) / 32);
    dfree(h, h->d_ctl, 1);
    dfree(h, h->vb.vseg, h->n);
    dfree(h, h->vb.newcap, h->n);
    dfree(h, h->vb.newoff, h->n);
    dfree(h, h->vb.part, std::max<uint64_t>(scan_parts(h->n) + 1, 8192));
    dfree(h, h->vb.big, h->n);
    dfree(h, h->vb.touched, h->n);
    if (h->h_ctl) cudaFreeHost(h->h_ctl);
    h->h_ctl = nullptr;
    for (auto& e : h->ev)
        if (e) cudaEventDestroy(e), e = nullptr;
    for (cudaEvent_t* e : {&h->ev_fork, &h->ev_valid, &h->ev_join})
        if (*e) cudaEventDestroy(*e), *e = nullptr;
    if (h->st2) cudaStreamSynchronize(h->st2), cudaStreamDestroy(h->st2), h->st2 = nullptr;
    dfree(h, h->d_trace, 4ull * h->trace_cap + 8);
    dfree(h, h->d_ring, h->ring_cap);
    if (h->sa) {
        h->dev_bytes -= sortagg_bytes(h->sa);
        sortagg_free(h->sa);
        h->sa = nullptr;
    }
    if (h->own_stream && h->st) cudaStreamDestroy(h->st);
    h->st = nullptr;
}

#ifndef PPR_RING_TAIL_DEFAULT
#define PPR_RING_TAIL_DEFAULT 16384
#endif
constexpr uint64_t kRingTailDefault = PPR_RING_TAIL_DEFAULT;  // entries
bool ring_fits(const ppr_ctx* h) { return (uint64_t)h->S * h->n <= (1ull << 27); }

ppr_status ensure_ring(ppr_ctx* h) {
    if (h->d_ring) return PPR_OK;
    const uint64_t cap = 2ull * h->S * h->n + 1024;
    if (dalloc(h, &h->d_ring, cap) != cudaSuccess) {
        set_err(h, "out of device memory for the async ring (%llu slots)", (unsigned long long)cap);
        return PPR_ENOMEM;
    }
    h->ring_cap = cap;
    cudaMemsetAsync(h->d_ring, 0xFF, sizeof(unsigned long long) * cap, h->st);
    return PPR_OK;
}

// PPR_MODE_SORTAGG: host-driven rounds (push_sortagg.cu); the statistics the
// persistent kernel would have accumulated are written into the control block
ppr_status run_push_sortagg(ppr_ctx* h, PushArgs& a, uint32_t* launches) {
    cudaError_t e = cudaMemcpyAsync(h->h_ctl, &h->d_ctl->st, sizeof(DevStats), cudaMemcpyDeviceToHost, h->st);
    if (e == cudaSuccess) e = cudaStreamSynchronize(h->st);
    if (e != cudaSuccess) return cuda_fail(h, e, "sortagg (control block)");
    if (h->h_ctl->err != KERR_OK) return PPR_OK;  // an earlier stage failed: finish() maps it
    SortAggStats out;
    out.active_pool = h->h_ctl->active_pool;
    const uint64_t before = sortagg_bytes(h->sa);
    e = sortagg_push(&h->sa, a, a.seed_v ? h->h_ctl->n_touched : 0, h->st, &out, launches);
    h->dev_bytes += sortagg_bytes(h->sa) - before;
    if (e == cudaErrorMemoryAllocation) {
        cudaGetLastError();
        set_err(h, "out of device memory for the sort-and-aggregate pairs");
        h->poisoned = true;
        return PPR_ENOMEM;
    }
    if (e != cudaSuccess) return cuda_fail(h, e, "sortagg push");
    struct {
        unsigned long long pushes, edges, max_frontier;
        unsigned iters[2];
    } w{out.pushes, out.edges, out.max_frontier, {out.iters[0], out.iters[1]}};
    static_assert(sizeof(w) == offsetof(DevStats, err), "DevStats prefix layout");
    cudaMemcpyAsync(&h->d_ctl->st, &w, sizeof w, cudaMemcpyHostToDevice, h->st);
    if (out.noconv) {
        const int k = KERR_NOCONV;
        cudaMemcpyAsync(&h->d_ctl->st.err, &k, sizeof k, cudaMemcpyHostToDevice, h->st);
    }
    e = cudaStreamSynchronize(h->st);
    if (e != cudaSuccess) return cuda_fail(h, e, "sortagg stats");
    return PPR_OK;
}

ppr_status run_push(ppr_ctx* h, PushArgs& a, uint32_t* launches) {
    if (h->mode == PPR_MODE_SORTAGG) return run_push_sortagg(h, a, launches);
    if (h->mode == PPR_MODE_ASYNC && !h->d_ring) {
        ppr_status rs = ensure_ring(h);
        if (rs != PPR_OK) return rs;
    }
    if (h->mode == PPR_MODE_OPT && h->hyb_thresh && !h->d_ring && ensure_ring(h) != PPR_OK) {
        h->hyb_thresh = 0;  // no room for the ring: rounds to the end
        h->err.clear();
    }
    a.ring = h->d_ring;
    a.ring_cap = h->ring_cap;
    a.hyb_thresh = h->mode == PPR_MODE_OPT ? h->hyb_thresh : 0;
    // every phase runs on the ring worklist from its seeds (RING_ALL default): with
    // lazy done-accounting (push.cu RING_LAZY) it beats frontier rounds on the
    // sparse LJ shape too (push 2.94 -> 2.88 ms); dense
    // graphs (>= 8 arcs per vertex) take the 3-chain walk there
    bool dense = false;
    {
        dense = (double)h->m >= 8.0 * (double)h->n;
        a.hyb_all = (a.hyb_thresh && (h->ring_all != 0)) ? 1 : 0;
    }
    // dense graphs on the ring: 3 edge chains per lane (push_u3.cu); sparse ones keep
    // the pipelined 2-chain walk; PPR_OPT_EDGE_CHAINS overrides
    const bool u3 = h->mode == PPR_MODE_OPT &&
                    (h->edge_chains == 0 ? (a.hyb_all != 0 && dense) : h->edge_chains == 3);
    // SHARED with a wave size: one launch per group of wave/32 source groups, so
    // each launch's residual rows stay L2-sized (PPR_OPT_WAVE)
    const uint32_t SG = (h->S + 31) / 32;
    const uint32_t gw = (h->mode == PPR_MODE_SHARED && h->wave) ? h->wave / 32 : SG;
    for (uint32_t g0 = 0; g0 < SG; g0 += gw) {
        a.g_lo = gw == SG ? 0u : g0;
        a.g_hi = gw == SG ? 0u : std::min(SG, g0 + gw);
        const bool chk = h->check_enq && h->mode == PPR_MODE_OPT;  // debug build of the Opt push
        cudaError_t e = chk  ? launch_push_chk(h->mode, a, h->num_sms, h->st)
                        : u3 ? launch_push_u3(h->mode, a, h->num_sms, h->st)
                             : launch_push(h->mode, a, h->num_sms, h->st);
        if (e != cudaSuccess) return cuda_fail(h, e, "push launch");
        ++*launches;
    }
    return PPR_OK;
}

// The device work of one batch after staging (captured into a CUDA graph and
// replayed, or launched directly): keys, two sorts on two streams, store,
// restore, push.
// PPR_DEBUG=1: report the first launch error of a batch with the step that raised it
inline void dbg_step(const char* what) {
    if (!dbg_on()) return;
    cudaError_t e = cudaPeekAtLastError();
    if (e != cudaSuccess) fprintf(stderr, "PPR_DEBUG: %s: %s\n", what, cudaGetErrorString(e));
}

ppr_status enqueue_batch(ppr_ctx* h, const uint32_t* is, const uint32_t* id, uint64_t n_ins,
                         const uint32_t* ds, const uint32_t* dd, uint64_t n_del, uint64_t N,
                         uint32_t* launches_out) {
    cudaStream_t st = h->st;
    uint32_t launches = 0;
    DevGraph dg = graph_of(h);
    BatchBufs& b = h->bb;
    launch_ctl_reset(h->d_ctl, st, &launches);
    dbg_step("launch_ctl_reset");
    launch_batch_keys(is, id, n_ins, ds, dd, n_del, h->undirected, h->n, b, 0, h->d_ctl, h->d_perm, st,
                      &launches);
    dbg_step("launch_batch_keys");
    // Fork: the store chain (sort by (v,u), heads, validate) stays on st; the
    // restore chain's sort by (u,v) and heads run on st2 meanwhile.
    cudaEventRecord(h->ev_fork, st);
    cudaStreamWaitEvent(h->st2, h->ev_fork, 0);
    cudaStream_t s2 = h->st2;
    int wv = radix_sort_pairs(b.kv[0], b.ov[0], b.kv[1], b.ov[1], N, h->shifts, h->npasses,
                              b.hist, st, &launches);
    dbg_step("radix_sort_pairs");
    int wu = radix_sort_pairs(b.ku[0], b.ou[0], b.ku[1], b.ou[1], N, h->shifts, h->npasses,
                              b.hist2, s2, &launches);
    dbg_step("radix_sort_pairs");
    const uint64_t* kv = b.kv[wv];
    const uint64_t* ku = b.ku[wu];
    cudaMemsetAsync(b.claim, 0, sizeof(uint32_t) * N, st);
    launch_heads(kv, b.ov[wv], N, b.rnv, b.vheads, &h->d_ctl->st.n_vheads, st, &launches);
    dbg_step("launch_heads");
    launch_heads(ku, b.ou[wu], N, b.rnu, b.uheads, &h->d_ctl->st.n_uheads, s2, &launches);
    dbg_step("launch_heads");
    // a1: graph store -- validation (deletion claims, rebuild decision) on the store branch
    launch_store_validate(dg, kv, N, b, h->vb, h->d_ctl, h->force_rebuild ? 1 : 0, st, &launches);
    dbg_step("launch_store_validate");
    // join: the in-place apply (a1) and the restore (a2) need the validation
    // (an invalid batch mutates nothing) and both sorts; one launch does both
    cudaEventRecord(h->ev_join, s2);
    cudaStreamWaitEvent(st, h->ev_join, 0);
    launch_apply_restore(dg, kv, ku, N, b, h->vb, h->d_ctl, st, &launches);
    dbg_step("launch_apply_restore");
    // sort/merge rebuild if a slab overflowed (exits at once otherwise), then
    // the reset of the v -> segment map
    StoreParams sp{h->slack, h->min_cap, h->pool_cap[0], h->pool_cap[1]};
    const cudaError_t erb = launch_store_rebuild(dg, kv, N, b, h->vb, sp, h->d_ctl, st, &launches,
                                                 /*finish=*/true);
    if (erb != cudaSuccess) return cuda_fail(h, erb, "store rebuild launch");
    launch_refresh_degrees(dg, h->vb, h->d_ctl, st, &launches);  // wide pool entries only
    *launches_out = launches;
    return PPR_OK;
}

}  // namespace

extern "C" {

const char* ppr_status_str(ppr_status s) {
    switch (s) {
        case PPR_OK: return "PPR_OK";
        case PPR_EINVAL: return "PPR_EINVAL";
        case PPR_ERANGE: return "PPR_ERANGE";
        case PPR_ENOENT: return "PPR_ENOENT";
        case PPR_ENOMEM: return "PPR_ENOMEM";
        case PPR_ECUDA: return "PPR_ECUDA";
        case PPR_EPOISONED: return "PPR_EPOISONED";
        case PPR_ENOCONV: return "PPR_ENOCONV";
    }
    return "PPR_UNKNOWN";
}

const char* ppr_last_error(const ppr_ctx* h) { return h ? h->err.c_str() : "null handle"; }

uint64_t ppr_device_bytes(const ppr_ctx* h) { return h ? h->dev_bytes : 0; }

ppr_status ppr_reset_persisting_l2(void) {
    return cudaCtxResetPersistingL2Cache() == cudaSuccess ? PPR_OK : PPR_ECUDA;
}

ppr_status ppr_create(const ppr_graph* g, const uint32_t* sources, uint32_t num_sources,
                      double alpha, double eps, const ppr_opts* opts, ppr_ctx** out,
                      ppr_batch_stats* stats) {
    if (!out) return PPR_EINVAL;
    *out = nullptr;
    if (!g || !sources || num_sources == 0 || g->n == 0) return PPR_EINVAL;
    if (!(alpha > 0.0 && alpha < 1.0) || !(eps > 0.0) || !std::isfinite(eps)) return PPR_EINVAL;
    if (g->m > 0 && (!g->src || !g->dst)) return PPR_EINVAL;
    if (g->n >= 0xFFFFFFFFu) return PPR_EINVAL;
    {
        std::vector<uint32_t> s(sources, sources + num_sources);
        for (uint32_t x : s)
            if (x >= g->n) return PPR_ERANGE;
        std::sort(s.begin(), s.end());
        if (std::adjacent_find(s.begin(), s.end()) != s.end()) return PPR_EINVAL;
    }
    for (uint64_t i = 0; i < g->m; i++)
        if (g->src[i] >= g->n || g->dst[i] >= g->n) return PPR_ERANGE;
    ppr_opts o{};
    o.device = 0;
    o.cuda_stream = nullptr;
    o.mode = PPR_MODE_OPT;
    o.slack = 0.25;
    o.min_cap = 4;
    o.relabel = -1;
    o.layout = PPR_LAYOUT_ARRAYS;
    o.l2_persist = -1;
    o.pool_degrees = -1;
    if (opts) o = *opts;
    if (o.mode < PPR_MODE_OPT || o.mode > PPR_MODE_SORTAGG || !(o.slack >= 0.0) ||
        o.min_cap == 0 || (o.layout != PPR_LAYOUT_ARRAYS && o.layout != PPR_LAYOUT_PACKED) ||
        o.pool_degrees < -1 || o.pool_degrees > 1)
        return PPR_EINVAL;

    ppr_ctx* h = new (std::nothrow) ppr_ctx();
    if (!h) return PPR_ENOMEM;
    h->device = o.device;
    h->n = g->n;
    h->S = num_sources;
    h->alpha = alpha;
    h->eps = eps;
    h->undirected = g->undirected ? 1 : 0;
    h->mode = o.mode;
    h->slack = o.slack;
    h->min_cap = o.min_cap;

    cudaError_t e = cudaSetDevice(h->device);
    if (e != cudaSuccess) {
        delete h;
        return PPR_EINVAL;
    }
    cudaDeviceGetAttribute(&h->num_sms, cudaDevAttrMultiProcessorCount, h->device);
    if (o.cuda_stream) {
        h->st = (cudaStream_t)o.cuda_stream;
    } else {
        e = cudaStreamCreateWithFlags(&h->st, cudaStreamNonBlocking);
        if (e != cudaSuccess) {
            delete h;
            return PPR_ECUDA;
        }
        h->own_stream = true;
    }
    for (auto& ev : h->ev) cudaEventCreate(&ev);
    cudaStreamCreateWithFlags(&h->st2, cudaStreamNonBlocking);
    cudaEventCreateWithFlags(&h->ev_fork, cudaEventDisableTiming);
    cudaEventCreateWithFlags(&h->ev_valid, cudaEventDisableTiming);
    cudaEventCreateWithFlags(&h->ev_join, cudaEventDisableTiming);
    h->npasses = key_shifts(ceil_log2(h->n), h->shifts);
    // hybrid tail (PPR_OPT_RING_TAIL): the ring costs
    // 16 B per (source, vertex), so it is only used up to 2^27 of them
    h->hyb_thresh = ring_fits(h) ? kRingTailDefault : 0;
    if (getenv("PPR_TRACE") && atoi(getenv("PPR_TRACE")) > 0) {
        h->trace_cap = 4096;
        dalloc(h, &h->d_trace, 4ull * h->trace_cap + 8);
    }

    const uint64_t Sn = (uint64_t)h->S * h->n;
    const uint64_t arcs_in = g->undirected ? 2 * g->m : g->m;
    // layout: one 32-byte record per vertex for single-source handles whose
    // pools fit 32-bit offsets; arrays (R, P as [S][n]) otherwise
    const double pool_bound = (1.0 + h->slack) * (double)arcs_in * 1.25 + 8.0 * h->n + 4096;
    // Default: arrays (R + d_out = 12 B/vertex stay L2-resident, see ppr_internal.cuh);
    // ppr_opts.layout = PPR_LAYOUT_PACKED selects the 32-byte records (measured slower).
    if (o.layout == PPR_LAYOUT_PACKED &&
        !(h->S == 1 && o.mode != PPR_MODE_SHARED && o.mode != PPR_MODE_SORTAGG && pool_bound < 4.0e9)) {
        destroy_all(h);
        delete h;
        return PPR_EINVAL;
    }
    const bool packed = o.layout == PPR_LAYOUT_PACKED;
    bool ok = packed ? dalloc(h, &h->d_rec, h->n) == cudaSuccess
                     : (dalloc(h, &h->d_hot, Sn + (h->n + 1) / 2 + 32) == cudaSuccess &&
                        dalloc(h, &h->d_slab, h->n) == cudaSuccess &&
                        dalloc(h, &h->d_cap, h->n) == cudaSuccess &&
                        dalloc(h, &h->d_P, Sn) == cudaSuccess);
    if (ok && !packed) {
        h->d_R = h->d_hot;
        h->d_dout = reinterpret_cast<uint32_t*>(h->d_hot + Sn);
        h->hot_bytes = sizeof(double) * Sn + sizeof(uint32_t) * h->n;
        // keep R and d_out (the random per-edge targets) resident in L2: the push
        // is bound by random fp64 atomics, ~3x faster on L2-resident lines.  Only
        // when the whole hot set fits the persisting set-aside (LJ 58 MB, Orkut
        // 37 MB of 79 MB): a window over a larger set (Twitter 480 MB) persists a
        // random hitRatio share of its lines and slows the push by 18%
        // (profiles/round1_l2win.md).  PPR_L2_PERSIST=0 / 1 forces it off / on.
        int maxp = 0, maxw = 0;
        cudaDeviceGetAttribute(&maxp, cudaDevAttrMaxPersistingL2CacheSize, h->device);
        cudaDeviceGetAttribute(&maxw, cudaDevAttrMaxAccessPolicyWindowSize, h->device);
        const bool want = o.l2_persist > 0 || (o.l2_persist < 0 && h->hot_bytes <= (uint64_t)maxp);
        // degrees cached in the pool entries iff R + d_out do not fit the persisting
        // set-aside (DRAM-resident gathers; ppr_internal.cuh PoolEnt)
        h->pool_wide = o.pool_degrees > 0 || (o.pool_degrees < 0 && h->hot_bytes > (uint64_t)maxp);
        if (h->pool_wide && prepare_refresh_degrees() != cudaSuccess) h->pool_wide = false;
        if (want && maxp > 0 && maxw > 0) {
            // the window travels with each push launch (launch attribute); the
            // caller's stream is left alone.  The device-wide set-aside is raised
            // while any handle on the device needs it (l2_acquire / l2_release).
            const size_t win = std::min<size_t>(h->hot_bytes, (size_t)maxw);
            const size_t setaside = std::min<size_t>(win, (size_t)maxp);
            h->l2_window = l2_acquire(h->device, setaside);
            h->l2_win_bytes = h->l2_window ? win : 0;
            h->l2_hit = (float)std::min(1.0, (double)setaside / (double)win);
            if (dbg_on())
                fprintf(stderr, "ppr: L2 window %zu B of %llu hot (max window %d, max set-aside %d), hit ratio %.3f\n",
                        win, (unsigned long long)h->hot_bytes, maxw, maxp, h->l2_hit);
        }
    }
    if (packed && o.pool_degrees > 0) {  // the packed records keep u32 in-list entries
        destroy_all(h);
        delete h;
        return PPR_EINVAL;
    }
    ok = ok &&
              dalloc(h, &h->d_sources, h->S) == cudaSuccess &&
              dalloc(h, &h->d_F[0], Sn) == cudaSuccess && dalloc(h, &h->d_F[1], Sn) == cudaSuccess &&
              dalloc(h, &h->d_W, Sn) == cudaSuccess &&
              dalloc(h, &h->d_bitmap, (Sn + 31) / 32) == cudaSuccess &&
              dalloc(h, &h->d_ctl, 1) == cudaSuccess && dalloc(h, &h->vb.vseg, h->n) == cudaSuccess &&
              dalloc(h, &h->vb.newcap, h->n) == cudaSuccess &&
              dalloc(h, &h->vb.newoff, h->n) == cudaSuccess &&
              dalloc(h, &h->vb.part, std::max<uint64_t>(scan_parts(h->n) + 1, 8192)) == cudaSuccess &&
              dalloc(h, &h->vb.big, h->n) == cudaSuccess &&
              dalloc(h, &h->vb.touched, h->n) == cudaSuccess &&
              cudaMallocHost(&h->h_ctl, sizeof(DevStats)) == cudaSuccess;
    uint32_t *d_src = nullptr, *d_dst = nullptr;
    ok = ok && dalloc(h, &d_src, g->m) == cudaSuccess && dalloc(h, &d_dst, g->m) == cudaSuccess;
    if (!ok) {
        dfree(h, d_src, g->m);
        dfree(h, d_dst, g->m);
        destroy_all(h);
        delete h;
        return PPR_ENOMEM;
    }
    uint32_t launches = 0;
    cudaStream_t st = h->st;
    record(h, 0);
    cudaMemsetAsync(h->d_ctl, 0, sizeof(DevCtl), st);
    if (packed) {
        cudaMemsetAsync(h->d_rec, 0, sizeof(VRec) * h->n, st);
    } else {
        cudaMemsetAsync(h->d_dout, 0, sizeof(uint32_t) * h->n, st);
        cudaMemsetAsync(h->d_slab, 0, sizeof(SlabRec) * h->n, st);
        cudaMemsetAsync(h->d_cap, 0, sizeof(uint32_t) * h->n, st);
        cudaMemsetAsync(h->d_P, 0, sizeof(double) * Sn, st);
        cudaMemsetAsync(h->d_R, 0, sizeof(double) * Sn, st);
    }
    cudaMemsetAsync(h->d_bitmap, 0, sizeof(uint32_t) * ((Sn + 31) / 32), st);
    cudaMemsetAsync(h->vb.vseg, 0xFF, sizeof(uint32_t) * h->n, st);
    cudaMemcpyAsync(h->d_sources, sources, sizeof(uint32_t) * h->S, cudaMemcpyHostToDevice, st);
    if (g->m) {
        cudaMemcpyAsync(d_src, g->src, sizeof(uint32_t) * g->m, cudaMemcpyHostToDevice, st);
        cudaMemcpyAsync(d_dst, g->dst, sizeof(uint32_t) * g->m, cudaMemcpyHostToDevice, st);
    }
    // auto: R + d_out exceed 48 MB, except for the SHARED push: clustering the hubs' S-wide
    // rows concentrates its row reductions on few L2 slices (32-source shard 37.7 ms relabelled
    // vs 25.4 ms not; 4 sources in Opt mode 12.3 vs 19.7 ms the other way round;
    // profiles/round1_spread3.md)
    const bool relabel = o.relabel > 0 ||
                         (o.relabel < 0 && o.mode != PPR_MODE_SHARED &&
                          8.0 * (double)Sn + 4.0 * h->n > 48.0 * 1024 * 1024);
    if (relabel) {  // degree-ordered internal ids
        uint64_t *k0 = nullptr, *k1 = nullptr;
        uint32_t *v0 = nullptr, *v1 = nullptr, *hist = nullptr;
        bool okr = dalloc(h, &h->d_perm, h->n) == cudaSuccess && dalloc(h, &h->d_inv, h->n) == cudaSuccess &&
                   dalloc(h, &k0, h->n) == cudaSuccess && dalloc(h, &k1, h->n) == cudaSuccess &&
                   dalloc(h, &v0, h->n) == cudaSuccess && dalloc(h, &v1, h->n) == cudaSuccess &&
                   dalloc(h, &hist, rs_hist_entries(h->n)) == cudaSuccess;
        if (okr) {
            launch_relabel(d_src, d_dst, g->m, h->undirected, h->n, h->vb.newcap, k0, v0, k1, v1, hist,
                           h->d_perm, h->d_inv, st, &launches);
            launch_map_ids(d_src, g->m, h->d_perm, st, &launches);
            launch_map_ids(d_dst, g->m, h->d_perm, st, &launches);
            launch_map_ids(h->d_sources, h->S, h->d_perm, st, &launches);
            cudaStreamSynchronize(st);
        }
        dfree(h, k0, h->n);
        dfree(h, k1, h->n);
        dfree(h, v0, h->n);
        dfree(h, v1, h->n);
        dfree(h, hist, rs_hist_entries(h->n));
        if (!okr) {
            dfree(h, d_src, g->m);
            dfree(h, d_dst, g->m);
            destroy_all(h);
            delete h;
            return PPR_ENOMEM;
        }
    }
    DevGraph dg = graph_of(h);
    launch_build_count(d_src, d_dst, g->m, h->undirected, dg, h->n, st, &launches);
    launch_caps_from_len(dg, h->vb, h->slack, h->min_cap, st, &launches);
    unsigned long long* d_total = &h->d_ctl->st.pool_top;
    exclusive_scan_u32(h->vb.newcap, h->vb.newoff, h->n, h->vb.part, d_total, st, &launches);
    unsigned long long total = 0;
    cudaMemcpyAsync(&total, d_total, sizeof total, cudaMemcpyDeviceToHost, st);
    e = cudaStreamSynchronize(st);
    if (e == cudaSuccess) e = cudaGetLastError();
    if (e != cudaSuccess) {
        dfree(h, d_src, g->m);
        dfree(h, d_dst, g->m);
        destroy_all(h);
        delete h;
        return PPR_ECUDA;
    }
    // both pools get the rebuild bound with headroom up front, so steady-state
    // batches never reallocate (ensure_alt_pool only grows them if m grows a lot)
    {
        const double need = std::ceil((1.0 + h->slack) * (double)arcs_in) +
                            (double)(h->min_cap + 1) * h->n + 1024;
        uint64_t cap = (uint64_t)(need + need / 4);
        if (cap < total + 1024) cap = total + 1024;
        if (cap > kPoolMaxEntries) cap = std::max<uint64_t>((uint64_t)need, total + 1024);
        h->pool_cap[0] = h->pool_cap[1] = cap;
    }
    if (h->pool_cap[0] > kPoolMaxEntries) {  // u32 slab offsets (SlabRec)
        dfree(h, d_src, g->m);
        dfree(h, d_dst, g->m);
        set_err(h, "the graph needs a slab pool beyond 2^32 - 1 entries");
        destroy_all(h);
        delete h;
        return PPR_ENOMEM;
    }
    if (dalloc(h, &h->d_pool[0], pool_words(h, h->pool_cap[0])) != cudaSuccess ||
        dalloc(h, &h->d_pool[1], pool_words(h, h->pool_cap[1])) != cudaSuccess) {
        dfree(h, d_src, g->m);
        dfree(h, d_dst, g->m);
        destroy_all(h);
        delete h;
        return PPR_ENOMEM;
    }
    // every slot starts POOL_EMPTY (slab slack stays empty; the degree refresh streams the pool)
    cudaMemsetAsync(h->d_pool[0], 0xFF, sizeof(PoolEnt) * pool_words(h, h->pool_cap[0]), st);
    cudaMemsetAsync(h->d_pool[1], 0xFF, sizeof(PoolEnt) * pool_words(h, h->pool_cap[1]), st);
    cudaMemcpyAsync(&h->d_ctl->st.pool_extent, &total, sizeof total, cudaMemcpyHostToDevice, st);
    dg = graph_of(h);
    launch_build_fill(d_src, d_dst, g->m, h->undirected, dg, h->vb, st, &launches);
    launch_init_state(dg, st, &launches);
    h->m = arcs_in;
    if (h->undirected) {  // self-loops count once
        // exact arc count = sum of in-degrees; computed by the scan of lengths below
    }
    record(h, 1);
    record(h, 2);
    // static PPR: push from the sources (P = 0, R = e_s)
    std::vector<unsigned long long> seeds(h->S);
    std::vector<uint32_t> isrc(h->S);  // internal ids of the sources
    cudaMemcpyAsync(isrc.data(), h->d_sources, sizeof(uint32_t) * h->S, cudaMemcpyDeviceToHost, st);
    cudaStreamSynchronize(st);
    for (uint32_t i = 0; i < h->S; i++) seeds[i] = ((unsigned long long)i << 32) | isrc[i];
    unsigned long long* d_seeds = nullptr;
    if (dalloc(h, &d_seeds, h->S) != cudaSuccess) {
        dfree(h, d_src, g->m);
        dfree(h, d_dst, g->m);
        destroy_all(h);
        delete h;
        return PPR_ENOMEM;
    }
    cudaMemcpyAsync(d_seeds, seeds.data(), sizeof(unsigned long long) * h->S,
                    cudaMemcpyHostToDevice, st);
    PushArgs a = push_args(h);
    a.seed_e = d_seeds;
    a.n_seed_e = h->S;
    ppr_status rs = run_push(h, a, &launches);
    record(h, 3);
    record(h, 4);
    if (rs == PPR_OK) rs = finish(h, "ppr_create");
    dfree(h, d_seeds, h->S);
    dfree(h, d_src, g->m);
    dfree(h, d_dst, g->m);
    if (rs != PPR_OK) {
        destroy_all(h);
        delete h;
        return rs;
    }
    if (h->undirected) {  // exact arc count (self-loops once)
        uint32_t* lens = nullptr;
        uint64_t mm = 0;
        if (dalloc(h, &lens, h->n) == cudaSuccess) {
            launch_len_to_u32(graph_of(h), lens, h->st, &launches);
            std::vector<uint32_t> hl(h->n);
            cudaMemcpyAsync(hl.data(), lens, sizeof(uint32_t) * h->n, cudaMemcpyDeviceToHost, h->st);
            cudaStreamSynchronize(h->st);
            for (uint32_t x : hl) mm += x;
            dfree(h, lens, h->n);
        }
        h->m = mm;
    }
    fill_stats(h, stats, launches, h->timing);
    if (stats) stats->touched = h->S;
    *out = h;
    return PPR_OK;
}

ppr_status ppr_destroy(ppr_ctx* h) {
    if (!h) return PPR_EINVAL;
    destroy_all(h);
    delete h;
    return PPR_OK;
}

ppr_status ppr_set_option(ppr_ctx* h, int key, int64_t value) {
    if (!h) return PPR_EINVAL;
    if (h->poisoned) return PPR_EPOISONED;
    switch (key) {
        case PPR_OPT_MODE:
            if (value < PPR_MODE_OPT || value > PPR_MODE_SORTAGG) return PPR_EINVAL;
            if ((value == PPR_MODE_SHARED || value == PPR_MODE_SORTAGG) && h->d_rec)
                return PPR_EINVAL;  // arrays layout only
            h->mode = (int)value;
            return PPR_OK;
        case PPR_OPT_PUSH: h->push_enabled = value != 0; return PPR_OK;
        case PPR_OPT_MAX_ITERS:
            if (value < 0 || value > 0xFFFFFFFFll) return PPR_EINVAL;
            h->max_iters = (uint32_t)value;
            return PPR_OK;
        case PPR_OPT_TIMING: h->timing = value != 0; return PPR_OK;
        case PPR_OPT_FORCE_REBUILD: h->force_rebuild = value != 0; return PPR_OK;
        case PPR_OPT_RING_TAIL:
            if (value < 0) return PPR_EINVAL;
            h->hyb_thresh = (value > 0 && ring_fits(h)) ? (uint64_t)value : 0;
            return PPR_OK;
        case PPR_OPT_RING_ALL:
            if (value < -1 || value > 1) return PPR_EINVAL;
            h->ring_all = (int)value;
            return PPR_OK;
        case PPR_OPT_EDGE_CHAINS:
            if (value != 0 && value != 2 && value != 3) return PPR_EINVAL;
            h->edge_chains = (int)value;
            return PPR_OK;
        case PPR_OPT_GRAPHS: h->graphs = value != 0; return PPR_OK;
        case PPR_OPT_CHECK_ENQUEUE: h->check_enq = value != 0; return PPR_OK;
        case PPR_OPT_WAVE:
            if (value < 0 || value % 32 != 0 || value > 0xFFFFFFFFll) return PPR_EINVAL;
            h->wave = (uint32_t)value;
            return PPR_OK;
        default: return PPR_EINVAL;
    }
}

ppr_status ppr_apply_batch(ppr_ctx* h, const uint32_t* ins_src, const uint32_t* ins_dst,
                           uint64_t n_ins, const uint32_t* del_src, const uint32_t* del_dst,
                           uint64_t n_del, int mem, ppr_batch_stats* stats) {
    if (!h) return PPR_EINVAL;
    if (h->poisoned) return PPR_EPOISONED;
    if (mem != PPR_MEM_HOST && mem != PPR_MEM_DEVICE) return PPR_EINVAL;
    if ((n_ins && (!ins_src || !ins_dst)) || (n_del && (!del_src || !del_dst))) return PPR_EINVAL;
    if (stats) memset(stats, 0, sizeof *stats);
    if (n_ins + n_del == 0) {
        if (stats) stats->num_arcs = h->m;
        return PPR_OK;
    }
    const uint64_t nupd = std::max(n_ins, n_del);
    const uint64_t N = (n_ins + n_del) * (h->undirected ? 2 : 1);
    ppr_status rs = ensure_batch(h, nupd, N);
    if (rs != PPR_OK) return rs;
    rs = ensure_alt_pool(h, (h->undirected ? 2 : 1) * n_ins);
    if (rs != PPR_OK) return rs;

    cudaStream_t st = h->st;
    uint32_t launches = 0;
    record(h, 0);
    // a0: stage the batch in the handle's buffers (H2D, or D2D when the work is a replayed graph)
    const bool use_graph = h->graphs && !h->d_trace;
    const uint32_t *is = ins_src, *id = ins_dst, *ds = del_src, *dd = del_dst;
    if (mem == PPR_MEM_HOST || use_graph) {
        const cudaMemcpyKind kind = mem == PPR_MEM_HOST ? cudaMemcpyHostToDevice : cudaMemcpyDeviceToDevice;
        uint32_t* pk = h->d_in[0];  // [ins_src | ins_dst | del_src | del_dst], packed by the counts
        uint32_t *pis = pk, *pid = pk + n_ins, *pds = pk + 2 * n_ins, *pdd = pk + 2 * n_ins + n_del;
        const bool packed = n_ins && n_del && ins_dst == ins_src + n_ins &&
                            del_src == ins_dst + n_ins && del_dst == del_src + n_del;
        if (packed) {  // the caller's arrays are one block laid out the same way: one copy
            cudaMemcpyAsync(pk, ins_src, 4 * (2 * n_ins + 2 * n_del), kind, st);
        } else {
            if (n_ins) {
                cudaMemcpyAsync(pis, ins_src, 4 * n_ins, kind, st);
                cudaMemcpyAsync(pid, ins_dst, 4 * n_ins, kind, st);
            }
            if (n_del) {
                cudaMemcpyAsync(pds, del_src, 4 * n_del, kind, st);
                cudaMemcpyAsync(pdd, del_dst, 4 * n_del, kind, st);
            }
        }
        is = pis;
        id = pid;
        ds = pds;
        dd = pdd;
    }
    if (h->mode == PPR_MODE_ASYNC && h->push_enabled) {
        rs = ensure_ring(h);
        if (rs != PPR_OK) return rs;
    }
    if (use_graph) {  // one graph per batch shape, replayed
        const GraphKey key{n_ins, n_del, h->push_enabled, h->mode, h->max_iters, h->timing,
                           h->force_rebuild, h->buf_epoch, h->pool_cap[0], h->pool_cap[1],
                           (const void*)h->d_pool[0], (const void*)h->d_pool[1]};
        if (!h->gexec || !(key == h->gkey)) {
            if (h->gexec) cudaGraphExecDestroy(h->gexec), h->gexec = nullptr;
            cudaGraph_t graph = nullptr;
            uint32_t glaunches = 0;
            cudaError_t e = cudaStreamBeginCapture(st, cudaStreamCaptureModeThreadLocal);
            ppr_status ers = PPR_OK;
            if (e == cudaSuccess) ers = enqueue_batch(h, is, id, n_ins, ds, dd, n_del, N, &glaunches);
            cudaError_t e2 = cudaStreamEndCapture(st, &graph);
            if (e == cudaSuccess) e = e2;
            if (e == cudaSuccess && ers == PPR_OK) e = cudaGraphInstantiate(&h->gexec, graph, 0);
            if (graph) cudaGraphDestroy(graph);
            if (e != cudaSuccess || ers != PPR_OK) {  // capture unsupported: run the stream path
                cudaGetLastError();
                h->gexec = nullptr;
                h->graphs = false;
                set_err(h, "graph capture failed (%s); using stream launches", cudaGetErrorString(e));
                h->poisoned = false;
            } else {
                h->gkey = key;
                h->glaunches = glaunches;
            }
        }
        if (h->gexec) {
            dbg_step("before graph launch");
            cudaError_t e = cudaGraphLaunch(h->gexec, st);
            if (e != cudaSuccess) return cuda_fail(h, e, "cudaGraphLaunch");
            launches = h->glaunches;
        } else {
            rs = enqueue_batch(h, is, id, n_ins, ds, dd, n_del, N, &launches);
            if (rs != PPR_OK) return rs;
        }
    } else {
        rs = enqueue_batch(h, is, id, n_ins, ds, dd, n_del, N, &launches);
        if (rs != PPR_OK) return rs;
    }
    // store and restore (two streams, joined) are timed together; the push is
    // one cooperative launch between its own events on the handle's stream
    record(h, 1);
    record(h, 2);
    if (h->push_enabled) {
        PushArgs a = push_args(h);
        a.seed_v = h->vb.touched;
        a.n_seed_v_dev = &h->d_ctl->st.n_touched;
        rs = run_push(h, a, &launches);
        dbg_step("push");
        if (rs != PPR_OK) return rs;
    }
    record(h, 3);
    record(h, 4);
    rs = finish(h, "ppr_apply_batch");
    dump_trace(h, "apply_batch");
    if (rs == PPR_OK) {
        h->m = (uint64_t)((long long)h->m + h->h_ctl->arc_delta);
        h->active = h->h_ctl->active_pool;
    }
    if (rs == PPR_OK || rs == PPR_ERANGE || rs == PPR_ENOENT)
        fill_stats(h, stats, launches, h->timing && rs == PPR_OK,
                   mem == PPR_MEM_HOST ? 8 * (n_ins + n_del) : 0);
    return rs;
}

ppr_status ppr_push(ppr_ctx* h, ppr_batch_stats* stats) {
    if (!h) return PPR_EINVAL;
    if (h->poisoned) return PPR_EPOISONED;
    uint32_t launches = 0;
    record(h, 0);
    record(h, 1);
    record(h, 2);
    launch_ctl_reset(h->d_ctl, h->st, &launches);
    PushArgs a = push_args(h);
    a.seed_all = 1;
    ppr_status rs = run_push(h, a, &launches);
    if (rs != PPR_OK) return rs;
    record(h, 3);
    record(h, 4);
    rs = finish(h, "ppr_push");
    if (rs == PPR_OK) fill_stats(h, stats, launches, h->timing);
    return rs;
}

ppr_status ppr_reset(ppr_ctx* h) {
    if (!h) return PPR_EINVAL;
    if (h->poisoned) return PPR_EPOISONED;
    uint32_t launches = 0;
    const uint64_t Sn = (uint64_t)h->S * h->n;
    if (h->d_rec) {
        launch_gather_rec(graph_of(h), nullptr, nullptr, nullptr, 1, nullptr, h->st, &launches);
    } else {
        cudaMemsetAsync(h->d_P, 0, sizeof(double) * Sn, h->st);
        cudaMemsetAsync(h->d_R, 0, sizeof(double) * Sn, h->st);
    }
    launch_init_state(graph_of(h), h->st, &launches);
    cudaError_t e = cudaStreamSynchronize(h->st);
    if (e == cudaSuccess) e = cudaGetLastError();
    if (e != cudaSuccess) return cuda_fail(h, e, "ppr_reset");
    return PPR_OK;
}

ppr_status ppr_query(ppr_ctx* h, uint32_t source_idx, double* P_out, double* R_out, int mem) {
    if (!h || (!P_out && !R_out)) return PPR_EINVAL;
    if (h->poisoned) return PPR_EPOISONED;
    if (source_idx >= h->S) return PPR_ERANGE;
    if (mem != PPR_MEM_HOST && mem != PPR_MEM_DEVICE) return PPR_EINVAL;
    const cudaMemcpyKind k = mem == PPR_MEM_HOST ? cudaMemcpyDeviceToHost : cudaMemcpyDeviceToDevice;
    const size_t off = (size_t)source_idx * h->n;
    cudaError_t e = cudaSuccess;
    if (h->d_rec) {  // gather out of the vertex records (through a device buffer for host output)
        double* tmp = nullptr;
        const bool host = mem == PPR_MEM_HOST;
        if (host && dalloc(h, &tmp, 2ull * h->n) != cudaSuccess) return PPR_ENOMEM;
        uint32_t launches = 0;
        double* dP = host ? (P_out ? tmp : nullptr) : P_out;
        double* dR = host ? (R_out ? tmp + h->n : nullptr) : R_out;
        launch_gather_rec(graph_of(h), dP, dR, nullptr, 0, h->d_perm, h->st, &launches);
        if (host && P_out) e = cudaMemcpyAsync(P_out, tmp, sizeof(double) * h->n, k, h->st);
        if (host && e == cudaSuccess && R_out)
            e = cudaMemcpyAsync(R_out, tmp + h->n, sizeof(double) * h->n, k, h->st);
        if (e == cudaSuccess) e = cudaStreamSynchronize(h->st);
        dfree(h, tmp, 2ull * h->n);
        if (e != cudaSuccess) return cuda_fail(h, e, "ppr_query");
        return PPR_OK;
    }
    if (h->S > 1 || h->d_perm) {  // vertex-major [n][S] / internal ids: gather through a device buffer
        double* tmp = nullptr;
        const bool host = mem == PPR_MEM_HOST;
        if (host && dalloc(h, &tmp, h->n) != cudaSuccess) return PPR_ENOMEM;
        uint32_t launches = 0;
        const double* srcs[2] = {h->d_P, h->d_R};
        double* outs[2] = {P_out, R_out};
        for (int q = 0; q < 2 && e == cudaSuccess; q++) {
            if (!outs[q]) continue;
            launch_gather_col(srcs[q], h->S, source_idx, h->n, host ? tmp : outs[q], h->d_perm, h->st,
                              &launches);
            if (host) e = cudaMemcpyAsync(outs[q], tmp, sizeof(double) * h->n, k, h->st);
            if (e == cudaSuccess) e = cudaStreamSynchronize(h->st);
        }
        dfree(h, tmp, h->n);
        if (e != cudaSuccess) return cuda_fail(h, e, "ppr_query");
        return PPR_OK;
    }
    if (P_out) e = cudaMemcpyAsync(P_out, h->d_P + off, sizeof(double) * h->n, k, h->st);
    if (e == cudaSuccess && R_out) e = cudaMemcpyAsync(R_out, h->d_R + off, sizeof(double) * h->n, k, h->st);
    if (e == cudaSuccess) e = cudaStreamSynchronize(h->st);
    if (e != cudaSuccess) return cuda_fail(h, e, "ppr_query");
    return PPR_OK;
}

ppr_status ppr_export_dout(ppr_ctx* h, uint32_t* dout_out) {
    if (!h || !dout_out) return PPR_EINVAL;
    if (h->poisoned) return PPR_EPOISONED;
    cudaError_t e = cudaSuccess;
    if (h->d_rec) {
        uint32_t* tmp = nullptr;
        uint32_t launches = 0;
        if (dalloc(h, &tmp, h->n) != cudaSuccess) return PPR_ENOMEM;
        launch_gather_rec(graph_of(h), nullptr, nullptr, tmp, 0, h->d_perm, h->st, &launches);
        e = cudaMemcpyAsync(dout_out, tmp, sizeof(uint32_t) * h->n, cudaMemcpyDeviceToHost, h->st);
        if (e == cudaSuccess) e = cudaStreamSynchronize(h->st);
        dfree(h, tmp, h->n);
        if (e != cudaSuccess) return cuda_fail(h, e, "ppr_export_dout");
        return PPR_OK;
    }
    if (h->d_perm) {
        uint32_t* tmp = nullptr;
        uint32_t launches = 0;
        if (dalloc(h, &tmp, h->n) != cudaSuccess) return PPR_ENOMEM;
        launch_gather_u32(h->d_dout, h->d_perm, h->n, tmp, h->st, &launches);
        e = cudaMemcpyAsync(dout_out, tmp, sizeof(uint32_t) * h->n, cudaMemcpyDeviceToHost, h->st);
        if (e == cudaSuccess) e = cudaStreamSynchronize(h->st);
        dfree(h, tmp, h->n);
        if (e != cudaSuccess) return cuda_fail(h, e, "ppr_export_dout");
        return PPR_OK;
    }
    e = cudaMemcpyAsync(dout_out, h->d_dout, sizeof(uint32_t) * h->n,
                                    cudaMemcpyDeviceToHost, h->st);
    if (e == cudaSuccess) e = cudaStreamSynchronize(h->st);
    if (e != cudaSuccess) return cuda_fail(h, e, "ppr_export_dout");
    return PPR_OK;
}

ppr_status ppr_export_edges(ppr_ctx* h, uint32_t* src_out, uint32_t* dst_out, uint64_t cap,
                            uint64_t* m_out) {
    if (!h || !m_out) return PPR_EINVAL;
    if (h->poisoned) return PPR_EPOISONED;
    *m_out = h->m;
    if (cap < h->m || (h->m && (!src_out || !dst_out))) return PPR_EINVAL;
    if (h->m == 0) return PPR_OK;
    uint32_t launches = 0;
    uint64_t* k[2] = {nullptr, nullptr};
    uint32_t* v[2] = {nullptr, nullptr};
    uint32_t* hist = nullptr;
    uint32_t* lens = nullptr;
    unsigned long long* off = nullptr;
    const uint64_t m = h->m;
    bool ok = dalloc(h, &k[0], m) == cudaSuccess && dalloc(h, &k[1], m) == cudaSuccess &&
              dalloc(h, &v[0], m) == cudaSuccess && dalloc(h, &v[1], m) == cudaSuccess &&
              dalloc(h, &hist, rs_hist_entries(m)) == cudaSuccess &&
              dalloc(h, &lens, h->n) == cudaSuccess && dalloc(h, &off, h->n) == cudaSuccess;
    ppr_status rs = PPR_OK;
    if (!ok) {
        rs = PPR_ENOMEM;
    } else {
        cudaStream_t st = h->st;
        DevGraph dg = graph_of(h);
        launch_len_to_u32(dg, lens, st, &launches);
        exclusive_scan_u32(lens, off, h->n, h->vb.part, &h->d_ctl->st.pool_top, st, &launches);
        launch_export(dg, (int)h->active, off, k[0], h->d_inv, st, &launches);
        cudaMemsetAsync(v[0], 0, sizeof(uint32_t) * m, st);
        int w = radix_sort_pairs(k[0], v[0], k[1], v[1], m, h->shifts, h->npasses, hist, st,
                                 &launches);
        std::vector<uint64_t> keys(m);
        cudaMemcpyAsync(keys.data(), k[w], sizeof(uint64_t) * m, cudaMemcpyDeviceToHost, st);
        cudaError_t e = cudaStreamSynchronize(st);
        if (e == cudaSuccess) e = cudaGetLastError();
        if (e != cudaSuccess) {
            rs = cuda_fail(h, e, "ppr_export_edges");
        } else {
            for (uint64_t i = 0; i < m; i++) {
                dst_out[i] = (uint32_t)(keys[i] >> 32);
                src_out[i] = (uint32_t)keys[i];
            }
        }
    }
    dfree(h, k[0], m);
    dfree(h, k[1], m);
    dfree(h, v[0], m);
    dfree(h, v[1], m);
    dfree(h, hist, rs_hist_entries(m));
    dfree(h, lens, h->n);
    dfree(h, off, h->n);
    return rs;
}

}  // extern "C"
