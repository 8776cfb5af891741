/*
 * ppr.h -- C ABI of libppr.so: batch-parallel maintenance of Personalized
 * PageRank (PPR) on a dynamic graph, on one NVIDIA B200 (sm_100a).
 *
 * The operation is the paper's problem statement (Guo, Li, Sha, Tan,
 * "Parallel Personalized PageRank on Dynamic Graphs", PVLDB 11(1) 2017;
 * cites "P:L" are lines of its text, PAPER.md):
 *   - an initial graph G0 and a sequence of update sets E_t of arcs
 *     (u, v, op), op in {insert, delete}
 *   - for each unit-vector source s, maintain an estimate P_s and a residual
 *     R_s satisfying the invariant (Eq. 2)
 *        P(v) + a R(v) = (1-a)/d(v) * sum_{x in N_out(v)} P(x) + a 1[v=s]
 *     and |R(v)| <= eps for all v, so |pi_s(v) - P(v)| <= eps.
 *   - per batch: restore the invariant for all k updates (Alg 1, P:185-196,
 *     in the batch closed form of Lemma 3's proof), then one
 *     two-phase (POS, NEG) parallel local push (Alg 3 P:454-480 / Alg 4
 *     P:1132-1157).
 *   - pi_s is read as the reverse-PPR fixed point a (I-(1-a) D^-1 A)^-1 e_s
 *     (reading R1; Eq. 1's W is Lemma 1's W^T = D^-1 A).
 *
 * Conventions for every call ("Boundary"):
 *   - Every call returns ppr_status; PPR_OK == 0.
 *   - Ownership: the caller owns every input array; it is consumed before
 *     the call returns and no pointer is retained.  The library owns all
 *     device state.  Output buffers are caller-allocated.
 *   - Memory kinds: `mem` = PPR_MEM_HOST for host pointers (pageable or
 *     pinned), PPR_MEM_DEVICE for device pointers on the handle's device,
 *     valid in stream order on the handle's stream.
 *   - Synchrony: calls return after the result is complete (the handle's
 *     stream is synchronised).
 *   - Validation happens before any mutation.  On PPR_EINVAL, PPR_ERANGE or
 *     PPR_ENOENT the state is unchanged.  A CUDA failure returns PPR_ECUDA
 *     and poisons the handle: every later call returns PPR_EPOISONED.
 *   - Semantics: arcs form a multiset (a duplicate insertion raises the
 *     multiplicity, Eq. 2 counts it); self-loops are allowed; the vertex set
 *     is fixed to [0, n) (a vertex with no arcs is "absent");
 *     within a batch insertions apply before deletions; an empty batch is a
 *     no-op.  Vertex ids are uint32_t < n.
 *   - Threading: a handle is bound to one device and is not thread-safe.
 */
#ifndef PPR_H
#define PPR_H

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef struct ppr_ctx ppr_ctx; /* opaque; owned by the library */

typedef enum {
    PPR_OK = 0,
    PPR_EINVAL = -1,    /* bad alpha / eps / n / sources / flags / option */
    PPR_ERANGE = -2,    /* a vertex id >= n */
    PPR_ENOENT = -3,    /* deletion of an arc absent after this batch's insertions */
    PPR_ENOMEM = -4,    /* device or host allocation failed (state unchanged) */
    PPR_ECUDA = -5,     /* CUDA error: the handle is poisoned */
    PPR_EPOISONED = -6, /* an earlier call poisoned the handle */
    PPR_ENOCONV = -7    /* push exceeded the iteration cap (handle poisoned) */
} ppr_status;

enum { PPR_MEM_HOST = 0, PPR_MEM_DEVICE = 1 };

/* Parallel push variants of Table 3. */
enum {
    PPR_MODE_OPT = 0,       /* eager propagation + local duplicate detection (Alg 4);
                               self-update fused with propagation (DESIGN.md K-PUSH) */
    PPR_MODE_EAGER = 1,     /* eager propagation, UniqueEnqueue via bitmap */
    PPR_MODE_DUPDETECT = 2, /* Alg 3 sessions + local duplicate detection */
    PPR_MODE_VANILLA = 3,   /* Alg 3 as printed: snapshot, barrier, propagate, UniqueEnqueue */
    PPR_MODE_ASYNC = 4,     /* Alg 4's operations without rounds: asynchronous ring worklist
                               (any push order is valid by Lemma 1; DESIGN.md K-ASYNC);
                               iters_pos/iters_neg are reported as 0 */
    PPR_MODE_EAGER_SCAN = 5, /* eager propagation; residual updates are fire-and-forget
                               reductions that mark touched vertices in a bitmap, and each
                               round's frontier comes from a warp-ballot/scan compaction of
                               that bitmap (DESIGN.md K-SCAN) */
    PPR_MODE_SHARED = 6,    /* multi-source: shared-adjacency push.  A frontier entry is a
                               (vertex, group of 32 sources); one warp reads N_in(u) once and
                               every lane pushes its own source's residual onto the shared
                               [n][S] row (coalesced reductions); bitmap dedup + compaction as
                               in EAGER_SCAN (DESIGN.md K-SHARED).  Any S >= 1; arrays layout */
    PPR_MODE_SORTAGG = 7    /* Alg 3 rounds with sort-and-aggregate propagation instead of
                               atomics (the alternative of P:433-442): pairs (v, (1-a)w_u/d(v))
                               are radix-sorted by v and each run is added to R(v) in
                               ascending-u order.  No atomics: bit-reproducible, and equal bit
                               for bit to a sequential Alg 3 round loop over the sorted frontier
                               when ids are not relabelled (ppr_opts.relabel = 0).  Host-driven
                               rounds; arrays layout (DESIGN.md K-SORTAGG) */
};

/* Graph for ppr_create: m arcs src[i] -> dst[i] on [0, n) (host pointers).
 * undirected = 1 expands each {src,dst} into two arcs (one for a self-loop),
 * P:868-870. */
typedef struct {
    uint32_t n;
    uint64_t m;
    const uint32_t *src;
    const uint32_t *dst;
    int undirected;
} ppr_graph;

/* Options for ppr_create; pass NULL for defaults. */
typedef struct {
    int device;          /* CUDA device ordinal (default 0) */
    void *cuda_stream;   /* cudaStream_t to run on; NULL: the library creates one */
    int mode;            /* PPR_MODE_* (default PPR_MODE_OPT) */
    double slack;        /* slab slack fraction (default 0.25) */
    uint32_t min_cap;    /* minimum slab capacity (default 4) */
    int relabel;         /* 1: vertices are renumbered internally by G0 out-degree (descending)
                            so the most-pushed-to residuals share cache lines; 0: identity;
                            -1 (default): relabel iff mode != PPR_MODE_SHARED and the residual
                            + out-degree arrays (8*S*n + 4*n bytes) exceed 48 MB, i.e. do not sit
                            in L2 anyway (measured: LJ-shaped 58 MB -12%, Twitter-shaped -60% per
                            batch, 4 sources in Opt mode -38%; Orkut-shaped 37 MB +11%, hot lines
                            concentrate on few L2 slices; SHARED 32-source shard +48%, the same
                            effect on the hubs' S-wide rows).
                            Every id at the boundary stays external. */
    int layout;          /* PPR_LAYOUT_ARRAYS (default): R / d_out / slab / P as separate arrays;
                            PPR_LAYOUT_PACKED: one 32-byte {R, P, off, len, d_out, cap} record per
                            vertex (single source, not SHARED / SORTAGG, pool < 2^32 entries;
                            otherwise PPR_EINVAL).  Measured slower on every shape. */
    int l2_persist;      /* persisting L2 access-policy window over R and d_out, passed with each
                            push launch: -1 (default) iff they fit the device's persisting
                            set-aside, 0 never, 1 always */
    int pool_degrees;    /* in-list (slab pool) entries: 1 = (d_out(u), u) pairs, so the push
                            reads each divisor d_out(u) with the entry (one dependent random access
                            per pushed edge fewer), kept exact by a streaming refresh after every
                            batch's restore; 0 = u32 ids and a d_out gather per pushed edge;
                            -1 (default): pairs iff R + d_out exceed the persisting L2 set-aside
                            (DRAM-resident: Twitter shape push -28%; L2-resident: LJ shape +6%).
                            1 with layout = PPR_LAYOUT_PACKED: PPR_EINVAL. */
} ppr_opts;

enum { PPR_LAYOUT_ARRAYS = 0, PPR_LAYOUT_PACKED = 1 };

/* Per-call statistics (filled by ppr_create, ppr_apply_batch, ppr_push). */
typedef struct {
    uint32_t iters_pos, iters_neg;  /* frontier rounds per phase */
    uint64_t pushes;                /* frontier vertices pushed (self-updates) */
    uint64_t pushed_edges;          /* neighbour propagations (atomic adds) */
    uint64_t max_frontier;          /* largest frontier seen */
    uint64_t touched;               /* distinct (u, source) restored this batch */
    uint64_t num_arcs;              /* arcs in the store after the call */
    uint32_t rebuilt;               /* 1 if the slab store was rebuilt */
    uint32_t kernel_launches;       /* kernels launched by this call */
    uint64_t h2d_bytes, d2h_bytes;  /* host<->device bytes this call copied */
    float ms_total;                 /* CUDA-event time of the call on the stream */
    float ms_store;                 /* CUDA events: batch staging through the store and restore
                                       branches (a0-a2; the restore branch runs concurrently) */
    float ms_restore;               /* device clock (%globaltimer): the Lemma 3 restore kernel
                                       alone (a2), first CTA start to last CTA end; inside ms_store */
    float ms_push;                  /* CUDA events around the push launch (a3-a6, both phases) */
    uint64_t walk_edges;            /* in-arc reads of the push: PPR_MODE_SHARED walks N_in(u) once
                                       per (source group, u), so walk_edges <= pushed_edges;
                                       other modes: = pushed_edges */
    float ms_push_pos, ms_push_neg; /* device clock inside the push launch: seed + rounds of the
                                       POS phase (a3-a4) and of the NEG phase (a5); 0 for
                                       PPR_MODE_SORTAGG (host-driven rounds) */
    uint64_t entries;               /* frontier entries processed: PPR_MODE_SHARED counts (vertex,
                                       32-source group) rows with a pushing lane; other modes:
                                       = pushes */
    uint64_t dup_enqueues;          /* with PPR_OPT_CHECK_ENQUEUE: enqueues of a (source, vertex)
                                       already in the frontier / worklist (0 otherwise) */
} ppr_batch_stats;

/* Creates a handle: builds the slab store for g, sets P_s = 0 and R_s = e_s
 * for every source (Eq. 2 holds trivially, Fig. 3 a(1)) and runs
 * the two-phase push to convergence (static PPR).
 * sources: num_sources distinct vertex ids < n (host pointer).
 * 0 < alpha < 1, eps > 0 finite.  stats may be NULL.
 * PPR_ENOMEM also when a slab pool would exceed 2^32 - 1 entries (slab
 * offsets are u32; the pool holds the arcs with slack, ~1.25 m + 5 n). */
ppr_status ppr_create(const ppr_graph *g, const uint32_t *sources, uint32_t num_sources,
                      double alpha, double eps, const ppr_opts *opts, ppr_ctx **out,
                      ppr_batch_stats *stats);

/* Applies one batch: n_ins insertions ins_src[i] -> ins_dst[i] and n_del
 * deletions del_src[i] -> del_dst[i] (arcs; undirected handles expand them),
 * restores the invariant at every touched vertex for every source, then runs
 * the two-phase push until |R| <= eps everywhere.  mem: PPR_MEM_HOST or
 * PPR_MEM_DEVICE for the four input arrays.  stats may be NULL.
 * PPR_ENOMEM if the graph grows past what the rebuild pool can hold (see
 * ppr_create); the handle's state is unchanged then. */
ppr_status ppr_apply_batch(ppr_ctx *h, const uint32_t *ins_src, const uint32_t *ins_dst,
                           uint64_t n_ins, const uint32_t *del_src, const uint32_t *del_dst,
                           uint64_t n_del, int mem, ppr_batch_stats *stats);

/* Runs the two-phase push from a full scan of V (Alg 3 lines 1 and 4).
 * Used after ppr_apply_batch with PPR_OPT_PUSH = 0.  stats may be NULL. */
ppr_status ppr_push(ppr_ctx *h, ppr_batch_stats *stats);

/* Resets every source to P_s = 0, R_s = e_s, which satisfies Eq. 2 for any
 * graph (Fig. 3 a(1)); the next ppr_push recomputes static PPR. */
ppr_status ppr_reset(ppr_ctx *h);

/* Copies P_s (and R_s if R_out != NULL) of source number source_idx (its
 * position in ppr_create's `sources`) into caller buffers of n doubles. */
ppr_status ppr_query(ppr_ctx *h, uint32_t source_idx, double *P_out, double *R_out, int mem);

/* Writes the arc multiset, sorted by (dst, src), into host buffers of `cap`
 * entries; *m_out = number of arcs (PPR_EINVAL if cap is too small, with
 * *m_out set). */
ppr_status ppr_export_edges(ppr_ctx *h, uint32_t *src_out, uint32_t *dst_out, uint64_t cap,
                            uint64_t *m_out);

/* Copies d_out (n uint32_t) into a host buffer. */
ppr_status ppr_export_dout(ppr_ctx *h, uint32_t *dout_out);

/* Runtime options. */
enum {
    PPR_OPT_MODE = 1,      /* PPR_MODE_* for later pushes */
    PPR_OPT_PUSH = 2,      /* 0: ppr_apply_batch stops after restore (tests); default 1 */
    PPR_OPT_MAX_ITERS = 3, /* stop each phase after this many rounds (0 = run to eps) */
    PPR_OPT_TIMING = 4,    /* 1: record per-phase CUDA events (default 1) */
    PPR_OPT_FORCE_REBUILD = 5, /* 1: every batch takes the sort/merge rebuild path */
    PPR_OPT_RING_TAIL = 6,   /* Opt: a phase whose frontier has shrunk (past its peak) to at most
                                this many entries finishes on the asynchronous ring worklist
                                (default 16384; 0: rounds to the end) */
    PPR_OPT_RING_ALL = 7,    /* Opt: whole phases on the ring from their seeds: -1 or 1 (default
                                -1: always), 0 never -- frontier rounds, the ring only for the
                                tail (needs RING_TAIL > 0) */
    PPR_OPT_EDGE_CHAINS = 8, /* Opt: independent edge chains per lane, 2 or 3 (0 = default: 3
                                when whole phases run on the ring and the graph has >= 8 arcs
                                per vertex, else 2) */
    PPR_OPT_GRAPHS = 9,      /* 1 (default): replay each batch shape's store/restore pipeline as
                                one CUDA graph; 0: launch the kernels one by one */
    PPR_OPT_CHECK_ENQUEUE = 11, /* PPR_MODE_OPT, debug: 1 = count enqueues of a (source, vertex)
                                   that is already queued (SURVEY 8(a) exactly-once enqueue of the
                                   fused self-update; ppr_batch_stats.dup_enqueues must stay 0).
                                   Uses the UniqueEnqueue bitmap as an in-queue flag; slower */
    PPR_OPT_WAVE = 10        /* PPR_MODE_SHARED: push the sources in waves of this many (a
                                multiple of 32; 0 = default: all in one launch), one push launch
                                per wave after the shared store/restore, so each launch's residual
                                rows stay L2-sized */
};
ppr_status ppr_set_option(ppr_ctx *h, int key, int64_t value);

/* Measurement utility: returns every persisting L2 line of the calling
 * thread's current device to normal (evictable) status, so that a following
 * L2 flush really empties the cache.  Handles keep their residual and
 * out-degree arrays in a persisting L2 window;
 * bench.py calls this before its between-step flush. */
ppr_status ppr_reset_persisting_l2(void);

/* Device memory held by the handle, in bytes. */
uint64_t ppr_device_bytes(const ppr_ctx *h);

ppr_status ppr_destroy(ppr_ctx *h);
const char *ppr_status_str(ppr_status s);
const char *ppr_last_error(const ppr_ctx *h);

#ifdef __cplusplus
}
#endif
#endif /* PPR_H */
