/*
 * oracle/ppr_oracle.h -- TEST INFRASTRUCTURE ONLY.
 *
 * Plain, slow, single-threaded fp64 CPU oracle for dynamic Personalized
 * PageRank maintenance (Guo, Li, Sha, Tan, PVLDB 11(1) 2017; PAPER.md).
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline /
 * --impl reference legs may load this library.  It shares no code, header,
 * constant or helper with the CUDA product path in
 * paper_journals_pvldb_guolst17_b200/csrc/, and it includes nothing from
 * include/.
 *
 * Citations: "P:L" = /root/reference/PAPER.md line L (read once, at design
 * time; nothing here reads it at run time).
 *
 *   Alg 1 RestoreInvariant ........ P:185-196 (decoded: minus signs were lost
 *                                   in extraction, readings R2,R3)
 *   Alg 2 SequentialLocalPush ..... P:293-304 (reading R6: snapshot r, zero R(u),
 *                                   then propagate, as Alg 3 P:469-471 does)
 *   Alg 3 ParallelLocalPush ....... P:454-480 (emulated as synchronous rounds)
 *   CPU-Seq / CPU-Base ............ P:1237-1245
 *   Eq. 2 invariant ............... P:305-312 (checked in oracle/exact.py)
 */
#ifndef PPR_ORACLE_H
#define PPR_ORACLE_H
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef struct oracle oracle;

/* return codes (the oracle's own; values mirror the documented ABI contract
 * in DESIGN.md so that tests can compare behaviour, but nothing is shared) */
#define ORC_OK 0
#define ORC_EINVAL (-1)
#define ORC_ERANGE (-2)
#define ORC_ENOENT (-3)
#define ORC_ENOMEM (-4)

/* push modes */
#define ORC_SEQ 0    /* CPU-Seq: Alg 1 per update, then Alg 2 FIFO */
#define ORC_BASE 1   /* CPU-Base: Alg 1 + Alg 2 after every single update */
#define ORC_JACOBI 2 /* Alg 3 emulation: synchronous rounds, ascending order */

/* Creates the state for graph (src[i] -> dst[i]), i < m, on vertices [0,n),
 * with S distinct sources.  P = 0, R = e_s for every source, which satisfies
 * Eq. 2 for any graph (Fig. 3 a(1)).  No push is run here: call
 * oracle_push to run the static computation. */
int oracle_create(uint32_t n, uint64_t m, const uint32_t *src, const uint32_t *dst,
                  const uint32_t *sources, uint32_t S, double alpha, double eps,
                  oracle **out);
void oracle_destroy(oracle *h);

/* Runs the two-phase push (POS then NEG) for every source.  The initial
 * frontier of each phase is every vertex meeting pushCond, scanned in
 * ascending id order (Alg 2 line 1 / Alg 3 line 1 literally).
 * max_steps < 0: run to convergence.  Otherwise stop after max_steps pushes
 * (ORC_SEQ) or rounds (ORC_JACOBI), for reproducing the traces of Fig. 3. */
int oracle_push(oracle *h, int mode, int64_t max_steps);

/* Applies one batch: insertions (in order) then deletions (in order), each
 * followed by Alg 1 with the post-update out-degree.  Validation happens
 * before any mutation (ids < n; each deletion matches an arc present after
 * this batch's insertions, multiset semantics); on failure nothing changes.
 * mode ORC_SEQ / ORC_JACOBI: one push (oracle_push) after all k restores
 * (batch processing) unless do_push == 0.
 * mode ORC_BASE: a push after every single update, seeded by {u}. */
int oracle_apply(oracle *h, const uint32_t *ins_src, const uint32_t *ins_dst, uint64_t n_ins,
                 const uint32_t *del_src, const uint32_t *del_dst, uint64_t n_del,
                 int mode, int do_push);

/* state access */
int oracle_set_state(oracle *h, uint32_t sidx, const double *P, const double *R);
int oracle_query(const oracle *h, uint32_t sidx, double *P, double *R);
uint64_t oracle_num_arcs(const oracle *h);
/* arcs sorted by (dst, src) ascending; returns number written (== num_arcs) */
uint64_t oracle_export(const oracle *h, uint32_t *src, uint32_t *dst);
void oracle_dout(const oracle *h, uint32_t *dout);

/* counters since the last oracle_reset_stats */
typedef struct {
    uint64_t pushes;        /* SeqPush / self-update count */
    uint64_t pushed_edges;  /* neighbour-propagation count */
    uint64_t rounds_pos, rounds_neg; /* ORC_JACOBI rounds (ORC_SEQ: 0) */
} oracle_stats;
void oracle_get_stats(const oracle *h, oracle_stats *st);
void oracle_reset_stats(oracle *h);

#ifdef __cplusplus
}
#endif
#endif
