/*
 * mcm.h -- C ABI of the B200 (sm_100a) push-relabel maximum-cardinality
 * bipartite matching library (Deveci, Kaya, Ucar, Catalyurek, ICPP 2013).
 *
 * Citations: P:a-b = lines a..b of the paper text (PAPER.md, LF numbering).
 *
 * Problem.  G = (V_R u V_C, E) bipartite; rows V_R = V1 (m of them),
 * columns V_C = V2 (n of them), matrix view P:115-118.  A matching M is a set of
 * vertex-disjoint edges; mcm_solve returns a maximum-cardinality matching
 * (|M| >= |M'| for every matching M').
 *
 * Method.  G-PR (Alg. 7): cheap initial matching, then a
 * loop of lock- and atomic-free concurrent push / double-push steps over the
 * active-column worklist (Alg. 8/9, worklist P:532-555, shrink
 * P:656-701), with periodic global relabelling by a level-synchronous BFS from the
 * unmatched rows (Alg. 4/5) scheduled by GETITERGR, gap
 * relabelling, and a final FIXMATCHING pass.  The whole loop
 * runs on the device in one persistent kernel; the only host synchronisation of a
 * solve is the final read of the cardinality.
 *
 * Conventions.  All ids are int32, 0-based.  Graph input is the CSR of the m x n
 * pattern (row u -> columns).  Unsorted adjacency and duplicate entries are
 * accepted (they change tie-breaks only).  m = 0, n = 0 or nnz = 0 is valid.
 * Limits: m + n + 2 < 2^31 and nnz < 2^31, else MCM_EINVAL.
 *
 * Memory.  The library performs NO device allocation: the caller provides one
 * device workspace of at least mcm_workspace_bytes() bytes (e.g. a torch uint8
 * tensor) that must outlive the handle.  indptr/indices are borrowed only for the
 * duration of mcm_create (they are copied and transposed into the workspace).
 * The handle itself is a small host object.
 *
 * Streams.  Every call enqueues its device work on the given stream; nothing
 * touches the legacy default stream or synchronises the device.  mcm_create
 * synchronises `stream` twice (the validation result, then the end of the
 * transpose); mcm_solve and the other device entry points once (to return their
 * result).  A handle is bound to the device current at mcm_create; calling
 * it with another device current returns MCM_EDEVICE.  One handle per host
 * thread (handles are not thread-safe).  After MCM_ECUDA the handle is poisoned:
 * every later call returns MCM_ECUDA.
 */
#ifndef MCM_H_
#define MCM_H_

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef struct mcm_ctx *mcm_handle_t;
typedef void *mcm_stream_t; /* a cudaStream_t (NULL = legacy default stream) */

enum {
  MCM_OK = 0,
  MCM_EINVAL = -1,    /* bad argument or malformed CSR (see mcm_create) */
  MCM_ECUDA = -2,     /* a CUDA runtime call failed; the handle is poisoned */
  MCM_ENOMEM = -3,    /* workspace smaller than mcm_workspace_bytes() */
  MCM_EDEVICE = -4,   /* called with a different current device than at create */
  MCM_ENOCONV = -5,   /* iteration cap (options.max_loops) exceeded */
  MCM_EINTERNAL = -6  /* internal consistency check failed (a bug) */
};

/* GR frequency strategy: adaptive = next GR after k*maxLevel loops,
 * fixed = every k loops. */
enum { MCM_GR_ADAPTIVE = 0, MCM_GR_FIXED = 1 };

/* Initial matching: cheap greedy on the device (reading R13), the
 * caller's matching in rmatch/cmatch, or empty.  GIVEN: every rmatch[u] must be
 * -1 or a column (< n) and every cmatch[v] -1 or a row (< m), else mcm_solve
 * returns MCM_EINVAL (checked on the device before any phase runs).  Pairs that
 * do not point back at each other are tolerated, with the paper's conventions: a
 * column whose row does not point back is unmatched (Alg. 6 l.3, reading R1); a
 * row whose column does not point back is repaired before the exactness guard's
 * GR (reading R27).  The pairs are not checked to be edges. */
enum { MCM_INIT_GREEDY = 0, MCM_INIT_GIVEN = 1, MCM_INIT_EMPTY = 2 };

typedef struct {
  double k;             /* GR frequency.  Adaptive: next GR after max(1, ceil(k*maxLevel))
                           loops; fixed: every max(1, (int)k) loops.  Default 0.4: the
                           paper's best is 0.7; with this build's early-stop
                           GR and tail mode 0.4 measured faster on C2-C4 (R23). */
  int32_t gr_strategy;  /* MCM_GR_ADAPTIVE (default) or MCM_GR_FIXED */
  int32_t shrink_min;   /* compact the worklist after a GR when |Ac| >= shrink_min
                           (G-PR-SHRKRNL); default 512;
                           < 0: never (G-PR-NoShr). */
  int32_t init;         /* MCM_INIT_GREEDY (default), MCM_INIT_GIVEN, MCM_INIT_EMPTY */
  int32_t gap;          /* gap relabelling (reading R14): 0 off (default), 1 on */
  int32_t final_check;  /* 1 (default): exactness guard -- one GR after termination;
                           any unmatched column it reaches is re-activated (R16). */
  int32_t dead_skip;    /* 1 (default): an active column whose label is already
                           >= m+n dies without scanning Gamma(v) (R19). */
  int32_t tail_max;     /* worklists of at most this many slots run on the tail group
                           (tail_ctas CTAs) instead of the whole grid (0 = off); default 32 */
  int32_t tail_f;       /* GR levels whose frontier has at most this many rows run on the
                           tail group (handed back to the grid above it, to the tail below
                           tail_f/2); 0 = 2 * tail_max; default 128 */
  int32_t compact_every;/* 1: compact the worklist at every fix step (an option beyond
                           the paper's post-GR shrink); default 0 */
  int32_t grid_ctas;    /* CTAs of the persistent kernel; 0 (default) = all co-resident */
  int32_t tail_ctas;    /* CTAs of the tail group: 1 (default) = one CTA (__syncthreads);
                           2..16 (power of 2) = a thread-block cluster with the hardware
                           cluster barrier (the grid then shrinks to whole clusters) */
  int32_t compact_adapt;/* 1 (default): compact the worklist at the next fix step when
                           fewer than 1/4 of its slots hold an active column */
  int32_t gr_early;     /* 1: a GR stops once every alive unmatched column has a label;
                           unreached vertices get the next level as a lower bound (R22);
                           default 1 (ignored when gap = 1); 0 = the paper's complete GR */
  int32_t serial;       /* 1 (tests): the fix and push steps run on one thread with the slots
                           in increasing order, GRs complete, no tail / adaptive compaction:
                           the trajectory of the serial simulator (oracle or_gpr_serial);
                           default 0 */
  int32_t sort_csc;     /* mcm_create: 1 = sort every Gamma(v) by row id (deterministic scan
                           order, needed for bit-exact serial runs); default 0 */
  int32_t bu_div;       /* direction-optimising GR: a BFS level whose frontier
                           has at least bu_div/8 adjacency entries per still-unlabelled
                           column and at least n/64 rows runs bottom-up (every unlabelled
                           column looks for a
                           neighbour at the current level); identical labels; default 16,
                           0 = top-down only */
  int32_t scan_rot;     /* 1: every push scan starts at a (column, loop)-dependent rotation of
                           Gamma(v) and wraps around -- a different but equally valid first
                           minimum (reading R11); default 0 */
  int32_t variant;      /* 0 (default): G-PR (Alg. 7, active-column worklist);
                           1: G-PR-First (Alg. 3 + Alg. 6: every column
                           tested every loop; the Fig. 1 ablation) */
  int32_t tail_chain;   /* single-CTA tail with at most 32 active columns: each column's lanes
                           runs a chain of double pushes (the displaced column is pushed next
                           by the same warp, its row claimed by CAS) instead of one push per
                           loop -- a build addition (R26); 0 = the paper's one push
                           per column per loop; default 256 = maximum pushes per chain */
  int32_t grid_chain;   /* the same push chains for grid loops with at most one active column per
                           two threads (rows claimed by CAS at gpu scope, re-scanned at gpu scope
                           after a lost claim); default 128 = maximum pushes per chain; 0 = the
                           paper's one push per column per loop */
  int64_t max_loops;    /* iteration cap; 0 = default (2*(m+n)+100000).  MCM_ENOCONV beyond */
  double gr_target;     /* early-stop GR (gr_early, R22/R28): the BFS stops once this
                           fraction of the alive unmatched columns carries a label; (0, 1];
                           default 0.6; 1.0 = every one (R22 alone); see gr_target_min */
  int32_t gr_target_min; /* gr_target applies only to GRs that start with at least this many
                           alive unmatched columns (fewer: every one must be labelled);
                           default 1024 */
  int32_t gr_concurrent; /* concurrent GR and push (the paper's future work; SURVEY
                           NEXT-2; an experiment): > 0 = a second persistent kernel on
                           this many CTAs runs complete GRs into shadow labels, on a stream of
                           the handle's own, while the solve kernel (the remaining CTAs) keeps
                           pushing; finished labels are installed at the next loop boundary.
                           The exactness guard keeps the result exact.  Ignored in serial mode
                           and for G-PR-First.  Default 0 (off). */
  int32_t perturb;      /* fault injection (tests only): each of the paper's
                           pushes (Alg. 9 l.14-18, not the push chains of R26) loses its row
                           store with probability perturb / 65536 (a counter hash of the
                           column and the loop): mu(v) <- u and Ap(i) <- w are written, the
                           row word keeps its old mate -- the outcome of losing the race for
                           u to another column.  The column is then active by
                           reading R1 and is pushed again; the rollback (Alg. 8 l.3-6),
                           FIXMATCHING and the exactness guard must still return
                           a maximum matching.  0..65536; default 0 (off). */
  int32_t gr_window;    /* windowed GR levels (a build addition; the paper's GR is level-synchronous,
                           Alg. 5): K > 1 = every CTA expands its share of a grid
                           frontier and the rows that share reaches, K levels deep, before the
                           next grid barrier; labels are lowered by CAS (label correcting), so
                           every label is the exact BFS distance at the window's end (DESIGN.md
                           R29).  0 or 1 = one level per barrier.  0..64 */
  int32_t gr_window_max; /* windows run for grid frontiers of at most this many rows (wider
                           levels are work-bound and stay level-synchronous) */
} mcm_options_t;

typedef struct {
  int64_t loops;             /* iterations of Alg. 7's while loop */
  int64_t gr_count;          /* global relabels (incl. the guard GR) */
  int64_t gr_levels;         /* sum over GRs of BFS row levels */
  int64_t pushes;            /* successful single/double pushes */
  int64_t blocked;           /* pushes refused by the iA test (Alg. 9 l.13) */
  int64_t dead;              /* columns declared unmatchable (mu = -2) */
  int64_t edges_scanned;     /* neighbours read by the push scans */
  int64_t slots;             /* worklist slots visited by fix steps */
  int64_t shrinks;           /* SHRKRNL compactions */
  int64_t gaps;              /* gap relabels applied */
  int64_t guard_reactivated; /* columns re-activated by the exactness guard */
  int64_t fixed_cols;        /* columns reset by FIXMATCHING */
  int64_t init_card;         /* |M0| */
  int64_t card;              /* |M| returned */
  int64_t tail_loops;        /* loops run in the single-CTA tail mode */
  int64_t grid_barriers;     /* grid-wide barriers executed */
  int64_t gr_rows;           /* rows expanded by all GR levels (frontier entries) */
  int64_t gr_edges;          /* adjacency entries read by all GR levels */
  int64_t gr_cols;           /* columns labelled by all GRs */
  int64_t greedy_edges;      /* adjacency entries read by the greedy initial matching */
  int64_t rows_repaired;     /* stale rows (mate not pointing back) re-attached or made unmatched before
                                the guard GR (R27) */
  int64_t tail_gr_levels;    /* GR levels run by the single-CTA tail (frontier in shared memory) */
  int64_t debug_violations;  /* consistency violations found by the debug checks (env MCM_DEBUG=1) */
  int64_t kernel_launches;   /* kernels launched by this handle's mcm_create plus by the last call (counted
                                at the launch sites: the create's setup kernels + one persistent kernel) */
  int64_t gr_window_levels;  /* BFS levels run inside windows (option gr_window; K per window) */
  double ms_init;            /* device time: initial matching + worklist build */
  double ms_gr;              /* device time in global relabels */
  double ms_loop;            /* device time in fix + push steps */
  double ms_total;           /* device time of the whole solve kernel */
  double ms_setup;           /* mcm_create: validation + copy + transpose (host-timed) */
  int32_t grid_ctas, threads_per_cta;
} mcm_stats_t;

/* Fill *o with the defaults above. */
void mcm_default_options(mcm_options_t *o);

/* Bytes of device workspace a handle for an (m, n, nnz) graph needs (256-B aligned
 * sub-buffers).  Returns 0 when the sizes are out of range. */
size_t mcm_workspace_bytes(int32_t m, int32_t n, int64_t nnz, const mcm_options_t *o);

/* Validate the CSR (indptr[0] = 0, non-decreasing, indptr[m] = nnz, 0 <= indices
 * < n; one O(m + nnz) device pass), copy it and build the CSC transpose in the
 * workspace.  indptr (m+1) and indices (nnz) are DEVICE pointers.  o = NULL means
 * defaults.  Returns MCM_OK and *out, or an error code (no handle is created). */
int mcm_create(const int32_t *indptr, const int32_t *indices, int32_t m, int32_t n, int64_t nnz, void *workspace,
               size_t ws_bytes, mcm_stream_t stream, const mcm_options_t *o, mcm_handle_t *out);

/* Run G-PR.  rmatch (m) and cmatch (n) are caller-owned DEVICE int32 buffers,
 * written on return: rmatch[u] = column or -1, cmatch[v] = row or -1, mutually
 * consistent (FIXMATCHING: the internal -2 "dead" mark never escapes).
 * With MCM_INIT_GIVEN they are also read as the initial matching.  Returns the
 * cardinality (>= 0) or a negative error code.  Synchronises `stream` once. */
int64_t mcm_solve(mcm_handle_t h, mcm_stream_t stream, int32_t *rmatch, int32_t *cmatch);

/* One call from HOST memory to HOST memory (the end-to-end path): copies the CSR
 * indptr (m+1) / indices (nnz) from the HOST straight into the workspace's CSR
 * copy, validates and transposes it there (as mcm_create), solves (as mcm_solve)
 * and copies the matching into the HOST arrays rmatch (m) / cmatch (n).  All
 * copies are enqueued on `stream` (asynchronous when the host arrays are pinned)
 * and the call synchronises `stream` twice (validation result, final
 * cardinality).  workspace: DEVICE, >= mcm_workspace_bytes(m, n, nnz, o); no
 * handle outlives the call.  o: NULL = defaults; init = MCM_INIT_GIVEN is not
 * supported here (MCM_EINVAL).  stats (may be NULL) receives the solve's
 * statistics.  Returns the cardinality or a negative error code (the CSR checks
 * of mcm_create apply). */
int64_t mcm_match_host(const int32_t *indptr, const int32_t *indices, int32_t m, int32_t n, int64_t nnz,
                       void *workspace, size_t ws_bytes, mcm_stream_t stream, const mcm_options_t *o,
                       int32_t *rmatch, int32_t *cmatch, mcm_stats_t *stats);

/* Global relabel (Alg. 4/5) of a given matching, run exactly as a solve
 * runs its GRs under the handle's options: grid BFS levels, single-CTA tail levels
 * with the frontier in shared memory (tail_max > 0 and frontiers of at most tail_f
 * rows, handed back to the grid above it), bottom-up levels (bu_div), and the
 * early stop of gr_early / gr_target / gr_target_min (R22 / R28).
 * rmatch (m) and cmatch (n) are DEVICE inputs with the paper's mu conventions
 * (column entries may be stale or -2; rows are authoritative; ranges as
 * for MCM_INIT_GIVEN, cmatch may also hold -2, else MCM_EINVAL).  Writes psi_row (m)
 * and psi_col (n) (DEVICE): the exact alternating BFS distance from the unmatched
 * rows for every vertex the BFS labelled; a vertex it did not reach gets m+n after
 * a complete GR, and the lower bound floor_row / floor_col after an early stop.
 * Returns maxLevel as GETITERGR uses it ((deepest row level) + 2, Alg. 4's final
 * cLevel; after an early stop at row level l: l + 4), or a negative error code.
 * info (may be NULL) receives 4 values: [0] the number of columns that are not
 * matched but got a finite label (> 0 iff an augmenting path exists, after a
 * complete GR), [1] floor_row, [2] floor_col (m+n after a complete GR), [3] the
 * BFS levels the single-CTA tail ran. */
int64_t mcm_global_relabel(mcm_handle_t h, mcm_stream_t stream, const int32_t *rmatch, const int32_t *cmatch,
                           int32_t *psi_row, int32_t *psi_col, int64_t *info);

/* The cheap initial matching alone (reading R13: every column
 * claims the first free row of Gamma(v) by CAS -- the phase a default mcm_solve
 * starts with).  Writes rmatch (m) / cmatch (n) (DEVICE) = M0, a valid maximal
 * matching, and returns |M0| or a negative error code.  Used for the paper's timing
 * protocol (the cheap matching excluded from the timed solve: feed M0 to
 * mcm_solve with MCM_INIT_GIVEN) and to test M0 on its own. */
int64_t mcm_initial_matching(mcm_handle_t h, mcm_stream_t stream, int32_t *rmatch, int32_t *cmatch);

/* ONE phase of the solve kernel on a caller-given state (test and inspection
 * entry point: the code a solve runs, not a re-implementation).
 *   unit  MCM_UNIT_FIX         G-PR-INITKRNL (Alg. 8): rollback of lost
 *                              pushes, iA marks; returns the active-slot count
 *         MCM_UNIT_SHRINK      G-PR-SHRKRNL: the same with the surviving
 *                              slots compacted in slot order; returns the new length
 *         MCM_UNIT_PUSH        G-PR-PUSHKRNL (Alg. 9; no push chains);
 *                              returns 0
 *         MCM_UNIT_FIXMATCHING FIXMATCHING: mu_col <- the output
 *                              convention (reading R15); returns |M|
 *   where MCM_WHERE_GRID (every CTA, the phase code of a wide loop) or
 *         MCM_WHERE_TAIL (CTA 0 alone with the worklist in shared memory when it
 *         fits, as the solve's tail mode runs it; the tail fix step always compacts,
 *         so FIX there behaves as SHRINK).  FIXMATCHING always runs on the grid.
 *   loop  the loop counter (iA marks, Alg. 9 l.13), 0 <= loop < 2^31
 *   len   worklist slots, 0 <= len <= n
 * In/out DEVICE int32 arrays: mu_row (m, -1 or a column), mu_col (n, -2, -1 or a
 * row), psi_row (m) and psi_col (n) (labels; < 0 or >= m+n mean m+n on input),
 * iA (n), Ac (len), Ap (len).  Out-of-range entries return MCM_EINVAL.  The
 * phase's statistics (pushes, blocked, dead, slots) are in mcm_get_stats. */
enum { MCM_UNIT_FIX = 0, MCM_UNIT_SHRINK = 1, MCM_UNIT_PUSH = 2, MCM_UNIT_FIXMATCHING = 3 };
enum { MCM_WHERE_GRID = 0, MCM_WHERE_TAIL = 1 };
int64_t mcm_unit_step(mcm_handle_t h, mcm_stream_t stream, int32_t unit, int32_t where, int64_t loop, int32_t len,
                      int32_t *mu_row, int32_t *mu_col, int32_t *psi_row, int32_t *psi_col, int32_t *iA, int32_t *Ac,
                      int32_t *Ap);

/* Gap relabelling (reading R14) of given labels, in place: psi_row (m)
 * and psi_col (n) are DEVICE int32 labels (values >= m+n, or < 0, mean infinite).
 * Counts the vertices of every finite label below H = min(m+n+2, 2^20); if some
 * label g below the largest finite label has no vertex, every label in (g, m+n)
 * becomes m+n (labels >= m+n are written back as m+n).  Returns g, or -1 when there
 * is no gap, or a negative error code below -1.  This is the same device routine
 * the solve applies once between two GRs when options.gap = 1. */
int64_t mcm_gap_relabel(mcm_handle_t h, mcm_stream_t stream, int32_t *psi_row, int32_t *psi_col);

/* ---- NEXT-4 (an EXPERIMENT, not on the solve path) ----
 * A 1D row-partitioned global relabel (Alg. 2 with the matched test of Alg. 5 l.6,
 * P:257-272, 401-410) whose BFS levels exchange the row frontier as a bitmap with
 * an all-gather (NCCL over NVLink in paper_conf_icpp_devecikuc13_b200/pgr.py).  It
 * exists to measure why replicas win: one collective per BFS level.
 *   nparts P >= 1 parts, this call's part p (0 <= p < P), words W >= 1 bitmap words
 *   (32 rows each) per part, with 32 W P >= m.  Part p owns rows [32 W p, 32 W (p+1))
 *   and the mate column of each owned row u with cmatch[rmatch[u]] = u (the column
 *   is matched, Alg. 5 l.6), plus the columns that are not matched in
 *   [ceil(n/P) p, ceil(n/P) (p+1)).
 *   Frontier buffers (DEVICE uint32): P slices of W + 1 words, part q's slice at
 *   word q (W + 1): W bitmap words (bit u mod 32 of word (u mod 32W) / 32 = row u
 *   is in the frontier) and one count word (rows the part added).  `slice` points
 *   at THIS part's slice (W + 1 words) of the buffer being built, `frontier` at the
 *   whole gathered buffer of the previous level.
 *   psi_row (m) / psi_col (n): DEVICE int32 labels; only owned entries are written
 *   after mcm_pgr_init (the elementwise minimum over the parts is the GR result:
 *   the exact BFS distance, m+n when unreached).  rmatch (m) / cmatch
 *   (n): DEVICE, the matching with the paper's mu conventions (cmatch may be stale
 *   or -2; rows are authoritative); entries out of range are treated as unmatched.
 * Both calls only enqueue work on `stream` (no synchronisation) and return MCM_OK
 * or a negative error code. */
/* Level 0 (Alg. 2 l.1-3): owned rows get 0 (unmatched) or m+n, every column m+n;
 * writes this part's slice of F_0. */
int mcm_pgr_init(mcm_handle_t h, mcm_stream_t stream, int32_t nparts, int32_t part, int32_t words,
                 const int32_t *rmatch, uint32_t *slice, int32_t *psi_row, int32_t *psi_col);
/* Level L >= 0 (row labels 2L form `frontier`): every unlabelled owned column v
 * with a row of Gamma(v) in the frontier gets 2L+1, its owned mate row 2L+2 (the
 * row joins this part's slice of F_{L+1}).  *reached_free (DEVICE uint64,
 * accumulated) += columns that are not matched and got a label. */
int mcm_pgr_level(mcm_handle_t h, mcm_stream_t stream, int32_t nparts, int32_t part, int32_t words, int32_t level,
                  const int32_t *rmatch, const int32_t *cmatch, const uint32_t *frontier, uint32_t *slice,
                  int32_t *psi_row, int32_t *psi_col, uint64_t *reached_free);

/* Replace the options of a handle (takes effect at the next solve). */
int mcm_set_options(mcm_handle_t h, const mcm_options_t *o);
int mcm_set_k(mcm_handle_t h, double k);

/* Statistics of the last mcm_solve. */
int mcm_get_stats(mcm_handle_t h, mcm_stats_t *out);

/* Free the host handle (the workspace stays the caller's). */
int mcm_destroy(mcm_handle_t h);

const char *mcm_strerror(int code);

/* sizeof(mcm_options_t) and sizeof(mcm_stats_t) as compiled into the library, so a
 * binding can verify its struct mirrors (returns MCM_OK). */
int mcm_abi_sizes(size_t *options_size, size_t *stats_size);

#ifdef __cplusplus
}
#endif
#endif /* MCM_H_ */
