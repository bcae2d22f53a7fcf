// solve.cuh -- the persistent G-PR kernel (Alg. 7) and its phases.
//
// One cooperative launch runs a whole solve: initial matching, worklist build,
// then Alg. 7's loop { GR when loop == iterGR; INIT/SHR fix step; PUSH; swap }
// with grid-wide barriers between dependent phases, the exactness guard, and
// FIXMATCHING.  Control state (loop, iterGR, |Ac|, ...) lives in registers and is
// updated identically by every thread from counters read after each barrier,
// so no CTA ever waits for another to broadcast a decision.
//
// Phase functions are templated on GRID: GRID=true spreads the items over all
// CTAs and separates phases with grid.sync(); GRID=false runs them on CTA 0
// alone with __syncthreads() (the "tail mode" used when the worklist is short --
// most of the paper's iterations have "only a few" active columns).
#pragma once
#include <cooperative_groups.h>
#include "device.cuh"

namespace cg = cooperative_groups;

#ifndef MCM_CHAIN_PLAIN
#define MCM_CHAIN_PLAIN 0
#endif
#ifndef MCM_FINE
#define MCM_FINE 0
#endif
// batch widths of the wide phases (independent items in flight per thread; capped
// by the register budget: 512 threads x 128 registers)
#ifndef MCM_RG
#define MCM_RG 4   // greedy: columns per lane
#endif
#ifndef MCM_EB
#define MCM_EB 4   // wide BFS level: adjacency entries per batch (two frontier entries per thread)
#endif
#ifndef MCM_PB
#define MCM_PB 2   // wide push: slots per thread
#endif
#ifndef MCM_BUFLUSH
#define MCM_BUFLUSH 16  // bottom-up BFS level: flush the staged frontier every this many tiles
#endif
#ifndef MCM_WFLUSH
#define MCM_WFLUSH 0  // wide BFS level: flush the staged frontier every this many tiles (0: once per level)
#endif
namespace mcm {

constexpr int NT = 512;          // threads per CTA
constexpr int NWARP = NT / 32;
constexpr int QCAP = 16384;      // shared staging (ints, 64 KB, dynamic smem): next BFS frontier, gap histogram
constexpr int QCAP4 = QCAP / 4;  // ... as int4 frontier entries
constexpr int TQ = QCAP4 / 2;    // tail: two shared int4 frontier buffers of TQ entries (alias q)
constexpr int TW = 1024;         // tail: shared worklist capacity (Ac / Ap)
constexpr int SMALL_DEG = 32;    // greedy: adjacency lists up to this length: one thread
constexpr int BIG_DEG = 64;      // GR / push: longer lists go to the whole warp
constexpr int HUGE_DEG = 512;    // push: longer lists go to the whole CTA
constexpr int MAXHUGE = 32;      // CTA-wide push list per tile
constexpr int HUGE_CTA = 4;      // at most this many per tile: one CTA-wide scan each; more: a warp each ...
constexpr int HUGE_WARP = 8192;  // ... unless longer than this
constexpr int KB = 4;            // neighbours in flight per lane (batched loads)
constexpr int SPLIT = 1024;      // GR: a frontier row's adjacency is split into ranges of at most this many

enum { MODE_SOLVE = 0, MODE_RELABEL = 1, MODE_GAP = 2, MODE_UNIT = 3, MODE_INIT = 4, MODE_CONC_GR = 5 };
// mcm_unit_step: one phase of the solve on a given state (include/mcm.h)
enum { UNIT_FIX = 0, UNIT_SHRINK = 1, UNIT_PUSH = 2, UNIT_FIXMATCHING = 3 };

// statistics slots (Ctrl::stat)
enum {
  ST_LOOPS, ST_GRS, ST_LEVELS, ST_PUSHES, ST_BLOCKED, ST_DEAD, ST_SCANNED, ST_SLOTS, ST_SHRINKS, ST_GAPS,
  ST_GUARD, ST_FIXED, ST_INITCARD, ST_CARD, ST_TAILLOOPS, ST_BARRIERS, ST_NS_INIT, ST_NS_GR, ST_NS_LOOP,
  ST_NS_TOTAL, ST_MAXLEVEL, ST_REACHED_FREE, ST_GR_ROWS, ST_GR_EDGES, ST_GR_COLS, ST_GREEDY_EDGES, ST_TRACE_N, ST_REPAIRED,
  ST_FLOOR_R, ST_FLOOR_C, ST_TAIL_LEVELS, ST_WINDOWS, ST_NSTAT = 32
};

struct Ctrl {
  u32 ring[4][8];          // per-phase counters, rotated (see Solver::barrier)
  u32 bar;                 // grid barrier word (device.cuh grid_sync)
  u32 pad0[3];
  long long stat[ST_NSTAT];
  int err;                 // 0 or an MCM_* code
  u32 gcnt;                // exactness-guard list cursor (monotonic within a solve)
  int gmax, gmin;          // gap relabel: largest finite label, smallest empty label
  u32 ndead;               // columns declared dead (mu = -2), net of guard re-activations
  int pad[11];
  long long dbg[8];        // debug checks: [0] count, [1] where, [2] loop, [3] vertex, [4] value
  // tail-mode handoff (tail group -> grid): reason, phase counter, Ctl image
  int ho_reason, ho_ph;
  long long ho[32];
  // concurrent GR (option gr_concurrent): handshake between the push
  // kernel and the GR kernel (fields of the GR kernel's own Ctrl block): requests
  // (push -> GR), completions and the epoch of the finished labels (GR -> push),
  // exit / exited, and the GR kernel's per-level frontier counters
  u32 creq, cdone, cexit, cexited, csbase, ccnt[4];
};

struct Params {
  int m, n, mode;
  const int *rptr, *radj, *cptr, *cadj;
  u64 *rowst, *colst;
  int *iA, *wl0, *wl1, *qa, *qb, *qc, *qd;  // qc, qd: int4 BFS frontiers
  int *ctacnt;
  int *dbgbuf;             // n ints (debug checks only)
  int tail_ctas;           // CTAs of the tail group (= cluster 0 when > 1)
  int tail_f;              // GR frontier limit of the tail group (0: 2 * tail_max)
  int *hist;               // gap relabel histogram (hist_len counters, zero between uses)
  int4 *ovf;               // per-CTA overflow regions of the BFS frontier staging
  long long ovf_len;       // entries in ovf
  int hist_len;
  int debug;
  long long *trace;        // optional phase trace: {tag, size, t_end_ns} triples (MCM_TRACE)
  long long *ctat;         // optional: per-CTA grid-barrier arrival times [phase][cta] (MCM_CTATIME)
  int ctat_n;
  int trace_cap;
  Ctrl *ctrl;
  // options
  double k, gr_target;
  int gr_target_min;
  int gr_fixed, shrink_min, init, gap, final_check, dead_skip, tail_max, compact_every, compact_adapt, gr_early;
  int serial;              // 1: fix/push by one thread in slot order (bit-exact vs the serial simulator)
  int variant;             // 0: G-PR (Alg. 7, worklist); 1: G-PR-First (Alg. 3 + Alg. 6, all columns)
  int tail_chain;          // single-CTA tail, <= chain_slots active columns: max pushes per chain (0: off)
  int chain_slots;
  int grid_chain;          // grid loops of <= 1/grid_chain_div slot per thread: max pushes per chain (0: off)
  int grid_chain_div;
  int bu_div;              // bottom-up BFS level rule (see use_bottom_up; 0: top-down only)
  int scan_rot;            // push scans start at a (column, loop)-dependent rotation (tie-break)
  int perturb;             // fault injection: a push loses its row store with probability perturb/65536
  int gr_window, gr_window_max;  // windowed GR levels (see gr_window_level): levels per window, frontier limit
  long long max_loops;
  // I/O
  const int *rmatch_in, *cmatch_in;
  int *rmatch_out, *cmatch_out;  // solve: matching; relabel: psi_row / psi_col
  // MODE_UNIT: labels in / out, and the phase to run (Ac / Ap / iA are copied into
  // wl0 / wl1 / iA by the host)
  int *psi_row_io, *psi_col_io;
  int unit_what, unit_where, unit_len;
  long long unit_loop;
  // concurrent GR (NEXT-2): CTAs of the GR kernel (0: off), its shadow labels, its
  // control block
  int conc;
  u32 *srow, *scol;
  Ctrl *ctrl2;
};

// per-CTA statistics accumulators (Smem::st), flushed at every barrier from
// per-thread 32-bit counters that live only within one phase
enum { SS_PUSH, SS_BLOCK, SS_DEAD, SS_SCAN, SS_SLOTS, SS_FREE, SS_GRROWS, SS_GREDGES, SS_GRCOLS, SS_GYEDGES, SS_N };
// control-loop statistics and the phase-trace cursor: kept by the lead thread
// (block 0, thread 0) only, in shared memory, so they hold no registers
struct LeadStats {
  long long grs, levels, shrinks, gaps, guard_re, loops, tail_loops, ns_gr, ns_loop, nbar, repaired, tail_levels,
      wlevels;
  int tn, ttag, tsz, pad;
};
struct Smem;
extern __shared__ Smem smem_dyn[];
struct Smem {
  u32 ts[SS_N][NT];        // per-thread statistics (thread-private slots: no atomics)
  LeadStats ld;
  u32 lvc[2];              // BFS level: [1] next-frontier adjacency entries (direction choice)
  u32 rp[8];               // phase counters of the last completed phase (loaded by thread 0)
  u32 bc;                  // broadcast slot (bcast_ld)
  int ho_reason, ho_ph;    // tail hand-over image (loaded by thread 0 after the barrier)
  long long ho[32];
  long long red[NWARP];
  int w[NWARP];
  alignas(16) int q[QCAP];
  int wl[2][TW];           // tail: the worklist (Ac/Ap) while the single-CTA tail owns it
  int4 huge[MAXHUGE];      // push: columns deferred to the CTA-wide scan {slot, v, s, e}
  u64 hugec[MAXHUGE];
  int huget[MAXHUGE];
  int nhuge;
  int4 lq[2][512];         // windowed GR (option gr_window): the CTA's local BFS queues
  int lqn[2];
  int lwdirty, lwmax;
  u32 nd;                  // push: columns declared dead in this tile (-> Ctrl::ndead)
  int chmax;               // push_chain: longest chain of the phase
  int qcnt, qbase, tmp;
};

// worklist / frontier loads: shared (tail residency) or global (bypass L1)
__device__ __forceinline__ int ld_wl(const int *p) { return __isShared(p) ? *p : __ldcg(p); }
__device__ __forceinline__ int4 ld_q(const int4 *p) { return __isShared(p) ? *p : __ldcg(p); }

__device__ __forceinline__ u64 gtime() {
  u64 t;
  asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
  return t;
}
// phase timers: only the lead thread (block 0, thread 0) reads the clock
__device__ __forceinline__ u64 tnow() { return (threadIdx.x == 0 && blockIdx.x == 0) ? gtime() : 0ull; }

// Compile-time feature set of a kernel instance.  The production solve kernel
// carries only what a default solve runs; the test / ablation / auxiliary paths
// (serial mode, G-PR-First, debug checks, gap relabelling, the label-only modes)
// live in a second instance, so they cost the hot kernel no code size (its
// instruction footprint is on the critical path of every short phase).
enum { F_SERIAL = 1, F_FIRST = 2, F_DEBUG = 4, F_GAP = 8, F_AUX = 16, F_BU = 32 };
constexpr int F_FAST = F_BU;
constexpr int F_ALL = F_SERIAL | F_FIRST | F_DEBUG | F_GAP | F_AUX | F_BU;

template <int F>
struct Solver {
  const Params &p;
  // vertex state (rowst, colst, iA): relaxed GPU-scope accesses (device.cuh, R17)
  __device__ __forceinline__ static u64 vld(const u64 *a) { return ldv(a); }
  __device__ __forceinline__ static int vld(const int *a) { return ldv(a); }
  __device__ __forceinline__ static void vst(u64 *a, u64 v) { stv(a, v); }
  __device__ __forceinline__ static void vst(int *a, int v) { stv(a, v); }
  // the dynamic shared block, named through a namespace-scope extern __shared__
  // array so every access compiles to a shared-space instruction (a Smem& member
  // made the staging atomics generic ATOM.E)
#define sm (smem_dyn[0])
  const int m, n, INF;
  // per-thread statistics: 32-bit thread-private slots in shared memory (Smem::ts),
  // summed at the end of the solve -- they hold no registers, need no atomics and
  // no per-phase reduction (a per-phase warp flush with 64-bit shared atomics, which
  // are CAS spin loops on sm_100, cost ~1 us per BFS level)
  int ph = 0;  // phase counter: identical in every thread
  __device__ __forceinline__ static bool lead() { return threadIdx.x == 0 && blockIdx.x == 0; }
  __device__ __forceinline__ static LeadStats &L() { return smem_dyn[0].ld; }
  __device__ __forceinline__ static u32 &S(int k) { return smem_dyn[0].ts[k][threadIdx.x]; }
  __device__ __forceinline__ void trace(int tag, int sz) {
    if (lead()) { L().ttag = tag; L().tsz = sz; }
  }
  __device__ __forceinline__ void tmark(int tag, int sz) { trace_rec(tag, sz); }
  __device__ __forceinline__ void trace_rec(int tag, int sz) {
    if (p.trace && lead() && L().tn < p.trace_cap) {
      const int tn = L().tn;
      p.trace[3 * tn] = tag; p.trace[3 * tn + 1] = sz; p.trace[3 * tn + 2] = (long long)gtime();
      L().tn = tn + 1;
    }
  }

  int ovf_r = 0;  // entries of this CTA's overflow region
  int n_iso = 0;  // rows without edges (excluded from U in solve mode)
  __device__ Solver(const Params &p_) : p(p_), m(p_.m), n(p_.n), INF(p_.m + p_.n) {
    ovf_r = (int)(p_.ovf_len / gridDim.x);
  }

  // ---------------------------------------------------------------- barriers
  // ring[ph & 3] collects the counts produced during phase ph; the consumer reads
  // it right after the barrier.  ring[(ph + 2) & 3] was produced two phases ago
  // and consumed at the start of the previous phase, so CTA 0 may clear it now.
  // RP: the next phase reads the counters of this one (ring_prev); loading them
  // is one more L2 round trip on the barrier's critical path, so barriers whose
  // successor does not need them skip it
  template <bool GRID, bool RP = true>
  __device__ __forceinline__ void barrier() {
    const u32 *rn = p.ctrl->ring[ph & 3];
    auto load_rp = [&] {
#pragma unroll
      for (int j = 0; j < 8; j++) sm.rp[j] = ld_rlx(rn + j);
    };
    if (GRID) {
      if (MCM_FINE) tmark(105, 0);
      if (p.ctat) {  // analysis only: when the CTA's last warp reached this barrier
        __syncthreads();
        if (threadIdx.x == 0 && ph < p.ctat_n) p.ctat[(long long)ph * gridDim.x + blockIdx.x] = (long long)gtime();
      }
      if (RP) grid_sync(&p.ctrl->bar, false, load_rp);
      else grid_sync(&p.ctrl->bar, false);
      if (lead()) L().nbar++;
    } else {
      if (p.tail_ctas > 1) {
        // tail group = thread-block cluster 0: hardware cluster barrier (release /
        // acquire at cluster scope covers the global writes of the cluster's CTAs)
        asm volatile("barrier.cluster.arrive.release.aligned;\n\tbarrier.cluster.wait.acquire.aligned;" ::: "memory");
      } else {
        __syncthreads();
      }
      if (RP) {
        if (threadIdx.x < 8) sm.rp[threadIdx.x] = ld_rlx(rn + threadIdx.x);
        __syncthreads();
      }
    }
    // phase trace: stamped after the barrier, so a phase's duration includes its
    // slowest CTA
    if (p.trace && lead()) trace_rec(L().ttag * 2 + (GRID ? 1 : 0), L().tsz);
    ph++;
    if (blockIdx.x == 0 && threadIdx.x == 0) {
      u32 *r = p.ctrl->ring[(ph + 2) & 3];
#pragma unroll
      for (int j = 0; j < 8; j++) r[j] = 0;
    }
  }
  __device__ __forceinline__ u32 *ring_now(int j) { return &p.ctrl->ring[ph & 3][j]; }
  // counter j of the phase completed by the last barrier (every barrier loads them)
  __device__ __forceinline__ u32 ring_prev(int j) const { return sm.rp[j]; }
  // a CTA-uniform global word, loaded once per CTA
  __device__ __forceinline__ u32 bcast_ld(const u32 *a) {
    __syncthreads();
    if (threadIdx.x == 0) sm.bc = ld_rlx(a);
    __syncthreads();
    return sm.bc;
  }

  template <bool GRID>
  __device__ __forceinline__ int cta() const { return blockIdx.x; }  // tail group = blocks [0, tail_ctas)
  template <bool GRID>
  __device__ __forceinline__ int ncta() const { return GRID ? gridDim.x : p.tail_ctas; }

  // CTA total -> ring counter j (one atomic per CTA)
  __device__ __forceinline__ void add_count(long long x, int j) {
    long long t = cta_sum<NT>(x, sm.red);
    if (threadIdx.x == 0 && t) atomicAdd(ring_now(j), (u32)t);
  }

  __device__ __forceinline__ bool col_unmatched(int v) const {
    // R1: mu(v) = -1, or mu(v) >= 0 and mu(mu(v)) != v.  mu(v) = -2 (dead) is inactive.
    int c = mu_of(vld(p.colst + v));
    if (c == -1) return true;
    if (c < 0) return false;
    return mu_of(vld(p.rowst + c)) != v;
  }

  // R1 for columns i0 .. i0+RB-1 (< hi): val[k] = the column if unmatched, else -1.
  // skip_iso: columns without any edge are left out as well (returns their count):
  // they can never be matched, and a first push would only declare them dead
  template <int RB>
  // consistent: every matched column's row points back (the device greedy's M0:
  // its row CAS precedes the column store), so R1 needs no row-word load
  __device__ __forceinline__ int cols_unmatched(int i0, int hi, int *val, bool skip_iso, bool consistent) const {
    u64 cw[RB], rw[RB];
    int cs[RB], ce[RB];
#pragma unroll
    for (int k = 0; k < RB; k++) cw[k] = i0 + k < hi ? vld(p.colst + i0 + k) : pack(-2, 0);
#pragma unroll
    for (int k = 0; k < RB; k++)
      rw[k] = (!consistent && mu_of(cw[k]) >= 0) ? vld(p.rowst + mu_of(cw[k])) : pack(i0 + k, 0);
#pragma unroll
    for (int k = 0; k < RB; k++) {
      const bool f = skip_iso && mu_of(cw[k]) == -1;
      cs[k] = f ? ld_ro(p.cptr + i0 + k) : 0;
      ce[k] = f ? ld_ro(p.cptr + i0 + k + 1) : 1;
    }
    int iso = 0;
#pragma unroll
    for (int k = 0; k < RB; k++) {
      const int c = mu_of(cw[k]);
      val[k] = (c == -1 || (c >= 0 && mu_of(rw[k]) != i0 + k)) ? i0 + k : -1;
      if (c == -1 && cs[k] == ce[k]) { val[k] = -1; iso++; }
    }
    return iso;
  }

  // ---------------------------------------------------------------- staging
  // BFS frontier entries are {row, rptr[row], rptr[row+1], 0}: the producer loads
  // the adjacency bounds of a row it discovers in parallel with its mate check, so
  // the next level starts one dependent load earlier.
  __device__ __forceinline__ void stage(int4 x, int4 *next, u32 *gcnt) {
    // warp-aggregated: one shared atomic per group of converged lanes
    cg::coalesced_group g = cg::coalesced_threads();
    int base = 0;
    if (g.thread_rank() == 0) base = atomicAdd(&sm.qcnt, (int)g.size());
    base = g.shfl(base, 0);
    int q = base + (int)g.thread_rank();
    if (q < (sq ? TQ : QCAP4)) {
      (sq ? sq_next : reinterpret_cast<int4 *>(sm.q))[q] = x;
    } else if (!sq && q - QCAP4 < ovf_r) {  // overflow: this CTA's private global region
      p.ovf[(long long)blockIdx.x * ovf_r + (q - QCAP4)] = x;
    } else {  // region full too: direct append, one global atomic per group
      cg::coalesced_group o = cg::coalesced_threads();
      u32 gb = 0;
      if (o.thread_rank() == 0) gb = atomicAdd(gcnt, (u32)o.size());
      gb = o.shfl(gb, 0);
      next[gb + o.thread_rank()] = x;
    }
  }
  // A row joins the next frontier as the edge range [s, e) of its adjacency; a
  // long list is split into ranges of SPLIT entries (w = 1 marks a continuation),
  // each expanded independently at the next level -- an R-MAT hub row (1.5 * 10^5
  // entries) on one warp held every level it appeared in for ~1.2 ms
  __device__ __forceinline__ void stage_row(int w, int s, int e, int4 *next, u32 *gcnt) {
    if (e - s <= SPLIT) {
      stage(make_int4(w, s, e, 0), next, gcnt);
      return;
    }
    for (int c = s; c < e; c += SPLIT) stage(make_int4(w, c, min(e, c + SPLIT), c > s), next, gcnt);
  }
  // one more alive unmatched column labelled by this GR (ring counter 2): warp-
  // aggregated into a per-CTA shared counter that flush() publishes once per level
  // (one global atomic per reached column put ~10^6 same-address atomics on one
  // L2 line in the first GRs of C3 / C4)
  __device__ __forceinline__ void count_free() {
    cg::coalesced_group g = cg::coalesced_threads();
    if (g.thread_rank() == 0) atomicAdd(&sm.lvc[0], (u32)g.size());
  }
  __device__ __forceinline__ void flush(int4 *next, u32 *gcnt) {
    if (sq) return;  // tail: the next frontier is the shared buffer itself
    __syncthreads();
    // one reservation per CTA and tile for the shared entries and the private
    // overflow region (wide levels would otherwise serialise on one counter)
    const int c = min(sm.qcnt, QCAP4), co = min(max(sm.qcnt - QCAP4, 0), ovf_r);
    if (threadIdx.x == 0) sm.qbase = (c + co) ? (int)atomicAdd(gcnt, (u32)(c + co)) : 0;
    __syncthreads();
    u32 fe = 0;  // adjacency entries of the next frontier (direction choice)
    for (int j = threadIdx.x; j < c; j += NT) {
      const int4 q = reinterpret_cast<const int4 *>(sm.q)[j];
      next[sm.qbase + j] = q;
      fe += (u32)(q.z - q.y);
    }
    for (int j = threadIdx.x; j < co; j += NT) {
      const int4 q = __ldcg(p.ovf + (long long)blockIdx.x * ovf_r + j);
      next[sm.qbase + c + j] = q;
      fe += (u32)(q.z - q.y);
    }
    if (fe_on) {  // the CTA's sum rides on the two barriers below
      fe = __reduce_add_sync(0xffffffffu, fe);
      if (lane_id() == 0 && fe) atomicAdd(&sm.lvc[1], fe);
    }
    __syncthreads();
    if (threadIdx.x == 0) {
      sm.qcnt = 0;
      if (sm.lvc[0]) {
        atomicAdd(ring_now(2), sm.lvc[0]);
        sm.lvc[0] = 0;
      }
      if (fe_on && sm.lvc[1]) {
        atomicAdd(ring_now(4), sm.lvc[1]);
        sm.lvc[1] = 0;
      }
    }
    __syncthreads();
  }

  // ---------------------------------------------------------------- stable compaction
  // Pass 1 of a stable compaction of items [0, len): f(i0, hi, val) fills val[k]
  // with the value to keep for item i0 + k (< hi) or -1 -- RB consecutive items per
  // thread, so f can issue each stage's loads for all of them at once.  Survivors
  // of CTA c's chunk go to T[lo_c + rank]; ctacnt[c] = count.  GRID=false: a single
  // CTA, written straight to `out` (a tile's reads finish before its writes -- the
  // scan's barrier separates them -- and writes never pass the tile being read).
  template <bool GRID, int RB, class Fn>
  __device__ int compact_pass1(int len, Fn f, int *T, int *out) {
    const int C = ncta<GRID>(), c = cta<GRID>();
    const int chunk = (len + C - 1) / C;
    const int lo = min(len, c * chunk), hi = min(len, lo + chunk);
    int run = 0;
    for (int t = lo; t < hi; t += NT * RB) {
      int val[RB];
      f(t + (int)threadIdx.x * RB, hi, val);
      int cnt = 0;
#pragma unroll
      for (int k = 0; k < RB; k++) cnt += val[k] != -1;
      int tot, r = cta_scan<NT>(cnt, sm.w, &tot);
      int *dst = (C > 1 ? T + lo : out) + run + r;
#pragma unroll
      for (int k = 0; k < RB; k++)
        if (val[k] != -1) *dst++ = val[k];
      run += tot;
    }
    if (C > 1 && threadIdx.x == 0) p.ctacnt[c] = run;
    return run;
  }
  // Pass 2 (after a barrier): move T[lo_c ..] to out[offset_c ..]; returns the total.
  template <bool GRID>
  __device__ int compact_pass2(int len, const int *T, int *out, int run1, int *out2 = nullptr) {
    const int C = ncta<GRID>(), c = cta<GRID>();
    if (C == 1) {
      if (out2)
        for (int j = threadIdx.x; j < run1; j += NT) out2[j] = __ldcg(out + j);
      return run1;
    }
    const int chunk = (len + C - 1) / C;
    const int lo = min(len, c * chunk);
    long long before = 0, total = 0;
    for (int j = threadIdx.x; j < C; j += NT) {
      int x = __ldcg(p.ctacnt + j);
      total += x;
      if (j < c) before += x;
    }
    before = cta_sum<NT>(before, sm.red);
    total = cta_sum<NT>(total, sm.red);
    int mine = __ldcg(p.ctacnt + c);
    for (int j = threadIdx.x; j < mine; j += NT) {
      int x = __ldcg(T + lo + j);
      out[before + j] = x;
      if (out2) out2[before + j] = x;
    }
    return (int)total;
  }

  // ---------------------------------------------------------------- init
  // Vertex state from the initial matching (GIVEN / RELABEL / UNIT: the caller's
  // arrays; else empty).  Labels start stale (psi = 0 < base), except in MODE_UNIT.
  // Returns this thread's count of out-of-range inputs.
  __device__ long long init_state() {
    const int G = gridDim.x * NT, g = blockIdx.x * NT + threadIdx.x;
    if (p.mode == MODE_GAP) {
      for (int u = g; u < m; u += G) {
        int l = p.rmatch_in[u];
        vst(p.rowst + u, pack(-1, (l >= 0 && l < INF) ? 1u + (u32)l : 0u));
      }
      for (int v = g; v < n; v += G) {
        int l = p.cmatch_in[v];
        vst(p.colst + v, pack(-1, (l >= 0 && l < INF) ? 1u + (u32)l : 0u));
      }
      return 0;
    }
    // a caller's matching (GIVEN solve, relabel, unit) is range-checked here: a bad
    // entry is counted (-> MCM_EINVAL after the barrier) and read as -1, so no
    // later phase can index outside rowst / colst.  Columns may carry the internal
    // -2 ("dead") mark in the relabel and unit modes only.
    const bool given = p.mode == MODE_RELABEL || p.mode == MODE_UNIT || (p.mode == MODE_SOLVE && p.init == 1);
    const int cmin = p.mode == MODE_SOLVE ? -1 : -2;
    const bool unit = p.mode == MODE_UNIT;
    long long bad = 0, dead = 0;
    for (int u = g; u < m; u += G) {
      int x = given ? p.rmatch_in[u] : -1;
      if (x < -1 || x >= n) { bad++; x = -1; }
      vst(p.rowst + u, pack(x, unit ? enc_label(p.psi_row_io[u]) : 0u));
    }
    for (int v = g; v < n; v += G) {
      int x = given ? p.cmatch_in[v] : -1;
      if (x < cmin || x >= m) { bad++; x = -1; }
      dead += x == -2;
      vst(p.colst + v, pack(x, unit ? enc_label(p.psi_col_io[v]) : 0u));
      if (!unit) p.iA[v] = -1;  // R12 (unit: the caller's iA)
    }
    if (unit)
      for (int i = g; i < p.unit_len; i += G) {
        const int a = p.wl0[i], b = p.wl1[i];
        bad += (a < -1 || a >= n) + (b < -1 || b >= n);
        if (a < -1 || a >= n) p.wl0[i] = -1;
        if (b < -1 || b >= n) p.wl1[i] = -1;
      }
    // relabel mode: -2 columns count as dead for the early-stop target (R22)
    dead = cta_sum<NT>(dead, sm.red);
    if (threadIdx.x == 0 && dead && p.mode == MODE_RELABEL) atomicAdd(&p.ctrl->ndead, (u32)dead);
    return bad;
  }
  // label l of a caller (MODE_UNIT) -> stored word value at base 1: 1 + l when
  // finite, 0 (stale = m+n) otherwise
  __device__ __forceinline__ u32 enc_label(int l) const { return (l >= 0 && l < INF) ? 1u + (u32)l : 0u; }

  // Cheap greedy matching on the device (reading R13): every column claims the
  // first free row of Gamma(v) with a CAS.  A column fails only when every
  // neighbour is taken, so the result is maximal.  (Outside the push loop, the
  // paper's atomic-free claim concerns the push-relabel steps.)
  __device__ void greedy() {
    // RG columns per lane (a warp tile of 32*RG columns): the bounds, the first KB
    // candidates and their row words of all RG columns are loaded stage by stage and
    // the RG claims issued together, so a thread keeps RG independent chains in
    // flight; a column whose first free candidate was taken meanwhile (or that has
    // none among its first KB) continues alone from there.
    constexpr int RG = MCM_RG;
    const int lane = lane_id();
    const int gw = (blockIdx.x * NT + threadIdx.x) >> 5, NWG = gridDim.x * NWARP;
    for (long long b = (long long)gw * 32 * RG; b < n; b += (long long)NWG * 32 * RG) {
      int v[RG], s[RG], e[RG];
#pragma unroll
      for (int k = 0; k < RG; k++) {
        const long long x = b + k * 32 + lane;
        v[k] = x < n ? (int)x : -1;
      }
#pragma unroll
      for (int k = 0; k < RG; k++) {
        s[k] = v[k] >= 0 ? ld_ro(p.cptr + v[k]) : 0;
        e[k] = v[k] >= 0 ? ld_ro(p.cptr + v[k] + 1) : 0;
      }
      int u[RG][KB];
      u64 rs[RG][KB];
      // lists longer than KB: the first KB candidates start at a column-dependent
      // rotation of Gamma(v) (reading R13), so the first claims of R-MAT columns,
      // whose lists all begin with the same few hub rows, spread over their rows; a
      // column whose candidates were all taken then walks its whole list from s
      int rot[RG];
#pragma unroll
      for (int k = 0; k < RG; k++) {
        const int d = e[k] - s[k];
        rot[k] = d > KB ? (int)(((u32)v[k] * 2654435761u) % (u32)d) : 0;
      }
#pragma unroll
      for (int k = 0; k < RG; k++)
#pragma unroll
        for (int q = 0; q < KB; q++) {
          const int d = e[k] - s[k];
          int x = rot[k] + q;
          if (x >= d) x -= d;
          u[k][q] = q < d ? ld_adj(p.cadj + s[k] + x) : -1;
        }
#pragma unroll
      for (int k = 0; k < RG; k++)
#pragma unroll
        for (int q = 0; q < KB; q++) rs[k][q] = u[k][q] >= 0 ? vld(p.rowst + u[k][q]) : 0ull;
      int pos[RG];
      bool done[RG];
      u64 exp_[RG], old[RG];
      int cu[RG];
#pragma unroll
      for (int k = 0; k < RG; k++) {
        int pick = -1;
#pragma unroll
        for (int q = KB - 1; q >= 0; q--)
          if (u[k][q] >= 0 && mu_of(rs[k][q]) == -1) pick = q;
        const int deg = e[k] - s[k];
        if (v[k] >= 0) S(SS_GYEDGES) += pick >= 0 ? pick + 1 : min(deg, KB);
        cu[k] = -1;
        exp_[k] = 0;
#pragma unroll
        for (int q = 0; q < KB; q++)
          if (q == pick) { cu[k] = u[k][q]; exp_[k] = rs[k][q]; }
        pos[k] = rot[k] ? s[k] : (pick >= 0 ? s[k] + pick + 1 : s[k] + KB);
      }
#pragma unroll
      for (int k = 0; k < RG; k++)
        old[k] = cu[k] >= 0 ? atomicCAS(p.rowst + cu[k], exp_[k], pack(v[k], psi_of(exp_[k]))) : ~exp_[k];
#pragma unroll
      for (int k = 0; k < RG; k++) {
        done[k] = cu[k] >= 0 && old[k] == exp_[k];
        if (done[k]) vst(p.colst + v[k], pack(cu[k], 0));
      }
#pragma unroll
      for (int k = 0; k < RG; k++) {
        if (v[k] >= 0 && e[k] - s[k] <= SMALL_DEG && !done[k]) {  // the rest of a short list, alone
          bool dn = false;
          for (int j0 = pos[k]; j0 < e[k] && !dn; j0 += KB) {
            int uu[KB];
            u64 rr[KB];
#pragma unroll
            for (int q = 0; q < KB; q++) uu[q] = j0 + q < e[k] ? ld_adj(p.cadj + j0 + q) : -1;
#pragma unroll
            for (int q = 0; q < KB; q++) rr[q] = uu[q] >= 0 ? vld(p.rowst + uu[q]) : 0ull;
#pragma unroll
            for (int q = 0; q < KB; q++) {
              if (dn || uu[q] < 0) continue;
              S(SS_GYEDGES)++;
              if (mu_of(rr[q]) != -1) continue;
              if (atomicCAS(p.rowst + uu[q], rr[q], pack(v[k], psi_of(rr[q]))) == rr[q]) {
                vst(p.colst + v[k], pack(uu[q], 0));
                dn = true;
              }
            }
          }
        }
        unsigned big = __ballot_sync(0xffffffffu, v[k] >= 0 && e[k] - s[k] > SMALL_DEG && !done[k] && pos[k] < e[k]);
        while (big) {  // the rest of a long list: the whole warp
          int bl = __ffs(big) - 1;
          big &= big - 1;
          int vb = __shfl_sync(0xffffffffu, v[k], bl);
          int sb = __shfl_sync(0xffffffffu, pos[k], bl), eb = __shfl_sync(0xffffffffu, e[k], bl);
          bool dn = false;
          for (int c0 = sb; c0 < eb && !dn; c0 += 32) {
            int j = c0 + lane;
            int uu = -1;
            u64 rr = 0;
            if (j < eb) { uu = ld_adj(p.cadj + j); rr = vld(p.rowst + uu); S(SS_GYEDGES)++; }
            unsigned cand = __ballot_sync(0xffffffffu, uu >= 0 && mu_of(rr) == -1);
            while (cand && !dn) {
              int l = __ffs(cand) - 1;
              cand &= cand - 1;
              int ok = 0;
              if (lane == l) {
                ok = atomicCAS(p.rowst + uu, rr, pack(vb, psi_of(rr))) == rr;
                if (ok) vst(p.colst + vb, pack(uu, 0));
              }
              dn = __shfl_sync(0xffffffffu, ok, l);
            }
          }
        }
      }
    }
  }

  // unmatched rows -> U (any order); ring j
  // solve mode: rows without any edge can never be matched nor reach a column, so
  // they stay out of U (their count goes to ring counter j+1)
  __device__ void build_unmatched_rows(int *U, int j) {
    // RB rows per thread per tile, all loads of a stage issued before any is used
    // (the vertex-state loads are volatile asm: written one item at a time they
    // would run as RB dependent round trips); one reservation per tile
    constexpr int RB = 8;
    long long iso = 0;
    for (long long t = (long long)blockIdx.x * NT * RB; t < m; t += (long long)gridDim.x * NT * RB) {
      int u[RB];
      u64 w[RB];
      int rs[RB], re[RB];
#pragma unroll
      for (int k = 0; k < RB; k++) {
        const long long x = t + k * NT + threadIdx.x;
        u[k] = x < m ? (int)x : -1;
      }
#pragma unroll
      for (int k = 0; k < RB; k++) w[k] = u[k] >= 0 ? vld(p.rowst + u[k]) : 0ull;
      const bool need_deg = p.mode == MODE_SOLVE;
#pragma unroll
      for (int k = 0; k < RB; k++) {
        const bool f = u[k] >= 0 && mu_of(w[k]) == -1 && need_deg;
        rs[k] = f ? ld_ro(p.rptr + u[k]) : 0;
        re[k] = f ? ld_ro(p.rptr + u[k] + 1) : 1;
      }
      int cnt = 0;
      unsigned fm = 0;
#pragma unroll
      for (int k = 0; k < RB; k++) {
        bool f = u[k] >= 0 && mu_of(w[k]) == -1;
        if (f && need_deg && rs[k] == re[k]) { f = false; iso++; }
        if (f) { fm |= 1u << k; cnt++; }
      }
      int tot, r = cta_scan<NT>(cnt, sm.w, &tot);
      if (threadIdx.x == 0) sm.qbase = tot ? (int)atomicAdd(ring_now(j), (u32)tot) : 0;
      __syncthreads();
      r += sm.qbase;
#pragma unroll
      for (int k = 0; k < RB; k++)
        if (fm >> k & 1) U[r++] = u[k];
    }
    add_count(iso, j + 1);
  }

  // ---------------------------------------------------------------- global relabel
  // One BFS level (Alg. 5, as a frontier expansion): every row u of
  // `cur` (label lvl) visits the unvisited columns v of Gamma(u): psi(v) = lvl+1;
  // if v is matched (mu(v) > -1 and mu(mu(v)) = v) its mate gets lvl+2 and joins
  // `next`.  A CAS claims each column once per GR, so each row joins once.
  // lvl == 0: `cur` is the unmatched-row list U; rows that got matched since are
  // dropped, the others get label 0 (INITRELABEL) and are written to
  // Uout (the filtered U).
  // Lanes per vertex for a phase over `items` vertices on `threads` threads: the
  // largest power of two <= 32 with items * G <= threads, so narrow frontiers and
  // short worklists spread each adjacency list over a lane group instead of
  // walking it one dependent load at a time.
  __device__ __forceinline__ static int pick_group(long long items, int threads) {
    int g = 1;
    while (g < 32 && items * (g * 2) <= threads) g <<= 1;
    return g;
  }
  __device__ __forceinline__ static unsigned group_mask(int G) {
    return G == 32 ? 0xffffffffu : (((1u << G) - 1u) << (lane_id() & ~(G - 1)));
  }

  // One BFS level (Alg. 5).  lvl == 0: `cur0` is the unmatched-row list U (rows
  // matched since are dropped, the others get label 0 and go to Uout); lvl > 0:
  // `cur4` holds the frontier entries of the previous level.
  template <bool GRID>
  __device__ void gr_level(const int *cur0, const int4 *cur4, int curlen, int lvl, u32 base, int4 *next, u32 *ncnt,
                           int *Uout, u32 *ucnt, int *guard, u32 *gcnt) {
    const int lane = lane_id();
    const u32 lc = base + lvl + 1, lr = base + lvl + 2;
    if (GRID && lvl > 0 && curlen > 2 * NT * ncta<GRID>()) {
      // wide level: two frontier entries per thread per tile, their adjacency
      // expanded as one list in batches of 2*KB (twice the loads in flight of a
      // one-entry tile; the kernel's register budget caps the batch)
      int wt = 0;
      for (int t = cta<GRID>() * 2 * NT; t < curlen; t += ncta<GRID>() * 2 * NT) {
        const int i0 = t + (int)threadIdx.x, i1 = i0 + NT;
        int4 q0 = i0 < curlen ? ld_q(cur4 + i0) : make_int4(-1, 0, 0, 0);
        int4 q1 = i1 < curlen ? ld_q(cur4 + i1) : make_int4(-1, 0, 0, 0);
        if (q0.x >= 0) { S(SS_GRROWS) += !(q0.w & 1); S(SS_GREDGES) += q0.z - q0.y; }
        if (q1.x >= 0) { S(SS_GRROWS) += !(q1.w & 1); S(SS_GREDGES) += q1.z - q1.y; }
        const bool big0 = q0.x >= 0 && q0.z - q0.y > BIG_DEG, big1 = q1.x >= 0 && q1.z - q1.y > BIG_DEG;
        expand_pair(big0 || q0.x < 0 ? 0 : q0.z - q0.y, q0.y, big1 || q1.x < 0 ? 0 : q1.z - q1.y, q1.y, lc, lr, next,
                    ncnt, guard, gcnt);
#pragma unroll
        for (int h = 0; h < 2; h++) {
          const int4 q = h ? q1 : q0;
          unsigned bigm = __ballot_sync(0xffffffffu, h ? big1 : big0);
          while (bigm) {  // long lists: the whole warp
            int bl = __ffs(bigm) - 1;
            bigm &= bigm - 1;
            int sb = __shfl_sync(0xffffffffu, q.y, bl), eb = __shfl_sync(0xffffffffu, q.z, bl);
            expand(sb + lane, eb, 32, lc, lr, next, ncnt, guard, gcnt, false);
          }
        }
        // every MCM_WFLUSH tiles (0: once per level): a flush is a few CTA barriers,
        // and without it a wide level's output overflows the shared staging into the
        // CTA's global overflow region (one more copy)
        if (MCM_WFLUSH > 0 && ++wt % (MCM_WFLUSH > 0 ? MCM_WFLUSH : 1) == 0) flush(next, ncnt);
      }
      flush(next, ncnt);
      return;
    }
    const int G = pick_group(curlen, ncta<GRID>() * NT);
    const int gl = lane & (G - 1), per_tile = NT / G;
    if (GRID && lvl > 0 && MCM_FINE) tmark(101, curlen);
    for (int t = cta<GRID>() * per_tile; t < curlen; t += ncta<GRID>() * per_tile) {
      int i = t + (int)threadIdx.x / G;
      int u = -1, s = 0, e = 0, cont = 0;
      if (lvl == 0) {
        u = (i < curlen) ? ld_cg(cur0 + i) : -1;
        bool keep = false;
        if (u >= 0) {
          if (mu_of(vld(p.rowst + u)) == -1) {
            if (gl == 0) vst(p.rowst + u, pack(-1, base));
            keep = gl == 0;
          } else {
            u = -1;
          }
        }
        if (keep) {  // filtered U: any order, one atomic per coalesced group (no CTA barrier;
                     // a per-tile CTA reservation measured 10% slower on C4, equal on C3 / C5)
          cg::coalesced_group kg = cg::coalesced_threads();
          u32 b = 0;
          if (kg.thread_rank() == 0) b = atomicAdd(ucnt, (u32)kg.size());
          Uout[kg.shfl(b, 0) + kg.thread_rank()] = u;
        }
        if (u >= 0) { s = ld_ro(p.rptr + u); e = ld_ro(p.rptr + u + 1); }
      } else if (i < curlen) {
        int4 q = ld_q(cur4 + i);
        u = q.x; s = q.y; e = q.z; cont = q.w & 1;
      }
      if (GRID && lvl > 0 && MCM_FINE && t == cta<GRID>() * per_tile) tmark(102, 0);
      if (u >= 0 && gl == 0) { S(SS_GRROWS) += !cont; S(SS_GREDGES) += e - s; }
      const bool big = u >= 0 && G < 32 && e - s > BIG_DEG;
      if (u >= 0 && !big) expand(s + gl, e, G, lc, lr, next, ncnt, guard, gcnt, G >= 4);
      unsigned bigm = __ballot_sync(0xffffffffu, big && gl == 0);
      while (bigm) {  // long lists: the whole warp
        int bl = __ffs(bigm) - 1;
        bigm &= bigm - 1;
        int sb = __shfl_sync(0xffffffffu, s, bl), eb = __shfl_sync(0xffffffffu, e, bl);
        expand(sb + lane, eb, 32, lc, lr, next, ncnt, guard, gcnt, false);
      }
      if (GRID && lvl > 0 && MCM_FINE && t == cta<GRID>() * per_tile) tmark(103, 0);
    }
    flush(next, ncnt);  // once per level
  }
  // Visit radj[j], j = j0, j0+step, ... < e, KB at a time.  A CAS claims each
  // column once per GR (so every row joins the next frontier once and every
  // reached unmatched column is counted once); the mate check and the mate's
  // adjacency bounds are loaded in the same round trip as the CAS (they depend only
  // on the column word), so a level costs: column loads -> {CAS, mate, bounds}.
  __device__ __forceinline__ void expand(int j0, int e, int step, u32 lc, u32 lr, int4 *next, u32 *ncnt, int *guard,
                                         u32 *gcnt, bool spec) {
    for (int j = j0; j < e; j += step * KB) {
      int v[KB];
      u64 cs[KB], old[KB], rw[KB];
      int rs[KB], re[KB];
#pragma unroll
      for (int k = 0; k < KB; k++) {
        int jj = j + k * step;
        v[k] = jj < e ? ld_adj(p.radj + jj) : -1;
      }
#pragma unroll
      for (int k = 0; k < KB; k++) cs[k] = v[k] >= 0 ? vld(p.colst + v[k]) : ~0ull;
      if (spec) {  // narrow level: mate loads ride along with the CAS (one round trip)
#pragma unroll
        for (int k = 0; k < KB; k++) {
          // unvisited in this GR <=> its label is from an older epoch (< base)
          const bool try_ = v[k] >= 0 && psi_of(cs[k]) < gr_base;
          const int w = mu_of(cs[k]);
          old[k] = try_ ? atomicCAS(p.colst + v[k], cs[k], pack(w, lc)) : ~cs[k];
          const bool go = try_ && w >= 0;
          rw[k] = go ? vld(p.rowst + w) : 0ull;
          rs[k] = go ? ld_ro(p.rptr + w) : 0;
          re[k] = go ? ld_ro(p.rptr + w + 1) : 0;
        }
      } else {  // wide level: only CAS winners load their mate (no wasted traffic)
#pragma unroll
        for (int k = 0; k < KB; k++) {
          const bool try_ = v[k] >= 0 && psi_of(cs[k]) < gr_base;
          old[k] = try_ ? atomicCAS(p.colst + v[k], cs[k], pack(mu_of(cs[k]), lc)) : ~cs[k];
        }
#pragma unroll
        for (int k = 0; k < KB; k++) {
          const int w = mu_of(cs[k]);
          const bool go = old[k] == cs[k] && w >= 0;
          rw[k] = go ? vld(p.rowst + w) : 0ull;
          rs[k] = go ? ld_ro(p.rptr + w) : 0;
          re[k] = go ? ld_ro(p.rptr + w + 1) : 0;
        }
      }
#pragma unroll
      for (int k = 0; k < KB; k++) {
        if (old[k] != cs[k]) continue;  // not claimed by this thread
        S(SS_GRCOLS)++;
        int w = mu_of(cs[k]);
        if (w >= 0 && mu_of(rw[k]) == v[k]) {  // matched: mu(v) > -1 and mu(mu(v)) = v
          vst(p.rowst + w, pack(v[k], lr));
          stage_row(w, rs[k], re[k], next, ncnt);
        } else {
          S(SS_FREE)++;
          if (guard) guard[atomicAdd(gcnt, 1u)] = v[k];
          if (mu_of(cs[k]) != -2) count_free();  // an alive unmatched column got its label
        }
      }
    }
  }
  // expand() over the concatenation of two adjacency ranges radj[s0, s0+d0) and
  // radj[s1, s1+d1), 2*KB entries per batch, wide-level claiming (only CAS winners
  // load their mate)
  __device__ __forceinline__ void expand_pair(int d0, int s0, int d1, int s1, u32 lc, u32 lr, int4 *next, u32 *ncnt,
                                              int *guard, u32 *gcnt) {
    constexpr int B = MCM_EB;
    const int tot = d0 + d1;
    for (int o = 0; o < tot; o += B) {
      int v[B];
      u64 cs[B], old[B], rw[B];
      int rs[B], re[B];
#pragma unroll
      for (int k = 0; k < B; k++) {
        const int x = o + k;
        v[k] = x < d0 ? ld_adj(p.radj + s0 + x) : (x < tot ? ld_adj(p.radj + s1 + (x - d0)) : -1);
      }
#pragma unroll
      for (int k = 0; k < B; k++) cs[k] = v[k] >= 0 ? vld(p.colst + v[k]) : ~0ull;
#pragma unroll
      for (int k = 0; k < B; k++) {
        const bool try_ = v[k] >= 0 && psi_of(cs[k]) < gr_base;
        old[k] = try_ ? atomicCAS(p.colst + v[k], cs[k], pack(mu_of(cs[k]), lc)) : ~cs[k];
      }
#pragma unroll
      for (int k = 0; k < B; k++) {
        const int w = mu_of(cs[k]);
        const bool go = old[k] == cs[k] && w >= 0;
        rw[k] = go ? vld(p.rowst + w) : 0ull;
        rs[k] = go ? ld_ro(p.rptr + w) : 0;
        re[k] = go ? ld_ro(p.rptr + w + 1) : 0;
      }
#pragma unroll
      for (int k = 0; k < B; k++) {
        if (old[k] != cs[k]) continue;  // not claimed by this thread
        S(SS_GRCOLS)++;
        const int w = mu_of(cs[k]);
        if (w >= 0 && mu_of(rw[k]) == v[k]) {  // matched: its mate joins the next level
          vst(p.rowst + w, pack(v[k], lr));
          stage_row(w, rs[k], re[k], next, ncnt);
        } else {
          S(SS_FREE)++;
          if (guard) guard[atomicAdd(gcnt, 1u)] = v[k];
          if (mu_of(cs[k]) != -2) count_free();
        }
      }
    }
  }
  // Bottom-up BFS level (direction-optimising GR): every column
  // not yet labelled in this GR looks for any row of Gamma(v) carrying the
  // current level `lvl`, stopping at the first one; a hit labels v lvl+1 and, if v
  // is matched, its mate lvl+2 (staged for the next level).  Produces exactly the
  // labels of the top-down level (BFS distances are unique) while reading a
  // fraction of the adjacency on wide levels.  One thread per column (no CAS:
  // each column is visited by its own thread); lists longer than BIG_DEG are
  // scanned by the whole warp with the same early exit.
  template <bool GRID>
  __device__ void gr_level_bu(int lvl, u32 base, int4 *next, u32 *ncnt, int *guard, u32 *gcnt) {
    const int lane = lane_id();
    const u32 lf = base + lvl, lc = base + lvl + 1, lr = base + lvl + 2;
    int bt = 0;
    for (int t = cta<GRID>() * NT; t < n; t += ncta<GRID>() * NT) {
      const int v = t + (int)threadIdx.x;
      u64 cs = 0;
      int s = 0, e = 0;
      bool open = false, hit = false;
      if (v < n) {
        cs = vld(p.colst + v);
        if (psi_of(cs) < base) {
          open = true;
          s = ld_ro(p.cptr + v);
          e = ld_ro(p.cptr + v + 1);
        }
      }
      if (open && e - s <= BIG_DEG) {
        for (int j = s; j < e && !hit; j += KB) {
          int x[KB];
          u64 rs[KB];
#pragma unroll
          for (int k = 0; k < KB; k++) x[k] = j + k < e ? ld_adj(p.cadj + j + k) : -1;
#pragma unroll
          for (int k = 0; k < KB; k++) rs[k] = x[k] >= 0 ? vld(p.rowst + x[k]) : 0ull;
#pragma unroll
          for (int k = 0; k < KB; k++) hit |= x[k] >= 0 && psi_of(rs[k]) == lf;
          S(SS_GREDGES) += min(KB, e - j);
        }
      }
      unsigned bigm = __ballot_sync(0xffffffffu, open && e - s > BIG_DEG);
      while (bigm) {  // long lists: the whole warp, exit at the first hit
        const int bl = __ffs(bigm) - 1;
        bigm &= bigm - 1;
        const int sb = __shfl_sync(0xffffffffu, s, bl), eb = __shfl_sync(0xffffffffu, e, bl);
        bool any = false;
        for (int c0 = sb; c0 < eb && !any; c0 += 32 * KB) {
          bool h = false;
#pragma unroll
          for (int k = 0; k < KB; k++) {
            const int jj = c0 + k * 32 + lane;
            if (jj < eb) h |= psi_of(vld(p.rowst + ld_adj(p.cadj + jj))) == lf;
          }
          any = __any_sync(0xffffffffu, h);
          if (lane == 0) S(SS_GREDGES) += min(32 * KB, eb - c0);
        }
        if (lane == bl) hit = any;
      }
      if (hit) {
        vst(p.colst + v, pack(mu_of(cs), lc));
        S(SS_GRCOLS)++;
        const int w = mu_of(cs);
        u64 rw = 0;
        int rs = 0, re = 0;
        if (w >= 0) { rw = vld(p.rowst + w); rs = ld_ro(p.rptr + w); re = ld_ro(p.rptr + w + 1); }
        if (w >= 0 && mu_of(rw) == v) {  // matched: its mate joins the next level
          vst(p.rowst + w, pack(v, lr));
          stage_row(w, rs, re, next, ncnt);
        } else {
          S(SS_FREE)++;
          if (guard) guard[atomicAdd(gcnt, 1u)] = v;
          if (w != -2) count_free();
        }
      }
      // every MCM_BUFLUSH tiles: a bottom-up level walks all n columns (C3: ~300
      // tiles per CTA), so its output would overflow the shared staging
      if (++bt % MCM_BUFLUSH == 0) flush(next, ncnt);
    }
    flush(next, ncnt);
  }
  // bottom-up when the frontier's adjacency entries reach bu_div/8 times the
  // columns still unlabelled (Beamer-style edge rule; frontier rows alone mislead on
  // low-degree road graphs)
  __device__ __forceinline__ bool use_bottom_up(long long fedges, long long unvisited, int nlen) const {
    return (F & F_BU) && p.bu_div > 0 && fedges * 8 >= unvisited * (long long)p.bu_div && (long long)nlen * 64 >= n;
  }

  u32 gr_base = 0;
  // Direction choice bookkeeping (bottom-up BFS levels): the adjacency entries of
  // the next frontier (ring counter 4) are summed only when the current frontier is
  // within a factor 4 of the bottom-up size threshold (flush, fe_on); the columns
  // labelled so far follow from counters the level produces anyway (next-frontier
  // rows + reached unmatched columns), so narrow levels pay nothing for it.
  bool fe_on = false;
  __device__ __forceinline__ void set_fe(long long nlen) {
    fe_on = (F & F_BU) && p.bu_div > 0 && nlen * 256 >= n;
  }
  int fl_r = 0, fl_c = 0;  // push: labels of vertices the last GR did not reach (set from Ctl)
  __device__ __forceinline__ int labf(u32 s, u32 base, int stale) const {
    return s >= base ? (int)min((u64)(s - base), (u64)INF + 1) : stale;
  }
  bool sq = false;          // tail GR: stage() writes straight into sq_next (shared)
  int4 *sq_next = nullptr;
  __device__ __forceinline__ int4 *sfr(int i) { return reinterpret_cast<int4 *>(sm.q) + i * TQ; }

  // Full GR (Alg. 4).  U/T: unmatched-row list and a free buffer
  // (swapped on return); Qa/Qb frontier buffers.  Returns maxLevel.
  // guard != nullptr: every reached column that is not matched is appended to
  // guard[0 .. gcount) (the exactness guard, R16).
  template <bool GRID>
  __device__ int global_relabel(int *&U, int &ulen, int *&T, int4 *Qa, int4 *Qb, u32 base, int *guard, int &gcount) {
    GRState g;
    gr_start<GRID>(g, U, ulen, T, Qa, base, guard);
    gr_levels<GRID>(g, base, Qa, Qb, guard, 0x7fffffff);
    gcount = (int)bcast_ld(&p.ctrl->gcnt);
    return g.deepest + 2;
  }

  // The GR as a resumable state machine, so that a CTA-local GR (tail mode) can
  // hand a frontier that grew too wide over to the whole grid mid-BFS.
  struct GRState {
    int lvl, deepest, nlen, cur_is_a, in_smem, reached, target, dirty;  // reached/target: early stop (R22)
                                                                        // dirty: a window left labels below
                                                                        // its end in the frontier
    long long fedges, visited;  // next frontier's adjacency entries; columns labelled in this GR
  };
  // level 0 (INITRELABEL + first expansion): U -> filtered U (in T, then swapped), frontier -> Qa
  template <bool GRID>
  __device__ void gr_start(GRState &g, int *&U, int &ulen, int *&T, int4 *Qa, u32 base, int *guard) {
    gr_base = base;
    u32 *gc = &p.ctrl->gcnt;  // zero here: reset one phase after its last use
    trace(1, ulen);
    set_fe(ulen);
    gr_level<GRID>(U, nullptr, ulen, 0, base, Qa, ring_now(0), T, ring_now(1), guard, gc);
    barrier<GRID>();
    g.nlen = (int)ring_prev(0);
    g.fedges = ring_prev(4);
    g.visited = (long long)g.nlen + ring_prev(2);
    g.reached = (int)ring_prev(2);
    ulen = (int)ring_prev(1);
    int *tmp = U; U = T; T = tmp;
    g.lvl = 0; g.deepest = 0; g.cur_is_a = 1;
  }
  // levels 2, 4, ... until the frontier is empty (returns true) or, before expanding
  // a level, the frontier exceeds `limit` (returns false; state kept for resuming).
  template <bool GRID>
  __device__ bool gr_levels(GRState &g, u32 base, int4 *Qa, int4 *Qb, int *guard, int limit) {
    gr_base = base;
    u32 *gc = &p.ctrl->gcnt;
    while (g.nlen > 0) {
      if (g.nlen > limit) return false;
      g.lvl += 2;
      g.deepest = g.lvl;
      int4 *cur = g.cur_is_a ? Qa : Qb, *nxt = g.cur_is_a ? Qb : Qa;
      trace(2, g.nlen);
      set_fe(g.nlen);
      if (GRID && use_bottom_up(g.fedges, (long long)n - g.visited, g.nlen))
        gr_level_bu<GRID>(g.lvl, base, nxt, ring_now(0), guard, gc);
      else
        gr_level<GRID>(nullptr, cur, g.nlen, g.lvl, base, nxt, ring_now(0), nullptr, nullptr, guard, gc);
      barrier<GRID>();
      g.nlen = (int)ring_prev(0);
      g.fedges = ring_prev(4);
      g.visited += (long long)g.nlen + ring_prev(2);
      g.cur_is_a ^= 1;
    }
    return true;
  }

  // ---------------------------------------------------------------- windowed GR levels
  // Option gr_window = K > 1 (a build addition; the paper's GR is level-synchronous,
  // Alg. 5): K BFS levels per grid barrier.  Every CTA expands its share of the
  // frontier (rows with label L0, entries carrying their label offset in .w, see
  // below) and then, without leaving the CTA, the rows that share discovers, level
  // after level (a shared-memory queue and CTA barriers), until every row it reached
  // with a label below Lend = L0 + 2K is expanded; rows reached with label Lend form
  // the next (global) frontier.  Because the CTAs run ahead of one another, a vertex
  // can first be reached by a longer path: labels are lowered by CAS (a column's
  // word, then its mate row's) and a row whose label was lowered is expanded again
  // with the smaller label (label correcting).  When every CTA's queue is empty (the
  // window's grid barrier) every vertex whose BFS distance is below Lend carries its
  // exact distance (its shortest path's rows were each expanded with their exact
  // label), and the frontier rows carry exactly Lend -- the state a level-synchronous
  // BFS reaches after the level of L0 + 2K - 2, so the early stop (R22 / R28), the
  // floors and maxLevel are as if the levels had run one by one.  A local queue that
  // overflows sends its row to the global frontier with its own label (.w offset)
  // and marks the window dirty: the next unit of GR work is then another window (its
  // L0 = Lend decodes the offsets), and no stop test or hand-over happens before a
  // clean window.  Frontier entry .w: bit 0 = continuation of a split row, the rest
  // = L0 - label (0 for every entry of a level-synchronous frontier).
  static constexpr int LQ = 512;
  __device__ __forceinline__ bool lower_ok(u64 w, u32 l) const { return psi_of(w) < gr_base || psi_of(w) > l; }
  // queue a row range for this CTA's next sub-level (label lab), or, when the queue
  // is full, for the next window (dirty)
  __device__ __forceinline__ void lpush(int4 x, int nb, int lab, int L0n, int4 *next, u32 *gcnt) {
    cg::coalesced_group g = cg::coalesced_threads();
    int b = 0;
    if (g.thread_rank() == 0) b = atomicAdd(&sm.lqn[nb], (int)g.size());
    b = g.shfl(b, 0) + (int)g.thread_rank();
    if (b < LQ) {
      x.w |= lab;
      sm.lq[nb][b] = x;
    } else {
      x.w |= L0n - lab;
      stage(x, next, gcnt);
      sm.lwdirty = 1;
    }
  }
  __device__ __forceinline__ void lpush_row(int w, int s, int e, int nb, int lab, int Lend, int4 *next, u32 *gcnt) {
    for (int c = s; c < e || c == s; c += SPLIT) {
      lpush(make_int4(w, c, min(e, c + SPLIT), c > s), nb, lab, Lend, next, gcnt);
      if (e - s <= SPLIT) break;
    }
  }
  // expand radj[j0, e) (stride `step`) of a row with label lab: columns get lab+1,
  // their mates lab+2 (queued below Lend, staged at Lend)
  __device__ __forceinline__ void expand_w(int j0, int e, int step, int lab, int Lend, int nb, int4 *next,
                                           u32 *ncnt) {
    const u32 lc = gr_base + (u32)lab + 1u, lr = lc + 1u;
    for (int j = j0; j < e; j += step * KB) {
      int v[KB], rs[KB], re[KB];
      u64 cs[KB], old[KB], rw[KB];
      bool won[KB];
#pragma unroll
      for (int k = 0; k < KB; k++) {
        int jj = j + k * step;
        v[k] = jj < e ? ld_adj(p.radj + jj) : -1;
      }
#pragma unroll
      for (int k = 0; k < KB; k++) cs[k] = v[k] >= 0 ? vld(p.colst + v[k]) : 0ull;
#pragma unroll
      for (int k = 0; k < KB; k++) {  // claim (lower) the column; the mate's word rides along
        const bool try_ = v[k] >= 0 && lower_ok(cs[k], lc);
        const int w = mu_of(cs[k]);
        old[k] = try_ ? atomicCAS(p.colst + v[k], cs[k], pack(w, lc)) : ~cs[k];
        const bool go = try_ && w >= 0;
        rw[k] = go ? vld(p.rowst + w) : 0ull;
        rs[k] = go ? ld_ro(p.rptr + w) : 0;
        re[k] = go ? ld_ro(p.rptr + w + 1) : 0;
      }
#pragma unroll
      for (int k = 0; k < KB; k++) {
        won[k] = old[k] == cs[k];
        if (!won[k] && v[k] >= 0 && old[k] != ~cs[k]) {  // lost a race: retry while still lower
          u64 cur = old[k];
          while (lower_ok(cur, lc)) {
            const u64 o = atomicCAS(p.colst + v[k], cur, pack(mu_of(cur), lc));
            if (o == cur) { won[k] = true; break; }
            cur = o;
          }
          if (won[k]) {
            cs[k] = cur;
            const int w = mu_of(cur);
            rw[k] = w >= 0 ? vld(p.rowst + w) : 0ull;
            rs[k] = w >= 0 ? ld_ro(p.rptr + w) : 0;
            re[k] = w >= 0 ? ld_ro(p.rptr + w + 1) : 0;
          }
        }
      }
#pragma unroll
      for (int k = 0; k < KB; k++) {  // lower the mate rows (all CASes in flight)
        const int w = mu_of(cs[k]);
        const bool mt = won[k] && w >= 0 && mu_of(rw[k]) == v[k];
        old[k] = (mt && lower_ok(rw[k], lr)) ? atomicCAS(p.rowst + w, rw[k], pack(v[k], lr)) : ~rw[k];
        if (won[k] && !mt) {  // an unmatched column (first label only: counted once)
          if (psi_of(cs[k]) < gr_base) {
            S(SS_FREE)++;
            if (mu_of(cs[k]) != -2) count_free();
          }
        }
        if (won[k] && psi_of(cs[k]) < gr_base) S(SS_GRCOLS)++;
      }
#pragma unroll
      for (int k = 0; k < KB; k++) {
        const int w = mu_of(cs[k]);
        if (!(won[k] && w >= 0 && mu_of(rw[k]) == v[k])) continue;
        bool low = old[k] == rw[k];
        if (!low && old[k] != ~rw[k]) {
          u64 cur = old[k];
          while (lower_ok(cur, lr)) {
            const u64 o = atomicCAS(p.rowst + w, cur, pack(v[k], lr));
            if (o == cur) { low = true; break; }
            cur = o;
          }
        }
        if (!low) continue;
        if (lab + 2 < Lend) {
          lpush_row(w, rs[k], re[k], nb, lab + 2, Lend, next, ncnt);
        } else {
          stage_row(w, rs[k], re[k], next, ncnt);
        }
      }
    }
  }
  // one entry (a row range with its label) by a lane group of G lanes; longer lists
  // by the whole warp
  __device__ __forceinline__ void win_entry(int4 q, bool ok, int lab, int G, int gl, int Lend, int nb, int4 *next,
                                            u32 *ncnt, int &mx) {
    const int lane = lane_id();
    if (ok && gl == 0) { S(SS_GRROWS) += !(q.w & 1); S(SS_GREDGES) += q.z - q.y; }
    if (ok) mx = max(mx, lab);
    const bool big = ok && G < 32 && q.z - q.y > BIG_DEG;
    if (ok && !big) expand_w(q.y + gl, q.z, G, lab, Lend, nb, next, ncnt);
    unsigned bigm = __ballot_sync(0xffffffffu, big && gl == 0);
    while (bigm) {
      int bl = __ffs(bigm) - 1;
      bigm &= bigm - 1;
      int sb = __shfl_sync(0xffffffffu, q.y, bl), eb = __shfl_sync(0xffffffffu, q.z, bl);
      int lb = __shfl_sync(0xffffffffu, lab, bl);
      expand_w(sb + lane, eb, 32, lb, Lend, nb, next, ncnt);
    }
  }
  // One window: the frontier cur4[0, curlen) (rows at L0, .w offsets) -> rows at
  // Lend in `next`.  Ring counters: 0 next-frontier length (stage/flush), 2 alive
  // unmatched columns labelled, 3 deepest expanded row label + 1, 4 next-frontier
  // adjacency entries (fe_on), 5 rows expanded inside the window, 6 dirty.
  __device__ void gr_window_level(const int4 *cur4, int curlen, int L0, int Lend, int4 *next, u32 *ncnt) {
    if (threadIdx.x == 0) { sm.lqn[0] = 0; sm.lqn[1] = 0; sm.lwdirty = 0; sm.lwmax = 0; }
    __syncthreads();
    int mx = -1;
    const int lane = lane_id();
    {
      const int G = pick_group(curlen, gridDim.x * NT);
      const int gl = lane & (G - 1), per_tile = NT / G;
      for (int t = blockIdx.x * per_tile; t < curlen; t += gridDim.x * per_tile) {
        const int i = t + (int)threadIdx.x / G;
        const bool ok = i < curlen;
        int4 q = ok ? ld_q(cur4 + i) : make_int4(-1, 0, 0, 0);
        win_entry(q, ok, L0 - (q.w & ~1), G, gl, Lend, 0, next, ncnt, mx);
      }
    }
    int cb = 0, rows = 0, nr = 0;
    for (;;) {
      __syncthreads();
      const int cnt = min(sm.lqn[cb], LQ);
      if (cnt == 0) break;
      rows += cnt;
      __syncthreads();
      if (threadIdx.x == 0) sm.lqn[cb ^ 1] = 0;
      __syncthreads();
      const int G = pick_group(cnt, NT);
      const int gl = lane & (G - 1), per_tile = NT / G;
      for (int t = 0; t < cnt; t += per_tile) {
        const int i = t + (int)threadIdx.x / G;
        const bool ok = i < cnt;
        int4 q = ok ? sm.lq[cb][i] : make_int4(-1, 0, 0, 0);
        win_entry(q, ok, q.w & ~1, G, gl, Lend, cb ^ 1, next, ncnt, mx);
      }
      cb ^= 1;
      nr++;
    }
    mx = __reduce_max_sync(0xffffffffu, mx);
    if (lane == 0 && mx >= 0) atomicMax(&sm.lwmax, mx + 1);
    flush(next, ncnt);  // (its barriers order the lwmax updates before thread 0 reads it)
    if (threadIdx.x == 0) {
      if (sm.lwmax) atomicMax(ring_now(3), (u32)sm.lwmax);
      if (rows) atomicAdd(ring_now(5), (u32)rows);
      if (sm.lwdirty) atomicAdd(ring_now(6), 1u);
      if (p.trace && nr) atomicMax(ring_now(7), (u32)nr);
    }
  }

  // ---------------------------------------------------------------- fix step
  // G-PR-INITKRNL (Alg. 8) for slot i: roll back a push that lost its
  // race (Ap(i) = v still unmatched => Ac(i) <- v, l.3-6), then mark the slot's
  // column active in this loop (l.8-11, reading R5: after the if/else).
  __device__ __forceinline__ int fix_slot(int i, int *Ac, const int *Ap, int loop) {
    int a;
    fix_slots<1>(i, i + 1, Ac, Ap, loop, &a);
    return a;
  }
  // slots i0 .. i0+RB-1 (< hi); val[k] = the slot's column after the fix, or -1.
  // Loads are issued stage by stage for all RB slots (Ap and Ac, then the rolled-
  // back columns' words, then their mates' words).
  template <int RB>
  __device__ __forceinline__ void fix_slots(int i0, int hi, int *Ac, const int *Ap, int loop, int *val) {
    int v[RB], a[RB];
    u64 cw[RB], rw[RB];
#pragma unroll
    for (int k = 0; k < RB; k++) {
      const bool ok = i0 + k < hi;
      v[k] = ok ? ld_wl(Ap + i0 + k) : -1;
      a[k] = ok ? ld_wl(Ac + i0 + k) : -1;
    }
#pragma unroll
    for (int k = 0; k < RB; k++) cw[k] = v[k] != -1 ? vld(p.colst + v[k]) : 0ull;
#pragma unroll
    for (int k = 0; k < RB; k++) rw[k] = (v[k] != -1 && mu_of(cw[k]) >= 0) ? vld(p.rowst + mu_of(cw[k])) : 0ull;
#pragma unroll
    for (int k = 0; k < RB; k++) {
      if (v[k] != -1) {  // l.3-6: roll back a push that lost its race (R1: v still unmatched)
        const int c = mu_of(cw[k]);
        if (c == -1 || (c >= 0 && mu_of(rw[k]) != v[k])) {
          Ac[i0 + k] = v[k];
          a[k] = v[k];
        }
      }
      if (a[k] != -1) vst(p.iA + a[k], loop);  // l.8-11 (R5)
      val[k] = a[k];
    }
  }

  template <bool GRID>
  __device__ void fix_plain(int len, int *Ac, const int *Ap, int loop, int j) {
    long long cnt = 0;
    if (GRID && len > 2 * NT * ncta<GRID>()) {  // wide: 4 slots per thread in flight
      for (int t = cta<GRID>() * NT * 4; t < len; t += ncta<GRID>() * NT * 4) {
        int val[4];
        fix_slots<4>(t + (int)threadIdx.x * 4, len, Ac, Ap, loop, val);
#pragma unroll
        for (int k = 0; k < 4; k++) cnt += val[k] != -1;
      }
    } else {
      for (int t = cta<GRID>() * NT; t < len; t += ncta<GRID>() * NT) {
        int i = t + threadIdx.x;
        if (i < len) cnt += fix_slot(i, Ac, Ap, loop) != -1;
      }
    }
    S(SS_SLOTS) += cnt;
    add_count(cnt, j);
  }

  // ---------------------------------------------------------------- push
  // G-PR-PUSHKRNL (Alg. 9) over slots [0, len).  Each column gets a lane
  // group (pick_group); lists longer than BIG_DEG go to the whole warp, lists longer
  // than HUGE_DEG to the whole CTA (a straggler column would otherwise hold up the
  // phase: C2's dense "rail" columns have 2,000 rows).  Every scan takes a
  // (label, position) minimum per step with the early exit at psi(v)-1 (R11).
  // iaw: iA(wb) when the caller loaded it already (push_wide), else IA_LOAD
  static constexpr int IA_LOAD = -0x7fffffff - 1;
  __device__ __forceinline__ void push_finalize(int i, int v, u64 cs, u64 best, int ub, int wb, int loop, u32 base,
                                                int *Ac, int *Ap, int iaw = IA_LOAD) {
    // (dead columns are counted for the early-stop GR target, R22)
    int psimin = best == ~0ull ? INF : (int)(best >> 32);
    if (psimin < INF) {                                 // l.12
      if (wb == -1 || (iaw == IA_LOAD ? vld(p.iA + wb) : iaw) != loop) {  // l.13
        // option perturb (F_AUX builds only): the row store is lost, as if another
        // column had won the race for ub; v stays active by R1
        if (!((F & F_AUX) && p.perturb &&
              (hash2((u32)v, (u32)loop) & 0xffffu) < (u32)p.perturb))
          vst(p.rowst + ub, pack(v, base + (u32)psimin + 2u));  // l.14, l.17
        vst(p.colst + v, pack(ub, base + (u32)psimin + 1u));  // l.15, l.16
        Ap[i] = wb;                                     // l.18 (R3)
        S(SS_PUSH)++;
      } else {
        Ap[i] = -1;                                     // R4: blocked
        S(SS_BLOCK)++;
      }
    } else {
      vst(p.colst + v, pack(-2, psi_of(cs)));        // l.20
      Ac[i] = -1;                                       // l.21
      Ap[i] = -1;                                       // l.22
      S(SS_DEAD)++;
      cg::coalesced_group g = cg::coalesced_threads();  // published once per tile (push)
      if (g.thread_rank() == 0) atomicAdd(&sm.nd, (u32)g.size());
    }
  }

  template <bool GRID>
  __device__ void push(int len, int *Ac, int *Ap, int loop, u32 base) {
    const int lane = lane_id();
    const int G = pick_group(len, ncta<GRID>() * NT);
    if (GRID && len > 2 * NT * ncta<GRID>()) {
      push_wide<GRID>(len, Ac, Ap, loop, base);
      return;
    }
    const int gl = lane & (G - 1), per_tile = NT / G;
    const unsigned gmask = group_mask(G);
    for (int t = cta<GRID>() * per_tile; t < len; t += ncta<GRID>() * per_tile) {
      int i = t + (int)threadIdx.x / G;
      int v = (i < len) ? ld_wl(Ac + i) : -1;
      int s = 0, e = 0, psiv = INF;
      u64 cs = 0;
      if (v >= 0) {
        cs = vld(p.colst + v);
        psiv = labf(psi_of(cs), base, fl_c);
        s = ld_ro(p.cptr + v);
        e = ld_ro(p.cptr + v + 1);
        if (p.dead_skip && psiv >= INF) e = s;  // R19: provably unmatchable
      }
      const int target = psiv - 1;
      const int rot = (p.scan_rot && e - s > 1) ? (int)(((u32)v * 2654435761u + (u32)loop * 2246822519u) % (u32)(e - s)) : 0;
      bool huge = v >= 0 && e - s > HUGE_DEG;
      if (huge && gl == 0) {  // defer to the CTA-wide pass below
        int q = atomicAdd(&sm.nhuge, 1);
        if (q < MAXHUGE) { sm.huge[q] = make_int4(i, v, s, e); sm.hugec[q] = cs; sm.huget[q] = target; }
        else huge = false;  // list full: the warp takes it
      }
      huge = __shfl_sync(gmask, huge, lane & ~(G - 1));
      const bool big = v >= 0 && !huge && G < 32 && e - s > BIG_DEG;
      u64 best = ~0ull;
      int ub = -1, wb = -1;
      if (v >= 0 && !big && !huge) scan(s, e, gl, G, gmask, target, base, best, ub, wb, rot);  // l.6-11
      unsigned bigm = __ballot_sync(0xffffffffu, big && gl == 0);
      while (bigm) {  // long lists: the whole warp
        int bl = __ffs(bigm) - 1;
        bigm &= bigm - 1;
        int sb = __shfl_sync(0xffffffffu, s, bl), eb = __shfl_sync(0xffffffffu, e, bl);
        int tb = __shfl_sync(0xffffffffu, target, bl);
        int rb = __shfl_sync(0xffffffffu, rot, bl);
        u64 b2;
        int u2, w2;
        scan(sb, eb, lane, 32, 0xffffffffu, tb, base, b2, u2, w2, rb);
        if (lane == bl) { best = b2; ub = u2; wb = w2; }
      }
      if (gl == 0 && !huge) {
        if (v >= 0) push_finalize(i, v, cs, best, ub, wb, loop, base, Ac, Ap);
        else if (i < len) Ap[i] = -1;                   // l.24
      }
    }
    push_huge(loop, base, Ac, Ap);
  }
  // The columns a push phase deferred to the CTA (lists longer than HUGE_DEG, at most
  // MAXHUGE per CTA and phase; beyond that the lane group / warp scans them itself):
  // pushed once at the end of the phase, so the tiles of a phase never wait for each
  // other.  With more than HUGE_CTA of them, those of at most HUGE_WARP entries get a
  // warp each (in parallel), the rest the whole CTA each (a warp walks ~128 entries
  // per round trip, the CTA ~2048: R-MAT hub columns of 10^5 entries on one warp held
  // the phase for ~1.2 ms).  Publishes the CTA's dead-column count.
  __device__ void push_huge(int loop, u32 base, int *Ac, int *Ap) {
    const int lane = lane_id();
    __syncthreads();
    const int nh = min(sm.nhuge, MAXHUGE);
    if (nh > HUGE_CTA) {
      for (int h = warp_id(); h < nh; h += NWARP) {
        const int4 hq = sm.huge[h];
        if (hq.w - hq.z > HUGE_WARP) continue;
        u64 hb;
        int hu, hw;
        scan(hq.z, hq.w, lane, 32, 0xffffffffu, sm.huget[h], base, hb, hu, hw);
        if (lane == 0) push_finalize(hq.x, hq.y, sm.hugec[h], hb, hu, hw, loop, base, Ac, Ap);
      }
    }
    for (int h = 0; h < nh; h++) {
      const int4 hq = sm.huge[h];
      if (nh > HUGE_CTA && hq.w - hq.z <= HUGE_WARP) continue;
      u64 hb;
      int hu, hw;
      scan_cta(hq.z, hq.w, sm.huget[h], base, hb, hu, hw);
      if (threadIdx.x == 0) push_finalize(hq.x, hq.y, sm.hugec[h], hb, hu, hw, loop, base, Ac, Ap);
    }
    __syncthreads();
    if (threadIdx.x == 0) {
      sm.nhuge = 0;
      if (sm.nd) { atomicAdd(&p.ctrl->ndead, sm.nd); sm.nd = 0; }
    }
    __syncthreads();
  }
  // PUSHKRNL on a wide worklist (more than two slots per thread): PB slots per
  // thread per tile, each stage's loads issued for all of them before any is used
  // -- Ac, then the column words and bounds, then the first KB neighbours and their
  // row words, then iA of the displaced columns -- so a thread keeps PB chains in
  // flight.  Short lists (<= BIG_DEG) whose first KB neighbours do not reach
  // psi(v)-1 continue alone (scan from s+KB, positions kept relative to s, so the
  // first-minimum tie-break of R11 is unchanged); longer lists take the warp / CTA
  // paths of push().
  template <bool GRID>
  __device__ void push_wide(int len, int *Ac, int *Ap, int loop, u32 base) {
    constexpr int PB = MCM_PB;
    const int lane = lane_id();
    for (int t = cta<GRID>() * NT * PB; t < len; t += ncta<GRID>() * NT * PB) {
      int i[PB], v[PB], s[PB], e[PB], tg[PB];
      u64 cs[PB];
#pragma unroll
      for (int k = 0; k < PB; k++) {
        i[k] = t + k * NT + (int)threadIdx.x;
        v[k] = i[k] < len ? ld_wl(Ac + i[k]) : -1;
      }
#pragma unroll
      for (int k = 0; k < PB; k++) {
        cs[k] = v[k] >= 0 ? vld(p.colst + v[k]) : 0ull;
        s[k] = v[k] >= 0 ? ld_ro(p.cptr + v[k]) : 0;
        e[k] = v[k] >= 0 ? ld_ro(p.cptr + v[k] + 1) : 0;
      }
#pragma unroll
      for (int k = 0; k < PB; k++) {
        const int psiv = labf(psi_of(cs[k]), base, fl_c);
        if (p.dead_skip && psiv >= INF) e[k] = s[k];  // R19
        tg[k] = psiv - 1;
      }
      int x[PB][KB];
      u64 rs[PB][KB];
#pragma unroll
      for (int k = 0; k < PB; k++)
#pragma unroll
        for (int q = 0; q < KB; q++)
          x[k][q] = (v[k] >= 0 && e[k] - s[k] <= BIG_DEG && s[k] + q < e[k]) ? ld_adj(p.cadj + s[k] + q) : -1;
#pragma unroll
      for (int k = 0; k < PB; k++)
#pragma unroll
        for (int q = 0; q < KB; q++) rs[k][q] = x[k][q] >= 0 ? vld(p.rowst + x[k][q]) : 0ull;
      u64 best[PB];
      int ub[PB], wb[PB];
#pragma unroll
      for (int k = 0; k < PB; k++) {
        best[k] = ~0ull;
        ub[k] = -1;
        wb[k] = -1;
#pragma unroll
        for (int q = 0; q < KB; q++) {
          if (x[k][q] < 0) continue;
          S(SS_SCAN)++;
          const int l = labf(psi_of(rs[k][q]), base, fl_r);
          const u64 kk = l < INF ? (((u64)(u32)l << 32) | (u32)q) : ~0ull;
          if (kk < best[k]) { best[k] = kk; ub[k] = x[k][q]; wb[k] = mu_of(rs[k][q]); }
        }
      }
#pragma unroll
      for (int k = 0; k < PB; k++) {  // short lists longer than KB without a hit: the rest, alone
        const int sk = s[k], ek = e[k];
        if (v[k] >= 0 && ek - sk > KB && ek - sk <= BIG_DEG && !(best[k] != ~0ull && (int)(best[k] >> 32) == tg[k])) {
          u64 b2;
          int u2, w2;
          scan(sk + KB, ek, 0, 1, 1u << lane, tg[k], base, b2, u2, w2);
          if (b2 != ~0ull) b2 += KB;  // position relative to s
          if (b2 < best[k]) { best[k] = b2; ub[k] = u2; wb[k] = w2; }
        }
      }
      // longer lists: the whole warp (BIG_DEG < deg <= HUGE_DEG) or the CTA (deferred)
#pragma unroll
      for (int k = 0; k < PB; k++) {
        bool huge = v[k] >= 0 && e[k] - s[k] > HUGE_DEG;
        if (huge) {
          int q = atomicAdd(&sm.nhuge, 1);
          if (q < MAXHUGE) { sm.huge[q] = make_int4(i[k], v[k], s[k], e[k]); sm.hugec[q] = cs[k]; sm.huget[q] = tg[k]; }
          else huge = false;
        }
        if (huge) v[k] = -2;  // finalized by the CTA pass
        unsigned bigm = __ballot_sync(0xffffffffu, v[k] >= 0 && e[k] - s[k] > BIG_DEG);
        while (bigm) {
          const int bl = __ffs(bigm) - 1;
          bigm &= bigm - 1;
          const int sb = __shfl_sync(0xffffffffu, s[k], bl), eb = __shfl_sync(0xffffffffu, e[k], bl);
          const int tb = __shfl_sync(0xffffffffu, tg[k], bl);
          u64 b2;
          int u2, w2;
          scan(sb, eb, lane, 32, 0xffffffffu, tb, base, b2, u2, w2);
          if (lane == bl) { best[k] = b2; ub[k] = u2; wb[k] = w2; }
        }
      }
      int ia[PB];
#pragma unroll
      for (int k = 0; k < PB; k++) ia[k] = (v[k] >= 0 && best[k] != ~0ull && wb[k] != -1) ? vld(p.iA + wb[k]) : -1;
#pragma unroll
      for (int k = 0; k < PB; k++) {
        if (v[k] >= 0) push_finalize(i[k], v[k], cs[k], best[k], ub[k], wb[k], loop, base, Ac, Ap, ia[k]);
        else if (v[k] == -1 && i[k] < len) Ap[i[k]] = -1;  // l.24
      }
    }
    push_huge(loop, base, Ac, Ap);
  }
  // Push chains (single-CTA tail, at most chain_slots active columns; reading R26, a
  // build addition).  In the paper's loop a double push hands the displaced column
  // w to the next loop, so an augmenting path of length L costs ~L/2 loops, each a
  // fix phase + a push phase (~4.4 us in the tail): C2's last augmentations walk
  // paths of 400-900 BFS levels that way.  Here one warp per slot performs the same
  // push operations (Alg. 9 l.4-18: first minimum-label neighbour, labels psimin+1 /
  // psimin+2) back to back: after displacing w it pushes w itself.  The row is
  // claimed with a CAS on its {mu, psi} word (re-read at gpu scope, so the
  // comparison is against L2's value), which makes every displacement exclusive --
  // the role the iA test and the rollback play for the atomic-free loop -- so the
  // slot leaves Ac(i) = -1 and Ap(i) = its current column (or -1 when the path
  // reached an unmatched row or the column died): the next fix step then marks
  // exactly the unfinished chains active and rolls nothing back.
  // Returns the longest chain (pushes), CTA-uniform: the caller advances `loop` by
  // it, so the GR schedule (iterGR = loop + k * maxLevel, counted in push rounds)
  // sees the same number of push rounds as the one-push-per-loop schedule -- without
  // that, a chain circling on stale labels ran ~5 * 10^4 pushes between two GRs.
  // GRID: the slots spread over all CTAs (grid_chain); the longest chain goes to
  // ring counter 5 and the caller reads it after the barrier (returns 0).
  // mu(c) <- r after a chain claimed row r for column c (R27).  The store is a CAS
  // against the word the chain read, so a late write cannot overwrite a newer one:
  // once another chain has displaced c from r (CAS on r's word) and pushed c on,
  // c's word belongs to that chain.  A failed CAS (a stale read, or the newer
  // write already landed) is retried only while r still holds c.
  __device__ __forceinline__ void chain_settle(int c, int r, u64 exp, u64 val, u64 ret) {
    while (ret != exp) {
      if (mu_of(ld_rlx(p.rowst + r)) != c) return;  // displaced: the newer push owns mu(c)
      exp = ret;
      ret = atomicCAS(p.colst + c, exp, val);
    }
  }
  template <bool GRID>
  __device__ int push_chain(int len, int *Ac, int *Ap, u32 base, int cap) {
    const int lane = lane_id();
    const int G = pick_group(len, ncta<GRID>() * NT), gl = lane & (G - 1), lead_lane = lane & ~(G - 1);
    const unsigned gmask = group_mask(G);
    const int per_tile = NT / G;
    for (int t = cta<GRID>() * per_tile; t < len; t += ncta<GRID>() * per_tile) {
    const int i = t + (int)threadIdx.x / G;
    if (i < len) {
      int cur = ld_wl(Ac + i), left = -1, retry = 0, step = 0;
      // the last push's mu(column) CAS, checked one scan later (its latency hides
      // behind the next column's loads): {column, row, expected, written, returned}
      int pc = -1, pr = -1;
      u64 pexp = 0, pnew = 0, pret = 0;
      // the next column's word and adjacency bounds, loaded by the group's lead lane
      // in the same round trip as the row claim (the displaced column is known from
      // the scan): one dependent round trip less per push
      bool have = false;
      u64 ncs = 0;
      int ns = 0, ne = 0;
      while (cur >= 0) {
        if (step >= cap || retry > 8) { left = cur; break; }
        const u64 cs = have ? ncs : vld(p.colst + cur);
        const int psiv = labf(psi_of(cs), base, fl_c);
        const int s = have ? ns : ld_ro(p.cptr + cur);
        int e = have ? ne : ld_ro(p.cptr + cur + 1);
        have = false;
        if (p.dead_skip && psiv >= INF) e = s;  // R19
        if (step > 0 && e - s > HUGE_DEG * G / 32) { left = cur; break; }  // a long list ends the chain
        u64 best, braw = 0;
        int ub, wb;
        scan(s, e, gl, G, gmask, psiv - 1, base, best, ub, wb, 0, retry > 0, &braw);  // l.4-11
        if (gl == 0 && pc >= 0) { chain_settle(pc, pr, pexp, pnew, pret); pc = -1; }
        const int psimin = best == ~0ull ? INF : (int)(best >> 32);
        if (psimin >= INF) {  // l.19-22: dead
          if (gl == 0) {
            vst(p.colst + cur, pack(-2, psi_of(cs)));
            S(SS_DEAD)++;
            atomicAdd(&sm.nd, 1u);
          }
          break;
        }
        int ok = 0;
        if (gl == 0) {
          if (wb >= 0) { ncs = vld(p.colst + wb); ns = ld_ro(p.cptr + wb); ne = ld_ro(p.cptr + wb + 1); }
          // claim the row against the word the scan read (gpu scope): it fails when
          // any push changed the row since
          ok = atomicCAS(p.rowst + ub, braw, pack(cur, base + (u32)psimin + 2u)) == braw;  // l.14, l.17
          if (ok) {  // l.15, l.16
            pc = cur; pr = ub; pexp = cs; pnew = pack(ub, base + (u32)psimin + 1u);
#if MCM_CHAIN_PLAIN  // A/B only: the plain store of the first round-1 build
            vst(p.colst + cur, pnew);
            pret = pexp;
#else
            pret = atomicCAS(p.colst + cur, pexp, pnew);
#endif
            S(SS_PUSH)++;
          }
        }
        if (!__shfl_sync(gmask, ok, lead_lane)) { retry++; continue; }  // the row changed: scan again
        retry = 0;
        step++;
        cur = wb;  // -1: single push, the path is complete
        ncs = __shfl_sync(gmask, ncs, lead_lane);
        ns = __shfl_sync(gmask, ns, lead_lane);
        ne = __shfl_sync(gmask, ne, lead_lane);
        have = true;
      }
      __syncwarp(gmask);  // every lane of the group has read Ac(i) before it is cleared
      if (gl == 0) {
        if (pc >= 0) chain_settle(pc, pr, pexp, pnew, pret);
        Ac[i] = -1;
        Ap[i] = left;
        atomicMax(&sm.chmax, step);
      }
    }
    }
    __syncthreads();
    if (GRID) {
      if (threadIdx.x == 0) {
        if (sm.chmax) atomicMax(ring_now(5), (u32)sm.chmax);
        if (sm.nd) { atomicAdd(&p.ctrl->ndead, sm.nd); sm.nd = 0; }
        sm.chmax = 0;
      }
      return 0;
    }
    const int mx = sm.chmax;
    if (threadIdx.x == 0 && sm.nd) { atomicAdd(&p.ctrl->ndead, sm.nd); sm.nd = 0; }
    __syncthreads();
    if (threadIdx.x == 0) sm.chmax = 0;
    return mx;
  }
  // scan() with the whole CTA: KB*NT neighbours per step; CTA-wide (label, position)
  // minimum through shared memory; returns the result in every thread.
  __device__ void scan_cta(int s, int e, int target, u32 base, u64 &best, int &bu, int &bw) {
    best = ~0ull;
    bu = -1;
    bw = -1;
    for (int c0 = s; c0 < e; c0 += NT * KB) {
      int x[KB];
      u64 rs[KB];
#pragma unroll
      for (int k = 0; k < KB; k++) {
        int jj = c0 + (int)threadIdx.x + k * NT;
        x[k] = jj < e ? ld_adj(p.cadj + jj) : -1;
      }
#pragma unroll
      for (int k = 0; k < KB; k++) rs[k] = x[k] >= 0 ? vld(p.rowst + x[k]) : 0ull;
      u64 key = ~0ull;
      int kx = -1, kw = -1;
#pragma unroll
      for (int k = 0; k < KB; k++) {
        if (x[k] < 0) continue;
        S(SS_SCAN)++;
        int l = labf(psi_of(rs[k]), base, fl_r);
        u64 kk = l < INF ? (((u64)(u32)l << 32) | (u32)(c0 + (int)threadIdx.x + k * NT - s)) : ~0ull;
        if (kk < key) { key = kk; kx = x[k]; kw = mu_of(rs[k]); }
      }
      u64 km = key;
#pragma unroll
      for (int o = 16; o > 0; o >>= 1) {
        u64 other = __shfl_xor_sync(0xffffffffu, km, o);
        km = other < km ? other : km;
      }
      __syncthreads();
      if (lane_id() == 0) sm.red[warp_id()] = (long long)km;
      __syncthreads();
      u64 kmin = ~0ull;
#pragma unroll
      for (int w = 0; w < NWARP; w++) kmin = min(kmin, (u64)sm.red[w]);
      if (kmin < best) {
        if (key == kmin) { sm.tmp = kx; sm.qbase = kw; }  // unique position: one writer
        __syncthreads();
        best = kmin;
        bu = sm.tmp;
        bw = sm.qbase;
      }
      if (best != ~0ull && (int)(best >> 32) == target) break;
    }
    __syncthreads();
  }
  // First minimum of psi over Gamma(v) = cadj[s, e) in adjacency order (Alg. 9
  // l.6-11): the G lanes of a group read KB*G consecutive neighbours per step, take
  // the (label, position) minimum and stop after the step in which the running
  // minimum reaches psi(v)-1 (reading R11).  best = (label << 32 | position) or ~0.
  // rot: the scan starts at position s + rot and wraps around (option scan_rot, a
  // free tie-break in parallel mode, R11: contenders for one low-label row spread
  // over the equally low rows instead of blocking each other)
  // fresh: row words at gpu scope (L2), for a push chain re-scanning after a lost CAS
  // raw (optional): the winner's row word as the scan read it (push chains CAS against it)
  __device__ __forceinline__ void scan(int s, int e, int gl, int G, unsigned gmask, int target, u32 base, u64 &best,
                                       int &bu, int &bw, int rot = 0, bool fresh = false, u64 *raw = nullptr) {
    best = ~0ull;
    bu = -1;
    bw = -1;
    const int len = e - s;
    for (int c0 = s; c0 < e; c0 += G * KB) {
      int x[KB];
      u64 rs[KB];
#pragma unroll
      for (int k = 0; k < KB; k++) {
        int jj = c0 + gl + k * G;
        int q = jj - s + rot;
        if (q >= len) q -= len;
        x[k] = jj < e ? ld_adj(p.cadj + s + q) : -1;
      }
#pragma unroll
      for (int k = 0; k < KB; k++) rs[k] = x[k] >= 0 ? (fresh ? ld_rlx(p.rowst + x[k]) : vld(p.rowst + x[k])) : 0ull;
      u64 key = ~0ull, kr = 0;
      int kx = -1, kw = -1;
#pragma unroll
      for (int k = 0; k < KB; k++) {
        if (x[k] < 0) continue;
        S(SS_SCAN)++;
        int l = labf(psi_of(rs[k]), base, fl_r);
        u64 kk = l < INF ? (((u64)(u32)l << 32) | (u32)(c0 + gl + k * G - s)) : ~0ull;
        if (kk < key) { key = kk; kx = x[k]; kw = mu_of(rs[k]); kr = rs[k]; }
      }
      u64 km = key;
      for (int o = G >> 1; o > 0; o >>= 1) {
        u64 other = __shfl_xor_sync(gmask, km, o, G);
        km = other < km ? other : km;
      }
      if (km < best) {
        int src = __ffs(__ballot_sync(gmask, key == km)) - 1;
        best = km;
        bu = __shfl_sync(gmask, kx, src);
        bw = __shfl_sync(gmask, kw, src);
        if (raw) *raw = __shfl_sync(gmask, kr, src);
      }
      if (best != ~0ull && (int)(best >> 32) == target) break;
    }
  }

  // ---------------------------------------------------------------- FIXMATCHING
  // mu(v) <- -1 for columns with mu(mu(v)) != v, fused with writing the
  // caller's rmatch / cmatch and counting |M| (rows are authoritative).
  __device__ void fixmatching(int j_card, int j_fixed) {
    const int G = gridDim.x * NT, g = blockIdx.x * NT + threadIdx.x;
    long long card = 0, fixed = 0;
    for (int u = g; u < m; u += G) {
      int c = mu_of(vld(p.rowst + u));
      // without the guard (final_check = 0) no repair pass ran (R27): a stale row is
      // reported unmatched, so the output stays a valid matching
      if (!p.final_check && c >= 0 && mu_of(vld(p.colst + c)) != u) c = -1;
      p.rmatch_out[u] = c;
      card += c >= 0;
    }
    for (int v = g; v < n; v += G) {
      int c = mu_of(vld(p.colst + v));
      int ok = (c >= 0 && mu_of(vld(p.rowst + c)) == v) ? c : -1;
      fixed += (c != -1 && ok == -1);
      p.cmatch_out[v] = ok;
    }
    add_count(card, j_card);
    add_count(fixed, j_fixed);
  }

  __device__ void write_labels(u32 base) {
    const int G = gridDim.x * NT, g = blockIdx.x * NT + threadIdx.x;
    for (int u = g; u < m; u += G) p.rmatch_out[u] = lab(psi_of(vld(p.rowst + u)), base, INF);
    for (int v = g; v < n; v += G) p.cmatch_out[v] = lab(psi_of(vld(p.colst + v)), base, INF);
  }

  __device__ int iter_gap(int maxLevel) const {
    // GETITERGR (reading R7)
    if (p.gr_fixed) { long long g = (long long)p.k; return (int)(g < 1 ? 1 : (g > (1 << 30) ? (1 << 30) : g)); }
    double g = ceil(p.k * (double)maxLevel);
    return (int)(g < 1 ? 1 : (g > (1 << 30) ? (1 << 30) : g));
  }

  // ---------------------------------------------------------------- debug checks
  __device__ void dbg_record(int where, long long loop, int x, int val) {
    unsigned long long c = atomicAdd((unsigned long long *)&p.ctrl->dbg[0], 1ull);
    if (c == 0) { p.ctrl->dbg[1] = where; p.ctrl->dbg[2] = loop; p.ctrl->dbg[3] = x; p.ctrl->dbg[4] = val; }
  }
  // rows: mu(u) = v >= 0  =>  mu(v) = u ;  worklist: no column twice
  __device__ void debug_check(int where, long long loop, const int *Ac, int len) {
    if (!(F & F_DEBUG) || !p.debug) return;
    const int G = gridDim.x * NT, g = blockIdx.x * NT + threadIdx.x;
    for (int u = g; u < m; u += G) {
      int c = mu_of(vld(p.rowst + u));
      if (c >= 0 && mu_of(vld(p.colst + c)) != u) dbg_record(where, loop, u, c);
    }
    for (int v = g; v < n; v += G) p.dbgbuf[v] = 0;
    barrier<true, false>();
    if (Ac)
      for (int i = g; i < len; i += G) {
        int v = __ldcg(Ac + i);
        if (v >= 0 && atomicAdd(p.dbgbuf + v, 1) != 0) dbg_record(100 + where, loop, v, i);
      }
    barrier<true, false>();
  }

  // ---------------------------------------------------------------- gap relabel
  // Reading R14 of P:95-96 (the paper names GPU gap relabelling but gives no
  // algorithm): count the vertices of every finite label l < H (rows carry even
  // labels, columns odd); if some label g < L_max (the largest finite label) has
  // no vertex, every label in (g, m+n) becomes m+n.  Valid because along any
  // residual path labels drop by at most one per step (neighbourhood invariant,
  // P:203-209, and psi(u) = psi(mu(u)) + 1 for matched rows), so a vertex above
  // the gap cannot reach an unmatched row (label 0).  g = 0 (no unmatched row
  // left) kills every active column.  Counting every vertex (dead columns
  // included) can only hide gaps, never invent one.  Grid phases; returns g or -1.
  __device__ int gap_relabel(u32 base) {
    const int G = gridDim.x * NT, g = blockIdx.x * NT + threadIdx.x;
    const int H = p.hist_len;
    Ctrl *c = p.ctrl;
    if (blockIdx.x == 0 && threadIdx.x == 0) c->gmin = 0x7fffffff;
    // per-CTA shared histogram of the low labels (the frontier staging buffer is
    // idle here), flushed with one global atomic per non-empty bin
    const int SH = min(QCAP, H);
    for (int l = threadIdx.x; l < SH; l += NT) sm.q[l] = 0;
    __syncthreads();
    int lmax = -1;
    for (int x = g; x < m + n; x += G) {
      u64 w = vld(x < m ? p.rowst + x : p.colst + (x - m));
      int l = lab(psi_of(w), base, INF);
      if (l < INF) {
        if (l < SH) atomicAdd(&sm.q[l], 1);
        else if (l < H) atomicAdd(p.hist + l, 1);
        lmax = max(lmax, l);
      }
    }
    __syncthreads();
    for (int l = threadIdx.x; l < SH; l += NT)
      if (sm.q[l]) atomicAdd(p.hist + l, sm.q[l]);
    __syncthreads();
    if (threadIdx.x == 0) sm.qcnt = 0;
    for (int o = 16; o > 0; o >>= 1) lmax = max(lmax, __shfl_xor_sync(0xffffffffu, lmax, o));
    if (lane_id() == 0 && lmax >= 0) atomicMax(&c->gmax, lmax);
    barrier<true, false>();
    const int L = min((int)bcast_ld((const u32 *)&c->gmax), H);
    int first = 0x7fffffff;
    for (int l = g; l < L; l += G)
      if (__ldcg(p.hist + l) == 0) { first = l; break; }
    for (int o = 16; o > 0; o >>= 1) first = min(first, __shfl_xor_sync(0xffffffffu, first, o));
    if (lane_id() == 0 && first != 0x7fffffff) atomicMin(&c->gmin, first);
    barrier<true, false>();
    const int gap = (int)bcast_ld((const u32 *)&c->gmin);
    if (blockIdx.x == 0 && threadIdx.x == 0) c->gmax = 0;
    long long killed = 0;
    if (gap != 0x7fffffff) {
      for (int x = g; x < m + n; x += G) {
        u64 *a = x < m ? p.rowst + x : p.colst + (x - m);
        u64 w = vld(a);
        int l = lab(psi_of(w), base, INF);
        if (l > gap && l < INF) { vst(a, pack(mu_of(w), 0)); killed++; }  // psi 0 < base: infinite
      }
    }
    for (int l = g; l < L; l += G) p.hist[l] = 0;
    barrier<true, false>();
    return gap == 0x7fffffff ? -1 : gap;
  }

  // ---------------------------------------------------------------- control state
  // Alg. 7's control registers.  Every thread holds an identical copy, updated from
  // values read after barriers; a tail episode publishes the tail group's copy.
  struct Ctl {
    long long loop, iterGR, gapAt;
    int len, ulen;
    u32 base;
    int shrink, compact_next, gr_active, ac0, u0;
    int cflags;            // concurrent GR (NEXT-2): bit 0 active, bit 1 the GR kernel's labels are ready
    int floor_r, floor_c;  // labels of vertices the last GR did not reach (m+n unless it stopped early)
    u32 creq;              // concurrent GR (NEXT-2): requests sent to the GR kernel
    GRState gst;
  };
  static_assert(sizeof(Ctl) % 8 == 0 && sizeof(Ctl) / 8 <= 32, "Ctl handoff image");
  __device__ __forceinline__ int *Acp(const Ctl &c) const { return c.ac0 ? p.wl0 : p.wl1; }
  __device__ __forceinline__ int *App(const Ctl &c) const { return c.ac0 ? p.wl1 : p.wl0; }
  __device__ __forceinline__ int *Ub(const Ctl &c) const { return c.u0 ? p.qa : p.qb; }
  __device__ __forceinline__ int *Tb(const Ctl &c) const { return c.u0 ? p.qb : p.qa; }
  __device__ __forceinline__ u32 stride() const { return (u32)(m + n + 2); }
  __device__ __forceinline__ int4 *Q4(int i) const { return reinterpret_cast<int4 *>(i ? p.qd : p.qc); }
  __device__ __forceinline__ bool base_overflow(const Ctl &c) const {
    return (u64)c.base + 2ull * stride() >= 0xfffffff0ull;
  }

  enum { R_NONE = 0, R_TERM = 1, R_GRID = 2, R_CAP = 4 };
  // gap relabel schedule (R14): once, halfway between two GRs
  __device__ __forceinline__ long long gap_at(long long loop, long long iterGR) const {
    return ((F & F_GAP) && p.gap && iterGR - loop >= 2) ? loop + (iterGR - loop) / 2 : -1;
  }
  // GR frontiers of at most tail_f() rows run on the tail group (hand-over back to
  // the grid when a frontier outgrows it, back to the tail below tail_f()/2)
  __device__ __forceinline__ bool early_gr() const { return p.gr_early && !p.gap; }
  __device__ __forceinline__ int tail_f() const { return p.tail_f > 0 ? p.tail_f : 2 * p.tail_max; }
  // the next GR unit is a window (gr_window_step) rather than one level
  __device__ __forceinline__ bool win_ok(const Ctl &c) const {
    return (F & F_AUX) && p.gr_window > 1 && (c.gst.dirty || (c.gst.nlen <= p.gr_window_max && !c.gst.in_smem &&
                                               !use_bottom_up(c.gst.fedges, (long long)n - c.gst.visited, c.gst.nlen)));
  }

  // ---------------------------------------------------------------- units of work
  // Single-CTA tail GR levels keep the frontier in shared memory: stage() writes
  // the next frontier straight into a shared buffer (no flush, no global queue);
  // entries beyond TQ overflow to the global queue.  After the level: no overflow
  // -> the frontier stays shared; overflow -> the shared part is appended to the
  // global queue (the frontier is then global, e.g. for a hand-over to the grid).
  __device__ void tail_sq_begin(int4 *dst) {
    sq = true;
    sq_next = dst;
    if (threadIdx.x == 0) sm.qcnt = 0;
    __syncthreads();
  }
  // call after the level's barrier.  Everything the tail level produced is counted
  // in shared memory (no L2 round trip after the tail's CTA barrier): sm.qcnt =
  // staged rows (those beyond TQ went to the global queue, in order of the
  // overflow counter), sm.lvc[0] = alive unmatched columns labelled (R22).
  __device__ void tail_sq_end(GRState &g, int4 *nxt_global, const int4 *nxt_shared) {
    sq = false;
    const int q = sm.qcnt, sc = min(q, TQ), ovf = q - sc;
    const int rc = (int)sm.lvc[0];
    if (ovf == 0) {
      g.nlen = sc;
      g.in_smem = 1;
    } else {
      for (int j = threadIdx.x; j < sc; j += NT) nxt_global[ovf + j] = nxt_shared[j];
      g.nlen = ovf + sc;
      g.in_smem = 0;
    }
    g.reached += rc;
    g.visited += rc;
    __syncthreads();
    if (threadIdx.x == 0) { sm.qcnt = 0; sm.lvc[0] = 0; }
    __syncthreads();
  }
  // a shared frontier must move to the global queue before the grid can see it
  __device__ void tail_sq_spill(GRState &g) {
    if (!g.in_smem) return;
    const int4 *src = sfr(g.cur_is_a ? 0 : 1);
    int4 *dst = Q4(g.cur_is_a ? 0 : 1);
    for (int j = threadIdx.x; j < g.nlen; j += NT) dst[j] = src[j];
    __syncthreads();
    g.in_smem = 0;
  }

  // GR bookkeeping once the BFS is over (Alg. 7 l.7-9 with GETITERGR, R7)
  __device__ void gr_finish(Ctl &c, bool early = false) {
    // complete BFS: unreached = infinite (Alg. 2); early stop (R22) after expanding
    // the rows of level l: unreached columns >= l+3, rows >= l+4 (lower bounds that
    // keep the neighbourhood invariant next to the unexpanded rows of level l+2)
    c.floor_c = early ? c.gst.lvl + 3 : INF;
    c.floor_r = early ? c.gst.lvl + 4 : INF;
    if (early) c.gst.deepest = c.gst.lvl + 2;
    int ml = c.gst.deepest + 2;
    if (lead()) { L().grs++; L().levels += ml / 2; }
    c.iterGR = c.loop + iter_gap(ml);
    c.gapAt = gap_at(c.loop, c.iterGR);
    c.shrink = 1;
    c.gr_active = 0;
    c.base += stride();
    if ((F & F_AUX) && (c.cflags & 1)) {  // NEXT-2: from now on the GR kernel relabels in the background
      c.iterGR = 0x3fffffffffffffffLL;
      conc_request(c);
    }
  }
  // GR level 0 (INITRELABEL via the epoch bump + first expansion)
  template <bool GRID>
  __device__ void gr_begin(Ctl &c) {
    u64 g0 = tnow();
    int *U = Ub(c), *T = Tb(c);
    if (!GRID && p.tail_ctas == 1) {  // single-CTA tail: the next frontier stays in shared memory
      tail_sq_begin(sfr(0));  // level 0 fills buffer "a" (gr_start sets cur_is_a = 1)
      gr_start<GRID>(c.gst, U, c.ulen, T, Q4(0), c.base, nullptr);
      tail_sq_end(c.gst, Q4(0), sfr(0));
    } else {
      gr_start<GRID>(c.gst, U, c.ulen, T, Q4(0), c.base, nullptr);
      c.gst.in_smem = 0;
    }
    c.u0 ^= 1;
    c.gr_active = 1;
    // early stop (R22): every alive unmatched column is active; stop once all of them
    // carry a label.  alive unmatched = n - matched - dead; matched = m - |U|.
    c.gst.target = early_gr() ? n - (m - n_iso - c.ulen) - (int)bcast_ld((const u32 *)&p.ctrl->ndead) : 0x7fffffff;
    if (p.gr_target < 1.0 && early_gr() && c.gst.target >= p.gr_target_min)  // R28
      c.gst.target = (int)ceil(p.gr_target * (double)c.gst.target);
    if (c.gst.nlen == 0) gr_finish(c);
    else if (c.gst.reached >= c.gst.target) gr_finish(c, true);
    if (lead()) L().ns_gr += (long long)(tnow() - g0);
  }
  // one BFS level (Alg. 5)
  template <bool GRID>
  __device__ void gr_step(Ctl &c) {
    u64 g0 = tnow();
    if (GRID && MCM_FINE) tmark(107, 0);
    GRState &g = c.gst;
    g.lvl += 2;
    g.deepest = g.lvl;
    int4 *cur = g.in_smem ? sfr(g.cur_is_a ? 0 : 1) : Q4(g.cur_is_a ? 0 : 1), *nxt = Q4(g.cur_is_a ? 1 : 0);
    gr_base = c.base;
    trace(2, g.nlen);
    const bool smemq = !GRID && p.tail_ctas == 1;
    if (smemq) tail_sq_begin(sfr(g.cur_is_a ? 1 : 0));
    set_fe(g.nlen);
    if (GRID && use_bottom_up(g.fedges, (long long)n - g.visited, g.nlen))
      gr_level_bu<GRID>(g.lvl, c.base, nxt, ring_now(0), nullptr, &p.ctrl->gcnt);
    else
      gr_level<GRID>(nullptr, cur, g.nlen, g.lvl, c.base, nxt, ring_now(0), nullptr, nullptr, nullptr, &p.ctrl->gcnt);
    if (smemq) {  // single-CTA tail: counts in shared memory, no ring read
      barrier<GRID, false>();
      g.fedges = 0;
      tail_sq_end(g, nxt, sfr(g.cur_is_a ? 1 : 0));
      g.visited += g.nlen;
    } else {
      barrier<GRID>();
      g.fedges = ring_prev(4);
      g.nlen = (int)ring_prev(0);
      g.in_smem = 0;
      g.reached += (int)ring_prev(2);
      g.visited += (long long)g.nlen + ring_prev(2);
    }
    g.cur_is_a ^= 1;
    if (g.nlen == 0) gr_finish(c);
    else if (g.reached >= g.target) gr_finish(c, true);
    if (GRID && MCM_FINE) tmark(106, 0);
    if (lead()) L().ns_gr += (long long)(tnow() - g0);
  }
  // K BFS levels in one grid phase (option gr_window; see gr_window_level)
  __device__ void gr_window_step(Ctl &c) {
    u64 g0 = tnow();
    GRState &g = c.gst;
    g.lvl += 2;  // the frontier's label L0
    const int L0 = g.lvl, Lend = L0 + 2 * p.gr_window;
    const int4 *cur = Q4(g.cur_is_a ? 0 : 1);
    int4 *nxt = Q4(g.cur_is_a ? 1 : 0);
    gr_base = c.base;
    trace(5, g.nlen);
    set_fe(g.nlen);
    gr_window_level(cur, g.nlen, L0, Lend, nxt, ring_now(0));
    barrier<true>();
    g.fedges = ring_prev(4);
    g.nlen = (int)ring_prev(0);
    g.in_smem = 0;
    g.reached += (int)ring_prev(2);
    g.visited += (long long)g.nlen + ring_prev(2) + ring_prev(5);
    const int mx = (int)ring_prev(3) - 1;  // deepest row label expanded
    if (mx > g.deepest) g.deepest = mx;
    g.dirty = ring_prev(6) != 0;
    g.lvl = Lend - 2;  // (clean) every row below Lend expanded, the frontier holds Lend
    g.cur_is_a ^= 1;
    if (lead()) L().wlevels += p.gr_window;
    if (g.nlen == 0) {
      // the BFS ended inside this window: a row expanded with a label that was
      // lowered later makes mx too large, so maxLevel comes from the final labels
      // (one pass over the rows; at most once per GR)
      const u32 b = c.base;
      u32 best = 0;
      for (long long u = (long long)blockIdx.x * NT + threadIdx.x; u < m; u += (long long)gridDim.x * NT) {
        const u32 ps = psi_of(vld(p.rowst + u));
        if (ps >= b && ps - b + 1u > best) best = ps - b + 1u;
      }
      best = __reduce_max_sync(0xffffffffu, best);
      if (lane_id() == 0 && best) atomicMax(ring_now(3), best);
      barrier<true>();
      g.deepest = (int)ring_prev(3) - 1;
    }
    if (p.trace) { tmark(150, (int)ring_prev(7)); tmark(151, (int)ring_prev(5)); tmark(152, g.dirty); }
    if (g.nlen == 0) gr_finish(c);
    else if (!g.dirty && g.reached >= g.target) gr_finish(c, true);
    if (lead()) L().ns_gr += (long long)(tnow() - g0);
  }
  // SHRKRNL: the fix step of every slot (fix_slots, Alg. 8) with the
  // surviving columns compacted to Ac[0 ..) in slot order (two passes over the CTAs'
  // chunks; T = scratch of len entries); returns the new length.
  template <bool GRID>
  __device__ int fix_compact(int len, int *Ac, const int *Ap, int lp, int *T) {
    if (lead()) S(SS_SLOTS) += len;
    const int r1 = (GRID && len > 2 * NT * ncta<GRID>())
                       ? compact_pass1<GRID, 4>(len, [&](int i0, int hi, int *val) { fix_slots<4>(i0, hi, Ac, Ap, lp, val); },
                                                T, Ac)
                       : compact_pass1<GRID, 1>(len, [&](int i0, int hi, int *val) { fix_slots<1>(i0, hi, Ac, Ap, lp, val); },
                                                T, Ac);
    barrier<GRID, false>();
    if (ncta<GRID>() == 1) return r1;
    len = compact_pass2<GRID>(len, T, Ac, r1);
    barrier<GRID, false>();  // Ac was rewritten by other CTAs: order it before PUSH
    return len;
  }
  // one iteration of Alg. 7 l.10-19: fix step (INITKRNL, or SHRKRNL = fix + stable
  // compaction), then PUSHKRNL and the Ac/Ap swap.  Returns false when the fix
  // step found no active column.  The tail group compacts at every step.
  template <bool GRID>
  __device__ bool loop_step(Ctl &c, int *Ac, int *Ap) {
    u64 l0 = tnow();
    const u32 cur = c.base - stride();  // epoch of the labels in use
    const int lp = (int)c.loop;
    int act;
    trace(3, c.len);
    if (!GRID || (c.shrink && p.shrink_min >= 0 && c.len >= p.shrink_min) || p.compact_every || c.compact_next) {
      c.len = fix_compact<GRID>(c.len, Ac, Ap, lp, Tb(c));
      act = c.len;
      if (c.shrink && lead()) L().shrinks++;
      c.shrink = 0;
      c.compact_next = 0;
    } else {
      fix_plain<true>(c.len, Ac, Ap, lp, 0);
      barrier<true>();
      act = (int)ring_prev(0);
      // adaptive compaction (beyond the paper's post-GR shrink): when most slots
      // are empty the next fix step compacts, so the tail group can take over
      if (p.compact_adapt && act > 0 && (long long)act * 4 < c.len && c.len > p.tail_max) c.compact_next = 1;
    }
    if (GRID) debug_check(3, c.loop, Ac, c.len);
    if (act == 0) {
      if (lead()) L().ns_loop += (long long)(tnow() - l0);
      return false;
    }
    trace(4, c.len);
    fl_r = c.floor_r;
    fl_c = c.floor_c;
    long long adv = 1;  // push rounds of this loop (R26: a chain counts its pushes)
    const bool chain_grid = GRID && p.grid_chain > 0 && (long long)c.len * p.grid_chain_div <= (long long)ncta<GRID>() * NT;
    if (!GRID && p.tail_chain > 0 && p.tail_ctas == 1 && c.len <= p.chain_slots) {
      adv = max(1, push_chain<false>(c.len, Ac, Ap, cur, p.tail_chain));
    } else if (chain_grid) {
      // the longest chain holds the phase: shorter chains on longer worklists
      const int cap = c.len <= 1024 ? p.grid_chain : max(8, (int)((long long)p.grid_chain * 1024 / c.len));
      push_chain<true>(c.len, Ac, Ap, cur, min(cap, p.grid_chain));
    } else {
      push<GRID>(c.len, Ac, Ap, lp, cur);
    }
    const bool poll = GRID && (F & F_AUX) && (c.cflags & 1);  // NEXT-2: one grid-uniform look at the GR kernel
    if (poll && lead()) st_rlx((int *)ring_now(6), ld_acq(&p.ctrl2->cdone) == c.creq ? 1 : 0);
    if (chain_grid || poll) {
      barrier<GRID, true>();
      if (chain_grid) adv = max(1, (int)ring_prev(5));
      if (chain_grid && p.trace) tmark(160, (int)ring_prev(5));
      if (poll && ring_prev(6)) c.cflags |= 2;
    } else {
      barrier<GRID, false>();
    }
    if (c.iterGR > c.loop && adv > c.iterGR - c.loop) adv = c.iterGR - c.loop;  // land on iterGR / gapAt
    if (c.gapAt > c.loop && adv > c.gapAt - c.loop) adv = c.gapAt - c.loop;
    if (GRID) debug_check(4, c.loop, nullptr, 0);
    c.ac0 ^= 1;      // l.18: swap Ac and Ap
    c.loop += adv;   // l.19
    if (lead()) { if (GRID) L().loops++; else L().tail_loops++; }
    if (lead()) L().ns_loop += (long long)(tnow() - l0);
    return true;
  }

  // ---------------------------------------------------------------- tail mode
  // All CTAs call.  The tail group (CTA 0, or cluster 0) runs units of work alone
  // with CTA (cluster) barriers -- fix/push loops on worklists of at most tail_max
  // slots, GR levels of at most tail_f() rows -- while the other CTAs wait at one
  // grid barrier; most of the paper's iterations have "only a few" active columns
  // (P:525-528).  It stops when a unit needs the grid (R_GRID), when no active
  // column is left (R_TERM) or at the iteration cap (R_CAP), publishes its Ctl and
  // every CTA adopts it after the barrier.
  // thread 0, after the barrier: the published hand-over image -> shared memory
  __device__ __forceinline__ void load_handover() {
    const Ctrl *x = p.ctrl;
    sm.ho_reason = (int)ld_rlx((const u32 *)&x->ho_reason);
    sm.ho_ph = (int)ld_rlx((const u32 *)&x->ho_ph);
#pragma unroll
    for (int j = 0; j < (int)(sizeof(Ctl) / 8); j++) sm.ho[j] = ld_rlx(&x->ho[j]);
  }
  __device__ __forceinline__ void adopt_handover(Ctl &c) {
    long long *dst = reinterpret_cast<long long *>(&c);
#pragma unroll
    for (int j = 0; j < (int)(sizeof(Ctl) / 8); j++) dst[j] = sm.ho[j];
  }
  __device__ int tail_episode(Ctl &c) {
    int reason = R_NONE;
    Ctrl *x = p.ctrl;
    if (blockIdx.x < p.tail_ctas) {
      const int up = tail_f();
      bool wl_smem = false;  // the worklist lives in sm.wl (single-CTA tail)
      auto wl_in = [&]() {
        if (wl_smem || p.tail_ctas != 1 || c.len > TW) return;
        for (int i = threadIdx.x; i < c.len; i += NT) { sm.wl[0][i] = __ldcg(p.wl0 + i); sm.wl[1][i] = __ldcg(p.wl1 + i); }
        __syncthreads();
        wl_smem = true;
      };
      auto wl_out = [&]() {
        if (!wl_smem) return;
        for (int i = threadIdx.x; i < c.len; i += NT) { p.wl0[i] = sm.wl[0][i]; p.wl1[i] = sm.wl[1][i]; }
        __syncthreads();
        wl_smem = false;
      };
      for (;;) {
        if (c.loop >= p.max_loops) { reason = R_CAP; break; }
        if (c.gr_active) {
          if (c.gst.nlen > up) { reason = R_GRID; break; }
          gr_step<false>(c);
          if (lead()) L().tail_levels++;
          continue;
        }
        if ((F & F_AUX) && p.mode == MODE_RELABEL && c.loop != c.iterGR) { reason = R_TERM; break; }  // GR done
        if ((F & F_AUX) && (c.cflags & 1) && bcast_ld(&p.ctrl2->cdone) == c.creq) {  // NEXT-2: install on the grid
          c.cflags |= 2;
          reason = R_GRID;
          break;
        }
        if (c.loop == c.gapAt) { reason = R_GRID; break; }
        if (c.loop == c.iterGR) {
          if (c.ulen > up || base_overflow(c)) { reason = R_GRID; break; }
          gr_begin<false>(c);
          continue;
        }
        if (c.len > p.tail_max) { reason = R_GRID; break; }
        wl_in();
        bool more = wl_smem ? loop_step<false>(c, sm.wl[c.ac0 ? 0 : 1], sm.wl[c.ac0 ? 1 : 0])
                            : loop_step<false>(c, Acp(c), App(c));
        if (!more) { reason = R_TERM; break; }
      }
      wl_out();
      tail_sq_spill(c.gst);
      if (threadIdx.x == 0 && blockIdx.x == 0) {
        x->ho_reason = reason;
        x->ho_ph = ph;
        const long long *src = reinterpret_cast<const long long *>(&c);
        for (int j = 0; j < (int)(sizeof(Ctl) / 8); j++) x->ho[j] = src[j];
        for (int j = 0; j < 4; j++)
          for (int q = 0; q < 8; q++) x->ring[j][q] = 0;
      }
    }
    grid_sync(&p.ctrl->bar, true, [&] { load_handover(); });
    if (lead()) L().nbar++;
    trace_rec(99, reason);
    reason = sm.ho_reason;
    ph = sm.ho_ph + 1;
    adopt_handover(c);
    return reason;
  }

  // Serial mode (tests): one thread runs the fix and push steps of Alg. 7 with the
  // slots in increasing order -- exactly the schedule of the oracle's serial
  // simulator (or_gpr_serial, test side) -- until a GR (which runs on the grid, as
  // always) or a gap relabel is due, or no active column is left.  Trajectory,
  // matching and counters are then bit-exact against the simulator.
  __device__ void serial_fix_push(Ctl &c, int &reason) {
    const u32 base = c.base - stride();
    for (;;) {
      if (c.loop >= p.max_loops) { reason = R_CAP; return; }
      if (c.loop == c.gapAt || c.loop == c.iterGR) { reason = R_GRID; return; }
      int *Ac = Acp(c), *Ap = App(c);
      const int loop = (int)c.loop;
      bool act = false;
      S(SS_SLOTS) += c.len;
      if (c.shrink && p.shrink_min >= 0 && c.len >= p.shrink_min) {  // SHRKRNL, slot order
        int out = 0;
        for (int i = 0; i < c.len; i++) {
          int v = Ap[i], a = Ac[i];
          if (v != -1 && col_unmatched(v)) a = v;
          if (a != -1) { vst(p.iA + a, loop); act = true; Ac[out++] = a; }
        }
        c.len = out;
        if (lead()) L().shrinks++;
        c.shrink = 0;
      } else {  // INITKRNL (Alg. 8)
        for (int i = 0; i < c.len; i++) {
          int v = Ap[i];
          if (v != -1 && col_unmatched(v)) Ac[i] = v;
          v = Ac[i];
          if (v != -1) { vst(p.iA + v, loop); act = true; }
        }
      }
      if (!act) { reason = R_TERM; return; }
      for (int i = 0; i < c.len; i++) {  // PUSHKRNL (Alg. 9)
        int v = Ac[i];
        if (v == -1) { Ap[i] = -1; continue; }
        u64 cs = vld(p.colst + v);
        int psiv = labf(psi_of(cs), base, INF);
        int s = ld_ro(p.cptr + v), e = ld_ro(p.cptr + v + 1);
        if (p.dead_skip && psiv >= INF) e = s;
        int psimin = INF, ub = -1, wb = -1;
        for (int j = s; j < e; j++) {
          int x = ld_adj(p.cadj + j);
          u64 rs = vld(p.rowst + x);
          int l = labf(psi_of(rs), base, INF);
          S(SS_SCAN)++;
          if (l < psimin) {
            psimin = l; ub = x; wb = mu_of(rs);
            if (psimin == psiv - 1) break;
          }
        }
        u64 best = psimin < INF ? ((u64)(u32)psimin << 32) : ~0ull;
        push_finalize(i, v, cs, best, ub, wb, loop, base, Ac, Ap);
      }
      c.ac0 ^= 1;
      c.loop++;
      if (lead()) L().loops++;
    }
  }
  __device__ int serial_episode(Ctl &c) {
    int reason = R_NONE;
    Ctrl *x = p.ctrl;
    if (threadIdx.x == 0 && blockIdx.x == 0) {
      serial_fix_push(c, reason);
      if (sm.nd) { atomicAdd(&p.ctrl->ndead, sm.nd); sm.nd = 0; }
      x->ho_reason = reason;
      x->ho_ph = ph;
      const long long *src = reinterpret_cast<const long long *>(&c);
      for (int j = 0; j < (int)(sizeof(Ctl) / 8); j++) x->ho[j] = src[j];
    }
    grid_sync(&p.ctrl->bar, false, [&] { load_handover(); });
    if (lead()) L().nbar++;
    reason = sm.ho_reason;
    adopt_handover(c);
    return reason;
  }

  // G-PR-First (Alg. 3 + Alg. 6; the Fig. 1 ablation,
  // SURVEY NEXT-1): every loop tests every column for activity (R1) and pushes the
  // active ones -- no worklist, no iA.  One thread per column, batched scan.
  __device__ bool first_step(Ctl &c) {
    u64 l0 = tnow();
    const u32 base = c.base - stride();
    const int G = gridDim.x * NT, g = blockIdx.x * NT + threadIdx.x;
    long long act = 0;
    fl_r = c.floor_r;
    fl_c = c.floor_c;
    for (int v = g; v < n; v += G) {
      u64 cs = vld(p.colst + v);
      int cm = mu_of(cs);
      bool active = cm == -1 || (cm >= 0 && mu_of(vld(p.rowst + cm)) != v);  // Alg. 6 l.3 (R1)
      if (!active) continue;
      act++;
      int psiv = labf(psi_of(cs), base, fl_c);
      int s = ld_ro(p.cptr + v), e = ld_ro(p.cptr + v + 1);
      if (p.dead_skip && psiv >= INF) e = s;
      u64 best;
      int ub, wb;
      scan(s, e, 0, 1, 1u << lane_id(), psiv - 1, base, best, ub, wb);  // l.5-12
      int psimin = best == ~0ull ? INF : (int)(best >> 32);
      if (psimin < INF) {                                             // l.13-17
        vst(p.rowst + ub, pack(v, base + (u32)psimin + 2u));
        vst(p.colst + v, pack(ub, base + (u32)psimin + 1u));
        S(SS_PUSH)++;
      } else {                                                        // l.18-19
        vst(p.colst + v, pack(-2, psi_of(cs)));
        S(SS_DEAD)++;
        atomicAdd(&p.ctrl->ndead, 1u);
      }
    }
    trace(4, n);
    add_count(act, 0);
    barrier<true>();
    const long long a = ring_prev(0);
    if (lead()) L().ns_loop += (long long)(tnow() - l0);
    if (a == 0) return false;
    c.loop++;
    if (lead()) L().loops++;
    return true;
  }

  // Stale rows (R27, build addition): at termination a row u with mu(u) = c whose
  // column does not point back (mu(c) != u).  The paper argues that only column
  // entries of mu can be inconsistent when the loop ends.  Push chains
  // (R26) claim rows by CAS and then set mu(c) by CAS (chain_settle); a late
  // setting can still lose against a newer push of c, and a caller's GIVEN matching
  // may hold such rows too.  A stale row would count in |M| and never start a BFS.
  // So before the guard's GR: if c's own row does not point back either, c is
  // re-attached to u (CAS on c's word, so one row wins when several hold c);
  // otherwise, or when the CAS loses, u is set unmatched.  The same pass rebuilds
  // the unmatched-row list U from scratch (every row unmatched after the repair,
  // isolated rows excepted, each once), so the guard's GR starts from every
  // unmatched row and U can never overflow.  One pass over the row words (plus the
  // mates' column words and the bounds of the unmatched rows).
  __device__ void repair_rows(Ctl &c) {
    int *U = Ub(c);
    long long repaired = 0;
    for (int t = blockIdx.x * NT; t < m; t += gridDim.x * NT) {
      const int u = t + (int)threadIdx.x;
      u64 w = 0, cw = 0;
      int cc = -1;
      bool stale = false, unm = false;
      if (u < m) {
        w = vld(p.rowst + u);
        cc = mu_of(w);
        if (cc >= 0) {
          cw = ld_rlx(p.colst + cc);
          stale = mu_of(cw) != u;
        } else {
          unm = true;
        }
      }
      if (stale) {
        const int u2 = mu_of(cw);
        const bool c_free = u2 < 0 || mu_of(ld_rlx(p.rowst + u2)) != cc;
        if (c_free && atomicCAS(p.colst + cc, cw, pack(u, psi_of(cw))) == cw) {
          if (u2 == -2) atomicSub(&p.ctrl->ndead, 1u);
        } else {
          vst(p.rowst + u, pack(-1, psi_of(w)));
          unm = true;
        }
        repaired++;
      }
      if (unm && ld_ro(p.rptr + u) == ld_ro(p.rptr + u + 1)) unm = false;  // isolated: never in U (n_iso)
      int tot, r = cta_rank<NT>(unm, sm.w, &tot);
      if (threadIdx.x == 0) sm.qbase = tot ? (int)atomicAdd(ring_now(6), (u32)tot) : 0;
      __syncthreads();
      if (unm) U[sm.qbase + r] = u;
    }
    add_count(repaired, 7);
    barrier<true>();
    c.ulen = (int)ring_prev(6);
    if (lead()) L().repaired += ring_prev(7);
  }

  // exactness guard (R16): one more GR; every unmatched column it reaches is
  // re-activated and the loop resumes (returns true); otherwise the labels certify
  // maximality (returns false).
  __device__ bool guard_step(Ctl &c) {
    if (!p.final_check) return false;
    u64 g0 = tnow();
    repair_rows(c);
    if (base_overflow(c)) { reset_labels(); c.base = 1; }
    int gcount = 0;
    int *Ac = Acp(c), *Ap = App(c);
    int *U = Ub(c), *T = Tb(c);
    int ml = global_relabel<true>(U, c.ulen, T, Q4(0), Q4(1), c.base, Ac, gcount);
    c.u0 ^= 1;
    if (lead()) { L().grs++; L().levels += ml / 2; }
    c.base += stride();
    if (lead()) L().ns_gr += (long long)(tnow() - g0);
    if (gcount == 0) return false;
    if (lead()) L().guard_re += gcount;
    for (int i = blockIdx.x * NT + threadIdx.x; i < gcount; i += gridDim.x * NT) {
      int v = __ldcg(Ac + i);
      u64 cs = vld(p.colst + v);
      if (mu_of(cs) == -2) atomicSub(&p.ctrl->ndead, 1u);
      vst(p.colst + v, pack(-1, psi_of(cs)));
      Ap[i] = v;
    }
    barrier<true, false>();
    if (blockIdx.x == 0 && threadIdx.x == 0) p.ctrl->gcnt = 0;  // every CTA read it before the barrier above
    c.len = gcount;
    c.floor_r = c.floor_c = INF;
    c.iterGR = c.loop + iter_gap(ml);
    c.gapAt = gap_at(c.loop, c.iterGR);
    c.shrink = 0;
    return true;
  }

  // ---------------------------------------------------------------- the solve
  __device__ __forceinline__ void run() {
    if ((F & F_AUX) && p.mode == MODE_CONC_GR) {  // the GR kernel of a concurrent solve
      conc_gr();
      return;
    }
    u64 t0 = tnow(), tA = t0;
    long long ns_init = 0;
    int *Ac = p.wl0, *Ap = p.wl1;
    int *U = p.qa, *T = p.qb;
    int4 *Qa = Q4(0), *Qb = Q4(1);
    if (threadIdx.x == 0) { sm.qcnt = 0; sm.nhuge = 0; sm.nd = 0; sm.chmax = 0; memset(&sm.ld, 0, sizeof(LeadStats)); }
    for (int k = 0; k < SS_N; k++) sm.ts[k][threadIdx.x] = 0;
    if (threadIdx.x < 2) sm.lvc[threadIdx.x] = 0;
    add_count(init_state(), 7);
    barrier<true>();
    if (ring_prev(7)) {  // a caller's array held an out-of-range entry
      if (lead()) {
        p.ctrl->err = -1;  // MCM_EINVAL
        if ((F & F_AUX) && p.conc > 0) st_rlx((int *)&p.ctrl2->cexit, 1);  // release the GR kernel
      }
      return;
    }
    if ((F & F_AUX) && p.mode == MODE_UNIT) {  // mcm_unit_step: one phase on the caller's state
      unit();
      finish_stats(0, 0, 0);
      return;
    }
    if ((p.mode == MODE_SOLVE && p.init == 0) || p.mode == MODE_INIT) {
      greedy();
      barrier<true, false>();
    }
    if ((F & F_AUX) && p.mode == MODE_INIT) {  // mcm_initial_matching: M0 out, |M0| -> ring 0
      fixmatching(0, 1);
      barrier<true>();
      finish_stats(0, 0, 0);
      return;
    }
    debug_check(1, -1, nullptr, 0);
    // unmatched rows -> U; unmatched columns (increasing id) -> Ac (R12)
    build_unmatched_rows(U, 0);
    // isolated columns stay out of the worklist and count as dead (R25), except in
    // serial mode (the simulator's worklist holds every unmatched column, R12) and
    // in G-PR-First (no worklist: its loop tests and kills them itself)
    const bool skip_iso = (p.mode == MODE_SOLVE || p.mode == MODE_RELABEL) && !((F & F_SERIAL) && p.serial) &&
                          !((F & F_FIRST) && p.variant == 1);
    long long iso_c = 0;
    const bool consistent = p.mode == MODE_SOLVE && p.init == 0;  // M0 from the device greedy
    int run1 = compact_pass1<true, 8>(
        n, [&](int i0, int hi, int *val) { iso_c += cols_unmatched<8>(i0, hi, val, skip_iso, consistent); }, T, Ac);
    iso_c = cta_sum<NT>(iso_c, sm.red);
    if (threadIdx.x == 0 && iso_c) atomicAdd(&p.ctrl->ndead, (u32)iso_c);
    barrier<true>();
    int ulen = (int)ring_prev(0);
    n_iso = (int)ring_prev(1);  // isolated rows (never in U)
    int len = compact_pass2<true>(n, T, Ac, run1, Ap);  // Ap = Ac (R12)
    long long init_card = (long long)m - n_iso - ulen;

    if ((F & F_AUX) && p.mode == MODE_GAP) {  // mcm_gap_relabel: labels in, labels out
      int gl = gap_relabel(1);
      write_labels(1);
      if (lead()) p.ctrl->stat[ST_MAXLEVEL] = gl;
      finish_stats(0, 0, 0);
      return;
    }
    if ((F & F_AUX) && p.mode == MODE_RELABEL) {  // mcm_global_relabel: one GR as a solve would run it
      relabel(ulen);
      finish_stats(0, 0, 0);
      return;
    }

    barrier<true, false>();
    debug_check(2, -1, Ac, len);
    ns_init = (long long)(tnow() - t0);

    Ctl c;
    memset(&c, 0, sizeof(c));
    c.len = len; c.ulen = ulen; c.base = 1; c.gapAt = -1; c.ac0 = 1; c.u0 = 1;  // loop = iterGR = 0
    c.floor_r = c.floor_c = INF;
    c.cflags = ((F & F_AUX) && p.conc > 0 && p.mode == MODE_SOLVE) ? 1 : 0;
    for (;;) {
      if (c.loop >= p.max_loops) {
        if (lead()) p.ctrl->err = -5;
        break;
      }
      if ((F & F_AUX) && (c.cflags & 2)) { conc_install(c); continue; }  // NEXT-2: the GR kernel's labels
      if ((F & F_SERIAL) && p.serial && !c.gr_active && c.loop != c.iterGR && c.loop != c.gapAt) {
        int r = serial_episode(c);
        if (r == R_CAP) {
          if (lead()) p.ctrl->err = -5;
          break;
        }
        if (r == R_TERM && !guard_step(c)) break;
        continue;
      }
      const int up = tail_f();
      bool tail_ok = p.tail_max > 0 &&
                     (c.gr_active ? (c.gst.nlen <= up / 2 && !c.gst.dirty)
                                  : (c.loop == c.gapAt ? false
                                                       : (c.loop == c.iterGR ? (c.ulen <= up && !base_overflow(c))
                                                                             : c.len <= p.tail_max)));
      if (tail_ok) {
        int r = tail_episode(c);
        if (r == R_CAP) {
          if (lead()) p.ctrl->err = -5;
          break;
        }
        if (r == R_TERM) {
          if (F & F_AUX) conc_stop(c);
          if (!guard_step(c)) break;
        }
        continue;
      }
      // one unit of grid work
      if (c.gr_active) {                                               // Alg. 5 level(s)
        if (win_ok(c)) gr_window_step(c);
        else gr_step<true>(c);
        continue;
      }
      if ((F & F_GAP) && c.loop == c.gapAt) {                          // gap relabel (R14)
        u64 g0 = tnow();
        if (gap_relabel(c.base - stride()) >= 0 && lead()) L().gaps++;
        c.gapAt = -1;
        if (lead()) L().ns_gr += (long long)(tnow() - g0);
        continue;
      }
      if (c.loop == c.iterGR) {                                        // Alg. 7 l.6-9
        if (base_overflow(c)) { reset_labels(); c.base = 1; }
        gr_begin<true>(c);
        continue;
      }
      if ((F & F_FIRST) && p.variant == 1) {                                             // G-PR-First (Alg. 3)
        if (!first_step(c) && !guard_step(c)) break;
        continue;
      }
      if (!loop_step<true>(c, Acp(c), App(c))) {                      // l.10-19 / termination
        if (F & F_AUX) conc_stop(c);
        if (!guard_step(c)) break;
      }
    }
    if (F & F_AUX) conc_stop(c);
    fixmatching(0, 1);                                                 // l.20
    barrier<true>();
    finish_stats(init_card, ns_init, (long long)(tnow() - tA));
  }

  // mcm_global_relabel (MODE_RELABEL): one GR on the caller's matching, run by the
  // same state machine as a solve's GR -- grid levels, single-CTA tail levels with
  // the frontier in shared memory (tail_max > 0, frontiers of at most tail_f rows,
  // hand-over both ways), bottom-up levels (bu_div), and the early stop of R22 /
  // R28 when gr_early is set (unreached vertices then carry the lower bounds
  // floor_r / floor_c instead of m+n).  Writes the decoded labels; stats slots:
  // maxLevel (as GETITERGR sees it), the floors and the levels run in the tail.
  __device__ void relabel(int ulen) {
    Ctl c;
    memset(&c, 0, sizeof(c));
    c.ulen = ulen; c.base = 1; c.gapAt = -1; c.ac0 = 1; c.u0 = 1;  // loop = iterGR = 0: the GR is due
    c.floor_r = c.floor_c = INF;
    const int up = tail_f();
    for (;;) {
      if (!c.gr_active && c.loop != c.iterGR) break;  // gr_finish moved iterGR past loop: done
      const bool tail_ok = p.tail_max > 0 && (c.gr_active ? (c.gst.nlen <= up / 2 && !c.gst.dirty) : c.ulen <= up);
      if (tail_ok) tail_episode(c);
      else if (c.gr_active && win_ok(c)) gr_window_step(c);
      else if (c.gr_active) gr_step<true>(c);
      else gr_begin<true>(c);
    }
    const u32 base = c.base - stride();  // gr_finish moved base to the next epoch
    const int G = gridDim.x * NT, g = blockIdx.x * NT + threadIdx.x;
    for (int u = g; u < m; u += G) p.rmatch_out[u] = labf(psi_of(vld(p.rowst + u)), base, c.floor_r);
    for (int v = g; v < n; v += G) p.cmatch_out[v] = labf(psi_of(vld(p.colst + v)), base, c.floor_c);
    if (lead()) {
      p.ctrl->stat[ST_MAXLEVEL] = c.gst.deepest + 2;
      p.ctrl->stat[ST_FLOOR_R] = c.floor_r;
      p.ctrl->stat[ST_FLOOR_C] = c.floor_c;
    }
    barrier<true, false>();
  }

  // mcm_unit_step (MODE_UNIT): ONE phase of the solve on the caller's state (mu,
  // labels at base 1, iA, Ac = wl0, Ap = wl1, loop), run by the code a solve runs:
  // on the grid (every CTA) or in the single-CTA tail (CTA 0, the worklist in
  // shared memory when it fits, as tail_episode keeps it).  Result -> stat slot
  // ST_MAXLEVEL: FIX the active-slot count, SHRINK the new length, FIXMATCHING |M|.
  __device__ void unit() {
    const u32 base = 1;
    fl_r = fl_c = INF;
    const int lp = (int)p.unit_loop, len = p.unit_len, what = p.unit_what;
    int *Ac = p.wl0, *Ap = p.wl1;
    long long r = 0;
    if (p.unit_where == 0 || what == UNIT_FIXMATCHING) {
      if (what == UNIT_FIX) {
        fix_plain<true>(len, Ac, Ap, lp, 0);
        barrier<true>();
        r = ring_prev(0);
      } else if (what == UNIT_SHRINK) {
        r = fix_compact<true>(len, Ac, Ap, lp, p.qb);
      } else if (what == UNIT_PUSH) {
        push<true>(len, Ac, Ap, lp, base);
        barrier<true, false>();
      } else {
        fixmatching(0, 1);
        barrier<true>();
        r = ring_prev(0);
      }
    } else {
      if (blockIdx.x == 0) {
        const bool sh = len <= TW;  // tail_episode's wl_in
        for (int i = threadIdx.x; sh && i < len; i += NT) { sm.wl[0][i] = __ldcg(Ac + i); sm.wl[1][i] = __ldcg(Ap + i); }
        __syncthreads();
        int *A = sh ? sm.wl[0] : Ac, *B = sh ? sm.wl[1] : Ap;
        if (what == UNIT_PUSH) push<false>(len, A, B, lp, base);
        else r = fix_compact<false>(len, A, B, lp, nullptr);  // the tail compacts at every fix step
        __syncthreads();
        for (int i = threadIdx.x; sh && i < len; i += NT) { Ac[i] = sm.wl[0][i]; Ap[i] = sm.wl[1][i]; }
        if (threadIdx.x == 0) {
          p.ctrl->ho_ph = ph;
          p.ctrl->ho[0] = r;
          for (int j = 0; j < 4; j++)
            for (int q = 0; q < 8; q++) p.ctrl->ring[j][q] = 0;
        }
      }
      grid_sync(&p.ctrl->bar, true, [&] { load_handover(); });
      ph = sm.ho_ph + 1;
      r = sm.ho[0];
    }
    const int G = gridDim.x * NT, g = blockIdx.x * NT + threadIdx.x;
    for (int u = g; u < m; u += G) {
      const u64 w = vld(p.rowst + u);
      if (what != UNIT_FIXMATCHING) p.rmatch_out[u] = mu_of(w);
      p.psi_row_io[u] = labf(psi_of(w), base, INF);
    }
    for (int v = g; v < n; v += G) {
      const u64 w = vld(p.colst + v);
      if (what != UNIT_FIXMATCHING) p.cmatch_out[v] = mu_of(w);
      p.psi_col_io[v] = labf(psi_of(w), base, INF);
    }
    if (lead()) p.ctrl->stat[ST_MAXLEVEL] = r;
    barrier<true, false>();
  }


  // ---------------------------------------------------------------- concurrent GR (NEXT-2)
  // The paper's future work: "concurrent execution of global-relabeling
  // and push-relabel kernels".  With option gr_concurrent = A > 0 a solve is two
  // co-resident persistent kernels on two streams: this GR kernel on A CTAs and the
  // push kernel (run()) on the rest.  The GR kernel waits for a request, runs a
  // complete level-synchronous BFS (Alg. 2 / 4-5 semantics) from the unmatched rows
  // of the CURRENT matching -- which the push kernel keeps changing: the mates are
  // read racily, so the labels describe a matching of a few loops ago -- into SHADOW
  // label arrays (srow / scol, epoch-tagged like the packed words), publishes them,
  // and waits again.  The push kernel keeps pushing on its installed labels and,
  // at its next loop boundary after a completion, installs the shadow labels into
  // the packed {mu, psi} words (pushes paused for that one pass) and requests the
  // next GR.  Labels from a stale matching can be wrong (a column may look dead, a
  // row may keep label 0 after it was matched): the exactness guard (R16) runs
  // after termination as always, so the cardinality stays exact.
  __device__ void conc_gr() {
    Ctrl *x = p.ctrl;  // this kernel's own control block
    const u32 sd = stride();
    u32 sbase = 1, gen = 0;
    int *Q[2] = {p.qc, p.qd};  // row frontiers (the push kernel uses qa / qb / wl0 / wl1)
    const int GT = gridDim.x * NT, gt = blockIdx.x * NT + threadIdx.x;
    int k = 0;  // level counter for the rotating frontier counters
    auto gsync = [&](int j) {   // barrier; sm.rp[0] = ccnt[j] afterwards
      grid_sync(&x->bar, false, [&] { sm.rp[0] = ld_rlx(&x->ccnt[j]); });
    };
    for (;;) {
      if (threadIdx.x == 0) {
        const u64 t0 = gtime();
        u32 r;
        for (;;) {
          r = ld_acq(&x->creq);
          if (r > gen || ld_rlx(&x->cexit)) break;
          if (gtime() - t0 > 4000000000ull) { r = 0; break; }  // 4 s without a request: the push kernel is gone
          __nanosleep(200);
        }
        sm.bc = (r > gen && !ld_rlx(&x->cexit)) ? r : 0u;
      }
      __syncthreads();
      const u32 r = sm.bc;
      __syncthreads();
      if (r == 0) break;
      gen = r;  // serve the latest request
      if ((u64)sbase + 2ull * sd >= 0xfffffff0ull) {  // epoch overflow: all shadow labels stale again
        for (int u = gt; u < m; u += GT) st_rlx((int *)p.srow + u, 0);
        for (int v = gt; v < n; v += GT) st_rlx((int *)p.scol + v, 0);
        gsync(0);
        sbase = 1;
      }
      // level 0: the unmatched rows (with an edge) of the current matching, label 0
      for (int t = blockIdx.x * NT; t < m; t += GT) {
        const int u = t + (int)threadIdx.x;
        bool f = false;
        if (u < m && mu_of(vld(p.rowst + u)) == -1 && ld_ro(p.rptr + u) < ld_ro(p.rptr + u + 1)) {
          st_rlx((int *)p.srow + u, (int)sbase);
          f = true;
        }
        if (f) {
          cg::coalesced_group g = cg::coalesced_threads();
          u32 b = 0;
          if (g.thread_rank() == 0) b = atomicAdd(&x->ccnt[k & 3], (u32)g.size());
          Q[0][g.shfl(b, 0) + g.thread_rank()] = u;
        }
      }
      gsync(k & 3);
      int nlen = (int)sm.rp[0], cur = 0;
      if (lead()) x->ccnt[(k + 2) & 3] = 0;
      k++;
      for (u32 lvl = 0; nlen > 0; lvl += 2) {
        const u32 lc = sbase + lvl + 1, lr = sbase + lvl + 2;
        constexpr int GL = 8;  // lanes per frontier row
        const int gl = lane_id() & (GL - 1);
        for (int t = blockIdx.x * (NT / GL); t < nlen; t += gridDim.x * (NT / GL)) {
          const int i = t + (int)threadIdx.x / GL;
          const int u = i < nlen ? __ldcg(Q[cur] + i) : -1;
          const int s0 = u >= 0 ? ld_ro(p.rptr + u) : 0, e0 = u >= 0 ? ld_ro(p.rptr + u + 1) : 0;
          for (int j = s0 + gl; j < e0; j += GL) {
            const int v = ld_adj(p.radj + j);
            const u32 sv = (u32)ld_rlx((const int *)p.scol + v);
            if (sv >= sbase || atomicCAS(p.scol + v, sv, lc) != sv) continue;  // visited, or claimed by another
            const int w = mu_of(vld(p.colst + v));
            if (w < 0 || mu_of(vld(p.rowst + w)) != v) continue;  // not matched (Alg. 5 l.6)
            st_rlx((int *)p.srow + w, (int)lr);
            cg::coalesced_group g = cg::coalesced_threads();
            u32 b = 0;
            if (g.thread_rank() == 0) b = atomicAdd(&x->ccnt[k & 3], (u32)g.size());
            Q[cur ^ 1][g.shfl(b, 0) + g.thread_rank()] = w;
          }
        }
        gsync(k & 3);
        nlen = (int)sm.rp[0];
        if (lead()) x->ccnt[(k + 2) & 3] = 0;
        k++;
        cur ^= 1;
      }
      // every CTA passed the last barrier: the labels are complete -> publish
      if (lead()) {
        for (int j = 0; j < 4; j++) x->ccnt[j] = 0;
        st_rlx((int *)&x->csbase, (int)sbase);
        __threadfence();
        asm volatile("st.release.gpu.global.u32 [%0], %1;" ::"l"(&x->cdone), "r"(gen) : "memory");
        L().grs++;
      }
      k = 0;
      sbase += sd;
      gsync(0);  // the counters are zero before anyone appends again
    }
    grid_sync(&x->bar, false);
    if (lead()) asm volatile("st.release.gpu.global.u32 [%0], %1;" ::"l"(&x->cexited), "r"(1u) : "memory");
  }
  // push kernel: the GR kernel finished the requested labels (CTA-uniform via sm.bc)
  __device__ bool conc_ready(const Ctl &c) {
    return (c.cflags & 1) && bcast_ld(&p.ctrl2->cdone) == c.creq;
  }
  __device__ void conc_request(Ctl &c) {
    c.creq++;
    if (lead()) asm volatile("st.release.gpu.global.u32 [%0], %1;" ::"l"(&p.ctrl2->creq), "r"(c.creq) : "memory");
  }
  // install the shadow labels into the packed words (every push-kernel CTA, pushes
  // paused at a loop boundary), move to the new epoch, request the next GR
  __device__ void conc_install(Ctl &c) {
    u64 g0 = tnow();
    const u32 sb = bcast_ld(&p.ctrl2->csbase);
    if (base_overflow(c)) { reset_labels(); c.base = 1; }
    const u32 nb = c.base;
    const int G = gridDim.x * NT, g = blockIdx.x * NT + threadIdx.x;
    for (int u = g; u < m; u += G) {
      const u32 sl = (u32)ld_rlx((const int *)p.srow + u);
      if (sl >= sb) vst(p.rowst + u, pack(mu_of(vld(p.rowst + u)), nb + (sl - sb)));
    }
    for (int v = g; v < n; v += G) {
      const u32 sl = (u32)ld_rlx((const int *)p.scol + v);
      if (sl >= sb) vst(p.colst + v, pack(mu_of(vld(p.colst + v)), nb + (sl - sb)));
    }
    barrier<true, false>();
    c.base += stride();
    c.floor_r = c.floor_c = INF;
    c.cflags &= ~2;
    c.shrink = 1;  // Alg. 7 l.9: the worklist is compacted after a GR
    if (lead()) { L().grs++; L().ns_gr += (long long)(tnow() - g0); }
    conc_request(c);
  }
  // stop the GR kernel (it finishes a running BFS first) before the queues it uses
  // are needed again (guard GR) or the solve ends
  __device__ void conc_stop(Ctl &c) {
    if (!(c.cflags & 1)) return;
    if (lead()) {
      asm volatile("st.release.gpu.global.u32 [%0], %1;" ::"l"(&p.ctrl2->cexit), "r"(1u) : "memory");
      const u64 t0 = gtime();
      while (!ld_acq(&p.ctrl2->cexited) && gtime() - t0 < 8000000000ull) __nanosleep(200);
    }
    barrier<true, false>();
    c.cflags = 0;
  }

  __device__ void reset_labels() {
    const int G = gridDim.x * NT, g = blockIdx.x * NT + threadIdx.x;
    for (int u = g; u < m; u += G) {
      u64 w = vld(p.rowst + u);
      vst(p.rowst + u, pack(mu_of(w), 0));
    }
    for (int v = g; v < n; v += G) { u64 w = vld(p.colst + v); vst(p.colst + v, pack(mu_of(w), 0)); }
    barrier<true, false>();
  }

  __device__ void finish_stats(long long init_card, long long ns_init, long long ns_total) {
    __syncthreads();
    const int slot[SS_N] = {ST_PUSHES, ST_BLOCKED, ST_DEAD, ST_SCANNED, ST_SLOTS, ST_REACHED_FREE,
                            ST_GR_ROWS, ST_GR_EDGES, ST_GR_COLS, ST_GREEDY_EDGES};
    for (int k = 0; k < SS_N; k++) {
      const long long t = cta_sum<NT>((long long)sm.ts[k][threadIdx.x], sm.red);
      if (threadIdx.x == 0 && t) atomicAdd((unsigned long long *)&p.ctrl->stat[slot[k]], (unsigned long long)t);
    }
    if (lead()) {
      long long *st = p.ctrl->stat;
      const LeadStats &l = L();
      st[ST_LOOPS] = l.loops + l.tail_loops; st[ST_GRS] = l.grs; st[ST_LEVELS] = l.levels; st[ST_SHRINKS] = l.shrinks;
      st[ST_GAPS] = l.gaps;
      st[ST_GUARD] = l.guard_re; st[ST_INITCARD] = init_card; st[ST_NS_INIT] = ns_init; st[ST_NS_GR] = l.ns_gr;
      st[ST_NS_LOOP] = l.ns_loop; st[ST_NS_TOTAL] = ns_total; st[ST_TAILLOOPS] = l.tail_loops;
      st[ST_BARRIERS] = l.nbar;
      st[ST_REPAIRED] = l.repaired;
      st[ST_TAIL_LEVELS] = l.tail_levels;
      st[ST_WINDOWS] = l.wlevels;
      st[ST_TRACE_N] = l.tn;
      if (p.mode == MODE_SOLVE || p.mode == MODE_INIT) {
        st[ST_CARD] = (long long)ring_prev(0);
        st[ST_FIXED] = (long long)ring_prev(1);
      }
    }
  }
};

#ifndef MCM_MINB
#define MCM_MINB 1
#endif
template <int F>
__global__ void __launch_bounds__(NT, MCM_MINB) gpr_kernel(const __grid_constant__ Params p) {
  Solver<F> s(p);
  s.run();
}

#undef sm
}  // namespace mcm
