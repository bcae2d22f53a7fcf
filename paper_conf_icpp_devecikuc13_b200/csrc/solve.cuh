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

namespace mcm {

constexpr int NT = 512;          // threads per CTA
constexpr int NWARP = NT / 32;
constexpr int QCAP = 4096;       // shared staging for the next BFS frontier
constexpr int SMALL_DEG = 32;    // greedy: adjacency lists up to this length: one thread
constexpr int BIG_DEG = 64;      // GR / push: longer lists go to the whole warp
constexpr int KB = 4;            // neighbours in flight per lane (batched loads)

enum { MODE_SOLVE = 0, MODE_RELABEL = 1, MODE_GAP = 2 };

// statistics slots (Ctrl::stat)
enum {
  ST_LOOPS, ST_GRS, ST_LEVELS, ST_PUSHES, ST_BLOCKED, ST_DEAD, ST_SCANNED, ST_SLOTS, ST_SHRINKS, ST_GAPS,
  ST_GUARD, ST_FIXED, ST_INITCARD, ST_CARD, ST_TAILLOOPS, ST_BARRIERS, ST_NS_INIT, ST_NS_GR, ST_NS_LOOP,
  ST_NS_TOTAL, ST_MAXLEVEL, ST_REACHED_FREE, ST_GR_ROWS, ST_GR_EDGES, ST_GR_COLS, ST_GREEDY_EDGES, ST_TRACE_N, ST_NSTAT = 32
};

struct Ctrl {
  u32 ring[4][4];          // per-phase counters, rotated (see Solver::barrier)
  u32 bar;                 // grid barrier word (device.cuh grid_sync)
  u32 pad0[3];
  long long stat[ST_NSTAT];
  int err;                 // 0 or an MCM_* code
  u32 gcnt;                // exactness-guard list cursor (monotonic within a solve)
  int gmax, gmin;          // gap relabel: largest finite label, smallest empty label
  int pad[12];
  long long dbg[8];        // debug checks: [0] count, [1] where, [2] loop, [3] vertex, [4] value
  // tail-mode handoff (CTA 0 -> grid)
  int ho_reason, ho_ph, ho_len, ho_ulen, ho_shrink, ho_ac0, ho_u0, ho_gl, ho_gd, ho_gn, ho_gc;
  u32 ho_base;
  long long ho_loop, ho_iter, ho_gapat;
};

struct Params {
  int m, n, mode;
  const int *rptr, *radj, *cptr, *cadj;
  u64 *rowst, *colst;
  int *iA, *wl0, *wl1, *qa, *qb, *qc, *qd;
  int *ctacnt;
  int *dbgbuf;             // n ints (debug checks only)
  int tail_ctas;           // CTAs of the tail group (= cluster 0 when > 1)
  int *hist;               // gap relabel histogram (hist_len counters, zero between uses)
  int hist_len;
  int debug;
  long long *trace;        // optional phase trace: {tag, size, t_end_ns} triples (MCM_TRACE)
  int trace_cap;
  Ctrl *ctrl;
  // options
  double k;
  int gr_fixed, shrink_min, init, gap, final_check, dead_skip, tail_max, compact_every, compact_adapt;
  long long max_loops;
  // I/O
  const int *rmatch_in, *cmatch_in;
  int *rmatch_out, *cmatch_out;  // solve: matching; relabel: psi_row / psi_col
};

struct Smem {
  long long red[NWARP];
  int w[NWARP];
  int q[QCAP];
  int qcnt, qbase, tmp;
};

__device__ __forceinline__ u64 gtime() {
  u64 t;
  asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
  return t;
}

struct Solver {
  const Params &p;
  Smem &sm;
  const int m, n, INF;
  // per-thread statistics (reduced at the end)
  long long s_push = 0, s_block = 0, s_dead = 0, s_scan = 0, s_slots = 0, s_free = 0;
  long long s_grrows = 0, s_gredges = 0, s_grcols = 0, s_gyedges = 0, s_gapkill = 0;
  int ph = 0;  // phase counter: identical in every thread
  long long nbar = 0;
  int ttag = 0, tsz = 0, tn = 0;  // phase trace (lead thread only)
  long long gaps_total = 0;
  __device__ __forceinline__ void trace(int tag, int sz) {
    ttag = tag; tsz = sz;
  }

  __device__ Solver(const Params &p_, Smem &sm_) : p(p_), sm(sm_), m(p_.m), n(p_.n), INF(p_.m + p_.n) {}

  // ---------------------------------------------------------------- barriers
  // ring[ph & 3] collects the counts produced during phase ph; the consumer reads
  // it right after the barrier.  ring[(ph + 2) & 3] was produced two phases ago
  // and consumed at the start of the previous phase, so CTA 0 may clear it now.
  template <bool GRID>
  __device__ __forceinline__ void barrier() {
    if (p.trace && threadIdx.x == 0 && blockIdx.x == 0 && tn < p.trace_cap) {
      p.trace[3 * tn] = ttag * 2 + (GRID ? 1 : 0); p.trace[3 * tn + 1] = tsz; p.trace[3 * tn + 2] = (long long)gtime();
      tn++;
    }
    if (GRID) {
      grid_sync(&p.ctrl->bar, false);
      nbar++;
    } else if (p.tail_ctas > 1) {
      // tail group = thread-block cluster 0: hardware cluster barrier (release /
      // acquire at cluster scope covers the global writes of the cluster's CTAs)
      asm volatile("barrier.cluster.arrive.release.aligned;\n\tbarrier.cluster.wait.acquire.aligned;" ::: "memory");
    } else {
      __syncthreads();
    }
    ph++;
    if (blockIdx.x == 0 && threadIdx.x == 0) {
      u32 *r = p.ctrl->ring[(ph + 2) & 3];
      r[0] = r[1] = r[2] = r[3] = 0;
    }
  }
  __device__ __forceinline__ u32 *ring_now(int j) { return &p.ctrl->ring[ph & 3][j]; }
  __device__ __forceinline__ u32 ring_prev(int j) { return ld_rlx(&p.ctrl->ring[(ph - 1) & 3][j]); }

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
    int c = mu_of(ld_rlx(p.colst + v));
    if (c == -1) return true;
    if (c < 0) return false;
    return mu_of(ld_rlx(p.rowst + c)) != v;
  }

  // ---------------------------------------------------------------- staging
  __device__ __forceinline__ void stage(int x, int *next, u32 *gcnt) {
    int q = atomicAdd(&sm.qcnt, 1);
    if (q < QCAP) sm.q[q] = x;
    else next[atomicAdd(gcnt, 1u)] = x;  // overflow: direct append
  }
  __device__ __forceinline__ void flush(int *next, u32 *gcnt) {
    __syncthreads();
    int c = min(sm.qcnt, QCAP);
    if (threadIdx.x == 0) sm.qbase = c ? (int)atomicAdd(gcnt, (u32)c) : 0;
    __syncthreads();
    for (int j = threadIdx.x; j < c; j += NT) next[sm.qbase + j] = sm.q[j];
    __syncthreads();
    if (threadIdx.x == 0) sm.qcnt = 0;
    __syncthreads();
  }

  // ---------------------------------------------------------------- stable compaction
  // Pass 1 of a stable compaction of items [0, len): f(i) returns the value to keep
  // or -1.  Survivors of CTA c's chunk go to T[lo_c + rank]; ctacnt[c] = count.
  // GRID=false: a single CTA, written straight to `out` (reads of a tile finish
  // before its writes, and writes never pass the tile being read).
  template <bool GRID, class F>
  __device__ int compact_pass1(int len, F f, int *T, int *out) {
    const int C = ncta<GRID>(), c = cta<GRID>();
    const int chunk = (len + C - 1) / C;
    const int lo = min(len, c * chunk), hi = min(len, lo + chunk);
    int run = 0;
    for (int t = lo; t < hi; t += NT) {
      int i = t + threadIdx.x;
      int val = (i < hi) ? f(i) : -1;
      int tot;
      int r = cta_rank<NT>(val != -1, sm.w, &tot);
      if (val != -1) (C > 1 ? T[lo + run + r] : out[run + r]) = val;
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
  // Vertex state from the initial matching (GIVEN / RELABEL: the caller's arrays;
  // else empty).  Labels start stale (psi = 0 < base).
  __device__ void init_state() {
    const int G = gridDim.x * NT, g = blockIdx.x * NT + threadIdx.x;
    if (p.mode == MODE_GAP) {
      for (int u = g; u < m; u += G) {
        int l = p.rmatch_in[u];
        st_rlx(p.rowst + u, pack(-1, (l >= 0 && l < INF) ? 1u + (u32)l : 0u));
      }
      for (int v = g; v < n; v += G) {
        int l = p.cmatch_in[v];
        st_rlx(p.colst + v, pack(-1, (l >= 0 && l < INF) ? 1u + (u32)l : 0u));
      }
      return;
    }
    const bool given = (p.mode == MODE_RELABEL) || (p.init == 1);
    for (int u = g; u < m; u += G) st_rlx(p.rowst + u, pack(given ? p.rmatch_in[u] : -1, 0));
    for (int v = g; v < n; v += G) {
      st_rlx(p.colst + v, pack(given ? p.cmatch_in[v] : -1, 0));
      p.iA[v] = -1;  // R12
    }
  }

  // Cheap greedy matching on the device (reading R13): every column claims the
  // first free row of Gamma(v) with a CAS.  A column fails only when every
  // neighbour is taken, so the result is maximal.  (Outside the push loop, the
  // paper's atomic-free claim concerns the push-relabel steps.)
  __device__ void greedy() {
    const int lane = lane_id();
    const int gw = (blockIdx.x * NT + threadIdx.x) >> 5, NWG = gridDim.x * NWARP;
    for (int b = gw * 32; b < n; b += NWG * 32) {
      int v = b + lane;
      int s = 0, e = 0;
      if (v < n) { s = ld_ro(p.cptr + v); e = ld_ro(p.cptr + v + 1); }
      if (v < n && e - s <= SMALL_DEG) {
        for (int j = s; j < e; j++) {
          int u = ld_ro(p.cadj + j);
          u64 rs = ld_rlx(p.rowst + u);
          s_gyedges++;
          if (mu_of(rs) != -1) continue;
          if (atomicCAS(p.rowst + u, rs, pack(v, psi_of(rs))) == rs) {
            st_rlx(p.colst + v, pack(u, 0));
            break;
          }
        }
      }
      unsigned big = __ballot_sync(0xffffffffu, v < n && e - s > SMALL_DEG);
      while (big) {
        int bl = __ffs(big) - 1;
        big &= big - 1;
        int vb = __shfl_sync(0xffffffffu, v, bl);
        int sb = __shfl_sync(0xffffffffu, s, bl), eb = __shfl_sync(0xffffffffu, e, bl);
        bool done = false;
        for (int c0 = sb; c0 < eb && !done; c0 += 32) {
          int j = c0 + lane;
          int u = -1;
          u64 rs = 0;
          if (j < eb) { u = ld_ro(p.cadj + j); rs = ld_rlx(p.rowst + u); s_gyedges++; }
          unsigned cand = __ballot_sync(0xffffffffu, u >= 0 && mu_of(rs) == -1);
          while (cand && !done) {
            int l = __ffs(cand) - 1;
            cand &= cand - 1;
            int ok = 0;
            if (lane == l) {
              ok = atomicCAS(p.rowst + u, rs, pack(vb, psi_of(rs))) == rs;
              if (ok) st_rlx(p.colst + vb, pack(u, 0));
            }
            done = __shfl_sync(0xffffffffu, ok, l);
          }
        }
      }
    }
  }

  // unmatched rows -> U (any order); ring j
  __device__ void build_unmatched_rows(int *U, int j) {
    for (int t = blockIdx.x * NT; t < m; t += gridDim.x * NT) {
      int u = t + threadIdx.x;
      bool f = u < m && mu_of(ld_rlx(p.rowst + u)) == -1;
      int tot, r = cta_rank<NT>(f, sm.w, &tot);
      if (threadIdx.x == 0) sm.qbase = tot ? (int)atomicAdd(ring_now(j), (u32)tot) : 0;
      __syncthreads();
      if (f) U[sm.qbase + r] = u;
    }
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

  template <bool GRID>
  __device__ void gr_level(const int *cur, int curlen, int lvl, u32 base, int *next, u32 *ncnt, int *Uout,
                           u32 *ucnt, int *guard, u32 *gcnt) {
    const int lane = lane_id();
    const u32 lc = base + lvl + 1, lr = base + lvl + 2;
    const int G = pick_group(curlen, ncta<GRID>() * NT);
    const int gl = lane & (G - 1), per_tile = NT / G;
    for (int t = cta<GRID>() * per_tile; t < curlen; t += ncta<GRID>() * per_tile) {
      int i = t + (int)threadIdx.x / G;
      int u = (i < curlen) ? ld_cg(cur + i) : -1;
      if (lvl == 0) {
        bool keep = false;
        if (u >= 0) {
          if (mu_of(ld_rlx(p.rowst + u)) == -1) {
            if (gl == 0) st_rlx(p.rowst + u, pack(-1, base));
            keep = gl == 0;
          } else {
            u = -1;
          }
        }
        int tot, r = cta_rank<NT>(keep, sm.w, &tot);
        if (threadIdx.x == 0) sm.tmp = tot ? (int)atomicAdd(ucnt, (u32)tot) : 0;
        __syncthreads();
        if (keep) Uout[sm.tmp + r] = u;
      }
      int s = 0, e = 0;
      if (u >= 0) {
        s = ld_ro(p.rptr + u);
        e = ld_ro(p.rptr + u + 1);
        if (gl == 0) { s_grrows++; s_gredges += e - s; }
      }
      const bool big = u >= 0 && G < 32 && e - s > BIG_DEG;
      if (u >= 0 && !big) expand(s + gl, e, G, lc, lr, next, ncnt, guard, gcnt);
      unsigned bigm = __ballot_sync(0xffffffffu, big && gl == 0);
      while (bigm) {  // long lists: the whole warp
        int bl = __ffs(bigm) - 1;
        bigm &= bigm - 1;
        int sb = __shfl_sync(0xffffffffu, s, bl), eb = __shfl_sync(0xffffffffu, e, bl);
        expand(sb + lane, eb, 32, lc, lr, next, ncnt, guard, gcnt);
      }
      flush(next, ncnt);
    }
  }
  // Visit radj[j], j = j0, j0+step, ... < e, KB at a time: the KB column loads, then
  // the KB claims (CAS), then the KB mate checks are each issued back to back.
  __device__ __forceinline__ void expand(int j0, int e, int step, u32 lc, u32 lr, int *next, u32 *ncnt, int *guard,
                                         u32 *gcnt) {
    for (int j = j0; j < e; j += step * KB) {
      int v[KB];
      u64 cs[KB], old[KB], rw[KB];
#pragma unroll
      for (int k = 0; k < KB; k++) {
        int jj = j + k * step;
        v[k] = jj < e ? ld_ro(p.radj + jj) : -1;
      }
#pragma unroll
      for (int k = 0; k < KB; k++) cs[k] = v[k] >= 0 ? ld_rlx(p.colst + v[k]) : ~0ull;
#pragma unroll
      for (int k = 0; k < KB; k++)  // visited in this GR <=> label carries the current epoch (>= base)
        old[k] = (v[k] >= 0 && psi_of(cs[k]) < gr_base) ? atomicCAS(p.colst + v[k], cs[k], pack(mu_of(cs[k]), lc))
                                                         : ~cs[k];
#pragma unroll
      for (int k = 0; k < KB; k++) {
        int w = mu_of(cs[k]);
        rw[k] = (old[k] == cs[k] && w >= 0) ? ld_rlx(p.rowst + w) : 0ull;
      }
#pragma unroll
      for (int k = 0; k < KB; k++) {
        if (old[k] != cs[k]) continue;  // not claimed by this thread
        s_grcols++;
        int w = mu_of(cs[k]);
        if (w >= 0 && mu_of(rw[k]) == v[k]) {
          st_rlx(p.rowst + w, pack(v[k], lr));
          stage(w, next, ncnt);
        } else {
          s_free++;
          if (guard) guard[atomicAdd(gcnt, 1u)] = v[k];
        }
      }
    }
  }
  u32 gr_base = 0;

  // Full GR (Alg. 4).  U/T: unmatched-row list and a free buffer
  // (swapped on return); Qa/Qb frontier buffers.  Returns maxLevel.
  // guard != nullptr: every reached column that is not matched is appended to
  // guard[0 .. gcount) (the exactness guard, R16).
  template <bool GRID>
  __device__ int global_relabel(int *&U, int &ulen, int *&T, int *Qa, int *Qb, u32 base, int *guard, int &gcount) {
    GRState g;
    gr_start<GRID>(g, U, ulen, T, Qa, base, guard);
    gr_levels<GRID>(g, base, Qa, Qb, guard, 0x7fffffff);
    gcount = (int)ld_rlx(&p.ctrl->gcnt);
    return g.deepest + 2;
  }

  // The GR as a resumable state machine, so that a CTA-local GR (tail mode) can
  // hand a frontier that grew too wide over to the whole grid mid-BFS.
  struct GRState {
    int lvl, deepest, nlen, cur_is_a;
  };
  // level 0 (INITRELABEL + first expansion): U -> filtered U (in T, then swapped), frontier -> Qa
  template <bool GRID>
  __device__ void gr_start(GRState &g, int *&U, int &ulen, int *&T, int *Qa, u32 base, int *guard) {
    gr_base = base;
    u32 *gc = &p.ctrl->gcnt;  // zero here: reset one phase after its last use
    trace(1, ulen);
    gr_level<GRID>(U, ulen, 0, base, Qa, ring_now(0), T, ring_now(1), guard, gc);
    barrier<GRID>();
    g.nlen = (int)ring_prev(0);
    ulen = (int)ring_prev(1);
    int *tmp = U; U = T; T = tmp;
    g.lvl = 0; g.deepest = 0; g.cur_is_a = 1;
  }
  // levels 2, 4, ... until the frontier is empty (returns true) or, before expanding
  // a level, the frontier exceeds `limit` (returns false; state kept for resuming).
  template <bool GRID>
  __device__ bool gr_levels(GRState &g, u32 base, int *Qa, int *Qb, int *guard, int limit) {
    gr_base = base;
    u32 *gc = &p.ctrl->gcnt;
    while (g.nlen > 0) {
      if (g.nlen > limit) return false;
      g.lvl += 2;
      g.deepest = g.lvl;
      int *cur = g.cur_is_a ? Qa : Qb, *nxt = g.cur_is_a ? Qb : Qa;
      trace(2, g.nlen);
      gr_level<GRID>(cur, g.nlen, g.lvl, base, nxt, ring_now(0), nullptr, nullptr, guard, gc);
      barrier<GRID>();
      g.nlen = (int)ring_prev(0);
      g.cur_is_a ^= 1;
    }
    return true;
  }

  // ---------------------------------------------------------------- fix step
  // G-PR-INITKRNL (Alg. 8) for slot i: roll back a push that lost its
  // race (Ap(i) = v still unmatched => Ac(i) <- v, l.3-6), then mark the slot's
  // column active in this loop (l.8-11, reading R5: after the if/else).
  __device__ __forceinline__ int fix_slot(int i, int *Ac, const int *Ap, int loop) {
    int v = ld_cg(Ap + i);
    int a;
    if (v != -1 && col_unmatched(v)) {
      Ac[i] = v;
      a = v;
    } else {
      a = ld_cg(Ac + i);
    }
    if (a != -1) st_rlx(p.iA + a, loop);
    return a;
  }

  template <bool GRID>
  __device__ void fix_plain(int len, int *Ac, const int *Ap, int loop, int j) {
    long long cnt = 0;
    for (int t = cta<GRID>() * NT; t < len; t += ncta<GRID>() * NT) {
      int i = t + threadIdx.x;
      if (i < len) cnt += fix_slot(i, Ac, Ap, loop) != -1;
    }
    s_slots += cnt;
    add_count(cnt, j);
  }

  // ---------------------------------------------------------------- push
  // G-PR-PUSHKRNL (Alg. 9) over slots [0, len).  Columns with short
  // lists scan alone; longer lists are scanned by the whole warp in chunks of 32
  // with a (label, position) min-reduction and the early exit at psi(v)-1 taken
  // per chunk (reading R11).
  template <bool GRID>
  __device__ void push(int len, int *Ac, int *Ap, int loop, u32 base) {
    const int lane = lane_id();
    const int G = pick_group(len, ncta<GRID>() * NT);
    const int gl = lane & (G - 1), per_tile = NT / G;
    const unsigned gmask = group_mask(G);
    for (int t = cta<GRID>() * per_tile; t < len; t += ncta<GRID>() * per_tile) {
      int i = t + (int)threadIdx.x / G;
      int v = (i < len) ? ld_cg(Ac + i) : -1;
      int s = 0, e = 0, psiv = INF;
      u64 cs = 0;
      if (v >= 0) {
        cs = ld_rlx(p.colst + v);
        psiv = lab(psi_of(cs), base, INF);
        s = ld_ro(p.cptr + v);
        e = ld_ro(p.cptr + v + 1);
        if (p.dead_skip && psiv >= INF) e = s;  // R19: provably unmatchable
      }
      const int target = psiv - 1;
      const bool big = v >= 0 && G < 32 && e - s > BIG_DEG;
      u64 best = ~0ull;
      int ub = -1, wb = -1;
      if (v >= 0 && !big) scan(s, e, gl, G, gmask, target, base, best, ub, wb);      // l.6-11
      unsigned bigm = __ballot_sync(0xffffffffu, big && gl == 0);
      while (bigm) {  // long lists: the whole warp
        int bl = __ffs(bigm) - 1;
        bigm &= bigm - 1;
        int sb = __shfl_sync(0xffffffffu, s, bl), eb = __shfl_sync(0xffffffffu, e, bl);
        int tb = __shfl_sync(0xffffffffu, target, bl);
        u64 b2;
        int u2, w2;
        scan(sb, eb, lane, 32, 0xffffffffu, tb, base, b2, u2, w2);
        if (lane == bl) { best = b2; ub = u2; wb = w2; }
      }
      if (gl != 0) continue;
      if (v >= 0) {
        int psimin = best == ~0ull ? INF : (int)(best >> 32);
        if (psimin < INF) {                                 // l.12
          if (wb == -1 || ld_rlx(p.iA + wb) != loop) {      // l.13
            st_rlx(p.rowst + ub, pack(v, base + (u32)psimin + 2u));  // l.14, l.17
            st_rlx(p.colst + v, pack(ub, base + (u32)psimin + 1u));  // l.15, l.16
            Ap[i] = wb;                                     // l.18 (R3)
            s_push++;
          } else {
            Ap[i] = -1;                                     // R4: blocked
            s_block++;
          }
        } else {
          st_rlx(p.colst + v, pack(-2, psi_of(cs)));        // l.20
          Ac[i] = -1;                                       // l.21
          Ap[i] = -1;                                       // l.22
          s_dead++;
        }
      } else if (i < len) {
        Ap[i] = -1;                                         // l.24
      }
    }
  }
  // First minimum of psi over Gamma(v) = cadj[s, e) in adjacency order (Alg. 9
  // l.6-11): the G lanes of a group read KB*G consecutive neighbours per step, take
  // the (label, position) minimum and stop after the step in which the running
  // minimum reaches psi(v)-1 (reading R11).  best = (label << 32 | position) or ~0.
  __device__ __forceinline__ void scan(int s, int e, int gl, int G, unsigned gmask, int target, u32 base, u64 &best,
                                       int &bu, int &bw) {
    best = ~0ull;
    bu = -1;
    bw = -1;
    for (int c0 = s; c0 < e; c0 += G * KB) {
      int x[KB];
      u64 rs[KB];
#pragma unroll
      for (int k = 0; k < KB; k++) {
        int jj = c0 + gl + k * G;
        x[k] = jj < e ? ld_ro(p.cadj + jj) : -1;
      }
#pragma unroll
      for (int k = 0; k < KB; k++) rs[k] = x[k] >= 0 ? ld_rlx(p.rowst + x[k]) : 0ull;
      u64 key = ~0ull;
      int kx = -1, kw = -1;
#pragma unroll
      for (int k = 0; k < KB; k++) {
        if (x[k] < 0) continue;
        s_scan++;
        int l = lab(psi_of(rs[k]), base, INF);
        u64 kk = l < INF ? (((u64)(u32)l << 32) | (u32)(c0 + gl + k * G - s)) : ~0ull;
        if (kk < key) { key = kk; kx = x[k]; kw = mu_of(rs[k]); }
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
      int c = mu_of(ld_rlx(p.rowst + u));
      p.rmatch_out[u] = c;
      card += c >= 0;
    }
    for (int v = g; v < n; v += G) {
      int c = mu_of(ld_rlx(p.colst + v));
      int ok = (c >= 0 && mu_of(ld_rlx(p.rowst + c)) == v) ? c : -1;
      fixed += (c != -1 && ok == -1);
      p.cmatch_out[v] = ok;
    }
    add_count(card, j_card);
    add_count(fixed, j_fixed);
  }

  __device__ void write_labels(u32 base) {
    const int G = gridDim.x * NT, g = blockIdx.x * NT + threadIdx.x;
    for (int u = g; u < m; u += G) p.rmatch_out[u] = lab(psi_of(ld_rlx(p.rowst + u)), base, INF);
    for (int v = g; v < n; v += G) p.cmatch_out[v] = lab(psi_of(ld_rlx(p.colst + v)), base, INF);
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
    if (!p.debug) return;
    const int G = gridDim.x * NT, g = blockIdx.x * NT + threadIdx.x;
    for (int u = g; u < m; u += G) {
      int c = mu_of(ld_rlx(p.rowst + u));
      if (c >= 0 && mu_of(ld_rlx(p.colst + c)) != u) dbg_record(where, loop, u, c);
    }
    for (int v = g; v < n; v += G) p.dbgbuf[v] = 0;
    barrier<true>();
    if (Ac)
      for (int i = g; i < len; i += G) {
        int v = __ldcg(Ac + i);
        if (v >= 0 && atomicAdd(p.dbgbuf + v, 1) != 0) dbg_record(100 + where, loop, v, i);
      }
    barrier<true>();
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
      u64 w = ld_rlx(x < m ? p.rowst + x : p.colst + (x - m));
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
    barrier<true>();
    const int L = min((int)ld_rlx((const u32 *)&c->gmax), H);
    int first = 0x7fffffff;
    for (int l = g; l < L; l += G)
      if (__ldcg(p.hist + l) == 0) { first = l; break; }
    for (int o = 16; o > 0; o >>= 1) first = min(first, __shfl_xor_sync(0xffffffffu, first, o));
    if (lane_id() == 0 && first != 0x7fffffff) atomicMin(&c->gmin, first);
    barrier<true>();
    const int gap = (int)ld_rlx((const u32 *)&c->gmin);
    if (blockIdx.x == 0 && threadIdx.x == 0) c->gmax = 0;
    long long killed = 0;
    if (gap != 0x7fffffff) {
      for (int x = g; x < m + n; x += G) {
        u64 *a = x < m ? p.rowst + x : p.colst + (x - m);
        u64 w = ld_rlx(a);
        int l = lab(psi_of(w), base, INF);
        if (l > gap && l < INF) { st_rlx(a, pack(mu_of(w), 0)); killed++; }  // psi 0 < base: infinite
      }
    }
    for (int l = g; l < L; l += G) p.hist[l] = 0;
    s_gapkill += killed;
    barrier<true>();
    return gap == 0x7fffffff ? -1 : gap;
  }

  // ---------------------------------------------------------------- tail mode
  enum { R_NONE = 0, R_TERM = 1, R_NEEDGR = 2, R_ESC = 3, R_CAP = 4, R_GAP = 5 };
  // gap relabel schedule (R14): once, halfway between two GRs
  __device__ __forceinline__ long long gap_at(long long loop, long long iterGR) const {
    return (p.gap && iterGR - loop >= 2) ? loop + (iterGR - loop) / 2 : -1;
  }
  __device__ __forceinline__ int tail_f() const { return p.tail_max * 2; }

  // All CTAs call.  CTA 0 runs Alg. 7 iterations alone -- fix with compaction at
  // every step, push, and GRs whose frontiers stay narrow -- with __syncthreads
  // between phases, while the other CTAs wait at one grid barrier.  The episode
  // ends when a GR needs the grid (too many unmatched rows, or a frontier that
  // grew past tail_f(): R_ESC hands the BFS state over), when no active column is
  // left (R_TERM) or at the iteration cap (R_CAP).  CTA 0 then publishes its
  // control registers and every CTA adopts them after the barrier.
  __device__ int tail_episode(long long &loop, long long &iterGR, long long &gapAt, int &len, int &ulen, u32 &base,
                              bool &shrink,
                              int *&Ac, int *&Ap, int *&U, int *&T, int *Qa, int *Qb, GRState &gst, long long &grs,
                              long long &levels, long long &shrinks, long long &tail_loops, long long &ns_gr,
                              long long &ns_loop) {
    const u32 stride = (u32)(m + n + 2);
    int reason = R_NONE;
    Ctrl *c = p.ctrl;
    if (blockIdx.x < p.tail_ctas) {
      const int limit = tail_f();
      for (;;) {
        if (loop >= p.max_loops) { reason = R_CAP; break; }
        if (loop == gapAt) { reason = R_GAP; break; }
        if (loop == iterGR) {
          if (ulen > limit || (u64)base + 2ull * stride >= 0xfffffff0ull) { reason = R_NEEDGR; break; }
          u64 g0 = gtime();
          gr_start<false>(gst, U, ulen, T, Qa, base, nullptr);
          bool done = gr_levels<false>(gst, base, Qa, Qb, nullptr, limit);
          ns_gr += (long long)(gtime() - g0);
          if (!done) { reason = R_ESC; break; }
          int ml = gst.deepest + 2;
          grs++; levels += ml / 2;
          iterGR = loop + iter_gap(ml);
          gapAt = gap_at(loop, iterGR);
          shrink = true;
          base += stride;
        }
        u64 l0 = gtime();
        const int lp = (int)loop;
        if (threadIdx.x == 0) s_slots += len;
        trace(3, len);
        int r1 = compact_pass1<false>(len, [&](int i) { return fix_slot(i, Ac, Ap, lp); }, T, Ac);
        barrier<false>();
        if (p.tail_ctas > 1) {
          len = compact_pass2<false>(len, T, Ac, r1);
          barrier<false>();
        } else {
          len = r1;
        }
        if (shrink) { shrinks++; shrink = false; }
        if (len == 0) { reason = R_TERM; ns_loop += (long long)(gtime() - l0); break; }
        trace(4, len);
        push<false>(len, Ac, Ap, lp, base - stride);
        barrier<false>();
        int *tmp = Ac; Ac = Ap; Ap = tmp;
        loop++;
        tail_loops++;
        ns_loop += (long long)(gtime() - l0);
      }
      if (threadIdx.x == 0) {
        c->ho_reason = reason; c->ho_ph = ph; c->ho_len = len; c->ho_ulen = ulen; c->ho_shrink = shrink;
        c->ho_ac0 = (Ac == p.wl0); c->ho_u0 = (U == p.qa); c->ho_loop = loop; c->ho_iter = iterGR;
        c->ho_base = base; c->ho_gapat = gapAt; c->ho_gl = gst.lvl; c->ho_gd = gst.deepest; c->ho_gn = gst.nlen; c->ho_gc = gst.cur_is_a;
        for (int j = 0; j < 4; j++) c->ring[j][0] = c->ring[j][1] = c->ring[j][2] = c->ring[j][3] = 0;
      }
    }
    if (p.trace && threadIdx.x == 0 && blockIdx.x == 0 && tn < p.trace_cap) {
      p.trace[3 * tn] = 99; p.trace[3 * tn + 1] = reason; p.trace[3 * tn + 2] = (long long)gtime();
      tn++;
    }
    grid_sync(&p.ctrl->bar, true);
    nbar++;
    reason = ld_rlx((const u32 *)&c->ho_reason);
    ph = (int)ld_rlx((const u32 *)&c->ho_ph) + 1;
    len = (int)ld_rlx((const u32 *)&c->ho_len);
    ulen = (int)ld_rlx((const u32 *)&c->ho_ulen);
    shrink = ld_rlx((const u32 *)&c->ho_shrink) != 0;
    bool ac0 = ld_rlx((const u32 *)&c->ho_ac0) != 0, u0 = ld_rlx((const u32 *)&c->ho_u0) != 0;
    Ac = ac0 ? p.wl0 : p.wl1; Ap = ac0 ? p.wl1 : p.wl0;
    U = u0 ? p.qa : p.qb; T = u0 ? p.qb : p.qa;
    loop = ld_rlx(&c->ho_loop);
    iterGR = ld_rlx(&c->ho_iter);
    gapAt = ld_rlx(&c->ho_gapat);
    base = ld_rlx(&c->ho_base);
    gst.lvl = (int)ld_rlx((const u32 *)&c->ho_gl); gst.deepest = (int)ld_rlx((const u32 *)&c->ho_gd);
    gst.nlen = (int)ld_rlx((const u32 *)&c->ho_gn); gst.cur_is_a = (int)ld_rlx((const u32 *)&c->ho_gc);
    return reason;
  }

  // ---------------------------------------------------------------- the solve
  __device__ void run() {
    const bool lead = blockIdx.x == 0 && threadIdx.x == 0;
    u64 t0 = gtime(), tA = t0;
    long long ns_gr = 0, ns_loop = 0, ns_init = 0;
    long long grs = 0, levels = 0, shrinks = 0, loops = 0, guard_re = 0;
    int *Ac = p.wl0, *Ap = p.wl1;
    int *U = p.qa, *T = p.qb, *Qa = p.qc, *Qb = p.qd;
    if (threadIdx.x == 0) sm.qcnt = 0;
    init_state();
    barrier<true>();
    if (p.mode == MODE_SOLVE && p.init == 0) {
      greedy();
      barrier<true>();
    }
    debug_check(1, -1, nullptr, 0);
    // unmatched rows -> U; unmatched columns (increasing id) -> Ac (R12)
    build_unmatched_rows(U, 0);
    int run1 = compact_pass1<true>(n, [&](int v) { return col_unmatched(v) ? v : -1; }, T, Ac);
    barrier<true>();
    int ulen = (int)ring_prev(0);
    int len = compact_pass2<true>(n, T, Ac, run1, Ap);  // Ap = Ac (R12)
    long long init_card = (long long)m - ulen;
    u32 base = 1;  // epoch of the next GR
    const u32 stride = (u32)(m + n + 2);

    if (p.mode == MODE_GAP) {  // mcm_gap_relabel: labels in, labels out
      int gl = gap_relabel(1);
      write_labels(1);
      if (lead) p.ctrl->stat[ST_MAXLEVEL] = gl;
      finish_stats(0, 0, 0, 0, 0, 0, 0, 0, 0, 0, 0);
      return;
    }
    if (p.mode == MODE_RELABEL) {
      int g;
      int ml = global_relabel<true>(U, ulen, T, Qa, Qb, base, nullptr, g);
      write_labels(base);
      if (lead) {
        p.ctrl->stat[ST_MAXLEVEL] = ml;
      }
      finish_stats(0, 0, 0, 0, 0, 0, 0, 0, 0, 0, 0);
      return;
    }

    barrier<true>();
    debug_check(2, -1, Ac, len);
    u64 t1 = gtime();
    ns_init = (long long)(t1 - t0);

    long long loop = 0, iterGR = 0, tail_loops = 0, gapAt = -1, gaps = 0;
    bool shrink = false, compact_next = false;
    GRState gst;
    int reason = R_NONE;
    for (;;) {
      if (loop >= p.max_loops) {
        if (lead) p.ctrl->err = -5;
        break;
      }
      bool terminated = false;
      reason = R_NONE;
      // ---- tail episode: a short worklist runs on CTA 0 alone (CTA barriers)
      if (p.tail_max > 0 && len <= p.tail_max && !(loop == iterGR && ulen > tail_f())) {
        reason = tail_episode(loop, iterGR, gapAt, len, ulen, base, shrink, Ac, Ap, U, T, Qa, Qb, gst, grs, levels,
                              shrinks, tail_loops, ns_gr, ns_loop);
        if (reason == R_CAP) {
          if (lead) p.ctrl->err = -5;
          break;
        }
        if (reason == R_TERM) terminated = true;
      }
      if (!terminated && loop == gapAt) {                              // gap relabel (R14)
        u64 g0 = gtime();
        if (gap_relabel(base - stride) >= 0) gaps++;
        gapAt = -1;
        ns_gr += (long long)(gtime() - g0);
        if (p.tail_max > 0 && len <= p.tail_max && loop != iterGR) continue;
      }
      if (!terminated) {
        if (reason == R_ESC || loop == iterGR) {                       // Alg. 7 l.6
          u64 g0 = gtime();
          int ml;
          if (reason == R_ESC) {  // a tail GR whose frontier grew too wide: finish it here
            gr_levels<true>(gst, base, Qa, Qb, nullptr, 0x7fffffff);
            ml = gst.deepest + 2;
          } else {
            if ((u64)base + 2ull * stride >= 0xfffffff0ull) { reset_labels(); base = 1; }
            int gdummy;
            ml = global_relabel<true>(U, ulen, T, Qa, Qb, base, nullptr, gdummy);   // l.7
          }
          grs++; levels += ml / 2;
          iterGR = loop + iter_gap(ml);                                // l.8
          gapAt = gap_at(loop, iterGR);
          shrink = true;                                               // l.9
          base += stride;
          ns_gr += (long long)(gtime() - g0);
          if (p.tail_max > 0 && len <= p.tail_max) continue;           // fix + push in the tail
        }
        const u32 cur = base - stride;  // epoch of the labels in use
        u64 l0 = gtime();
        int act;
        if ((shrink && p.shrink_min >= 0 && len >= p.shrink_min) || p.compact_every || compact_next) {  // l.11
          const int lp = (int)loop;
          int r1 = compact_pass1<true>(len, [&](int i) { return fix_slot(i, Ac, Ap, lp); }, T, Ac);
          s_slots += 0;
          if (lead) s_slots += len;
          barrier<true>();
          len = compact_pass2<true>(len, T, Ac, r1);                   // SHRKRNL
          act = len;
          if (shrink) shrinks++;
          shrink = false;                                              // l.13
          compact_next = false;
          // Ac was rewritten by CTAs other than the pushing one: order it before PUSH
          barrier<true>();
        } else {
          trace(3, len);
          fix_plain<true>(len, Ac, Ap, (int)loop, 0);                  // l.15
          barrier<true>();
          act = (int)ring_prev(0);
          // adaptive compaction (beyond the paper's post-GR shrink): when most slots
          // are empty, the next fix step compacts, so the tail group can take over
          if (p.compact_adapt && act > 0 && (long long)act * 4 < len && len > p.tail_max) compact_next = true;
        }
        debug_check(3, loop, Ac, len);
        if (act != 0) {
          trace(4, len);
          push<true>(len, Ac, Ap, (int)loop, cur);                     // l.17
          barrier<true>();
          debug_check(4, loop, nullptr, 0);
          int *tmp = Ac; Ac = Ap; Ap = tmp;                            // l.18
          loop++;                                                      // l.19
          loops++;
          ns_loop += (long long)(gtime() - l0);
          continue;
        }
        ns_loop += (long long)(gtime() - l0);
      }
      // ---- no active column left (l.5 / l.16)
      if (!p.final_check) break;
      // exactness guard (R16): one more GR; every unmatched column it reaches is
      // re-activated and the loop resumes; otherwise psi certifies maximality.
      u64 g0 = gtime();
      if ((u64)base + 2ull * stride >= 0xfffffff0ull) { reset_labels(); base = 1; }
      int gcount = 0;
      int ml = global_relabel<true>(U, ulen, T, Qa, Qb, base, Ac, gcount);
      grs++; levels += ml / 2;
      base += stride;
      ns_gr += (long long)(gtime() - g0);
      if (gcount == 0) break;
      guard_re += gcount;
      for (int i = blockIdx.x * NT + threadIdx.x; i < gcount; i += gridDim.x * NT) {
        int v = __ldcg(Ac + i);
        u64 cs = ld_rlx(p.colst + v);
        st_rlx(p.colst + v, pack(-1, psi_of(cs)));
        Ap[i] = v;
      }
      barrier<true>();
      if (lead) p.ctrl->gcnt = 0;  // every CTA read it before the barrier above
      len = gcount;
      iterGR = loop + iter_gap(ml);
      gapAt = gap_at(loop, iterGR);
      shrink = false;
    }
    loops += tail_loops;
    gaps_total = gaps;
    fixmatching(0, 1);                                                 // l.20
    barrier<true>();
    finish_stats(loops, grs, levels, shrinks, guard_re, init_card, ns_init, ns_gr, ns_loop, (long long)(gtime() - tA),
                 tail_loops);
  }

  __device__ void reset_labels() {
    const int G = gridDim.x * NT, g = blockIdx.x * NT + threadIdx.x;
    for (int u = g; u < m; u += G) { u64 w = ld_rlx(p.rowst + u); st_rlx(p.rowst + u, pack(mu_of(w), 0)); }
    for (int v = g; v < n; v += G) { u64 w = ld_rlx(p.colst + v); st_rlx(p.colst + v, pack(mu_of(w), 0)); }
    barrier<true>();
  }

  __device__ void finish_stats(long long loops, long long grs, long long levels, long long shrinks, long long guard_re,
                               long long init_card, long long ns_init, long long ns_gr, long long ns_loop,
                               long long ns_total, long long tail_loops) {
    long long v[10] = {s_push, s_block, s_dead, s_scan, s_slots, s_free, s_grrows, s_gredges, s_grcols, s_gyedges};
    const int slot[10] = {ST_PUSHES, ST_BLOCKED, ST_DEAD, ST_SCANNED, ST_SLOTS, ST_REACHED_FREE,
                          ST_GR_ROWS, ST_GR_EDGES, ST_GR_COLS, ST_GREEDY_EDGES};
    for (int k = 0; k < 10; k++) {
      long long t = cta_sum<NT>(v[k], sm.red);
      if (threadIdx.x == 0 && t) atomicAdd((unsigned long long *)&p.ctrl->stat[slot[k]], (unsigned long long)t);
    }
    if (blockIdx.x == 0 && threadIdx.x == 0) {
      long long *st = p.ctrl->stat;
      st[ST_LOOPS] = loops; st[ST_GRS] = grs; st[ST_LEVELS] = levels; st[ST_SHRINKS] = shrinks;
      st[ST_GAPS] = gaps_total;
      st[ST_GUARD] = guard_re; st[ST_INITCARD] = init_card; st[ST_NS_INIT] = ns_init; st[ST_NS_GR] = ns_gr;
      st[ST_NS_LOOP] = ns_loop; st[ST_NS_TOTAL] = ns_total; st[ST_TAILLOOPS] = tail_loops;
      st[ST_BARRIERS] = nbar;
      st[ST_TRACE_N] = tn;
      if (p.mode == MODE_SOLVE) {
        st[ST_CARD] = (long long)ld_rlx(&p.ctrl->ring[(ph - 1) & 3][0]);
        st[ST_FIXED] = (long long)ld_rlx(&p.ctrl->ring[(ph - 1) & 3][1]);
      }
    }
  }
};

#ifndef MCM_MINB
#define MCM_MINB 1
#endif
__global__ void __launch_bounds__(NT, MCM_MINB) gpr_kernel(Params p) {
  __shared__ Smem sm;
  Solver s(p, sm);
  s.run();
}

}  // namespace mcm
