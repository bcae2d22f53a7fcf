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
constexpr int SMALL_DEG = 32;    // adjacency lists up to this length: one thread

enum { MODE_SOLVE = 0, MODE_RELABEL = 1 };

// statistics slots (Ctrl::stat)
enum {
  ST_LOOPS, ST_GRS, ST_LEVELS, ST_PUSHES, ST_BLOCKED, ST_DEAD, ST_SCANNED, ST_SLOTS, ST_SHRINKS, ST_GAPS,
  ST_GUARD, ST_FIXED, ST_INITCARD, ST_CARD, ST_TAILLOOPS, ST_BARRIERS, ST_NS_INIT, ST_NS_GR, ST_NS_LOOP,
  ST_NS_TOTAL, ST_MAXLEVEL, ST_REACHED_FREE, ST_NSTAT = 32
};

struct Ctrl {
  u32 ring[4][4];          // per-phase counters, rotated (see Solver::barrier)
  long long stat[ST_NSTAT];
  int err;                 // 0 or an MCM_* code
  u32 gcnt;                // exactness-guard list cursor (monotonic within a solve)
  int pad[14];
  long long dbg[8];        // debug checks: [0] count, [1] where, [2] loop, [3] vertex, [4] value
};

struct Params {
  int m, n, mode;
  const int *rptr, *radj, *cptr, *cadj;
  u64 *rowst, *colst;
  int *iA, *wl0, *wl1, *qa, *qb, *qc, *qd;
  int *ctacnt;
  int *dbgbuf;             // n ints (debug checks only)
  int debug;
  Ctrl *ctrl;
  // options
  double k;
  int gr_fixed, shrink_min, init, gap, final_check, dead_skip, tail_max, compact_every;
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
  int ph = 0;  // phase counter: identical in every thread
  long long nbar = 0;

  __device__ Solver(const Params &p_, Smem &sm_) : p(p_), sm(sm_), m(p_.m), n(p_.n), INF(p_.m + p_.n) {}

  // ---------------------------------------------------------------- barriers
  // ring[ph & 3] collects the counts produced during phase ph; the consumer reads
  // it right after the barrier.  ring[(ph + 2) & 3] was produced two phases ago
  // and consumed at the start of the previous phase, so CTA 0 may clear it now.
  template <bool GRID>
  __device__ __forceinline__ void barrier() {
    if (GRID) {
      cg::this_grid().sync();
      nbar++;
    } else {
      __syncthreads();
    }
    ph++;
    if (GRID ? (blockIdx.x == 0 && threadIdx.x == 0) : (threadIdx.x == 0)) {
      u32 *r = p.ctrl->ring[(ph + 2) & 3];
      r[0] = r[1] = r[2] = r[3] = 0;
    }
    if (!GRID) __syncthreads();
  }
  __device__ __forceinline__ u32 *ring_now(int j) { return &p.ctrl->ring[ph & 3][j]; }
  __device__ __forceinline__ u32 ring_prev(int j) { return ld_acq(&p.ctrl->ring[(ph - 1) & 3][j]); }

  template <bool GRID>
  __device__ __forceinline__ int cta() const { return GRID ? blockIdx.x : 0; }
  template <bool GRID>
  __device__ __forceinline__ int ncta() const { return GRID ? gridDim.x : 1; }

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
      if (val != -1) (GRID ? T[lo + run + r] : out[run + r]) = val;
      run += tot;
    }
    if (GRID && threadIdx.x == 0) p.ctacnt[c] = run;
    return run;
  }
  // Pass 2 (after a barrier): move T[lo_c ..] to out[offset_c ..]; returns the total.
  template <bool GRID>
  __device__ int compact_pass2(int len, const int *T, int *out, int run1, int *out2 = nullptr) {
    if (!GRID) return run1;
    const int C = gridDim.x, c = blockIdx.x;
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
          if (j < eb) { u = ld_ro(p.cadj + j); rs = ld_rlx(p.rowst + u); }
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
  template <bool GRID>
  __device__ void gr_level(const int *cur, int curlen, int lvl, u32 base, int *next, u32 *ncnt, int *Uout,
                           u32 *ucnt, int *guard, u32 *gcnt) {
    const int lane = lane_id();
    const u32 lc = base + lvl + 1, lr = base + lvl + 2;
    for (int t = cta<GRID>() * NT; t < curlen; t += ncta<GRID>() * NT) {
      int i = t + threadIdx.x;
      int u = (i < curlen) ? ld_cg(cur + i) : -1;
      if (lvl == 0) {
        bool keep = false;
        if (u >= 0) {
          if (mu_of(ld_rlx(p.rowst + u)) == -1) {
            st_rlx(p.rowst + u, pack(-1, base));
            keep = true;
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
      if (u >= 0) { s = ld_ro(p.rptr + u); e = ld_ro(p.rptr + u + 1); }
      if (u >= 0 && e - s <= SMALL_DEG)
        for (int j = s; j < e; j++) visit(ld_ro(p.radj + j), lc, lr, next, ncnt, guard, gcnt);
      unsigned big = __ballot_sync(0xffffffffu, u >= 0 && e - s > SMALL_DEG);
      while (big) {
        int bl = __ffs(big) - 1;
        big &= big - 1;
        int sb = __shfl_sync(0xffffffffu, s, bl), eb = __shfl_sync(0xffffffffu, e, bl);
        for (int j = sb + lane; j < eb; j += 32) visit(ld_ro(p.radj + j), lc, lr, next, ncnt, guard, gcnt);
      }
      flush(next, ncnt);
    }
  }
  __device__ __forceinline__ void visit(int v, u32 lc, u32 lr, int *next, u32 *ncnt, int *guard, u32 *gcnt) {
    u64 cs = ld_rlx(p.colst + v);
    // visited in this GR <=> its label carries the current epoch (>= base)
    if (psi_of(cs) >= gr_base) return;
    u64 nw = pack(mu_of(cs), lc);
    if (atomicCAS(p.colst + v, cs, nw) != cs) return;
    int w = mu_of(cs);
    if (w >= 0) {
      u64 rw = ld_rlx(p.rowst + w);
      if (mu_of(rw) == v) {
        st_rlx(p.rowst + w, pack(v, lr));
        stage(w, next, ncnt);
        return;
      }
    }
    s_free++;
    if (guard) guard[atomicAdd(gcnt, 1u)] = v;
  }
  u32 gr_base = 0;

  // Full GR (Alg. 4).  U/T: unmatched-row list and a free buffer
  // (swapped on return); Qa/Qb frontier buffers.  Returns maxLevel.
  // guard != nullptr: every reached column that is not matched is appended to
  // guard[0 .. gcount) (the exactness guard, R16).
  template <bool GRID>
  __device__ int global_relabel(int *&U, int &ulen, int *&T, int *Qa, int *Qb, u32 base, int *guard, int &gcount) {
    gr_base = base;
    u32 *gc = &p.ctrl->gcnt;  // zero here: reset one phase after its last use
    gr_level<GRID>(U, ulen, 0, base, Qa, ring_now(0), T, ring_now(1), guard, gc);
    barrier<GRID>();
    int nlen = (int)ring_prev(0);
    ulen = (int)ring_prev(1);
    int *tmp = U; U = T; T = tmp;
    int deepest = 0, lvl = 0;
    int *cur = Qa, *nxt = Qb;
    while (nlen > 0) {
      lvl += 2;
      deepest = lvl;
      gr_level<GRID>(cur, nlen, lvl, base, nxt, ring_now(0), nullptr, nullptr, guard, gc);
      barrier<GRID>();
      nlen = (int)ring_prev(0);
      int *t2 = cur; cur = nxt; nxt = t2;
    }
    gcount = (int)ld_acq(gc);
    return deepest + 2;
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
    for (int t = cta<GRID>() * NT; t < len; t += ncta<GRID>() * NT) {
      int i = t + threadIdx.x;
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
      int psimin = INF, ub = -1, wb = -1;
      const int target = psiv - 1;
      if (v >= 0 && e - s <= SMALL_DEG) {
        for (int j = s; j < e; j++) {                       // l.6
          int x = ld_ro(p.cadj + j);
          u64 rs = ld_rlx(p.rowst + x);
          int l = lab(psi_of(rs), base, INF);
          s_scan++;
          if (l < psimin) {                                 // l.7
            psimin = l; ub = x; wb = mu_of(rs);             // l.8-9, R3
            if (psimin == target) break;                    // l.10-11
          }
        }
      }
      unsigned big = __ballot_sync(0xffffffffu, v >= 0 && e - s > SMALL_DEG);
      while (big) {
        int bl = __ffs(big) - 1;
        big &= big - 1;
        int sb = __shfl_sync(0xffffffffu, s, bl), eb = __shfl_sync(0xffffffffu, e, bl);
        int tb = __shfl_sync(0xffffffffu, target, bl);
        u64 best = ~0ull;
        int bu = -1, bw = -1;
        for (int c0 = sb; c0 < eb; c0 += 32) {
          int j = c0 + lane;
          u64 key = ~0ull;
          int x = -1, w = -1;
          if (j < eb) {
            x = ld_ro(p.cadj + j);
            u64 rs = ld_rlx(p.rowst + x);
            int l = lab(psi_of(rs), base, INF);
            w = mu_of(rs);
            if (l < INF) key = ((u64)(u32)l << 32) | (u32)(j - sb);
            s_scan++;
          }
          u64 kmin = key;
#pragma unroll
          for (int o = 16; o > 0; o >>= 1) {
            u64 other = __shfl_xor_sync(0xffffffffu, kmin, o);
            kmin = other < kmin ? other : kmin;
          }
          if (kmin < best) {
            int src = (int)((u32)kmin - (u32)(c0 - sb));
            best = kmin;
            bu = __shfl_sync(0xffffffffu, x, src);
            bw = __shfl_sync(0xffffffffu, w, src);
          } else if (kmin != ~0ull) {
            // keep the earlier minimum (first in adjacency order)
          }
          if (best != ~0ull && (int)(best >> 32) == tb) break;
        }
        if (lane == bl) {
          if (best != ~0ull) { psimin = (int)(best >> 32); ub = bu; wb = bw; }
        }
      }
      if (v >= 0) {
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

    long long loop = 0, iterGR = 0;
    bool shrink = false;
    for (;;) {
      if (loop >= p.max_loops) {
        if (lead) p.ctrl->err = -5;
        break;
      }
      if (loop == iterGR) {                                            // Alg. 7 l.6
        u64 g0 = gtime();
        if ((u64)base + 2ull * stride >= 0xfffffff0ull) { reset_labels(); base = 1; }
        int gdummy;
        int ml = global_relabel<true>(U, ulen, T, Qa, Qb, base, nullptr, gdummy);   // l.7
        grs++; levels += ml / 2;
        iterGR = loop + iter_gap(ml);                                  // l.8
        shrink = true;                                                 // l.9
        base += stride;
        ns_gr += (long long)(gtime() - g0);
      }
      const u32 cur = base - stride;  // epoch of the labels in use
      u64 l0 = gtime();
      int act;
      if ((shrink && p.shrink_min >= 0 && len >= p.shrink_min) || p.compact_every) {  // l.11
        const int lp = (int)loop;
        int r1 = compact_pass1<true>(len, [&](int i) { return fix_slot(i, Ac, Ap, lp); }, T, Ac);
        barrier<true>();
        len = compact_pass2<true>(len, T, Ac, r1);                     // SHRKRNL
        act = len;
        s_slots += r1;
        if (shrink) shrinks++;
        shrink = false;                                                // l.13
        // Ac was rewritten by CTAs other than the pushing one: order it before PUSH
        barrier<true>();
      } else {
        fix_plain<true>(len, Ac, Ap, (int)loop, 0);                    // l.15
        barrier<true>();
        act = (int)ring_prev(0);
      }
      debug_check(3, loop, Ac, len);
      if (act == 0) {                                                  // l.5 / l.16
        ns_loop += (long long)(gtime() - l0);
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
        shrink = false;
        continue;
      }
      push<true>(len, Ac, Ap, (int)loop, cur);                         // l.17
      barrier<true>();
      debug_check(4, loop, nullptr, 0);
      int *tmp = Ac; Ac = Ap; Ap = tmp;                                // l.18
      loop++;                                                          // l.19
      loops++;
      ns_loop += (long long)(gtime() - l0);
    }
    fixmatching(0, 1);                                                 // l.20
    barrier<true>();
    finish_stats(loops, grs, levels, shrinks, guard_re, init_card, ns_init, ns_gr, ns_loop, (long long)(gtime() - tA),
                 0);
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
    long long v[7] = {s_push, s_block, s_dead, s_scan, s_slots, s_free, 0};
    const int slot[6] = {ST_PUSHES, ST_BLOCKED, ST_DEAD, ST_SCANNED, ST_SLOTS, ST_REACHED_FREE};
    for (int k = 0; k < 6; k++) {
      long long t = cta_sum<NT>(v[k], sm.red);
      if (threadIdx.x == 0 && t) atomicAdd((unsigned long long *)&p.ctrl->stat[slot[k]], (unsigned long long)t);
    }
    if (blockIdx.x == 0 && threadIdx.x == 0) {
      long long *st = p.ctrl->stat;
      st[ST_LOOPS] = loops; st[ST_GRS] = grs; st[ST_LEVELS] = levels; st[ST_SHRINKS] = shrinks;
      st[ST_GUARD] = guard_re; st[ST_INITCARD] = init_card; st[ST_NS_INIT] = ns_init; st[ST_NS_GR] = ns_gr;
      st[ST_NS_LOOP] = ns_loop; st[ST_NS_TOTAL] = ns_total; st[ST_TAILLOOPS] = tail_loops;
      st[ST_BARRIERS] = nbar;
      if (p.mode == MODE_SOLVE) {
        st[ST_CARD] = (long long)ld_acq(&p.ctrl->ring[(ph - 1) & 3][0]);
        st[ST_FIXED] = (long long)ld_acq(&p.ctrl->ring[(ph - 1) & 3][1]);
      }
    }
  }
};

__global__ void __launch_bounds__(NT, 2) gpr_kernel(Params p) {
  __shared__ Smem sm;
  Solver s(p, sm);
  s.run();
}

}  // namespace mcm
