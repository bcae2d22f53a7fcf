// device.cuh -- memory-model helpers, packed vertex state, warp/CTA primitives.
//
// Vertex state: every row u and every column v
// owns one 64-bit word {mu (low 32, int32), psi (high 32, uint32)}.  The paper
// keeps mu and psi in two arrays; packing them makes the row update
// of a push ( mu(u) <- v, psi(u) <- psimin+2, Alg. 9 l.14/l.17 ) ONE single-copy-
// atomic store, so a concurrent reader never sees a label from one push and a
// mate from another, and the label gather of the scan returns mu(u) for free.
//
// Labels are epoch-tagged: psi stores base + label, where `base` grows by m+n+2
// at every global relabel; a stored value below the current base is stale and
// decodes to "infinite" (m+n).  This replaces INITRELABEL's O(m+n)
// reset (Alg. 4 l.1) by an O(1) bump, so a GR touches only what it
// reaches.
//
// Racy words (vertex state, iA) are read and written with ld/st.relaxed.gpu:
// single-copy atomic, non-RMW -- the push loop stays atomic-free in the paper's
// sense and is well defined under the PTX memory model.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

namespace mcm {

typedef unsigned long long u64;
typedef unsigned int u32;

__device__ __forceinline__ u64 ld_rlx(const u64 *p) {
  u64 v;
  asm volatile("ld.relaxed.gpu.global.b64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void st_rlx(u64 *p, u64 v) {
  asm volatile("st.relaxed.gpu.global.b64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ int ld_rlx(const int *p) {
  int v;
  asm volatile("ld.relaxed.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void st_rlx(int *p, int v) {
  asm volatile("st.relaxed.gpu.global.b32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
// read-only graph arrays (never written during a solve)
__device__ __forceinline__ int ld_ro(const int *p) { return __ldg(p); }
// counter hash of two words (fault injection, option perturb)
__device__ __forceinline__ u32 hash2(u32 a, u32 b) {
  u32 x = a * 0x9E3779B1u ^ (b + 0x7F4A7C15u) * 0x85EBCA77u;
  x ^= x >> 15; x *= 0x2C1B3C6Du; x ^= x >> 12; x *= 0x297A2D39u; x ^= x >> 15;
  return x;
}
// adjacency lists (radj / cadj): streamed, read-only.  (L2 evict_first hints on
// these, and evict_last on the vertex state, were measured in round 2: within
// noise on C2-C5, profiles/r02_l2hint_ab.txt; not kept.)
__device__ __forceinline__ int ld_adj(const int *p) { return __ldg(p); }
// phase-to-phase mutable arrays (worklists, queues): bypass L1
__device__ __forceinline__ int ld_cg(const int *p) { return __ldcg(p); }
__device__ __forceinline__ u32 ld_rlx(const u32 *p) {
  u32 v;
  asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ long long ld_rlx(const long long *p) {
  long long v;
  asm volatile("ld.relaxed.gpu.global.b64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
// Vertex-state accessors (reading R17).  Every access to a racy vertex-state word
// (rowst / colst / iA) is a relaxed access at GPU scope: any two of them, from
// any two CTAs, are morally strong, so the PTX memory model gives each aligned
// 32- or 64-bit access single-copy atomicity (a reader never sees half of one
// packed {mu, psi} store and half of another) and the racy pushes of the paper
// are data-race free in the model's sense.  A CTA-scope (L1-
// cacheable) variant was measured in round 2 against this one on C2-C5
// (tools/ab_scope.sh, profiles/r02_scope_ab.txt): every median within the
// run-to-run spread, so the kernel keeps only the GPU-scope accessors.
__device__ __forceinline__ u64 ldv(const u64 *p) { return ld_rlx(p); }
__device__ __forceinline__ void stv(u64 *p, u64 v) { st_rlx(p, v); }
__device__ __forceinline__ int ldv(const int *p) { return ld_rlx(p); }
__device__ __forceinline__ void stv(int *p, int v) { st_rlx(p, v); }
__device__ __forceinline__ u32 ld_acq(const u32 *p) {
  u32 v;
  asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}

__device__ __forceinline__ u64 pack(int mu, u32 psi) { return (u64)(u32)mu | ((u64)psi << 32); }
__device__ __forceinline__ int mu_of(u64 w) { return (int)(u32)(w & 0xffffffffull); }
__device__ __forceinline__ u32 psi_of(u64 w) { return (u32)(w >> 32); }
// decoded label: stale (below base) = INF
__device__ __forceinline__ int lab(u32 s, u32 base, int INF) {
  return s >= base ? (int)min((u64)(s - base), (u64)INF + 1) : INF;
}

// Grid-wide barrier for a co-resident (cooperatively launched) grid.  One atomic
// per CTA on a single word: CTA 0 adds 2^31 - (G-1), every other CTA adds 1, so
// bit 31 flips exactly when the last CTA arrives (the low 31 bits return to 0).
// The waiting thread polls with relaxed loads -- an acquire load per poll would
// emit CCTL.IVALL and keep invalidating the L1 of every co-resident CTA (spills
// and read-only graph lines included) -- optionally backing off with nanosleep,
// and issues one gpu-scope fence after the flip.
//
// `post` runs in thread 0 after the barrier, before the CTA is released: it
// loads the CTA-uniform words the next phase needs (phase counters, hand-over
// state) into shared memory.  Every thread loading them itself put 16 warps x
// 148 CTAs of requests on one L2 line after every barrier (~1.2 us per phase).
template <class Post>
__device__ __forceinline__ void grid_sync(u32 *bar, bool sleepy, Post post) {
  __syncthreads();
  if (threadIdx.x == 0) {
    u32 nb = (blockIdx.x == 0) ? (0x80000000u - (gridDim.x - 1)) : 1u;
    __threadfence();
    u32 old = atomicAdd(bar, nb);
    u32 ns = 16;
    while (((ld_rlx(bar) ^ old) & 0x80000000u) == 0) {
      if (sleepy) {
        __nanosleep(ns);
        if (ns < 2048) ns <<= 1;
      }
    }
    __threadfence();
    post();
  }
  __syncthreads();
}
__device__ __forceinline__ void grid_sync(u32 *bar, bool sleepy) {
  grid_sync(bar, sleepy, [] {});
}

__device__ __forceinline__ int lane_id() { return threadIdx.x & 31; }
__device__ __forceinline__ int warp_id() { return threadIdx.x >> 5; }

// ---------------------------------------------------------------- CTA reductions
// All threads of the CTA must call these (they contain __syncthreads).
template <int NT>
__device__ __forceinline__ long long cta_sum(long long x, long long *s_red) {
  constexpr int NW = NT / 32;
#pragma unroll
  for (int o = 16; o > 0; o >>= 1) x += __shfl_xor_sync(0xffffffffu, x, o);
  __syncthreads();
  if (lane_id() == 0) s_red[warp_id()] = x;
  __syncthreads();
  long long t = 0;
#pragma unroll
  for (int w = 0; w < NW; w++) t += s_red[w];
  return t;
}

// Stable CTA-wide exclusive scan of a 0/1 flag.  Returns this thread's rank among
// flagged threads (in thread order); *total = number of flagged threads.
template <int NT>
__device__ __forceinline__ int cta_rank(bool flag, int *s_w, int *total) {
  constexpr int NW = NT / 32;
  unsigned b = __ballot_sync(0xffffffffu, flag);
  int lane = lane_id(), w = warp_id();
  int r = __popc(b & ((1u << lane) - 1u));
  __syncthreads();
  if (lane == 0) s_w[w] = __popc(b);
  __syncthreads();
  int off = 0, tot = 0;
#pragma unroll
  for (int i = 0; i < NW; i++) {
    int c = s_w[i];
    off += (i < w) ? c : 0;
    tot += c;
  }
  *total = tot;
  return off + r;
}

// Stable CTA-wide exclusive scan of a per-thread count (thread order); *total =
// the CTA's sum.
template <int NT>
__device__ __forceinline__ int cta_scan(int x, int *s_w, int *total) {
  constexpr int NW = NT / 32;
  const int lane = lane_id(), w = warp_id();
  int inc = x;
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    int y = __shfl_up_sync(0xffffffffu, inc, o);
    if (lane >= o) inc += y;
  }
  __syncthreads();
  if (lane == 31) s_w[w] = inc;
  __syncthreads();
  int off = 0, tot = 0;
#pragma unroll
  for (int i = 0; i < NW; i++) {
    int c = s_w[i];
    off += (i < w) ? c : 0;
    tot += c;
  }
  *total = tot;
  return off + inc - x;
}

}  // namespace mcm
