// api.cu -- the C ABI of include/mcm.h: workspace layout, graph ingest (validate,
// copy, CSC transpose) and the cooperative launch of the persistent G-PR kernel.
#include <cuda_runtime.h>
#include <nvtx3/nvToolsExt.h>
#include <chrono>
#include <cmath>
#include <cstdio>
#include <cstring>
#include <cstdlib>
#include <new>
#include <memory>
#include <algorithm>
#include <vector>

// NVTX ranges (SURVEY.md 5 "tracing"): one per host-visible step of the path
// (validation + copy, CSC transpose, each kernel launch by mode, host copies);
// the phases inside the persistent kernel are traced by MCM_TRACE instead.
struct NvtxRange {
  explicit NvtxRange(const char *name) { nvtxRangePushA(name); }
  ~NvtxRange() { nvtxRangePop(); }
  NvtxRange(const NvtxRange &) = delete;
  NvtxRange &operator=(const NvtxRange &) = delete;
};

#include "../../include/mcm.h"
#include "solve.cuh"

using namespace mcm;

namespace {

constexpr int SCAN_B = 2048;  // items per scan block
constexpr int MAX_CTAS = 4096;

size_t align256(size_t x) { return (x + 255) & ~(size_t)255; }

struct Layout {
  size_t ctrl, ovf, rptr, radj, cptr, cadj, rowst, colst, iA, wl0, wl1, q[4], ctacnt, bsum, hist, outr, outc, dbg, ctrl2,
      srow, scol, total;
  int hist_len;
};

Layout layout(int32_t m, int32_t n, int64_t nnz) {
  Layout L;
  size_t o = 0;
  auto take = [&](size_t bytes) { size_t r = o; o += align256(bytes > 0 ? bytes : 1); return r; };
  size_t mx = (size_t)(m > n ? m : n) + 1;
  L.ctrl = take(sizeof(Ctrl));
  L.ovf = take(sizeof(int4) * mx);
  L.rptr = take(sizeof(int) * ((size_t)m + 1));
  L.radj = take(sizeof(int) * (size_t)nnz);
  L.cptr = take(sizeof(int) * ((size_t)n + 1));
  L.cadj = take(sizeof(int) * (size_t)nnz);
  L.rowst = take(sizeof(u64) * (size_t)m);
  L.colst = take(sizeof(u64) * (size_t)n);
  L.iA = take(sizeof(int) * (size_t)n);
  L.wl0 = take(sizeof(int) * (size_t)n);
  L.wl1 = take(sizeof(int) * (size_t)n);
  // q2, q3: int4 BFS frontiers -- every row at most once per GR, plus the extra
  // ranges of rows whose adjacency is split (stage_row)
  for (int i = 0; i < 4; i++)
    L.q[i] = take(i < 2 ? sizeof(int) * mx : sizeof(int4) * (mx + (size_t)nnz / SPLIT + 1));
  L.ctacnt = take(sizeof(int) * MAX_CTAS);
  L.bsum = take(sizeof(int) * ((size_t)n / SCAN_B + 2));
  L.hist_len = (int)std::min<long long>((long long)m + n + 2, 1 << 20);
  L.hist = take(sizeof(int) * (size_t)L.hist_len);
  L.outr = take(sizeof(int) * (size_t)m);  // mcm_match_host: device copy of the matching
  L.outc = take(sizeof(int) * (size_t)n);
  L.dbg = take(sizeof(int) * ((size_t)n + 1) + (getenv("MCM_TRACE") ? (size_t)atoi(getenv("MCM_TRACE")) * 24 : 0));
  // concurrent GR (option gr_concurrent): the GR kernel's control block and shadow labels
  L.ctrl2 = take(sizeof(Ctrl));
  L.srow = take(sizeof(u32) * (size_t)m);
  L.scol = take(sizeof(u32) * (size_t)n);
  L.total = o;
  return L;
}

// ---------------------------------------------------------------- setup kernels
// One pass over the caller's CSR: validation (indptr[0] = 0, non-decreasing, indptr[m] = nnz, 0 <= indices < n), the copy into the
// workspace (copy = 0: it is already there, mcm_match_host) and the column degrees
// cnt[0..n) for the transpose -- the three used to be three passes over indices.
__global__ void k_ingest(const int *indptr, const int *indices, int m, int n, long long nnz, int *rptr, int *radj,
                         int *cnt, int *err, int copy) {
  const long long g = (long long)blockIdx.x * blockDim.x + threadIdx.x, G = (long long)gridDim.x * blockDim.x;
  if (g == 0 && (indptr[0] != 0 || (long long)indptr[m] != nnz)) atomicOr(err, 1);
  for (long long u = g; u <= m; u += G) {
    const int x = indptr[u];
    if (copy) rptr[u] = x;
    if (u < m && x > indptr[u + 1]) atomicOr(err, 2);
  }
  const bool vec = ((reinterpret_cast<size_t>(indices) | reinterpret_cast<size_t>(radj)) & 15) == 0;
  const long long n4 = vec ? nnz / 4 : 0;
  for (long long q = g; q < n4; q += G) {  // 4 entries per thread, 16-byte loads
    const int4 x = __ldg(reinterpret_cast<const int4 *>(indices) + q);
    if (copy) reinterpret_cast<int4 *>(radj)[q] = x;
    const int v[4] = {x.x, x.y, x.z, x.w};
#pragma unroll
    for (int k = 0; k < 4; k++) {
      if (v[k] < 0 || v[k] >= n) atomicOr(err, 4);
      else atomicAdd(cnt + v[k], 1);
    }
  }
  for (long long e = 4 * n4 + g; e < nnz; e += G) {
    const int v = __ldg(indices + e);
    if (copy) radj[e] = v;
    if (v < 0 || v >= n) atomicOr(err, 4);
    else atomicAdd(cnt + v, 1);
  }
}

// exclusive scan, 3 phases: block sums, scan of block sums (one CTA), block scans
__global__ void k_scan_sums(const int *in, int len, int *bsum) {
  __shared__ long long red[32];
  int b = blockIdx.x, lo = b * SCAN_B;
  long long s = 0;
  for (int i = lo + threadIdx.x; i < min(len, lo + SCAN_B); i += blockDim.x) s += in[i];
  for (int o = 16; o > 0; o >>= 1) s += __shfl_xor_sync(0xffffffffu, s, o);
  if ((threadIdx.x & 31) == 0) red[threadIdx.x >> 5] = s;
  __syncthreads();
  if (threadIdx.x == 0) {
    long long t = 0;
    for (int w = 0; w < (int)(blockDim.x >> 5); w++) t += red[w];
    bsum[b] = (int)t;
  }
}
__global__ void k_scan_bsum(int *bsum, int nb) {
  // one CTA of 1024 threads, sequential chunks
  __shared__ int s[1024];
  __shared__ int carry;
  if (threadIdx.x == 0) carry = 0;
  __syncthreads();
  for (int base = 0; base < nb; base += 1024) {
    int i = base + threadIdx.x;
    int x = i < nb ? bsum[i] : 0;
    s[threadIdx.x] = x;
    __syncthreads();
    for (int o = 1; o < 1024; o <<= 1) {
      int y = threadIdx.x >= o ? s[threadIdx.x - o] : 0;
      __syncthreads();
      s[threadIdx.x] += y;
      __syncthreads();
    }
    if (i < nb) bsum[i] = carry + s[threadIdx.x] - x;  // exclusive
    __syncthreads();
    if (threadIdx.x == 1023) carry += s[1023];
    __syncthreads();
  }
}
__global__ void k_scan_apply(const int *in, int len, const int *bsum, int *out, int total_slot) {
  // block of 1024 threads, SCAN_B = 2 items per thread
  __shared__ int s[1024];
  int b = blockIdx.x, lo = b * SCAN_B;
  int i0 = lo + 2 * threadIdx.x, i1 = i0 + 1;
  int x0 = i0 < len ? in[i0] : 0, x1 = i1 < len ? in[i1] : 0;
  s[threadIdx.x] = x0 + x1;
  __syncthreads();
  for (int o = 1; o < 1024; o <<= 1) {
    int y = threadIdx.x >= o ? s[threadIdx.x - o] : 0;
    __syncthreads();
    s[threadIdx.x] += y;
    __syncthreads();
  }
  int ex = bsum[b] + s[threadIdx.x] - x0 - x1;
  if (i0 < len) out[i0] = ex;
  if (i1 < len) out[i1] = ex + x0;
  if (total_slot >= 0 && b == gridDim.x - 1 && threadIdx.x == 1023) out[total_slot] = ex + x0 + x1;
}

// scatter rows into Gamma(v) lists, edge-parallel: warp w owns entries
// [w*32*SC_K, (w+1)*32*SC_K), lane l the entries base + k*32 + l (coalesced);
// each lane finds the row of its first entry by binary search in rptr and then
// walks forward, so a hub row (R-MAT: 1.5e5 entries) is spread over many warps.
constexpr int SC_K = 8;
// optional: sort every Gamma(v) by row id (insertion sort, thread per column; tests)
__global__ void k_sort_segments(const int *cptr, int *cadj, int n) {
  for (long long v = (long long)blockIdx.x * blockDim.x + threadIdx.x; v < n; v += (long long)gridDim.x * blockDim.x) {
    int s = cptr[v], e = cptr[v + 1];
    for (int i = s + 1; i < e; i++) {
      int x = cadj[i], j = i - 1;
      while (j >= s && cadj[j] > x) { cadj[j + 1] = cadj[j]; j--; }
      cadj[j + 1] = x;
    }
  }
}
__global__ void k_scatter(const int *rptr, const int *radj, int m, long long nnz, int *cursor, int *cadj) {
  const int lane = threadIdx.x & 31;
  const long long warps = ((long long)gridDim.x * blockDim.x) >> 5;
  for (long long w = ((long long)blockIdx.x * blockDim.x + threadIdx.x) >> 5; w * 32 * SC_K < nnz; w += warps) {
    const long long base = w * 32 * SC_K;
    long long e = base + lane;
    if (e >= nnz) continue;
    int lo = 0, hi = m - 1;  // largest r with rptr[r] <= e
    while (lo < hi) {
      int mid = (lo + hi + 1) >> 1;
      if (__ldg(rptr + mid) <= e) lo = mid; else hi = mid - 1;
    }
    int r = lo, rend = __ldg(rptr + r + 1);
#pragma unroll 4
    for (int k = 0; k < SC_K; k++, e += 32) {
      if (e >= nnz) break;
      while (e >= rend) rend = __ldg(rptr + (++r) + 1);
      cadj[atomicAdd(cursor + __ldg(radj + e), 1)] = r;
    }
  }
}

}  // namespace

struct mcm_ctx {
  int dev = 0, sms = 0;
  int32_t m = 0, n = 0;
  int64_t nnz = 0;
  mcm_options_t opt;
  char *ws = nullptr;
  Layout L;
  int grid = 0, max_grid = 0;
  bool poisoned = false;
  mcm_stats_t stats;
  double ms_setup = 0;
  int create_launches = 0;
  cudaStream_t s2 = nullptr;  // concurrent GR: the GR kernel's stream (created on first use)
  cudaEvent_t e1 = nullptr, e2 = nullptr;
  ~mcm_ctx() {
    if (s2) cudaStreamDestroy(s2);
    if (e1) cudaEventDestroy(e1);
    if (e2) cudaEventDestroy(e2);
  }
  Ctrl host_ctrl;
};

#define CK(x)                                  \
  do {                                         \
    cudaError_t e_ = (x);                      \
    if (e_ != cudaSuccess) {                   \
      if (h) h->poisoned = true;               \
      last_cuda_error = e_;                    \
      return MCM_ECUDA;                        \
    }                                          \
  } while (0)

static thread_local cudaError_t last_cuda_error = cudaSuccess;

extern "C" {

void mcm_default_options(mcm_options_t *o) {
  if (!o) return;
  memset(o, 0, sizeof(*o));
  o->k = 0.4;  // the paper's best is 0.7; this build's measured best (R23)
  o->gr_strategy = MCM_GR_ADAPTIVE;
  o->shrink_min = 512;
  o->init = MCM_INIT_GREEDY;
  o->gap = 0;
  o->final_check = 1;
  o->dead_skip = 1;
  o->tail_max = 32;
  o->tail_f = 128;
  o->tail_ctas = 1;
  o->compact_adapt = 1;
  o->gr_early = 1;
  o->bu_div = 16;
  o->compact_every = 0;
  o->grid_ctas = 0;
  o->max_loops = 0;
  o->gr_target = 0.6;
  o->gr_target_min = 1024;
  o->tail_chain = 256;
  o->grid_chain = 128;
  o->gr_window = 0;
  o->gr_window_max = 16384;
}

static bool sizes_ok(int32_t m, int32_t n, int64_t nnz) {
  return m >= 0 && n >= 0 && nnz >= 0 && (int64_t)m + n + 2 < ((int64_t)1 << 31) && nnz < ((int64_t)1 << 31);
}

size_t mcm_workspace_bytes(int32_t m, int32_t n, int64_t nnz, const mcm_options_t *) {
  if (!sizes_ok(m, n, nnz)) return 0;
  return layout(m, n, nnz).total;
}

const char *mcm_strerror(int code) {
  switch (code) {
    case MCM_OK: return "ok";
    case MCM_EINVAL: return "invalid argument or malformed CSR";
    case MCM_ECUDA: return cudaGetErrorString(last_cuda_error);
    case MCM_ENOMEM: return "workspace too small";
    case MCM_EDEVICE: return "wrong current device for this handle";
    case MCM_ENOCONV: return "iteration cap exceeded";
    case MCM_EINTERNAL: return "internal error";
    default: return "unknown error";
  }
}

static int check_opts(const mcm_options_t *o) {
  if (!o) return MCM_OK;
  if (!(o->k > 0) || !std::isfinite(o->k)) return MCM_EINVAL;
  if (!(o->gr_target > 0) || !(o->gr_target <= 1.0) || o->gr_target_min < 0) return MCM_EINVAL;
  if (o->gr_strategy != MCM_GR_ADAPTIVE && o->gr_strategy != MCM_GR_FIXED) return MCM_EINVAL;
  if (o->init < 0 || o->init > 2) return MCM_EINVAL;
  if (o->grid_ctas < 0 || o->grid_ctas > MAX_CTAS || o->tail_max < 0 || o->tail_f < 0 || o->max_loops < 0)
    return MCM_EINVAL;
  if (o->tail_ctas < 1 || o->tail_ctas > 16 || (o->tail_ctas & (o->tail_ctas - 1))) return MCM_EINVAL;
  if (o->variant < 0 || o->variant > 1 || o->bu_div < 0 || o->tail_chain < 0 || o->grid_chain < 0) return MCM_EINVAL;
  if (o->gr_concurrent < 0 || o->gr_concurrent > MAX_CTAS) return MCM_EINVAL;
  if (o->perturb < 0 || o->perturb > 65536) return MCM_EINVAL;
  if (o->gr_window < 0 || o->gr_window > 64 || o->gr_window_max < 0) return MCM_EINVAL;
  return MCM_OK;
}

// from_host: indptr / indices are HOST arrays, copied straight into the workspace's
// CSR copy (mcm_match_host); else DEVICE arrays (mcm_create)
static int create_impl(const int32_t *indptr, const int32_t *indices, int32_t m, int32_t n, int64_t nnz,
                       void *workspace, size_t ws_bytes, mcm_stream_t stream_, const mcm_options_t *o,
                       mcm_handle_t *out, bool from_host) {
  mcm_ctx *h = nullptr;
  if (!out || !sizes_ok(m, n, nnz) || !indptr || (nnz > 0 && !indices) || !workspace) return MCM_EINVAL;
  if (check_opts(o) != MCM_OK) return MCM_EINVAL;
  *out = nullptr;
  Layout L = layout(m, n, nnz);
  if (ws_bytes < L.total) return MCM_ENOMEM;
  cudaStream_t st = (cudaStream_t)stream_;
  NvtxRange r_create(from_host ? "mcm_create(host CSR)" : "mcm_create");
  auto t0 = std::chrono::steady_clock::now();
  h = new (std::nothrow) mcm_ctx();
  if (!h) return MCM_ENOMEM;
  std::unique_ptr<mcm_ctx> guard(h);
  h->m = m; h->n = n; h->nnz = nnz; h->L = L; h->ws = (char *)workspace;
  if (o) h->opt = *o; else mcm_default_options(&h->opt);
  CK(cudaGetDevice(&h->dev));
  CK(cudaDeviceGetAttribute(&h->sms, cudaDevAttrMultiProcessorCount, h->dev));
  int per_sm = 0;
  CK(cudaFuncSetAttribute(gpr_kernel<F_FAST>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sizeof(Smem)));
  CK(cudaFuncSetAttribute(gpr_kernel<F_ALL>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sizeof(Smem)));
  CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, gpr_kernel<F_ALL>, NT, sizeof(Smem)));
  if (per_sm < 1) return MCM_EINTERNAL;
  h->max_grid = h->sms * (per_sm > 2 ? 2 : per_sm);  // one or two CTAs per SM (MCM_MINB)
  if (h->max_grid > MAX_CTAS) h->max_grid = MAX_CTAS;

  char *ws = h->ws;
  Ctrl *ctrl = (Ctrl *)(ws + L.ctrl);
  int *err = &ctrl->err;
  int *rptr = (int *)(ws + L.rptr), *radj = (int *)(ws + L.radj);
  CK(cudaMemsetAsync(ctrl, 0, sizeof(Ctrl), st));
  if (from_host) {  // H2D straight into the CSR copy, validated there
    CK(cudaMemcpyAsync(rptr, indptr, sizeof(int) * ((size_t)m + 1), cudaMemcpyHostToDevice, st));
    if (nnz) CK(cudaMemcpyAsync(radj, indices, sizeof(int) * (size_t)nnz, cudaMemcpyHostToDevice, st));
  }
  const int32_t *vp = from_host ? rptr : indptr, *vi = from_host ? radj : indices;
  int *cnt = (int *)(ws + L.q[0]), *cursor = (int *)(ws + L.q[1]), *bsum = (int *)(ws + L.bsum);
  CK(cudaMemsetAsync(cnt, 0, sizeof(int) * ((size_t)n + 1), st));
  int vb = (int)std::min<long long>(std::max<long long>((nnz + 1023) / 1024, (m + 255) / 256 + 1), 148 * 8);
  k_ingest<<<vb, 256, 0, st>>>(vp, vi, m, n, nnz, rptr, radj, cnt, err, from_host ? 0 : 1);
  int nlaunch = 1;  // kernels this create launched (mcm_stats_t.kernel_launches)
  CK(cudaGetLastError());
  int herr = 0;
  CK(cudaMemcpyAsync(&herr, err, sizeof(int), cudaMemcpyDeviceToHost, st));
  CK(cudaStreamSynchronize(st));
  if (herr) return MCM_EINVAL;

  int *cptr = (int *)(ws + L.cptr), *cadj = (int *)(ws + L.cadj);
  NvtxRange r_csc("mcm_create: CSC transpose");
  // CSC by counting sort (Gamma(v) for the push, Alg. 9 l.6): degrees
  // (k_ingest), exclusive scan, scatter.  (Rejected alternatives, measured: a
  // pass-blocked scatter keeping each pass's cadj segment in L2, 5.3 ms on C4, round
  // 1; a bucketed two-pass transpose, 6.2-8.7 ms on C4 and a slower C3 trajectory,
  // round 2 -- DESIGN.md §7.)
  int nsb = (n + SCAN_B - 1) / SCAN_B;
  if (nsb == 0) nsb = 1;
  k_scan_sums<<<nsb, 512, 0, st>>>(cnt, n, bsum);
  k_scan_bsum<<<1, 1024, 0, st>>>(bsum, nsb);
  k_scan_apply<<<nsb, 1024, 0, st>>>(cnt, n, bsum, cptr, n);
  nlaunch += 3;
  CK(cudaGetLastError());
  if (n == 0) CK(cudaMemsetAsync(cptr, 0, sizeof(int), st));
  CK(cudaMemcpyAsync(cursor, cptr, sizeof(int) * ((size_t)n + 1), cudaMemcpyDeviceToDevice, st));
  if (nnz) {
    long long warps = (nnz + 32 * SC_K - 1) / (32 * SC_K);
    int sb = (int)std::min<long long>((warps + 7) / 8, 148 * 32);
    k_scatter<<<sb, 256, 0, st>>>(rptr, radj, m, nnz, cursor, cadj);
    nlaunch++;
    CK(cudaGetLastError());
    if (h->opt.sort_csc) {
      k_sort_segments<<<(n + 255) / 256, 256, 0, st>>>(cptr, cadj, n);
      nlaunch++;
      CK(cudaGetLastError());
    }
  }
  CK(cudaMemsetAsync(ws + L.hist, 0, sizeof(int) * (size_t)L.hist_len, st));  // zero between gap uses
  CK(cudaStreamSynchronize(st));
  h->ms_setup = std::chrono::duration<double, std::milli>(std::chrono::steady_clock::now() - t0).count();
  memset(&h->stats, 0, sizeof(h->stats));
  h->create_launches = nlaunch;
  *out = guard.release();
  return MCM_OK;
}

int mcm_create(const int32_t *indptr, const int32_t *indices, int32_t m, int32_t n, int64_t nnz, void *workspace,
               size_t ws_bytes, mcm_stream_t stream, const mcm_options_t *o, mcm_handle_t *out) {
  return create_impl(indptr, indices, m, n, nnz, workspace, ws_bytes, stream, o, out, false);
}

// MODE_UNIT: the phase to run, the caller's label arrays, and the device copies
// of the caller's iA / Ac / Ap into the workspace (before the kernel) and back
// (after it)
struct UnitArgs {
  int what, where, len;
  long long loop;
  int32_t *psi_r, *psi_c, *iA, *Ac, *Ap;
};

// host_r / host_c (optional): HOST buffers the outputs are copied into before the
// single synchronisation
static int64_t launch(mcm_ctx *h, cudaStream_t st, int mode, const int32_t *rin, const int32_t *cin, int32_t *out_r,
                      int32_t *out_c, int32_t *host_r = nullptr, int32_t *host_c = nullptr,
                      const UnitArgs *ua = nullptr) {
  if (h->poisoned) return MCM_ECUDA;
  static const char *const mode_name[] = {"mcm_solve", "mcm_global_relabel", "mcm_gap_relabel", "mcm_unit_step",
                                          "mcm_initial_matching", "mcm_solve"};
  NvtxRange r_launch(mode_name[mode >= 0 && mode <= MODE_CONC_GR ? mode : 0]);
  int dev = -1;
  CK(cudaGetDevice(&dev));
  if (dev != h->dev) return MCM_EDEVICE;
  const Layout &L = h->L;
  char *ws = h->ws;
  Params p;
  memset(&p, 0, sizeof(p));
  p.m = h->m; p.n = h->n; p.mode = mode;
  p.rptr = (const int *)(ws + L.rptr); p.radj = (const int *)(ws + L.radj);
  p.cptr = (const int *)(ws + L.cptr); p.cadj = (const int *)(ws + L.cadj);
  p.rowst = (u64 *)(ws + L.rowst); p.colst = (u64 *)(ws + L.colst);
  p.iA = (int *)(ws + L.iA); p.wl0 = (int *)(ws + L.wl0); p.wl1 = (int *)(ws + L.wl1);
  p.qa = (int *)(ws + L.q[0]); p.qb = (int *)(ws + L.q[1]); p.qc = (int *)(ws + L.q[2]); p.qd = (int *)(ws + L.q[3]);
  p.ctacnt = (int *)(ws + L.ctacnt);
  p.ctrl = (Ctrl *)(ws + L.ctrl);
  p.dbgbuf = (int *)(ws + L.dbg);
  p.hist = (int *)(ws + L.hist);
  p.ovf = (int4 *)(ws + L.ovf);
  p.ovf_len = (long long)((h->m > h->n ? h->m : h->n) + 1);
  p.hist_len = L.hist_len;
  p.debug = getenv("MCM_DEBUG") ? atoi(getenv("MCM_DEBUG")) : 0;
  // MCM_TRACE=<n>: record up to n phase boundaries into the (otherwise idle during
  // a solve) debug buffer; dumped to MCM_TRACE_FILE after the solve (analysis only)
  int tcap = getenv("MCM_TRACE") ? atoi(getenv("MCM_TRACE")) : 0;
  if (tcap > 0) {
    size_t room = (h->L.total - h->L.dbg) / (3 * sizeof(long long));
    if ((size_t)tcap > room) tcap = (int)room;
    p.trace = (long long *)(ws + L.dbg);
    p.trace_cap = tcap;
    // MCM_CTATIME=<phases> (with MCM_TRACE): every CTA's arrival time at the grid
    // barriers of the first <phases> phases, after the trace records; dumped to
    // MCM_CTATIME_FILE (analysis of load imbalance only, tools/cta_imbalance.py)
    const int cn = getenv("MCM_CTATIME") ? atoi(getenv("MCM_CTATIME")) : 0;
    const size_t left = (h->L.total - h->L.dbg) / sizeof(long long) - 3 * (size_t)tcap;
    if (cn > 0 && h->max_grid > 0) {
      p.ctat = p.trace + 3 * (size_t)tcap;
      p.ctat_n = (int)std::min<size_t>((size_t)cn, left / (size_t)h->max_grid);
    }
  }
  const mcm_options_t &o = h->opt;
  p.k = o.k; p.gr_fixed = o.gr_strategy == MCM_GR_FIXED; p.shrink_min = o.shrink_min; p.init = o.init;
  p.gap = o.gap; p.final_check = o.final_check; p.dead_skip = o.dead_skip; p.tail_max = o.tail_max;
  p.compact_every = o.compact_every;
  p.compact_adapt = o.compact_adapt;
  p.gr_early = o.gr_early;
  p.gr_target = o.gr_target;
  p.gr_target_min = o.gr_target_min;
  p.serial = o.serial;
  p.variant = o.variant;
  p.tail_chain = o.tail_chain;
  p.perturb = o.perturb;
  p.gr_window = o.gr_window;
  p.gr_window_max = o.gr_window_max;
  // worklists of at most this many slots run as push chains (lanes per slot from the
  // count); MCM_CHAIN_SLOTS: analysis knob
  // (analysis knobs, clamped: 0..TW slots; a divisor of at least 1)
  p.chain_slots = std::min(std::max(getenv("MCM_CHAIN_SLOTS") ? atoi(getenv("MCM_CHAIN_SLOTS")) : 32, 0), TW);
  p.grid_chain = o.grid_chain;
  p.grid_chain_div = std::max(getenv("MCM_GRID_CHAIN_DIV") ? atoi(getenv("MCM_GRID_CHAIN_DIV")) : 2, 1);
  p.bu_div = o.bu_div;
  p.scan_rot = o.serial ? 0 : o.scan_rot;
  if (o.variant == 1) {  // G-PR-First: no worklist, so no tail group either
    p.tail_max = 0;
    p.serial = 0;
  }
  if (o.serial) {  // the simulator's schedule: complete GRs, no tail, no adaptive compaction, no chains
    p.tail_max = 0;
    p.grid_chain = 0;
    p.gr_early = 0;
    p.compact_adapt = 0;
    p.compact_every = 0;
    p.gr_window = 0;
  }
  p.tail_f = o.tail_f;
  p.max_loops = o.max_loops > 0 ? o.max_loops : 2LL * ((long long)h->m + h->n) + 100000;
  p.rmatch_in = rin; p.cmatch_in = cin; p.rmatch_out = out_r; p.cmatch_out = out_c;
  if (ua) {
    p.unit_what = ua->what; p.unit_where = ua->where; p.unit_len = ua->len; p.unit_loop = ua->loop;
    p.psi_row_io = ua->psi_r; p.psi_col_io = ua->psi_c;
    if (h->n) CK(cudaMemcpyAsync(p.iA, ua->iA, sizeof(int) * (size_t)h->n, cudaMemcpyDeviceToDevice, st));
    if (ua->len) {
      CK(cudaMemcpyAsync(p.wl0, ua->Ac, sizeof(int) * (size_t)ua->len, cudaMemcpyDeviceToDevice, st));
      CK(cudaMemcpyAsync(p.wl1, ua->Ap, sizeof(int) * (size_t)ua->len, cudaMemcpyDeviceToDevice, st));
    }
  }
  int C = mode == MODE_UNIT ? 1 : o.tail_ctas;  // a unit's tail is CTA 0 alone
  // the lean production instance unless a feature only the full one carries is on
  // (a cluster tail group spans several SMs' L1s: it needs gpu-scope vertex state)
  const bool conc = mode == MODE_SOLVE && o.gr_concurrent > 0 && !o.serial && !o.variant;
  void (*kern)(const Params) = (mode != MODE_SOLVE || o.serial || o.variant || o.gap || p.debug || C > 1 || conc || o.perturb || o.gr_window > 1)
                                   ? gpr_kernel<F_ALL>
                                   : gpr_kernel<F_FAST>;
  if (o.grid_ctas > 0 && o.grid_ctas < C) C = 1;  // too few CTAs for a cluster: one-CTA tail group
  int maxg = h->max_grid;
  if (C > 1) {
    // co-resident clusters of C CTAs (the tail group is cluster 0)
    if (C > 8) CK(cudaFuncSetAttribute(kern, cudaFuncAttributeNonPortableClusterSizeAllowed, 1));
    cudaLaunchConfig_t q = {};
    cudaLaunchAttribute qa[1];
    qa[0].id = cudaLaunchAttributeClusterDimension;
    qa[0].val.clusterDim.x = C; qa[0].val.clusterDim.y = 1; qa[0].val.clusterDim.z = 1;
    q.gridDim = dim3(C); q.blockDim = dim3(NT); q.attrs = qa; q.numAttrs = 1;
    q.dynamicSmemBytes = sizeof(Smem);
    int ncl = 0;
    CK(cudaOccupancyMaxActiveClusters(&ncl, kern, &q));
    if (ncl < 1) return MCM_EINTERNAL;
    maxg = std::min(maxg, ncl * C);
  }
  int grid = o.grid_ctas > 0 ? std::min(o.grid_ctas, maxg) : maxg;
  grid = (grid / C) * C;
  if (grid < C) return MCM_EINVAL;
  p.tail_ctas = C;
  h->grid = grid;
  CK(cudaMemsetAsync(p.ctrl, 0, sizeof(Ctrl), st));
  if (conc) {
    // NEXT-2: the GR kernel on its own stream (ordered after everything enqueued on
    // `st` so far), co-resident with the solve kernel, which keeps the other CTAs
    const int A = std::min(o.gr_concurrent, grid - C);
    if (A < 1) return MCM_EINVAL;
    if (!h->s2) CK(cudaStreamCreateWithFlags(&h->s2, cudaStreamNonBlocking));
    if (!h->e1) CK(cudaEventCreateWithFlags(&h->e1, cudaEventDisableTiming));
    if (!h->e2) CK(cudaEventCreateWithFlags(&h->e2, cudaEventDisableTiming));
    Ctrl *c2 = (Ctrl *)(ws + L.ctrl2);
    p.ctrl2 = c2;
    p.srow = (u32 *)(ws + L.srow);
    p.scol = (u32 *)(ws + L.scol);
    CK(cudaMemsetAsync(c2, 0, sizeof(Ctrl), st));
    CK(cudaMemsetAsync(p.srow, 0, sizeof(u32) * (size_t)h->m, st));
    CK(cudaMemsetAsync(p.scol, 0, sizeof(u32) * (size_t)h->n, st));
    CK(cudaEventRecord(h->e1, st));
    CK(cudaStreamWaitEvent(h->s2, h->e1, 0));
    Params pg = p;
    pg.mode = MODE_CONC_GR;
    pg.ctrl = c2;
    cudaLaunchConfig_t cg2 = {};
    cudaLaunchAttribute a2[1];
    a2[0].id = cudaLaunchAttributeCooperative;
    a2[0].val.cooperative = 1;
    cg2.gridDim = dim3(A); cg2.blockDim = dim3(NT); cg2.dynamicSmemBytes = sizeof(Smem); cg2.stream = h->s2;
    cg2.attrs = a2; cg2.numAttrs = 1;
    CK(cudaLaunchKernelEx(&cg2, gpr_kernel<F_ALL>, pg));
    grid -= A;
    p.conc = A;
    h->grid = grid;
  }
  cudaLaunchConfig_t cfg = {};
  cudaLaunchAttribute at[2];
  at[0].id = cudaLaunchAttributeCooperative;
  at[0].val.cooperative = 1;
  at[1].id = cudaLaunchAttributeClusterDimension;
  at[1].val.clusterDim.x = C; at[1].val.clusterDim.y = 1; at[1].val.clusterDim.z = 1;
  cfg.gridDim = dim3(grid); cfg.blockDim = dim3(NT); cfg.dynamicSmemBytes = sizeof(Smem); cfg.stream = st;
  cfg.attrs = at; cfg.numAttrs = C > 1 ? 2 : 1;
  CK(cudaLaunchKernelEx(&cfg, kern, p));
  if (conc) {  // the solve's results are read after both kernels ended
    CK(cudaEventRecord(h->e2, h->s2));
    CK(cudaStreamWaitEvent(st, h->e2, 0));
  }
  if (ua) {
    if (h->n) CK(cudaMemcpyAsync(ua->iA, p.iA, sizeof(int) * (size_t)h->n, cudaMemcpyDeviceToDevice, st));
    if (ua->len) {
      CK(cudaMemcpyAsync(ua->Ac, p.wl0, sizeof(int) * (size_t)ua->len, cudaMemcpyDeviceToDevice, st));
      CK(cudaMemcpyAsync(ua->Ap, p.wl1, sizeof(int) * (size_t)ua->len, cudaMemcpyDeviceToDevice, st));
    }
  }
  if (host_r && h->m) CK(cudaMemcpyAsync(host_r, out_r, sizeof(int32_t) * (size_t)h->m, cudaMemcpyDeviceToHost, st));
  if (host_c && h->n) CK(cudaMemcpyAsync(host_c, out_c, sizeof(int32_t) * (size_t)h->n, cudaMemcpyDeviceToHost, st));
  CK(cudaMemcpyAsync(&h->host_ctrl, p.ctrl, sizeof(Ctrl), cudaMemcpyDeviceToHost, st));
  CK(cudaStreamSynchronize(st));
  const Ctrl &c = h->host_ctrl;
  mcm_stats_t &s = h->stats;
  memset(&s, 0, sizeof(s));
  const long long *x = c.stat;
  s.loops = x[ST_LOOPS]; s.gr_count = x[ST_GRS]; s.gr_levels = x[ST_LEVELS]; s.pushes = x[ST_PUSHES];
  s.blocked = x[ST_BLOCKED]; s.dead = x[ST_DEAD]; s.edges_scanned = x[ST_SCANNED]; s.slots = x[ST_SLOTS];
  s.shrinks = x[ST_SHRINKS]; s.gaps = x[ST_GAPS]; s.guard_reactivated = x[ST_GUARD]; s.fixed_cols = x[ST_FIXED];
  s.init_card = x[ST_INITCARD]; s.card = x[ST_CARD]; s.tail_loops = x[ST_TAILLOOPS]; s.grid_barriers = x[ST_BARRIERS];
  s.gr_rows = x[ST_GR_ROWS]; s.gr_edges = x[ST_GR_EDGES]; s.gr_cols = x[ST_GR_COLS];
  s.greedy_edges = x[ST_GREEDY_EDGES]; s.rows_repaired = x[ST_REPAIRED]; s.tail_gr_levels = x[ST_TAIL_LEVELS];
  s.debug_violations = c.dbg[0];
  s.gr_window_levels = x[ST_WINDOWS];
  s.kernel_launches = h->create_launches + 1;  // the create's kernels + this call's one persistent kernel
  s.ms_init = x[ST_NS_INIT] * 1e-6; s.ms_gr = x[ST_NS_GR] * 1e-6; s.ms_loop = x[ST_NS_LOOP] * 1e-6;
  s.ms_total = x[ST_NS_TOTAL] * 1e-6; s.ms_setup = h->ms_setup; s.grid_ctas = grid; s.threads_per_cta = NT;
  if (p.debug && c.dbg[0])
    fprintf(stderr, "[mcm debug] %lld violations; first: where=%lld loop=%lld x=%lld val=%lld\n", c.dbg[0], c.dbg[1],
            c.dbg[2], c.dbg[3], c.dbg[4]);
  if (p.trace && getenv("MCM_TRACE_FILE")) {
    long long tn = c.stat[ST_TRACE_N];
    std::vector<long long> buf(3 * (size_t)tn);
    cudaMemcpy(buf.data(), p.trace, buf.size() * sizeof(long long), cudaMemcpyDeviceToHost);
    FILE *f = fopen(getenv("MCM_TRACE_FILE"), "wb");
    if (f) { fwrite(buf.data(), sizeof(long long), buf.size(), f); fclose(f); }
  }
  if (p.ctat && getenv("MCM_CTATIME_FILE")) {
    std::vector<long long> buf((size_t)p.ctat_n * h->grid);
    cudaMemcpy(buf.data(), p.ctat, buf.size() * sizeof(long long), cudaMemcpyDeviceToHost);
    FILE *f = fopen(getenv("MCM_CTATIME_FILE"), "wb");
    if (f) {
      const long long hdr[2] = {p.ctat_n, h->grid};
      fwrite(hdr, sizeof(long long), 2, f);
      fwrite(buf.data(), sizeof(long long), buf.size(), f);
      fclose(f);
    }
  }
  if (c.err) return c.err;
  if (mode == MODE_RELABEL || mode == MODE_GAP || mode == MODE_UNIT) return x[ST_MAXLEVEL];
  return x[ST_CARD];
}

int64_t mcm_solve(mcm_handle_t h, mcm_stream_t stream, int32_t *rmatch, int32_t *cmatch) {
  if (!h) return MCM_EINVAL;
  if ((h->m > 0 && !rmatch) || (h->n > 0 && !cmatch)) return MCM_EINVAL;
  return launch(h, (cudaStream_t)stream, MODE_SOLVE, rmatch, cmatch, rmatch, cmatch);
}

int64_t mcm_match_host(const int32_t *indptr, const int32_t *indices, int32_t m, int32_t n, int64_t nnz,
                       void *workspace, size_t ws_bytes, mcm_stream_t stream, const mcm_options_t *o, int32_t *rmatch,
                       int32_t *cmatch, mcm_stats_t *stats) {
  if ((m > 0 && !rmatch) || (n > 0 && !cmatch)) return MCM_EINVAL;
  if (o && o->init == MCM_INIT_GIVEN) return MCM_EINVAL;  // no device copy of a given matching on this path
  NvtxRange r_e2e("mcm_match_host");
  mcm_handle_t h = nullptr;
  int rc = create_impl(indptr, indices, m, n, nnz, workspace, ws_bytes, stream, o, &h, true);
  if (rc != MCM_OK) return rc;
  std::unique_ptr<mcm_ctx> guard(h);
  int32_t *dr = (int32_t *)(h->ws + h->L.outr), *dc = (int32_t *)(h->ws + h->L.outc);
  int64_t card = launch(h, (cudaStream_t)stream, MODE_SOLVE, dr, dc, dr, dc, rmatch, cmatch);
  if (stats) *stats = h->stats;
  return card;
}

int64_t mcm_global_relabel(mcm_handle_t h, mcm_stream_t stream, const int32_t *rmatch, const int32_t *cmatch,
                           int32_t *psi_row, int32_t *psi_col, int64_t *info) {
  if (!h) return MCM_EINVAL;
  if ((h->m > 0 && (!rmatch || !psi_row)) || (h->n > 0 && (!cmatch || !psi_col))) return MCM_EINVAL;
  int64_t r = launch(h, (cudaStream_t)stream, MODE_RELABEL, rmatch, cmatch, psi_row, psi_col);
  if (r >= 0 && info) {
    const long long *x = h->host_ctrl.stat;
    info[0] = x[ST_REACHED_FREE]; info[1] = x[ST_FLOOR_R]; info[2] = x[ST_FLOOR_C]; info[3] = x[ST_TAIL_LEVELS];
  }
  return r;
}

int64_t mcm_initial_matching(mcm_handle_t h, mcm_stream_t stream, int32_t *rmatch, int32_t *cmatch) {
  if (!h) return MCM_EINVAL;
  if ((h->m > 0 && !rmatch) || (h->n > 0 && !cmatch)) return MCM_EINVAL;
  return launch(h, (cudaStream_t)stream, MODE_INIT, nullptr, nullptr, rmatch, cmatch);
}

int64_t mcm_unit_step(mcm_handle_t h, mcm_stream_t stream, int32_t unit, int32_t where, int64_t loop, int32_t len,
                      int32_t *mu_row, int32_t *mu_col, int32_t *psi_row, int32_t *psi_col, int32_t *iA, int32_t *Ac,
                      int32_t *Ap) {
  if (!h || unit < MCM_UNIT_FIX || unit > MCM_UNIT_FIXMATCHING || (where != MCM_WHERE_GRID && where != MCM_WHERE_TAIL))
    return MCM_EINVAL;
  if (loop < 0 || loop > 0x7fffffffLL || len < 0 || len > h->n) return MCM_EINVAL;
  if ((h->m > 0 && (!mu_row || !psi_row)) || (h->n > 0 && (!mu_col || !psi_col || !iA)) || (len > 0 && (!Ac || !Ap)))
    return MCM_EINVAL;
  UnitArgs ua{unit, where, len, loop, psi_row, psi_col, iA, Ac, Ap};
  return launch(h, (cudaStream_t)stream, MODE_UNIT, mu_row, mu_col, mu_row, mu_col, nullptr, nullptr, &ua);
}

// NEXT-4 experiment (pgr.cu): partitioned GR levels on the handle's CSC
int mcm_internal_pgr_init(int m, int n, int P, int p, int W, const int *rmatch, uint32_t *slice, int *psi_row,
                          int *psi_col, cudaStream_t st);
int mcm_internal_pgr_level(int m, int n, int P, int p, int W, int L, const int *cptr, const int *cadj,
                           const int *rmatch, const int *cmatch, const uint32_t *F, uint32_t *slice, int *psi_row,
                           int *psi_col, unsigned long long *counts, cudaStream_t st);

static bool pgr_args_ok(const mcm_ctx *h, int32_t nparts, int32_t part, int32_t words) {
  if (nparts < 1 || part < 0 || part >= nparts || words < 1) return false;
  return (int64_t)words * 32 * nparts >= h->m && (int64_t)words * nparts * 33 < ((int64_t)1 << 31);
}

int mcm_pgr_init(mcm_handle_t h, mcm_stream_t stream, int32_t nparts, int32_t part, int32_t words,
                 const int32_t *rmatch, uint32_t *slice, int32_t *psi_row, int32_t *psi_col) {
  if (!h || !pgr_args_ok(h, nparts, part, words) || !slice || (h->m > 0 && (!rmatch || !psi_row)) ||
      (h->n > 0 && !psi_col))
    return MCM_EINVAL;
  if (h->poisoned) return MCM_ECUDA;
  NvtxRange r("mcm_pgr_init");
  if (int rc = mcm_internal_pgr_init(h->m, h->n, nparts, part, words, rmatch, slice, psi_row, psi_col,
                                     (cudaStream_t)stream)) {
    h->poisoned = true;
    last_cuda_error = (cudaError_t)rc;
    return MCM_ECUDA;
  }
  return MCM_OK;
}

int mcm_pgr_level(mcm_handle_t h, mcm_stream_t stream, int32_t nparts, int32_t part, int32_t words, int32_t level,
                  const int32_t *rmatch, const int32_t *cmatch, const uint32_t *frontier, uint32_t *slice,
                  int32_t *psi_row, int32_t *psi_col, uint64_t *reached_free) {
  if (!h || !pgr_args_ok(h, nparts, part, words) || !frontier || !slice || !reached_free || level < 0 ||
      2LL * level + 2 >= (int64_t)h->m + h->n + 2 || (h->m > 0 && (!rmatch || !psi_row)) ||
      (h->n > 0 && (!cmatch || !psi_col)))
    return MCM_EINVAL;
  if (h->poisoned) return MCM_ECUDA;
  NvtxRange r("mcm_pgr_level");
  const Layout &L = h->L;
  if (int rc = mcm_internal_pgr_level(h->m, h->n, nparts, part, words, level, (const int *)(h->ws + L.cptr),
                             (const int *)(h->ws + L.cadj), rmatch, cmatch, frontier, slice, psi_row, psi_col,
                             (unsigned long long *)reached_free, (cudaStream_t)stream)) {
    h->poisoned = true;
    last_cuda_error = (cudaError_t)rc;
    return MCM_ECUDA;
  }
  return MCM_OK;
}

int64_t mcm_gap_relabel(mcm_handle_t h, mcm_stream_t stream, int32_t *psi_row, int32_t *psi_col) {
  if (!h) return MCM_EINVAL;
  if ((h->m > 0 && !psi_row) || (h->n > 0 && !psi_col)) return MCM_EINVAL;
  return launch(h, (cudaStream_t)stream, MODE_GAP, psi_row, psi_col, psi_row, psi_col);
}

int mcm_set_options(mcm_handle_t h, const mcm_options_t *o) {
  if (!h || !o || check_opts(o) != MCM_OK) return MCM_EINVAL;
  h->opt = *o;
  return MCM_OK;
}

int mcm_set_k(mcm_handle_t h, double k) {
  if (!h || !(k > 0) || !std::isfinite(k)) return MCM_EINVAL;
  h->opt.k = k;
  return MCM_OK;
}

int mcm_get_stats(mcm_handle_t h, mcm_stats_t *out) {
  if (!h || !out) return MCM_EINVAL;
  *out = h->stats;
  return MCM_OK;
}

int mcm_abi_sizes(size_t *options_size, size_t *stats_size) {
  if (options_size) *options_size = sizeof(mcm_options_t);
  if (stats_size) *stats_size = sizeof(mcm_stats_t);
  return MCM_OK;
}

int mcm_destroy(mcm_handle_t h) {
  if (!h) return MCM_EINVAL;
  delete h;
  return MCM_OK;
}

}  // extern "C"
