// pgr.cu -- SURVEY NEXT-4 (an experiment, clearly labelled): a 1D row-partitioned
// global relabel (Alg. 2 with the matched test of Alg. 5 l.6)
// whose BFS levels exchange the row frontier as a bitmap by an all-gather.
//
// Partition (P ranks, rank p, W words of 32 rows per rank):
//   * rank p owns rows [32 W p, min(m, 32 W (p+1))): their labels, and the label of
//     the mate column v = mu(u) of every owned row u with mu(v) = u (the column is
//     matched, Alg. 5 l.6 -- rows are authoritative);
//   * rank p owns the columns that are not matched in [CB p, min(n, CB (p+1))),
//     CB = ceil(n / P) (the BFS reaches them but they extend no path).
// Level L (row labels 2L are the frontier F_L): every unlabelled owned vertex pulls
// -- a column v gets 2L+1 iff some row of Gamma(v) is in F_L (the BFS distance,
// P:248-256), and its mate row 2L+2 (the row joins F_{L+1}).  Each rank writes its
// own slice of the next frontier: W bitmap words followed by one count word (the
// rows it added), so after the all-gather every rank holds F_{L+1} and every
// count and stops when they sum to 0 -- no other collective per level.
//
// The gathered buffer is P slices of W + 1 words: row u's bit is word
// (u / 32W) (W + 1) + (u mod 32W) / 32, bit u mod 32.
#include <cuda_runtime.h>
#include <cstdint>

namespace pgr {

__device__ __forceinline__ bool in_frontier(const uint32_t *F, int u, int W) {
  const int r = u / (32 * W), o = u - r * 32 * W;
  return (__ldg(F + (long long)r * (W + 1) + (o >> 5)) >> (o & 31)) & 1u;
}

// Level 0: owned rows get 0 (unmatched, Alg. 2 l.1) or m+n (l.3); every other row
// and every column m+n (l.2) -- each part fills the whole arrays, so the elementwise
// minimum over the parts is the GR result.
__global__ void k_init(int m, int n, int P, int p, int W, const int *rmatch, uint32_t *slice, int *psi_row,
                       int *psi_col) {
  const int INF = m + n;
  const long long lane = threadIdx.x & 31;
  const long long gt = blockIdx.x * (long long)blockDim.x + threadIdx.x, nt = (long long)gridDim.x * blockDim.x;
  const long long gw = gt >> 5, nw = nt >> 5;
  const long long r0 = (long long)p * 32 * W, r1 = r0 + 32LL * W;
  for (long long wi = gw; wi < W; wi += nw) {
    const long long u = r0 + wi * 32 + lane;
    const bool src = u < m && rmatch[u] == -1;
    const unsigned b = __ballot_sync(0xffffffffu, src);
    if (lane == 0) {
      slice[wi] = b;
      if (b) atomicAdd(slice + W, (uint32_t)__popc(b));
    }
  }
  for (long long u = gt; u < m; u += nt) psi_row[u] = (u >= r0 && u < r1 && rmatch[u] == -1) ? 0 : INF;
  for (long long v = gt; v < n; v += nt) psi_col[v] = INF;
}

// does some row of Gamma(v) = cadj[s, e) lie in F?
__device__ __forceinline__ bool pull(const int *cadj, int s, int e, const uint32_t *F, int W) {
  for (int j = s; j < e; j++)
    if (in_frontier(F, __ldg(cadj + j), W)) return true;
  return false;
}

// One level: see the file comment.  counts[0] += columns not matched that got a
// label (reached free columns, for the guard's test and the oracle's pin).
__global__ void k_level(int m, int n, int P, int p, int W, int L, const int *cptr, const int *cadj,
                        const int *rmatch, const int *cmatch, const uint32_t *F, uint32_t *slice, int *psi_row,
                        int *psi_col, unsigned long long *counts) {
  const int INF = m + n;
  const long long lane = threadIdx.x & 31;
  const long long gt = blockIdx.x * (long long)blockDim.x + threadIdx.x;
  const long long gw = gt >> 5, nw = ((long long)gridDim.x * blockDim.x) >> 5;
  // owned rows and their mate columns: one warp per bitmap word
  for (long long wi = gw; wi < W; wi += nw) {
    const long long u = (long long)p * 32 * W + wi * 32 + lane;
    bool add = false;
    if (u < m && psi_row[u] == INF) {
      const int v = rmatch[u];
      if (v >= 0 && v < n && cmatch[v] == (int)u && pull(cadj, __ldg(cptr + v), __ldg(cptr + v + 1), F, W)) {
        psi_col[v] = 2 * L + 1;  // Alg. 2 l.8
        psi_row[u] = 2 * L + 2;  // l.10
        add = true;
      }
    }
    const unsigned b = __ballot_sync(0xffffffffu, add);
    if (lane == 0) {
      slice[wi] = b;
      if (b) atomicAdd(slice + W, (uint32_t)__popc(b));
    }
  }
  // owned columns that are not matched
  const long long CB = ((long long)n + P - 1) / P;
  const long long c0 = CB * p, c1 = CB * (p + 1) < n ? CB * (p + 1) : n;
  unsigned long long fr = 0;
  for (long long v = c0 + gt; v < c1; v += (long long)gridDim.x * blockDim.x) {
    if (psi_col[v] != INF) continue;
    const int w = cmatch[v];
    if (w >= 0 && w < m && rmatch[w] == (int)v) continue;  // matched: the row's owner labels it
    if (pull(cadj, __ldg(cptr + v), __ldg(cptr + v + 1), F, W)) {
      psi_col[v] = 2 * L + 1;
      fr++;
    }
  }
  fr = __reduce_add_sync(0xffffffffu, (unsigned)fr);
  if (lane == 0 && fr) atomicAdd(counts, fr);
}

}  // namespace pgr

// internal launchers (called by api.cu's mcm_pgr_* with the handle's CSC); return a
// cudaError_t (0 = cudaSuccess); C linkage, declared in api.cu
extern "C" {
int mcm_internal_pgr_init(int m, int n, int P, int p, int W, const int *rmatch, uint32_t *slice, int *psi_row,
                          int *psi_col, cudaStream_t st) {
  cudaError_t e = cudaMemsetAsync(slice + W, 0, sizeof(uint32_t), st);
  if (e != cudaSuccess) return (int)e;
  long long work = (long long)W * 32 > n ? (long long)W * 32 : n;
  if (work < m) work = m;
  const int blocks = (int)((work + 255) / 256 < 148 * 8 ? (work + 255) / 256 + 1 : 148 * 8);
  pgr::k_init<<<blocks, 256, 0, st>>>(m, n, P, p, W, rmatch, slice, psi_row, psi_col);
  return (int)cudaGetLastError();
}

int mcm_internal_pgr_level(int m, int n, int P, int p, int W, int L, const int *cptr, const int *cadj,
                           const int *rmatch, const int *cmatch, const uint32_t *F, uint32_t *slice, int *psi_row,
                           int *psi_col, unsigned long long *counts, cudaStream_t st) {
  cudaError_t e = cudaMemsetAsync(slice + W, 0, sizeof(uint32_t), st);
  if (e != cudaSuccess) return (int)e;
  const long long CB = ((long long)n + P - 1) / P;
  const long long work = (long long)W * 32 > CB ? (long long)W * 32 : CB;
  const int blocks = (int)((work + 255) / 256 < 148 * 8 ? (work + 255) / 256 + 1 : 148 * 8);
  pgr::k_level<<<blocks, 256, 0, st>>>(m, n, P, p, W, L, cptr, cadj, rmatch, cmatch, F, slice, psi_row, psi_col,
                                       counts);
  return (int)cudaGetLastError();
}
}  // extern "C"
