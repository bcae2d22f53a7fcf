// Latency of the operations on the G-PR critical path (one thread, dependent chains).
#include <cstdio>
#include <cuda_runtime.h>
typedef unsigned long long u64;
__device__ __forceinline__ u64 ld_rlx(const u64 *p) { u64 v; asm volatile("ld.relaxed.gpu.global.b64 %0, [%1];" : "=l"(v) : "l"(p) : "memory"); return v; }
__device__ __forceinline__ u64 gt() { u64 t; asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t)); return t; }
__global__ void k(u64 *a, int *b, int iters, double *out) {
  // a: 8M u64 random cycle; b: 8M int random cycle
  u64 p = 0; u64 t0, t1;
  // warm
  for (int i = 0; i < 1000; i++) p = __ldcg(a + (p & ((1 << 23) - 1)));
  t0 = clock64(); for (int i = 0; i < iters; i++) p = ld_rlx(a + (p & ((1 << 23) - 1))); t1 = clock64();
  out[0] = (double)(t1 - t0) / iters;
  t0 = clock64(); for (int i = 0; i < iters; i++) p = __ldcg(a + (p & ((1 << 23) - 1))); t1 = clock64();
  out[1] = (double)(t1 - t0) / iters;
  int q = (int)p & 0xff;
  t0 = clock64(); for (int i = 0; i < iters; i++) q = __ldg(b + (q & ((1 << 23) - 1))); t1 = clock64();
  out[2] = (double)(t1 - t0) / iters;
  t0 = clock64(); for (int i = 0; i < iters; i++) { u64 x = a[p & ((1 << 23) - 1)]; p = atomicCAS(a + (x & ((1 << 23) - 1)), x, x); } t1 = clock64();
  out[3] = (double)(t1 - t0) / iters;  // load + CAS chain
  t0 = clock64(); for (int i = 0; i < iters; i++) { p = atomicAdd((unsigned long long*)(a + (p & ((1 << 23) - 1))), 0ull); } t1 = clock64();
  out[4] = (double)(t1 - t0) / iters;  // atomic round trip
  __shared__ int s[32];
  t0 = clock64(); for (int i = 0; i < iters; i++) { q = atomicAdd(&s[q & 31], 1); } t1 = clock64();
  out[5] = (double)(t1 - t0) / iters;
  u64 g0 = gt(); for (int i = 0; i < iters; i++) p = ld_rlx(a + (p & ((1 << 23) - 1))); u64 g1 = gt();
  out[6] = (double)(g1 - g0) / iters;  // ns per relaxed load
  out[7] = (double)(p + q);
}
int main() {
  size_t n = 1 << 23;
  u64 *h = (u64 *)malloc(n * 8); int *hb = (int *)malloc(n * 4);
  unsigned long long x = 88172645463325252ull; 
  int *perm = (int *)malloc(n * 4);
  for (size_t i = 0; i < n; i++) perm[i] = (int)i;
  for (size_t i = n - 1; i > 0; i--) { x ^= x << 13; x ^= x >> 7; x ^= x << 17; size_t j = x % (i + 1); int t = perm[i]; perm[i] = perm[j]; perm[j] = t; }
  for (size_t i = 0; i < n; i++) { h[perm[i]] = perm[(i + 1) % n]; hb[perm[i]] = perm[(i + 1) % n]; }
  u64 *a; int *b; double *o; cudaMalloc(&a, n * 8); cudaMalloc(&b, n * 4); cudaMalloc(&o, 64);
  cudaMemcpy(a, h, n * 8, cudaMemcpyHostToDevice); cudaMemcpy(b, hb, n * 4, cudaMemcpyHostToDevice);
  k<<<1, 1>>>(a, b, 2000, o); cudaDeviceSynchronize();
  k<<<1, 1>>>(a, b, 20000, o); cudaDeviceSynchronize();
  double r[8]; cudaMemcpy(r, o, 64, cudaMemcpyDeviceToHost);
  printf("64MB working set (L2-resident after warm): cycles per dependent op\n");
  printf(" ld.relaxed.gpu %.0f | ld.cg %.0f | ldg(nc) %.0f | ld+CAS %.0f | atomicAdd %.0f | smem atomic %.0f | relaxed ns %.1f\n",
         r[0], r[1], r[2], r[3], r[4], r[5], r[6]);
  printf("err %s\n", cudaGetErrorString(cudaGetLastError()));
}
