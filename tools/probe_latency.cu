// Latency probe: kernel launch, CUDA graph node, grid barrier, single-CTA barrier.
// Build: nvcc -O3 -gencode arch=compute_100a,code=sm_100a -o probe tools/probe_latency.cu
#include <cstdio>
#include <cuda_runtime.h>
#include <cooperative_groups.h>
namespace cg = cooperative_groups;

__global__ void empty_k(int* p) { if (threadIdx.x == 0 && blockIdx.x == 0 && p) p[0]++; }

__device__ __forceinline__ unsigned ld_acq(const unsigned* p) {
  unsigned v; asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory"); return v; }

// sense/generation grid barrier
__device__ void gbar(unsigned* cnt, unsigned* gen, unsigned nblk) {
  __syncthreads();
  if (threadIdx.x == 0) {
    unsigned g = ld_acq(gen);
    __threadfence();
    unsigned old = atomicAdd(cnt, 1u);
    if (old == nblk - 1) { atomicExch(cnt, 0u); __threadfence(); atomicAdd(gen, 1u); }
    else { while (ld_acq(gen) == g) { } }
  }
  __syncthreads();
}

__global__ void gbar_k(unsigned* cnt, unsigned* gen, int iters) {
  for (int i = 0; i < iters; i++) gbar(cnt, gen, gridDim.x);
}
__global__ void cg_k(int iters) {
  cg::grid_group g = cg::this_grid();
  for (int i = 0; i < iters; i++) g.sync();
}
__global__ void cta_k(int iters, int* out) {
  __shared__ int s;
  int acc = 0;
  for (int i = 0; i < iters; i++) { if (threadIdx.x == 0) s = i; __syncthreads(); acc += s; __syncthreads(); }
  if (threadIdx.x == 0) out[0] = acc;
}
// dependent global-load chain latency (pointer chase) in L2 and DRAM
__global__ void chase_k(const int* next, int iters, int* out) {
  int p = 0;
  for (int i = 0; i < iters; i++) p = __ldcg(next + p);
  out[0] = p;
}

int main() {
  cudaDeviceProp pr; cudaGetDeviceProperties(&pr, 0);
  int l2; cudaDeviceGetAttribute(&l2, cudaDevAttrL2CacheSize, 0);
  printf("device %s SMs %d L2 %d MB smem/blk optin %zu clock %d kHz\n", pr.name, pr.multiProcessorCount, l2 >> 20, pr.sharedMemPerBlockOptin, pr.clockRate);
  cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b); float ms;
  int* d; cudaMalloc(&d, 1 << 20);
  const int N = 2000;
  for (int w = 0; w < 100; w++) empty_k<<<148, 512>>>(d);
  cudaEventRecord(a);
  for (int i = 0; i < N; i++) empty_k<<<148, 512>>>(d);
  cudaEventRecord(b); cudaEventSynchronize(b); cudaEventElapsedTime(&ms, a, b);
  printf("stream launch back-to-back: %.3f us/kernel\n", ms * 1000 / N);
  // graph of N kernels
  cudaStream_t s; cudaStreamCreate(&s); cudaGraph_t gr; cudaGraphExec_t ge;
  cudaStreamBeginCapture(s, cudaStreamCaptureModeGlobal);
  for (int i = 0; i < 200; i++) empty_k<<<148, 512, 0, s>>>(d);
  cudaStreamEndCapture(s, &gr); cudaGraphInstantiate(&ge, gr, 0);
  cudaGraphLaunch(ge, s); cudaStreamSynchronize(s);
  cudaEventRecord(a, s);
  for (int i = 0; i < 10; i++) cudaGraphLaunch(ge, s);
  cudaEventRecord(b, s); cudaEventSynchronize(b); cudaEventElapsedTime(&ms, a, b);
  printf("graph node: %.3f us/kernel\n", ms * 1000 / 2000);
  unsigned* bar; cudaMalloc(&bar, 256); cudaMemset(bar, 0, 256);
  for (int bpsm = 1; bpsm <= 2; bpsm++) {
    int nb = pr.multiProcessorCount * bpsm;
    int it = 2000;
    void* args[] = {&bar, nullptr, &it};
    unsigned* gen = bar + 32; args[1] = &gen;
    cudaLaunchCooperativeKernel((void*)gbar_k, nb, 512, args, 0, 0); cudaDeviceSynchronize();
    cudaEventRecord(a);
    cudaLaunchCooperativeKernel((void*)gbar_k, nb, 512, args, 0, 0);
    cudaEventRecord(b); cudaEventSynchronize(b); cudaEventElapsedTime(&ms, a, b);
    printf("custom grid barrier %d CTAs: %.3f us/barrier (%s)\n", nb, ms * 1000 / it, cudaGetErrorString(cudaGetLastError()));
    void* args2[] = {&it};
    cudaLaunchCooperativeKernel((void*)cg_k, nb, 512, args2, 0, 0); cudaDeviceSynchronize();
    cudaEventRecord(a);
    cudaLaunchCooperativeKernel((void*)cg_k, nb, 512, args2, 0, 0);
    cudaEventRecord(b); cudaEventSynchronize(b); cudaEventElapsedTime(&ms, a, b);
    printf("cg grid.sync %d CTAs: %.3f us/barrier (%s)\n", nb, ms * 1000 / it, cudaGetErrorString(cudaGetLastError()));
  }
  cta_k<<<1, 512>>>(10000, d); cudaDeviceSynchronize();
  cudaEventRecord(a); cta_k<<<1, 512>>>(100000, d); cudaEventRecord(b); cudaEventSynchronize(b); cudaEventElapsedTime(&ms, a, b);
  printf("single-CTA 512t: %.4f us per 2x__syncthreads\n", ms * 1000 / 100000);
  // pointer chase
  for (size_t bytes : {(size_t)1 << 20, (size_t)1 << 26, (size_t)1 << 30}) {
    size_t n = bytes / 4; int* h = (int*)malloc(bytes); 
    // random cycle
    unsigned long long x = 88172645463325252ull;
    int* perm = (int*)malloc(bytes);
    for (size_t i = 0; i < n; i++) perm[i] = (int)i;
    for (size_t i = n - 1; i > 0; i--) { x ^= x << 13; x ^= x >> 7; x ^= x << 17; size_t j = x % (i + 1); int t = perm[i]; perm[i] = perm[j]; perm[j] = t; }
    for (size_t i = 0; i < n; i++) h[perm[i]] = perm[(i + 1) % n];
    int* dn; cudaMalloc(&dn, bytes); cudaMemcpy(dn, h, bytes, cudaMemcpyHostToDevice);
    chase_k<<<1, 1>>>(dn, 1000, d); cudaDeviceSynchronize();
    cudaEventRecord(a); chase_k<<<1, 1>>>(dn, 20000, d); cudaEventRecord(b); cudaEventSynchronize(b); cudaEventElapsedTime(&ms, a, b);
    printf("pointer chase %zu MB: %.1f ns/load\n", bytes >> 20, ms * 1e6 / 20000);
    cudaFree(dn); free(h); free(perm);
  }
  printf("err: %s\n", cudaGetErrorString(cudaGetLastError()));
  return 0;
}
