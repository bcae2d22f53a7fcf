// Probe: grid-barrier variants and memory-scope latencies on B200 (sm_100a).
// Build: nvcc -O3 -gencode arch=compute_100a,code=sm_100a -o tools/probe_sync tools/probe_sync.cu
//
//  A  current build: __threadfence + atomicAdd (returns) + relaxed poll + __threadfence
//  B  red.release.gpu (no return) on a monotonic counter, relaxed poll to a known
//     target, fence.acq_rel.gpu after the flip
//  C  as B, acquire poll
//  D  as B with the arrival replaced by atom.add.release (returning)
//  then dependent-load chains: ld.relaxed.gpu vs ld.relaxed.cta (re-read after a
//  store by the same CTA) vs ld.global.ca, and atomicAdd / CAS round trips.
#include <cstdio>
#include <cuda_runtime.h>

typedef unsigned u32;
typedef unsigned long long u64;

__device__ __forceinline__ u32 ld_rlx(const u32 *p) {
  u32 v;
  asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ u32 ld_acq(const u32 *p) {
  u32 v;
  asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void red_rel(u32 *p, u32 v) {
  asm volatile("red.release.gpu.global.add.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
__device__ __forceinline__ u32 atom_rel(u32 *p, u32 v) {
  u32 o;
  asm volatile("atom.release.gpu.global.add.u32 %0, [%1], %2;" : "=r"(o) : "l"(p), "r"(v) : "memory");
  return o;
}
__device__ __forceinline__ void fence_acqrel() { asm volatile("fence.acq_rel.gpu;" ::: "memory"); }

__device__ void bar_A(u32 *bar) {
  __syncthreads();
  if (threadIdx.x == 0) {
    u32 nb = (blockIdx.x == 0) ? (0x80000000u - (gridDim.x - 1)) : 1u;
    __threadfence();
    u32 old = atomicAdd(bar, nb);
    while (((ld_rlx(bar) ^ old) & 0x80000000u) == 0) {
    }
    __threadfence();
  }
  __syncthreads();
}
template <int V>
__device__ void bar_B(u32 *bar, u32 &target) {
  __syncthreads();
  target += gridDim.x;
  if (threadIdx.x == 0) {
    if (V == 3) (void)atom_rel(bar, 1u);
    else red_rel(bar, 1u);
    if (V == 2) {
      while ((int)(ld_acq(bar) - target) < 0) {
      }
    } else {
      while ((int)(ld_rlx(bar) - target) < 0) {
      }
      fence_acqrel();
    }
  }
  __syncthreads();
}

__global__ void kA(u32 *bar, int it) {
  for (int i = 0; i < it; i++) bar_A(bar);
}
template <int V>
__global__ void kB(u32 *bar, int it) {
  u32 t = 0;
  for (int i = 0; i < it; i++) bar_B<V>(bar, t);
}

// dependent chains (one thread)
__global__ void chase_gpu(u32 *a, int it, u32 *out) {
  u32 x = 0;
  for (int i = 0; i < it; i++) asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(x) : "l"(a + x) : "memory");
  out[0] = x;
}
__global__ void chase_cta(u32 *a, int it, u32 *out) {
  u32 x = 0;
  for (int i = 0; i < it; i++) asm volatile("ld.relaxed.cta.global.u32 %0, [%1];" : "=r"(x) : "l"(a + x) : "memory");
  out[0] = x;
}
__global__ void chase_ca(u32 *a, int it, u32 *out) {
  u32 x = 0;
  for (int i = 0; i < it; i++) asm volatile("ld.global.ca.u32 %0, [%1];" : "=r"(x) : "l"(a + x) : "memory");
  out[0] = x;
}
// store then dependent re-load by the same thread, cta scope: does L1 serve it?
__global__ void st_ld_cta(u32 *a, int it, u32 *out) {
  u32 x = 0;
  for (int i = 0; i < it; i++) {
    asm volatile("st.relaxed.cta.global.u32 [%0], %1;" ::"l"(a + (x & 1023)), "r"(x + 1) : "memory");
    asm volatile("ld.relaxed.cta.global.u32 %0, [%1];" : "=r"(x) : "l"(a + (x & 1023)) : "memory");
  }
  out[0] = x;
}
__global__ void st_ld_gpu(u32 *a, int it, u32 *out) {
  u32 x = 0;
  for (int i = 0; i < it; i++) {
    asm volatile("st.relaxed.gpu.global.u32 [%0], %1;" ::"l"(a + (x & 1023)), "r"(x + 1) : "memory");
    asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(x) : "l"(a + (x & 1023)) : "memory");
  }
  out[0] = x;
}
__global__ void atom_chain(u32 *a, int it, u32 *out) {
  u32 x = 0;
  for (int i = 0; i < it; i++) x = atomicAdd(a + (x & 1023), 1u) & 1023;
  out[0] = x;
}
__global__ void cas_chain(u32 *a, int it, u32 *out) {
  u32 x = 0;
  for (int i = 0; i < it; i++) x = atomicCAS(a + (x & 1023), x, x + 1) & 1023;
  out[0] = x;
}
__global__ void fence_chain(u32 *a, int it, u32 *out) {
  u32 x = 0;
  for (int i = 0; i < it; i++) {
    asm volatile("st.relaxed.gpu.global.u32 [%0], %1;" ::"l"(a + (i & 1023)), "r"(x) : "memory");
    __threadfence();
    x++;
  }
  out[0] = x;
}
__global__ void fence_ar_chain(u32 *a, int it, u32 *out) {
  u32 x = 0;
  for (int i = 0; i < it; i++) {
    asm volatile("st.relaxed.gpu.global.u32 [%0], %1;" ::"l"(a + (i & 1023)), "r"(x) : "memory");
    fence_acqrel();
    x++;
  }
  out[0] = x;
}

__global__ void gt_res(u64 *out) {
  u64 prev, t;
  asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(prev));
  int k = 0;
  for (int i = 0; i < 1000000 && k < 16; i++) {
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
    if (t != prev) { out[k++] = t - prev; prev = t; }
  }
}

int main() {
  cudaDeviceProp pr;
  cudaGetDeviceProperties(&pr, 0);
  printf("device %s SMs %d\n", pr.name, pr.multiProcessorCount);
  cudaEvent_t a, b;
  cudaEventCreate(&a);
  cudaEventCreate(&b);
  float ms;
  u32 *bar, *buf, *out;
  cudaMalloc(&bar, 4096);
  cudaMalloc(&buf, 64 << 20);
  cudaMalloc(&out, 64);
  const int nb = pr.multiProcessorCount, it = 4000;
  auto timeit = [&](const char *name, void *fn) {
    cudaMemset(bar, 0, 4096);
    int i2 = it;
    void *args[] = {&bar, &i2};
    cudaLaunchCooperativeKernel(fn, nb, 512, args, 0, 0);
    cudaDeviceSynchronize();
    cudaMemset(bar, 0, 4096);
    cudaEventRecord(a);
    cudaLaunchCooperativeKernel(fn, nb, 512, args, 0, 0);
    cudaEventRecord(b);
    cudaEventSynchronize(b);
    cudaEventElapsedTime(&ms, a, b);
    printf("%-48s %.3f us/barrier (%s)\n", name, ms * 1000 / it, cudaGetErrorString(cudaGetLastError()));
  };
  timeit("A fence+atomicAdd+rlx poll+fence", (void *)kA);
  timeit("B red.release + rlx poll + fence.acq_rel", (void *)kB<1>);
  timeit("C red.release + acquire poll", (void *)kB<2>);
  timeit("D atom.release + rlx poll + fence.acq_rel", (void *)kB<3>);

  // pointer-chase arrays: random cycle over 1 MB (L2 resident) and a 4 KB one (L1)
  for (size_t bytes : {(size_t)4096, (size_t)1 << 20, (size_t)32 << 20}) {
    size_t n = bytes / 4;
    u32 *h = (u32 *)malloc(bytes), *perm = (u32 *)malloc(bytes);
    for (size_t i = 0; i < n; i++) perm[i] = (u32)i;
    u64 x = 88172645463325252ull;
    for (size_t i = n - 1; i > 0; i--) {
      x ^= x << 13; x ^= x >> 7; x ^= x << 17;
      size_t j = x % (i + 1);
      u32 t = perm[i]; perm[i] = perm[j]; perm[j] = t;
    }
    for (size_t i = 0; i < n; i++) h[perm[i]] = perm[(i + 1) % n];
    cudaMemcpy(buf, h, bytes, cudaMemcpyHostToDevice);
    struct { const char *nm; void (*f)(u32 *, int, u32 *); } ks[] = {
        {"ld.relaxed.gpu", chase_gpu}, {"ld.relaxed.cta", chase_cta}, {"ld.global.ca", chase_ca}};
    for (auto &k : ks) {
      const int n2 = 20000;
      k.f<<<1, 1>>>(buf, 2000, out);
      cudaDeviceSynchronize();
      cudaEventRecord(a);
      k.f<<<1, 1>>>(buf, n2, out);
      cudaEventRecord(b);
      cudaEventSynchronize(b);
      cudaEventElapsedTime(&ms, a, b);
      printf("chase %-16s %8zu B: %.1f ns/load\n", k.nm, bytes, ms * 1e6 / n2);
    }
    free(h);
    free(perm);
  }
  cudaMemset(buf, 0, 1 << 20);
  struct { const char *nm; void (*f)(u32 *, int, u32 *); } ks2[] = {
      {"st+ld relaxed.cta (same addr)", st_ld_cta}, {"st+ld relaxed.gpu (same addr)", st_ld_gpu},
      {"atomicAdd chain", atom_chain},          {"atomicCAS chain", cas_chain},
      {"st + __threadfence", fence_chain},      {"st + fence.acq_rel.gpu", fence_ar_chain}};
  for (auto &k : ks2) {
    const int n2 = 20000;
    k.f<<<1, 1>>>(buf, 2000, out);
    cudaDeviceSynchronize();
    cudaEventRecord(a);
    k.f<<<1, 1>>>(buf, n2, out);
    cudaEventRecord(b);
    cudaEventSynchronize(b);
    cudaEventElapsedTime(&ms, a, b);
    printf("%-40s %.1f ns/iter\n", k.nm, ms * 1e6 / n2);
  }
  {
    u64 *d, h[16] = {0};
    cudaMalloc(&d, sizeof(h));
    cudaMemset(d, 0, sizeof(h));
    gt_res<<<1, 1>>>(d);
    cudaMemcpy(h, d, sizeof(h), cudaMemcpyDeviceToHost);
    printf("globaltimer deltas (ns):");
    for (int i = 0; i < 16; i++) printf(" %llu", h[i]);
    printf("\n");
  }
  printf("err: %s\n", cudaGetErrorString(cudaGetLastError()));
  return 0;
}
