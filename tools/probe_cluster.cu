// Probe: cooperative launch + thread-block clusters; cluster.sync latency.
#include <cstdio>
#include <cuda_runtime.h>
#include <cooperative_groups.h>
namespace cg = cooperative_groups;
__global__ void k(int iters, int *out) {
  cg::cluster_group cl = cg::this_cluster();
  for (int i = 0; i < iters; i++) cl.sync();
  if (threadIdx.x == 0) out[blockIdx.x] = cl.block_rank();
}
__global__ void kg(int iters, int *out) {
  cg::grid_group g = cg::this_grid();
  for (int i = 0; i < iters; i++) g.sync();
  if (threadIdx.x == 0) out[blockIdx.x] = 1;
}
int main() {
  int *d; cudaMalloc(&d, 1 << 20);
  cudaFuncSetAttribute(k, cudaFuncAttributeNonPortableClusterSizeAllowed, 1);
  cudaFuncSetAttribute(kg, cudaFuncAttributeNonPortableClusterSizeAllowed, 1);
  for (int cs : {2, 4, 8, 16}) {
    for (int coop = 0; coop < 2; coop++) {
      cudaLaunchConfig_t cfg = {};
      cfg.blockDim = dim3(512); cfg.dynamicSmemBytes = 0; cfg.stream = 0;
      cudaLaunchAttribute at[2];
      at[0].id = cudaLaunchAttributeClusterDimension; at[0].val.clusterDim.x = cs; at[0].val.clusterDim.y = 1; at[0].val.clusterDim.z = 1;
      at[1].id = cudaLaunchAttributeCooperative; at[1].val.cooperative = coop;
      cfg.attrs = at; cfg.numAttrs = 2;
      int ncl = 0;
      cfg.gridDim = dim3(cs);
      cudaError_t e0 = cudaOccupancyMaxActiveClusters(&ncl, (void*)k, &cfg);
      cfg.gridDim = dim3(ncl * cs);
      int iters = 20000;
      cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b);
      cudaError_t e1 = cudaLaunchKernelEx(&cfg, k, iters, d);
      cudaDeviceSynchronize();
      cudaEventRecord(a);
      cudaError_t e2 = cudaLaunchKernelEx(&cfg, k, iters, d);
      cudaEventRecord(b); cudaEventSynchronize(b);
      float ms; cudaEventElapsedTime(&ms, a, b);
      printf("cluster %2d coop %d: max active clusters %d (%s) grid %d: cluster.sync %.3f us (%s %s)\n", cs, coop, ncl,
             cudaGetErrorString(e0), ncl * cs, ms * 1000 / iters, cudaGetErrorString(e1), cudaGetErrorString(e2));
      if (coop) {
        int it2 = 2000;
        cudaLaunchKernelEx(&cfg, kg, it2, d);
        cudaDeviceSynchronize();
        cudaEventRecord(a);
        cudaError_t e3 = cudaLaunchKernelEx(&cfg, kg, it2, d);
        cudaEventRecord(b); cudaEventSynchronize(b);
        cudaEventElapsedTime(&ms, a, b);
        printf("     grid.sync with clusters: %.3f us (%s)\n", ms * 1000 / it2, cudaGetErrorString(e3));
      }
    }
  }
  return 0;
}
