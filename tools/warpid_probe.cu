// warpid_probe.cu -- which SM sub-partition (scheduler) does each warp of a
// 5-warp CTA land on, with 4 co-resident CTAs per SM (the median kernel's
// shape)?  %warpid % 4 is taken as the sub-partition.  Prints, per warp index
// within the CTA, how many warps landed on each of the 4 sub-partitions.
// nvcc -gencode arch=compute_100a,code=sm_100a -o tools/warpid_probe tools/warpid_probe.cu
#include <cstdio>
#include <cuda_runtime.h>

__global__ void __launch_bounds__(160, 4) probe(int* out, long long spin) {
  __shared__ int pad[12 * 1024];  // ~48 KB: at most 4 CTAs per SM
  unsigned wid, smid;
  asm volatile("mov.u32 %0, %%warpid;" : "=r"(wid));
  asm volatile("mov.u32 %0, %%smid;" : "=r"(smid));
  const long long t0 = clock64();
  while (clock64() - t0 < spin) {
  }
  if ((threadIdx.x & 31) == 0) {
    const int w = threadIdx.x >> 5;
    out[(blockIdx.x * 5 + w) * 2] = (int)wid;
    out[(blockIdx.x * 5 + w) * 2 + 1] = (int)smid + pad[threadIdx.x & 7] * 0;
  }
}

int main() {
  int sms = 0;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  const int grid = 4 * sms;
  int* d;
  cudaMalloc(&d, grid * 5 * 2 * sizeof(int));
  cudaFuncSetAttribute(probe, cudaFuncAttributePreferredSharedMemoryCarveout, 100);
  probe<<<grid, 160>>>(d, 2000000);
  int* h = new int[grid * 5 * 2];
  cudaMemcpy(h, d, grid * 5 * 2 * sizeof(int), cudaMemcpyDeviceToHost);
  int cnt[5][4] = {};
  for (int b = 0; b < grid; ++b)
    for (int w = 0; w < 5; ++w) cnt[w][h[(b * 5 + w) * 2] % 4]++;
  printf("warp-in-CTA: count per sub-partition (warpid %% 4) over %d CTAs\n", grid);
  for (int w = 0; w < 5; ++w) printf("  warp %d: %5d %5d %5d %5d\n", w, cnt[w][0], cnt[w][1], cnt[w][2], cnt[w][3]);
  printf("first CTAs (warpid of warps 0..4, smid):\n");
  for (int b = 0; b < 8; ++b)
    printf("  cta %d: %d %d %d %d %d  sm %d\n", b, h[b * 10], h[b * 10 + 2], h[b * 10 + 4], h[b * 10 + 6], h[b * 10 + 8],
           h[b * 10 + 1]);
  return 0;
}
