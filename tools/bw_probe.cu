// bw_probe.cu -- HBM bandwidth of read-only, write-only and mixed streams on B200.
// For k in {0, 1/4, 1/2, 3/4, 1}: read k*N floats (every row of a fraction of
// rows, like row perforation) and write N floats.  Prints GB/s of (read + write).
#include <cstdio>
#include <cuda_runtime.h>
__global__ void mix(const float4* __restrict__ in, float4* __restrict__ out, long long n4, int keep_num,
                    int keep_den, int row4) {
  // "rows" of row4 float4; a row is read iff (row % keep_den) < keep_num; every row is written
  for (long long i = blockIdx.x * (long long)blockDim.x + threadIdx.x; i < n4; i += (long long)gridDim.x * blockDim.x) {
    const long long row = i / row4;
    float4 v = make_float4(1.f, 2.f, 3.f, 4.f);
    if ((int)(row % keep_den) < keep_num) v = __ldcs(in + i);
    __stcs(out + i, v);
  }
}
__global__ void readonly(const float4* __restrict__ in, long long n4, float* sink) {
  float acc = 0.f;
  for (long long i = blockIdx.x * (long long)blockDim.x + threadIdx.x; i < n4; i += (long long)gridDim.x * blockDim.x) {
    float4 v = __ldcs(in + i);
    acc += v.x + v.y + v.z + v.w;
  }
  if (acc == 12345.f) sink[0] = acc;
}
int main() {
  const long long N = 1ll << 28;  // 1 GiB of floats per buffer
  float4 *a, *b;
  float* sink;
  cudaMalloc(&a, N * 4);
  cudaMalloc(&b, N * 4);
  cudaMalloc(&sink, 4);
  cudaMemset(a, 0, N * 4);
  cudaEvent_t e0, e1;
  cudaEventCreate(&e0);
  cudaEventCreate(&e1);
  const int grid = 148 * 16, blk = 256, row4 = 1024;  // 16 KB rows
  auto timeit = [&](auto f) {
    for (int w = 0; w < 3; ++w) f();
    cudaEventRecord(e0);
    for (int r = 0; r < 10; ++r) f();
    cudaEventRecord(e1);
    cudaEventSynchronize(e1);
    float ms;
    cudaEventElapsedTime(&ms, e0, e1);
    return ms / 10;
  };
  float ms = timeit([&] { readonly<<<grid, blk>>>(a, N / 4, sink); });
  printf("read-only      : %8.1f GB/s\n", N * 4 / ms / 1e6);
  int kn[] = {0, 1, 1, 3, 1}, kd[] = {1, 4, 2, 4, 1};
  for (int t = 0; t < 5; ++t) {
    ms = timeit([&] { mix<<<grid, blk>>>(a, b, N / 4, kn[t], kd[t], row4); });
    const double k = (double)kn[t] / kd[t];
    printf("read %4.2f + write 1: %8.3f ms  %8.1f GB/s (read+write), write-only rate %8.1f GB/s\n", k, ms,
           (k + 1.0) * N * 4 / ms / 1e6, N * 4 / ms / 1e6);
  }
  return 0;
}
