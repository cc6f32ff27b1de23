// bw_probe3.cu -- mixed read/write stream: effect of the per-CTA block shape
// (block = bw bytes wide x bh rows of a 16-KB-pitch image; rows kept per k)
#include <cstdio>
#include <cuda_runtime.h>
__global__ void mix_block(const float4* __restrict__ in, float4* __restrict__ out, int rows, int pitch4, int bw4,
                          int bh, int keep_num, int keep_den) {
  const int nbx = pitch4 / bw4, nby = (rows + bh - 1) / bh, nb = nbx * nby;
  for (int b = blockIdx.x; b < nb; b += gridDim.x) {
    const int bx = b % nbx, by = b / nbx;
    for (int r = by * bh; r < min(rows, by * bh + bh); ++r) {
      const bool keep = (r % keep_den) < keep_num;
      for (int c = threadIdx.x; c < bw4; c += blockDim.x) {
        const long long i = (long long)r * pitch4 + bx * bw4 + c;
        float4 v = make_float4(1.f, 2.f, 3.f, 4.f);
        if (keep) v = __ldcs(in + i);
        __stcs(out + i, v);
      }
    }
  }
}
int main() {
  const long long N = 1ll << 28;  // floats
  const int pitch4 = 1024;  // 4096 floats per row = 1024 float4 = 16 KB
  const int rows = (int)(N / 4 / pitch4);
  float4 *a, *b;
  cudaMalloc(&a, N * 4); cudaMalloc(&b, N * 4); cudaMemset(a, 0, N * 4); cudaMemset(b, 0, N * 4);
  cudaEvent_t e0, e1; cudaEventCreate(&e0); cudaEventCreate(&e1);
  auto timeit = [&](auto f) { for (int w = 0; w < 2; ++w) f(); cudaEventRecord(e0); for (int r = 0; r < 5; ++r) f();
    cudaEventRecord(e1); cudaEventSynchronize(e1); float ms; cudaEventElapsedTime(&ms, e0, e1); return ms / 5; };
  int kn[] = {1, 1, 1}, kd[] = {1, 2, 4};
  int shapes[][2] = {{1024, 64}, {256, 128}, {256, 256}, {256, 1024}, {64, 256}, {512, 128}, {1024, 16}};
  for (int t = 0; t < 3; ++t) {
    const double k = (double)kn[t] / kd[t];
    for (auto& sh : shapes) {
      for (int cpsm : {4, 8}) {
        float ms = timeit([&] { mix_block<<<148 * cpsm, 256>>>(a, b, rows, pitch4, sh[0], sh[1], kn[t], kd[t]); });
        if (cudaGetLastError() != cudaSuccess) { printf("launch error\n"); return 1; }
        printf("read %.2f block %5d B x %4d rows  ctas/sm %d: %7.3f ms %7.1f GB/s\n", k, sh[0] * 16, sh[1], cpsm, ms,
               (k + 1) * N * 4 / ms / 1e6);
      }
    }
  }
  return 0;
}
