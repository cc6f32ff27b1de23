// bw_probe2.cu -- does the store policy / burst grouping change the mixed-stream ceiling?
#include <cstdio>
#include <cuda_runtime.h>
template <int MODE>
__global__ void mix(const float4* __restrict__ in, float4* __restrict__ out, long long n4, int keep_num, int keep_den,
                    int row4) {
  for (long long i = blockIdx.x * (long long)blockDim.x + threadIdx.x; i < n4; i += (long long)gridDim.x * blockDim.x) {
    const long long row = i / row4;
    float4 v = make_float4(1.f, 2.f, 3.f, 4.f);
    if ((int)(row % keep_den) < keep_num) v = MODE == 2 ? in[i] : __ldcs(in + i);
    if (MODE == 0) __stcs(out + i, v);
    else if (MODE == 1) out[i] = v;
    else if (MODE == 2) __stwt(out + i, v);
    else asm volatile("st.global.L1::no_allocate.v4.f32 [%0], {%1,%2,%3,%4};" ::"l"(out + i), "f"(v.x), "f"(v.y), "f"(v.z), "f"(v.w));
  }
}
// blocked: each CTA streams its own contiguous 1 MB chunk (row-major like a CTA strip) -- reads and writes local
__global__ void mix_chunk(const float4* __restrict__ in, float4* __restrict__ out, long long n4, int keep_num,
                          int keep_den, int row4, long long chunk4) {
  for (long long c0 = blockIdx.x * chunk4; c0 < n4; c0 += (long long)gridDim.x * chunk4)
    for (long long i = c0 + threadIdx.x; i < c0 + chunk4 && i < n4; i += blockDim.x) {
      const long long row = i / row4;
      float4 v = make_float4(1.f, 2.f, 3.f, 4.f);
      if ((int)(row % keep_den) < keep_num) v = __ldcs(in + i);
      __stcs(out + i, v);
    }
}
int main() {
  const long long N = 1ll << 28;
  float4 *a, *b;
  cudaMalloc(&a, N * 4); cudaMalloc(&b, N * 4); cudaMemset(a, 0, N * 4); cudaMemset(b, 0, N * 4);
  cudaEvent_t e0, e1; cudaEventCreate(&e0); cudaEventCreate(&e1);
  auto timeit = [&](auto f) { for (int w = 0; w < 3; ++w) f(); cudaEventRecord(e0); for (int r = 0; r < 10; ++r) f();
    cudaEventRecord(e1); cudaEventSynchronize(e1); float ms; cudaEventElapsedTime(&ms, e0, e1); return ms / 10; };
  const int grid = 148 * 16, blk = 256, row4 = 1024;
  int kn[] = {1, 1, 1}, kd[] = {1, 2, 4};
  const char* names[] = {"stcs", "st", "ld/stwt", "st.na"};
  for (int t = 0; t < 3; ++t) {
    const double k = (double)kn[t] / kd[t];
    float ms[5];
    ms[0] = timeit([&] { mix<0><<<grid, blk>>>(a, b, N / 4, kn[t], kd[t], row4); });
    ms[1] = timeit([&] { mix<1><<<grid, blk>>>(a, b, N / 4, kn[t], kd[t], row4); });
    ms[2] = timeit([&] { mix<2><<<grid, blk>>>(a, b, N / 4, kn[t], kd[t], row4); });
    ms[3] = timeit([&] { mix<3><<<grid, blk>>>(a, b, N / 4, kn[t], kd[t], row4); });
    ms[4] = timeit([&] { mix_chunk<<<148 * 8, 512>>>(a, b, N / 4, kn[t], kd[t], row4, 65536); });
    for (int m = 0; m < 5; ++m)
      printf("read %.2f: %-10s %7.3f ms  %7.1f GB/s\n", k, m < 4 ? names[m] : "chunked1MB", ms[m], (k + 1) * N * 4 / ms[m] / 1e6);
  }
  return 0;
}
