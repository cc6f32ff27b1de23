// bwprobe.cu -- measurement tool (not part of the method): achievable HBM
// bandwidth of a plain streaming kernel with a given read/write mix, the same
// access shape as a perforated stencil: every output element is written once;
// an input element is read iff its row (row scheme) or its granule (column
// scheme) is kept -- kept fraction keep_num/keep_den.  Used by bench.py to put
// the perforated kernels next to the best a trivial kernel does with the same
// bytes.
#include <cuda_runtime.h>

#include <cstdint>

__global__ void bwp_mix(const float4* __restrict__ in, float4* __restrict__ out, long long n4, int keep_num,
                        int keep_den, int unit4, int n_in) {
  for (long long i = blockIdx.x * (long long)blockDim.x + threadIdx.x; i < n4;
       i += (long long)gridDim.x * blockDim.x) {
    const long long u = i / unit4;
    float4 v = make_float4(1.f, 2.f, 3.f, 4.f);
    if ((int)(u % keep_den) < keep_num) {
      v = __ldcs(in + i);
      if (n_in > 1) {  // second input (Hotspot power) at the same offset of the next buffer
        const float4 w = __ldcs(in + n4 + i);
        v.x += w.x;
      }
    }
    __stcs(out + i, v);
  }
}

extern "C" {
// Time one pass: n_out bytes written, keep_num/keep_den of the input units
// (unit_bytes each; 16 KB = row-like, 128 B = granule-like) read from n_in
// arrays of the same size.  Buffers are caller-provided device memory:
// in: n_in * n_out bytes, out: n_out bytes.  Returns milliseconds (best of reps).
float bwp_time_ms(const void* in, void* out, long long n_out_bytes, int keep_num, int keep_den,
                  int unit_bytes, int n_in, int reps, void* stream) {
  cudaStream_t s = (cudaStream_t)stream;
  const long long n4 = n_out_bytes / 16;
  const int unit4 = unit_bytes / 16 > 0 ? unit_bytes / 16 : 1;
  int dev = 0, sms = 148;
  cudaGetDevice(&dev);
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
  const int grid = sms * 16, blk = 256;
  cudaEvent_t e0, e1;
  cudaEventCreate(&e0);
  cudaEventCreate(&e1);
  float best = 1e30f;
  for (int r = 0; r < reps + 2; ++r) {
    cudaEventRecord(e0, s);
    bwp_mix<<<grid, blk, 0, s>>>((const float4*)in, (float4*)out, n4, keep_num, keep_den, unit4, n_in);
    cudaEventRecord(e1, s);
    cudaEventSynchronize(e1);
    float ms;
    cudaEventElapsedTime(&ms, e0, e1);
    if (r >= 2 && ms < best) best = ms;
  }
  cudaEventDestroy(e0);
  cudaEventDestroy(e1);
  return cudaGetLastError() == cudaSuccess ? best : -1.f;
}
}
