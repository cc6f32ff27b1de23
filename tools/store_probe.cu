// store_probe.cu -- measurement tool (not part of the method): does the store
// flavour change the HBM ceiling of a perforated stencil's byte mix?  Every
// output row (16 KB) is written once; the kept fraction of input rows is read
// (row scheme, skip 1/2 or none).  Store variants: 0 st.global.v4, 1
// st.global.L1::no_allocate.v4 (the kernels'), 2 st.global.cs.v4, 3 L2
// evict_first cache hint, 4 TMA bulk store of a shared-memory row
// (cp.async.bulk.global.shared::cta), 5 L2 evict_last hint.
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o store_probe store_probe.cu
#include <cuda_runtime.h>

#include <cstdint>
#include <cstdio>

__device__ __forceinline__ void st_v(int mode, float4* p, float4 v, uint64_t pol) {
  if (mode == 0) *p = v;
  else if (mode == 1)
    asm volatile("st.global.L1::no_allocate.v4.f32 [%0], {%1,%2,%3,%4};" ::"l"(p), "f"(v.x), "f"(v.y), "f"(v.z),
                 "f"(v.w) : "memory");
  else if (mode == 2) __stcs(p, v);
  else
    asm volatile("st.global.L2::cache_hint.v4.f32 [%0], {%1,%2,%3,%4}, %5;" ::"l"(p), "f"(v.x), "f"(v.y), "f"(v.z),
                 "f"(v.w), "l"(pol) : "memory");
}

// CTA streams rows r = blockIdx.x, += gridDim.x; row = W4 float4
__global__ void probe(const float4* __restrict__ in, float4* __restrict__ out, int rows, int W4, int keep_den,
                      int mode) {
  extern __shared__ float4 sbuf[];
  uint64_t pol = 0;
  if (mode == 3) asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(pol));
  if (mode == 5) asm volatile("createpolicy.fractional.L2::evict_last.b64 %0, 1.0;" : "=l"(pol));
  for (int r = blockIdx.x; r < rows; r += gridDim.x) {
    const bool kept = keep_den <= 1 || (r % keep_den) != keep_den - 1;
    if (mode == 4) {
      for (int c = threadIdx.x; c < W4; c += blockDim.x) {
        float4 v = make_float4(1.f, 2.f, 3.f, 4.f);
        if (kept) v = __ldcs(in + (long long)r * W4 + c);
        sbuf[c] = v;
      }
      asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
      __syncthreads();
      if (threadIdx.x == 0) {
        asm volatile("cp.async.bulk.global.shared::cta.bulk_group [%0], [%1], %2;" ::"l"(out + (long long)r * W4),
                     "r"((uint32_t)__cvta_generic_to_shared(sbuf)), "r"((uint32_t)(W4 * 16))
                     : "memory");
        asm volatile("cp.async.bulk.commit_group;");
        asm volatile("cp.async.bulk.wait_group.read 0;" ::: "memory");
      }
      __syncthreads();
    } else {
      for (int c = threadIdx.x; c < W4; c += blockDim.x) {
        float4 v = make_float4(1.f, 2.f, 3.f, 4.f);
        if (kept) v = __ldcs(in + (long long)r * W4 + c);
        st_v(mode, out + (long long)r * W4 + c, v, pol);
      }
    }
  }
  if (mode == 4 && threadIdx.x == 0) asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");
}

int main() {
  const int W4 = 1024, rows = 65536;  // 16 KB rows, 1 GiB
  float4 *in, *out;
  cudaMalloc(&in, (size_t)rows * W4 * 16);
  cudaMalloc(&out, (size_t)rows * W4 * 16);
  cudaMemset(in, 0, (size_t)rows * W4 * 16);
  cudaFuncSetAttribute(probe, cudaFuncAttributeMaxDynamicSharedMemorySize, 64 * 1024);
  int sms = 148;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  cudaEvent_t e0, e1;
  cudaEventCreate(&e0);
  cudaEventCreate(&e1);
  const char* names[] = {"st.v4", "st.L1::no_allocate", "st.cs", "st.L2 evict_first", "TMA bulk store", "st.L2 evict_last"};
  for (int den : {1, 2, 4}) {
    for (int mode = 0; mode < 6; ++mode) {
      float best = 1e30f;
      for (int cps : {4, 8}) {
        for (int rep = 0; rep < 6; ++rep) {
          cudaEventRecord(e0);
          probe<<<sms * cps, 256, mode == 4 ? W4 * 16 : 0>>>(in, out, rows, W4, den, mode);
          cudaEventRecord(e1);
          cudaEventSynchronize(e1);
          float ms;
          cudaEventElapsedTime(&ms, e0, e1);
          if (rep > 0 && ms < best) best = ms;
        }
      }
      const double kept = den <= 1 ? 1.0 : (double)(den - 1) / den;
      const double bytes = (double)rows * W4 * 16 * (1.0 + kept);
      printf("skip 1/%d %-20s %.3f ms  %.0f GB/s  (err %s)\n", den, names[mode], best, bytes / best / 1e6,
             cudaGetErrorString(cudaGetLastError()));
    }
  }
  return 0;
}
