// tma_probe.cu -- standalone check of the tensor-tile maps libkperf's TMA cell
// loader encodes (column runs; every den-th cell by traversal stride), outside
// the kernel, on a synthetic ramp image.  nvcc -arch=sm_100a tma_probe.cu -o tma_probe
#include <cuda.h>
#include <cudaTypedefs.h>
#include <cuda_runtime.h>

#include <cstdio>
#include <vector>

__device__ __forceinline__ unsigned su32(const void* p) { return (unsigned)__cvta_generic_to_shared(p); }

__global__ void probe(const __grid_constant__ CUtensorMap tm, int c0, int c1, int c2, int bytes, float* out) {
  __shared__ __align__(128) float buf[8192];
  __shared__ __align__(8) unsigned long long bar;
  if (threadIdx.x == 0) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(su32(&bar)));
    asm volatile("fence.mbarrier_init.release.cluster;");
  }
  __syncthreads();
  if (threadIdx.x == 0) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(su32(&bar)), "r"(bytes));
    asm volatile(
        "cp.async.bulk.tensor.3d.shared::cluster.global.tile.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3, %4}], [%5];" ::"r"(
            su32(buf)),
        "l"(reinterpret_cast<unsigned long long>(&tm)), "r"(c0), "r"(c1), "r"(c2), "r"(su32(&bar))
        : "memory");
  }
  unsigned ok = 0;
  while (!ok)
    asm volatile("{\n .reg .pred p;\n mbarrier.try_wait.parity.shared::cta.b64 p, [%1], 0;\n selp.u32 %0, 1, 0, p;\n}"
                 : "=r"(ok)
                 : "r"(su32(&bar)));
  for (int i = threadIdx.x; i < bytes / 4; i += blockDim.x) out[i] = buf[i];
}

int main() {
  const int W = 2048, H = 16;
  std::vector<float> h(W * H);
  for (int i = 0; i < W * H; ++i) h[i] = (float)i;
  float *d, *o;
  cudaMalloc(&d, W * H * 4);
  cudaMalloc(&o, 8192 * 4);
  cudaMemcpy(d, h.data(), W * H * 4, cudaMemcpyHostToDevice);
  void* f = nullptr;
  cudaDriverEntryPointQueryResult q;
  cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &f, cudaEnableDefault, &q);
  auto enc = reinterpret_cast<PFN_cuTensorMapEncodeTiled_v12000>(f);
  struct Case {
    const char* name;
    cuuint64_t dims[3], strides[2];
    cuuint32_t box[3], es[3];
    int c0, c1, c2, nelem;
  };
  const int G = 32;
  Case cases[] = {
      {"col runs den2", {32, (cuuint64_t)W / 64, H}, {64 * 4, (cuuint64_t)W * 4}, {32, 18, 1}, {1, 1, 1}, 0, -1, 3, 32 * 18},
      {"stride-2 cells", {32, (cuuint64_t)W / 32, H}, {32 * 4, (cuuint64_t)W * 4}, {32, 36, 1}, {1, 2, 1}, 0, -2, 3, 32 * 18},
      {"stride-2 cells start 1", {32, (cuuint64_t)W / 32, H}, {32 * 4, (cuuint64_t)W * 4}, {32, 36, 1}, {1, 2, 1}, 0, 1, 3, 32 * 18},
      {"stride-1 cells", {32, (cuuint64_t)W / 32, H}, {32 * 4, (cuuint64_t)W * 4}, {32, 18, 1}, {1, 1, 1}, 0, 1, 3, 32 * 18},
  };
  for (auto& c : cases) {
    CUtensorMap tm;
    CUresult r = enc(&tm, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 3, d, c.dims, c.strides, c.box, c.es,
                     CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_128B,
                     CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    cudaMemset(o, 0xff, 8192 * 4);
    probe<<<1, 128>>>(tm, c.c0, c.c1, c.c2, c.nelem * 4, o);
    cudaError_t e = cudaDeviceSynchronize();
    std::vector<float> got(c.nelem);
    cudaMemcpy(got.data(), o, c.nelem * 4, cudaMemcpyDeviceToHost);
    printf("%-24s encode %d launch %s  first cells:", c.name, (int)r, cudaGetErrorString(e));
    for (int k = 0; k < 4; ++k) printf(" [%g]", got[k * G]);
    printf("\n");
    if (e != cudaSuccess) return 1;
  }
  return 0;
}
