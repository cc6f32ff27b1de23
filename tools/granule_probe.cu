// granule_probe.cu -- which skipped stride actually saves DRAM bytes?
// Reads every other chunk of S bytes (S = 16..512) of a 1 GiB buffer;
// ncu's dram__bytes_read.sum / bytes requested tells the fill granule.
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>
__global__ void probe(const uint4* __restrict__ in, unsigned long long n16, int chunk16, unsigned* sink) {
  unsigned acc = 0;
  for (unsigned long long i = blockIdx.x * (unsigned long long)blockDim.x + threadIdx.x; i < n16;
       i += (unsigned long long)gridDim.x * blockDim.x) {
    if (((i / chunk16) & 1) == 0) { uint4 v = in[i]; acc ^= v.x ^ v.y ^ v.z ^ v.w; }
  }
  if (acc == 0x12345678u) sink[0] = acc;
}
int main() {
  const size_t bytes = 1ull << 30;
  uint4* d; unsigned* s;
  cudaMalloc(&d, bytes); cudaMalloc(&s, 4); cudaMemset(d, 1, bytes);
  for (int c = 1; c <= 32; c *= 2) {
    probe<<<148 * 16, 256>>>(d, bytes / 16, c, s);
    cudaDeviceSynchronize();
    printf("chunk %d B launched\n", c * 16);
  }
  return 0;
}
