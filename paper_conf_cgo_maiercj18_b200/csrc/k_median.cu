// k_median.cu -- instantiations of the perforated stencil kernel for AppMedian.
#include "kernel.cuh"
namespace kp {
cudaError_t launch_median(int scheme, int recon, const KParams& p, unsigned grid, size_t smem, cudaStream_t s) {
  return launch_app<AppMedian, kNCW>(scheme, recon, p, grid, smem, s);
}
}  // namespace kp
