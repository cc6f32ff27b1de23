// k_gauss1.cu -- instantiations of the perforated stencil kernel for AppGauss<1>.
#include "kernel.cuh"
namespace kp {
cudaError_t launch_gauss1(int scheme, int recon, const KParams& p, unsigned grid, size_t smem, cudaStream_t s) {
  return launch_app<AppGauss<1>, kNCW>(scheme, recon, p, grid, smem, s);
}
cudaError_t launch_gauss1_n2(int scheme, int recon, const KParams& p, unsigned grid, size_t smem, cudaStream_t s) {
  return launch_app<AppGauss<1>, 2>(scheme, recon, p, grid, smem, s);
}
}  // namespace kp
