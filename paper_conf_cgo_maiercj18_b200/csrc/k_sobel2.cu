// k_sobel2.cu -- instantiations of the perforated stencil kernel for AppSobel<2>.
#include "kernel.cuh"
namespace kp {
cudaError_t launch_sobel2(int scheme, int recon, const KParams& p, unsigned grid, size_t smem, cudaStream_t s) {
  return launch_app<AppSobel<2>, kNCW>(scheme, recon, p, grid, smem, s);
}
cudaError_t launch_sobel2_n2(int scheme, int recon, const KParams& p, unsigned grid, size_t smem, cudaStream_t s) {
  return launch_app<AppSobel<2>, 2>(scheme, recon, p, grid, smem, s);
}
}  // namespace kp
