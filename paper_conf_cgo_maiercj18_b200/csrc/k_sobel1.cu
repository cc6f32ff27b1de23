// k_sobel1.cu -- instantiations of the perforated stencil kernel for AppSobel<1>.
#include "kernel.cuh"
namespace kp {
cudaError_t launch_sobel1(int scheme, int recon, const KParams& p, unsigned grid, size_t smem, cudaStream_t s) {
  return launch_app<AppSobel<1>, kNCW>(scheme, recon, p, grid, smem, s);
}
cudaError_t launch_sobel1_n2(int scheme, int recon, const KParams& p, unsigned grid, size_t smem, cudaStream_t s) {
  return launch_app<AppSobel<1>, 2>(scheme, recon, p, grid, smem, s);
}
}  // namespace kp
