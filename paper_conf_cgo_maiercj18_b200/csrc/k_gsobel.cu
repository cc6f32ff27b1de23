// k_gsobel.cu -- instantiations of the perforated stencil kernel for AppGaussSobel.
#include "kernel.cuh"
namespace kp {
cudaError_t launch_gsobel(int scheme, int recon, const KParams& p, unsigned grid, size_t smem, cudaStream_t s) {
  return launch_app<AppGaussSobel, kNCW>(scheme, recon, p, grid, smem, s);
}
cudaError_t launch_gsobel_n3(int scheme, int recon, const KParams& p, unsigned grid, size_t smem, cudaStream_t s) {
  return launch_app<AppGaussSobel, 3>(scheme, recon, p, grid, smem, s);
}
}  // namespace kp
