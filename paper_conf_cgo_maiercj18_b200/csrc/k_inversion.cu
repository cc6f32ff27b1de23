// k_inversion.cu -- instantiations of the perforated stencil kernel for AppInversion.
#include "kernel.cuh"
namespace kp {
cudaError_t launch_inversion(int scheme, int recon, const KParams& p, unsigned grid, size_t smem, cudaStream_t s) {
  return launch_app<AppInversion, kNCW>(scheme, recon, p, grid, smem, s);
}
}  // namespace kp
