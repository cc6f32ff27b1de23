// k_hotspot.cu -- instantiations of the perforated stencil kernel for AppHotspot.
#include "kernel.cuh"
namespace kp {
cudaError_t launch_hotspot(int scheme, int recon, const KParams& p, unsigned grid, size_t smem, cudaStream_t s) {
  return launch_app<AppHotspot, kNCW>(scheme, recon, p, grid, smem, s);
}
}  // namespace kp
