/*
 * synth_gen.cu -- host and device drivers for the seeded synthetic inputs of
 * synth.h.  Host functions are plain loops; device functions launch one
 * thread per pixel.  Both evaluate the same integer functions, so the images
 * are bit-identical (checked by tests/test_synth.py and the GPU tests).
 *
 * This library is input plumbing only: it contains none of the method's
 * arithmetic (no mask, reconstruction, stencil or error).
 */
#include "synth.h"
#include <cuda_runtime.h>
#include <stdint.h>

extern "C" {

/* ---- host ---------------------------------------------------------------- */
int synth_image_f32_host(int cls, unsigned long long seed, int W, int H, float* out) {
  for (int64_t y = 0; y < H; ++y)
    for (int64_t x = 0; x < W; ++x)
      out[y * W + x] = (float)synth_pixel(cls, seed, x, y, W, H);
  return 0;
}

int synth_image_u8_host(int cls, unsigned long long seed, int W, int H, uint8_t* out) {
  for (int64_t y = 0; y < H; ++y)
    for (int64_t x = 0; x < W; ++x)
      out[y * W + x] = (uint8_t)synth_pixel(cls, seed, x, y, W, H);
  return 0;
}

int synth_hotspot_host(unsigned long long seed, int W, int H, float* T, float* P) {
  for (int64_t y = 0; y < H; ++y)
    for (int64_t x = 0; x < W; ++x) {
      T[y * W + x] = (float)synth_hotspot_t64(seed, x, y) * (1.0f / 64.0f);
      P[y * W + x] = (float)synth_hotspot_p17(seed ^ 0xB0B0ull, x, y, W, H) * (1.0f / 131072.0f);
    }
  return 0;
}

/* ---- device -------------------------------------------------------------- */
}  // extern "C"

template <typename T>
__global__ void synth_image_kernel(int cls, unsigned long long seed0, int W, int H, int frames, T* out) {
  const int64_t n = (int64_t)W * H;
  const int64_t total = n * frames;
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < total;
       i += (int64_t)gridDim.x * blockDim.x) {
    const int64_t f = i / n, r = i - f * n;
    const int64_t y = r / W, x = r - y * W;
    out[i] = (T)synth_pixel(cls, seed0 + (unsigned long long)f, x, y, W, H);
  }
}

__global__ void synth_hotspot_kernel(unsigned long long seed, int W, int H, float* T, float* P) {
  const int64_t total = (int64_t)W * H;
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < total;
       i += (int64_t)gridDim.x * blockDim.x) {
    const int64_t y = i / W, x = i - y * W;
    T[i] = (float)synth_hotspot_t64(seed, x, y) * (1.0f / 64.0f);
    P[i] = (float)synth_hotspot_p17(seed ^ 0xB0B0ull, x, y, W, H) * (1.0f / 131072.0f);
  }
}

/* rows [y0, y0 + h) of the global H x W hotspot grid (band generation) */
__global__ void synth_hotspot_band_kernel(unsigned long long seed, int W, int H, int y0, int h,
                                          float* T, float* P) {
  const int64_t total = (int64_t)W * h;
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < total;
       i += (int64_t)gridDim.x * blockDim.x) {
    const int64_t yy = i / W, x = i - yy * W;
    const int64_t y = y0 + yy;
    T[i] = (float)synth_hotspot_t64(seed, x, y) * (1.0f / 64.0f);
    P[i] = (float)synth_hotspot_p17(seed ^ 0xB0B0ull, x, y, W, H) * (1.0f / 131072.0f);
  }
}

static int grid_for(int64_t total) {
  int64_t g = (total + 255) / 256;
  if (g > 148 * 64) g = 148 * 64;
  return (int)(g < 1 ? 1 : g);
}

extern "C" {

/* frames consecutive W x H images, frame f uses seed0 + f */
int synth_image_f32_device(int cls, unsigned long long seed0, int W, int H, int frames, float* out,
                           void* stream) {
  synth_image_kernel<float><<<grid_for((int64_t)W * H * frames), 256, 0, (cudaStream_t)stream>>>(
      cls, seed0, W, H, frames, out);
  return (int)cudaGetLastError();
}

int synth_image_u8_device(int cls, unsigned long long seed0, int W, int H, int frames, uint8_t* out,
                          void* stream) {
  synth_image_kernel<uint8_t><<<grid_for((int64_t)W * H * frames), 256, 0, (cudaStream_t)stream>>>(
      cls, seed0, W, H, frames, out);
  return (int)cudaGetLastError();
}

int synth_hotspot_device(unsigned long long seed, int W, int H, float* T, float* P, void* stream) {
  synth_hotspot_kernel<<<grid_for((int64_t)W * H), 256, 0, (cudaStream_t)stream>>>(seed, W, H, T, P);
  return (int)cudaGetLastError();
}

int synth_hotspot_band_device(unsigned long long seed, int W, int H, int y0, int h, float* T, float* P,
                              void* stream) {
  synth_hotspot_band_kernel<<<grid_for((int64_t)W * h), 256, 0, (cudaStream_t)stream>>>(seed, W, H, y0, h,
                                                                                       T, P);
  return (int)cudaGetLastError();
}

}  // extern "C"
