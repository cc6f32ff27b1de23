// kernel.cuh -- the perforated stencil kernel template and its launcher.
// See engine.cuh for the design; apps.cuh for the stencil stages.
#pragma once
#include <cuda_runtime.h>

#include "apps.cuh"
#include "engine.cuh"

namespace kp {

template <class App, int SCHEME, int RECON, int NCW>
__global__ void __launch_bounds__(32 * (NCW + 1)) perf_kernel(const __grid_constant__ KParams p) {
  using T = typename App::T;
  using VTT = VT<T>;
  using Vec = typename VTT::Vec;
  constexpr int V = VTT::V;
  constexpr int TW = NCW * 32 * V;
  extern __shared__ __align__(128) uint8_t smem[];
  uint64_t* full = reinterpret_cast<uint64_t*>(smem);
  uint64_t* empty = full + p.nr;
  T* ring = reinterpret_cast<T*>(smem + ((2 * p.nr * 8 + 127) & ~127));
  const int slot_elems = p.row_elems * App::NIN;

  int b = blockIdx.x;
  const int strip = b % p.n_strips;
  b /= p.n_strips;
  const int seg = b % p.n_segs;
  const int frame = b / p.n_segs;
  const int x0 = strip * TW;
  const int ys = p.y_begin + seg * p.seg_h;
  const int ye = min(ys + p.seg_h, p.y_end);
  const Mask m{p.num, p.den, p.keep_one};
  const RowPlan rp = make_row_plan<SCHEME>(p, m, ys, ye, App::VR);
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;

  if (threadIdx.x == 0) {
    for (int s = 0; s < p.nr; ++s) {
      mbar_init(&full[s], p.loader == L_BULK ? 1u : 32u);
      mbar_init(&empty[s], (uint32_t)NCW);
    }
    mbar_fence_init();
  }
  __syncthreads();

  if (warp == 0) {  // (Ia) data perforation: only kept samples leave HBM
    producer<T, SCHEME, App::NIN, NCW>(p, m, rp, x0, frame, full, empty, ring);
    return;
  }

  // ---------------- consumers: (Ib) reconstruction + kernel execution -------
  const int w = warp - 1;
  const int xw = x0 + w * 32 * V;
  const int base = x0 - p.hx;
  const int xc = xw + lane * V;
  const ChunkInfo cc = make_chunk<SCHEME>(p, m, xc, V);
  const ChunkInfo ce = make_chunk<SCHEME>(p, m, lane < 16 ? xw - V : xw + 32 * V, V);
  App app;
  app.init(p);
  T* outp = static_cast<T*>(p.out) + (long long)frame * p.out_fstride;
  const int nmask = p.nr - 1;

  int ready = -1, released = 0;
  int y_prev = -1, ym = 0, yq = 0;
  for (int vy = ys - App::VR; vy < ye + App::VR; ++vy) {
    const int y = clampi(vy, rp.lim_lo, rp.lim_hi);
    if (y != y_prev) {  // y % den and y / den, incrementally
      if (y_prev >= 0 && y == y_prev + 1) {
        if (++ym == m.den) { ym = 0; ++yq; }
      } else {
        ym = y % m.den;
        yq = y / m.den;
      }
      y_prev = y;
    }
    RowCtx rc;
    rc.y = y;
    rc.ym = ym;
    rc.kept = 1;
    rc.has_a = rc.has_b = 0;
    rc.da = rc.db = 1;
    rc.slot_a = rc.slot_b = 0;
    int need_hi, need_lo;
    if (SCHEME == S_ROW) {
      rc.kept = m.phase_kept(ym);
      if (rc.kept) {
        const int id = (m.keep_one ? yq : yq * (m.den - 1) + ym) - rp.ord_lo;
        rc.slot_c = id & nmask;
        need_hi = need_lo = id;
      } else {
        rc.da = m.dlo(ym);
        rc.db = m.dhi(ym);
        rc.has_a = (y - rc.da) >= rp.lim_lo && (y - rc.da) >= rp.lo;
        rc.has_b = (y + rc.db) <= rp.lim_hi && (y + rc.db) <= rp.hi;
        const int ida = (m.keep_one ? yq : yq * (m.den - 1) + m.den - 2) - rp.ord_lo;
        const int idb = (m.keep_one ? yq + 1 : (yq + 1) * (m.den - 1)) - rp.ord_lo;
        rc.slot_a = ida & nmask;
        rc.slot_b = idb & nmask;
        rc.slot_c = rc.slot_a;
        need_hi = rc.has_b ? idb : ida;
        need_lo = rc.has_a ? ida : idb;
      }
    } else if (SCHEME == S_CHECKER) {
      rc.slot_c = (y - rp.lo) & nmask;
      need_hi = min(y + m.den - 1, rp.hi) - rp.lo;
      need_lo = max(y - (m.den - 1), rp.lo) - rp.lo;
    } else {
      rc.slot_c = (y - rp.lo) & nmask;
      need_hi = need_lo = y - rp.lo;
    }
    // release ring slots no consumer row will read again, then wait for the rows needed now
    if (released < need_lo) {
      __syncwarp();
      for (; released < need_lo; ++released)
        if (lane == 0) mbar_arrive(&empty[released & nmask]);
    }
    for (; ready < need_hi;) {
      ++ready;
      mbar_wait(&full[ready & nmask], (ready >> p.nr_log2) & 1);
    }
    const Vec c = rebuild_chunk<T, SCHEME, RECON>(p, m, rp, rc, cc, ring, slot_elems, base, 0);
    const Vec e = rebuild_chunk<T, SCHEME, RECON>(p, m, rp, rc, ce, ring, slot_elems, base, 0);
    Vec c2;
    if (App::NIN > 1) c2 = rebuild_chunk<T, SCHEME, RECON>(p, m, rp, rc, cc, ring, slot_elems, base, p.row_elems);
    else c2 = c;
    const Vec o = app.row(c, e, c2, lane, vy, xc, p);
    const int yo = vy - App::VR;
    if (yo >= ys && xc < p.W) {  // kernel execution result -> output buffer
      T* dst = outp + (long long)(yo - p.out_row0) * p.W + xc;
      if (p.vec_io && xc + V <= p.W) {
        const uint4 u = *reinterpret_cast<const uint4*>(&o);
        st_global_v4(dst, u.x, u.y, u.z, u.w);
      } else {
#pragma unroll
        for (int i = 0; i < V; ++i)
          if (xc + i < p.W) dst[i] = VTT::get(o, i);
      }
    }
  }
  // every issued copy must land before the CTA retires
  for (; ready < rp.nload - 1;) {
    ++ready;
    mbar_wait(&full[ready & nmask], (ready >> p.nr_log2) & 1);
  }
}

template <class App, int SCHEME, int RECON, int NCW>
cudaError_t launch_one(const KParams& p, unsigned grid, size_t smem, cudaStream_t s) {
  auto k = perf_kernel<App, SCHEME, RECON, NCW>;
  static bool attr = false;
  if (!attr) {
    cudaError_t e = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, 227 * 1024);
    if (e != cudaSuccess) return e;
    attr = true;
  }
  k<<<grid, 32 * (NCW + 1), smem, s>>>(p);
  return cudaGetLastError();
}

template <class App, int NCW>
cudaError_t launch_app(int scheme, int recon, const KParams& p, unsigned grid, size_t smem, cudaStream_t s) {
  switch (scheme * 2 + recon) {
    case S_NONE * 2 + R_NN:
    case S_NONE * 2 + R_LI: return launch_one<App, S_NONE, R_NN, NCW>(p, grid, smem, s);
    case S_ROW * 2 + R_NN: return launch_one<App, S_ROW, R_NN, NCW>(p, grid, smem, s);
    case S_ROW * 2 + R_LI: return launch_one<App, S_ROW, R_LI, NCW>(p, grid, smem, s);
    case S_COL * 2 + R_NN: return launch_one<App, S_COL, R_NN, NCW>(p, grid, smem, s);
    case S_COL * 2 + R_LI: return launch_one<App, S_COL, R_LI, NCW>(p, grid, smem, s);
    case S_CHECKER * 2 + R_NN: return launch_one<App, S_CHECKER, R_NN, NCW>(p, grid, smem, s);
    case S_CHECKER * 2 + R_LI: return launch_one<App, S_CHECKER, R_LI, NCW>(p, grid, smem, s);
  }
  return cudaErrorInvalidValue;
}

// per-app launchers (one translation unit each, compiled in parallel)
cudaError_t launch_gauss1(int, int, const KParams&, unsigned, size_t, cudaStream_t);
cudaError_t launch_gauss2(int, int, const KParams&, unsigned, size_t, cudaStream_t);
cudaError_t launch_sobel1(int, int, const KParams&, unsigned, size_t, cudaStream_t);
cudaError_t launch_sobel2(int, int, const KParams&, unsigned, size_t, cudaStream_t);
cudaError_t launch_median(int, int, const KParams&, unsigned, size_t, cudaStream_t);
cudaError_t launch_hotspot(int, int, const KParams&, unsigned, size_t, cudaStream_t);
cudaError_t launch_gsobel(int, int, const KParams&, unsigned, size_t, cudaStream_t);
cudaError_t launch_inversion(int, int, const KParams&, unsigned, size_t, cudaStream_t);

constexpr int kNCW = 4;  // consumer warps per CTA (tile width 512 fp32 / 2048 u8 columns)

}  // namespace kp
