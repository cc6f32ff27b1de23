// apps.cuh -- the unchanged application stencils (Sec. 6.1, :589-629),
// applied to the rebuilt rows as a register sliding window.
//
// Each App consumes one rebuilt input row per call (the lane's V samples `c`,
// its warp-edge chunk `e`, and for Hotspot the power row `c2`) and produces the
// lane's V outputs of row (vy - VR).  Horizontal neighbours come from the
// adjacent lanes by warp shuffles; lane 0 / lane 31 take them from `e`.
// Border handling is clamp-to-edge on the rebuilt image (R8).
#pragma once
#include "engine.cuh"

namespace kp {

constexpr unsigned FULLMASK = 0xFFFFFFFFu;

__device__ __forceinline__ float f4(const float4& v, int i) { return VT<float>::get(v, i); }

// x[0 .. 4+2RH): samples at columns xc-RH .. xc+3+RH of the rebuilt row
template <int RH>
__device__ __forceinline__ void ext_row(const float4& c, const float4& e, int lane, float (&x)[4 + 2 * RH]) {
#pragma unroll
  for (int i = 0; i < 4; ++i) x[RH + i] = f4(c, i);
#pragma unroll
  for (int k = 1; k <= RH; ++k) {
    float l = __shfl_up_sync(FULLMASK, f4(c, 4 - k), 1);
    float r = __shfl_down_sync(FULLMASK, f4(c, k - 1), 1);
    if (lane == 0) l = f4(e, 4 - k);
    if (lane == 31) r = f4(e, k - 1);
    x[RH - k] = l;
    x[RH + 3 + k] = r;
  }
}

// binomial taps [1,2,1] / [1,4,6,4,1] and derivative taps [-1,0,1] / [-1,-2,0,2,1]
template <int R>
__device__ __forceinline__ float smooth(const float* x) {
  if (R == 1) return fmaf(2.f, x[1], x[0] + x[2]);
  return fmaf(6.f, x[2], fmaf(4.f, x[1] + x[3], x[0] + x[4]));
}
template <int R>
__device__ __forceinline__ float deriv(const float* x) {
  if (R == 1) return x[2] - x[0];
  return fmaf(2.f, x[3] - x[1], x[4] - x[0]);
}

// ---------------------------------------------------------------------------
template <int R>
struct AppGauss {  // K1 Gaussian, binomial (2R+1)^2, fp32
  using T = float;
  static constexpr int VR = R, NIN = 1;
  float h[2 * R + 1][4];
  __device__ void init(const KParams&) {}
  __device__ __forceinline__ float4 row(const float4& c, const float4& e, const float4&, int lane, int, int,
                                        const KParams&) {
    float x[4 + 2 * R];
    ext_row<R>(c, e, lane, x);
#pragma unroll
    for (int k = 0; k < 2 * R; ++k)
#pragma unroll
      for (int i = 0; i < 4; ++i) h[k][i] = h[k + 1][i];
#pragma unroll
    for (int i = 0; i < 4; ++i) h[2 * R][i] = smooth<R>(x + i);
    constexpr float scale = R == 1 ? 1.f / 16.f : 1.f / 256.f;
    float o[4];
#pragma unroll
    for (int i = 0; i < 4; ++i) {
      float col[2 * R + 1];
#pragma unroll
      for (int k = 0; k <= 2 * R; ++k) col[k] = h[k][i];
      o[i] = smooth<R>(col) * scale;
    }
    return make_float4(o[0], o[1], o[2], o[3]);
  }
};

template <int R>
struct AppSobel {  // K5 Sobel, |(Gx, Gy)|, fp32
  using T = float;
  static constexpr int VR = R, NIN = 1;
  float sx[2 * R + 1][4], dx[2 * R + 1][4];
  __device__ void init(const KParams&) {}
  __device__ __forceinline__ float4 row(const float4& c, const float4& e, const float4&, int lane, int, int,
                                        const KParams&) {
    float x[4 + 2 * R];
    ext_row<R>(c, e, lane, x);
#pragma unroll
    for (int k = 0; k < 2 * R; ++k)
#pragma unroll
      for (int i = 0; i < 4; ++i) { sx[k][i] = sx[k + 1][i]; dx[k][i] = dx[k + 1][i]; }
#pragma unroll
    for (int i = 0; i < 4; ++i) { sx[2 * R][i] = smooth<R>(x + i); dx[2 * R][i] = deriv<R>(x + i); }
    float o[4];
#pragma unroll
    for (int i = 0; i < 4; ++i) {
      float cs[2 * R + 1], cd[2 * R + 1];
#pragma unroll
      for (int k = 0; k <= 2 * R; ++k) { cs[k] = sx[k][i]; cd[k] = dx[k][i]; }
      const float gx = smooth<R>(cd);  // vertical smoothing of the horizontal derivative
      const float gy = deriv<R>(cs);   // vertical derivative of the horizontal smoothing
      o[i] = sqrtf(fmaf(gx, gx, gy * gy));
    }
    return make_float4(o[0], o[1], o[2], o[3]);
  }
};

struct AppInversion {  // K2 Inversion, 255 - x
  using T = float;
  static constexpr int VR = 0, NIN = 1;
  __device__ void init(const KParams&) {}
  __device__ __forceinline__ float4 row(const float4& c, const float4&, const float4&, int, int, int,
                                        const KParams&) {
    return make_float4(255.f - c.x, 255.f - c.y, 255.f - c.z, 255.f - c.w);
  }
};

// ---------------------------------------------------------------------------
// K4 Hotspot (Rodinia 2D transient thermal step), T and P rebuilt alike.
struct AppHotspot {
  using T = float;
  static constexpr int VR = 1, NIN = 2;
  float tn[4], tc[6], pc[4];  // row vy-2 (centre), row vy-1 (centre + W/E halo), power of row vy-1
  float sdc, rx1, ry1, rz1, amb;
  __device__ void init(const KParams& p) { sdc = p.sdc; rx1 = p.rx1; ry1 = p.ry1; rz1 = p.rz1; amb = p.amb; }
  __device__ __forceinline__ float4 row(const float4& c, const float4& e, const float4& c2, int lane, int, int,
                                        const KParams&) {
    float x[6];
    ext_row<1>(c, e, lane, x);
    float o[4];
#pragma unroll
    for (int i = 0; i < 4; ++i) {
      const float t = tc[i + 1], ts = x[i + 1], tN = tn[i], te = tc[i + 2], tw = tc[i];
      o[i] = t + sdc * (pc[i] + (ts + tN - 2.0f * t) * ry1 + (te + tw - 2.0f * t) * rx1 + (amb - t) * rz1);
    }
#pragma unroll
    for (int i = 0; i < 4; ++i) { tn[i] = tc[i + 1]; pc[i] = f4(c2, i); }
#pragma unroll
    for (int i = 0; i < 6; ++i) tc[i] = x[i];
    return make_float4(o[0], o[1], o[2], o[3]);
  }
};

// ---------------------------------------------------------------------------
// Gaussian5 -> Sobel3 fused (the C5 pipeline).  The Gaussian row stays in
// registers; Sobel clamps in the Gaussian image (G(-1) = G(0), G(W) = G(W-1)).
struct AppGaussSobel {
  using T = float;
  static constexpr int VR = 3, NIN = 1;
  float h[5][5];             // horizontal Gaussian of the last 5 input rows: 4 lane columns + 1 edge column
  float gs[3][6];            // last 3 Gaussian rows, lane columns -1..4
  __device__ void init(const KParams&) {}
  __device__ __forceinline__ void push_g(const float (&g)[6]) {
#pragma unroll
    for (int k = 0; k < 2; ++k)
#pragma unroll
      for (int i = 0; i < 6; ++i) gs[k][i] = gs[k + 1][i];
#pragma unroll
    for (int i = 0; i < 6; ++i) gs[2][i] = g[i];
  }
  __device__ __forceinline__ float4 row(const float4& c, const float4& e, const float4&, int lane, int vy,
                                        int xc, const KParams& p) {
    float x[4 + 4];  // columns xc-2 .. xc+5
    ext_row<2>(c, e, lane, x);
    // edge column: lanes < 16 -> xw - 1 (from e = xw-4..xw-1 and c), lanes >= 16 -> xw + 32*4 (e = next 4)
    // only lane 0 / lane 31 use it; both are computed from e and the lane's own c.
    float he;
    if (lane < 16) {  // column xc-1 for lane 0: samples xc-3 .. xc+1
      float t[5] = {f4(e, 1), f4(e, 2), f4(e, 3), f4(c, 0), f4(c, 1)};
      he = smooth<2>(t);
    } else {          // column xc+4 for lane 31: samples xc+2 .. xc+6
      float t[5] = {f4(c, 2), f4(c, 3), f4(e, 0), f4(e, 1), f4(e, 2)};
      he = smooth<2>(t);
    }
#pragma unroll
    for (int k = 0; k < 4; ++k)
#pragma unroll
      for (int i = 0; i < 5; ++i) h[k][i] = h[k + 1][i];
#pragma unroll
    for (int i = 0; i < 4; ++i) h[4][i] = smooth<2>(x + i);
    h[4][4] = he;
    float gv[5];
#pragma unroll
    for (int i = 0; i < 5; ++i) {
      float col[5];
#pragma unroll
      for (int k = 0; k < 5; ++k) col[k] = h[k][i];
      gv[i] = smooth<2>(col) * (1.f / 256.f);
    }
    // Gaussian row gy = vy - 2 at columns xc-1 .. xc+4
    float g[6];
#pragma unroll
    for (int i = 0; i < 4; ++i) g[i + 1] = gv[i];
    float gl = __shfl_up_sync(FULLMASK, gv[3], 1);
    float gr = __shfl_down_sync(FULLMASK, gv[0], 1);
    if (lane == 0) gl = gv[4];
    if (lane == 31) gr = gv[4];
    g[0] = gl;
    g[5] = gr;
    // clamp in the Gaussian image: columns < 0 -> column 0, columns >= W -> column W-1
    if (xc <= 0) g[0] = g[1];
    const int cl = p.W - 1 - xc;  // local index of column W-1
    if (cl < 4) {
      float gw = g[0];
#pragma unroll
      for (int k = 0; k < 5; ++k) if (k == cl + 1) gw = g[k];
#pragma unroll
      for (int k = 1; k < 6; ++k) if (k > cl + 1) g[k] = gw;
    }
    // rows: G(-1) = G(0), G(H) = G(H-1)
    const int gy = vy - 2;
    if (gy == 0) { push_g(g); push_g(g); }
    else if (gy > 0 && gy < p.Hg) push_g(g);
    else if (gy >= p.Hg) { float last[6];
#pragma unroll
      for (int i = 0; i < 6; ++i) last[i] = gs[2][i];
      push_g(last); }
    else if (gy < -1) push_g(g);  // warm-up (shifted out before use)
    float o[4];
#pragma unroll
    for (int i = 0; i < 4; ++i) {
      const float d0 = gs[0][i + 2] - gs[0][i], d1 = gs[1][i + 2] - gs[1][i], d2 = gs[2][i + 2] - gs[2][i];
      const float gx = fmaf(2.f, d1, d0 + d2);
      const float s0 = fmaf(2.f, gs[0][i + 1], gs[0][i] + gs[0][i + 2]);
      const float s2 = fmaf(2.f, gs[2][i + 1], gs[2][i] + gs[2][i + 2]);
      const float gyv = s2 - s0;
      o[i] = sqrtf(fmaf(gx, gx, gyv * gyv));
    }
    return make_float4(o[0], o[1], o[2], o[3]);
  }
};

// ---------------------------------------------------------------------------
// K3 Median 3x3, u8: column sort of the 3-row window, then
// med9 = med3(max of column minima, med3 of column medians, min of column maxima)
// on packed u16x2 lanes (VIMNMX.U16x2), 2 pixels per instruction.
struct AppMedian {
  using T = uint8_t;
  static constexpr int VR = 1, NIN = 1;
  uint32_t r0[10], r1[10];  // previous two rows: word -1 (col -1 in the high half), words 0..7, word 8 (col 16 low)
  __device__ void init(const KParams&) {}
  __device__ __forceinline__ static uint32_t med3(uint32_t a, uint32_t b, uint32_t c) {
    return vmax2(vmin2(a, b), vmin2(vmax2(a, b), c));
  }
  __device__ __forceinline__ uint4 row(const uint4& c, const uint4& e, const uint4&, int lane, int, int,
                                       const KParams&) {
    uint32_t lft = __shfl_up_sync(FULLMASK, c.w, 1);
    uint32_t rgt = __shfl_down_sync(FULLMASK, c.x, 1);
    if (lane == 0) lft = e.w;
    if (lane == 31) rgt = e.x;
    uint32_t r2[10];
    r2[0] = __byte_perm(lft, 0, 0x4344);  // byte 3 -> high half: (0, col -1)
    const uint32_t cw[4] = {c.x, c.y, c.z, c.w};
#pragma unroll
    for (int k = 0; k < 4; ++k) {
      r2[1 + 2 * k] = __byte_perm(cw[k], 0, 0x4140);
      r2[2 + 2 * k] = __byte_perm(cw[k], 0, 0x4342);
    }
    r2[9] = __byte_perm(rgt, 0, 0x4440);  // byte 0 -> low half: (col 16, 0)
    // column sort of rows (r0, r1, r2) per word
    uint32_t lo[10], md[10], hi[10];
#pragma unroll
    for (int k = 0; k < 10; ++k) {
      const uint32_t t1 = vmin2(r0[k], r1[k]), t2 = vmax2(r0[k], r1[k]);
      lo[k] = vmin2(t1, r2[k]);
      const uint32_t t3 = vmax2(t1, r2[k]);
      md[k] = vmin2(t2, t3);
      hi[k] = vmax2(t2, t3);
    }
    // shifted-by-one-column words S_k = (col 2k+1, col 2k+2), k = -1..7 stored at [k+1]
    uint32_t out[8];
#pragma unroll
    for (int k = 0; k < 8; ++k) {
      const uint32_t ll = __byte_perm(lo[k], lo[k + 1], 0x5432), lr = __byte_perm(lo[k + 1], lo[k + 2], 0x5432);
      const uint32_t ml = __byte_perm(md[k], md[k + 1], 0x5432), mr = __byte_perm(md[k + 1], md[k + 2], 0x5432);
      const uint32_t hl = __byte_perm(hi[k], hi[k + 1], 0x5432), hr = __byte_perm(hi[k + 1], hi[k + 2], 0x5432);
      const uint32_t mx = vmax2(vmax2(ll, lo[k + 1]), lr);
      const uint32_t mn = vmin2(vmin2(hl, hi[k + 1]), hr);
      const uint32_t mm = med3(ml, md[k + 1], mr);
      out[k] = med3(mx, mm, mn);
    }
#pragma unroll
    for (int k = 0; k < 10; ++k) { r0[k] = r1[k]; r1[k] = r2[k]; }
    return make_uint4(__byte_perm(out[0], out[1], 0x6420), __byte_perm(out[2], out[3], 0x6420),
                      __byte_perm(out[4], out[5], 0x6420), __byte_perm(out[6], out[7], 0x6420));
  }
};

}  // namespace kp
