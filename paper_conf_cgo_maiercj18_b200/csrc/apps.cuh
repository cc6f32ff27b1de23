// apps.cuh -- the unchanged application stencils (Sec. 6.1, :589-629),
// applied to the rebuilt rows as a register sliding window.
//
// Each App consumes one rebuilt input row per call: the lane's V samples `c`,
// the warp-edge fragment `e` (EW samples left of the warp for lanes < 16,
// right of it for lanes >= 16; already clamped at image borders) and, for
// Hotspot, the power row `c2`.  It returns the lane's V outputs of row
// (vy - VR).  Horizontal neighbours come from adjacent lanes by warp
// shuffles; lane 0 / lane 31 take them from `e`.  The vertical window is a
// ring of NWIN register rows indexed by the compile-time phase U, so the
// caller unrolls its row loop NWIN times and no register moves are needed.
// Border handling is clamp-to-edge on the rebuilt image (R8).
#pragma once
#include "engine.cuh"
#include "fold.cuh"

#ifndef KPERF_ULI
#define KPERF_ULI 0
#endif
#ifndef KPERF_IPROD
#define KPERF_IPROD 0  // inline producer (PERF_KEY_PRODUCER 2) compiled in: slower and a bigger hot loop
#endif
#ifndef KPERF_GS_ULI
#define KPERF_GS_ULI 1
#endif
#ifndef KPERF_FOLD_EDGE
#define KPERF_FOLD_EDGE 1  // Gaussian / Sobel: the frame's first / last segments fold too (kernel.cuh)
#endif
#ifndef KPERF_GS_IPROD
#define KPERF_GS_IPROD 0
#endif
#ifndef KPERF_GS_FOLD_ROT
#define KPERF_GS_FOLD_ROT 1  // folded C5 loop: one kept row per iteration, register ring shifted (I-cache)
#endif
#ifndef KPERF_GS_MINB
#define KPERF_GS_MINB 3  // fused pipeline: CTAs per SM the registers are budgeted for
#endif

namespace kp {

constexpr unsigned FULLMASK = 0xFFFFFFFFu;

// x[0 .. V+2RH): samples at columns xc-RH .. xc+V-1+RH of the rebuilt row
// hf: bit 0 / bit 1 = the lane's left / right edge is a Stencil1 tile border:
// the halo there is rebuilt by NN from the tile (the lane's own edge sample).
template <int RH, int EW, int V>
__device__ __forceinline__ void ext_row(const Frag<float, V>& c, const Frag<float, EW>& e, int lane, uint32_t hf,
                                        float (&x)[V + 2 * RH]) {
  static_assert(RH <= EW, "edge fragment too small");
#pragma unroll
  for (int i = 0; i < V; ++i) x[RH + i] = c.v[i];
#pragma unroll
  for (int k = 1; k <= RH; ++k) {
    float l = __shfl_up_sync(FULLMASK, c.v[V - k], 1);
    float r = __shfl_down_sync(FULLMASK, c.v[k - 1], 1);
    if (lane == 0) l = e.v[EW - k];
    if (lane == 31) r = e.v[k - 1];
    if (hf & 1u) l = c.v[0];
    if (hf & 2u) r = c.v[V - 1];
    x[RH - k] = l;
    x[RH + V - 1 + k] = r;
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

// the same passes on the output column pair (2j, 2j+1), x = &x[2j]: per column
// the operations and their order are those of smooth / deriv (bit-identical),
// issued as paired fp32 ops (FADD2 / FFMA2) where both operands sit in aligned
// register pairs -- x[2j] is aligned when R = 2 (x[R + i] = c.v[i]), x[2j + 1]
// when R = 1 -- and as scalar ops otherwise.  Gaussian5: 5 instructions per
// column pair instead of 8.
template <int R>
__device__ __forceinline__ f2 smooth_pair(const float* x) {
  if (R == 1) return fma2(splat2(2.f), pk2(x[1], x[2]), pk2(x[0] + x[2], x[1] + x[3]));
  const f2 a = add2(pk2(x[0], x[1]), pk2(x[4], x[5]));
  const f2 b = pk2(x[1] + x[3], x[2] + x[4]);
  return fma2(splat2(6.f), pk2(x[2], x[3]), fma2(splat2(4.f), b, a));
}
template <int R>
__device__ __forceinline__ f2 deriv_pair(const float* x) {
  if (R == 1) return pk2(x[2] - x[0], x[3] - x[1]);
  return fma2(splat2(2.f), pk2(x[3] - x[1], x[4] - x[2]), sub2(pk2(x[4], x[5]), pk2(x[0], x[1])));
}

// vertical taps of the folded apps (fold.cuh)
template <int R>
struct BinomTaps;  // binomial smoothing, optionally scaled
template <>
struct BinomTaps<1> {
  static constexpr float v[3] = {1.f, 2.f, 1.f};
  static constexpr float g[3] = {1.f / 16, 2.f / 16, 1.f / 16};  // Gaussian 3x3 incl. its 1/16
};
template <>
struct BinomTaps<2> {
  static constexpr float v[5] = {1.f, 4.f, 6.f, 4.f, 1.f};
  static constexpr float g[5] = {1.f / 256, 4.f / 256, 6.f / 256, 4.f / 256, 1.f / 256};
};
template <int R>
struct DerivTaps;
template <>
struct DerivTaps<1> {
  static constexpr float v[3] = {-1.f, 0.f, 1.f};
};
template <>
struct DerivTaps<2> {
  static constexpr float v[5] = {-1.f, -2.f, 0.f, 2.f, 1.f};
};

// output pair j of a folded row: sum over kept rows t of w(PH, t) * ring[slot(t)][j]
// (compile-time weights of table TAB, kept rows relative to the arrival U)
template <const FoldTab& TAB, int TMAX, int RK, int U, int PH, int NJ>
__device__ __forceinline__ f2 fold_dot(const f2 (&ring)[8][NJ], int j) {
  f2 acc = splat2(0.f);
  static_for<0, 2 * kFoldT + 1>([&](auto tc) {
    constexpr int t = decltype(tc)::value - kFoldT;
    constexpr float w = TAB.w[PH][t + kFoldT];
    if constexpr (w != 0.f) acc = fma2(splat2(w), ring[fold_slot<RK>(U, t - TMAX)][j], acc);
  });
  return acc;
}
template <const FoldTab& TAB, int TMAX, int RK, int U, int PH>
__device__ __forceinline__ float fold_dot1(const float (&ring)[8]) {
  float acc = 0.f;
  static_for<0, 2 * kFoldT + 1>([&](auto tc) {
    constexpr int t = decltype(tc)::value - kFoldT;
    constexpr float w = TAB.w[PH][t + kFoldT];
    if constexpr (w != 0.f) acc = fmaf(w, ring[fold_slot<RK>(U, t - TMAX)], acc);
  });
  return acc;
}

// ---------------------------------------------------------------------------
template <int R>
struct AppGauss {  // K1 Gaussian, binomial (2R+1)^2, fp32
  using T = float;
  static constexpr bool ULI = KPERF_ULI;
  static constexpr bool IPROD = KPERF_IPROD;
  static constexpr int V = 8, EW = 2, VR = R, NIN = 1, NWIN = 2 * R + 1, MINB = 4;
  f2 h[NWIN][V / 2];  // horizontal results, column pairs (FADD2/FFMA2 vertical pass)
  __device__ void init(const KParams&) {}
  // folded row scheme (fold.cuh): vertical binomial taps incl. the 1/16, 1/256 scale
  static constexpr bool FOLD = true, FOLD_ROT = false, FOLD_EDGE = KPERF_FOLD_EDGE;
  template <int DEN, int RECON>
  struct Fold {
    static constexpr FoldTab tab = fold_tab<DEN, RECON>(BinomTaps<R>::g);
    static constexpr FoldTab tabs[1] = {tab};
    static constexpr FoldSched<DEN> sch = fold_sched<DEN>(tabs, 1);
    static_assert(fold_sched_ok(sch), "fold schedule");
  };
  f2 fk[8][V / 2];  // kept rows' horizontal results, ring
  template <int S>
  __device__ __forceinline__ void fold_h(const Frag<float, V>& c, const Frag<float, EW>& e, int lane, uint32_t hf) {
    float x[V + 2 * R];
    ext_row<R, EW, V>(c, e, lane, hf, x);
#pragma unroll
    for (int j = 0; j < V / 2; ++j) fk[S][j] = smooth_pair<R>(x + 2 * j);
  }
  template <class F, int RK, int U, int PH, class Store>
  __device__ __forceinline__ void fold_emit(int q, int ys, int ye, int, int, const KParams&, Store&& st) {
    if (q < ys || q >= ye) return;
    Frag<float, V> o;
#pragma unroll
    for (int j = 0; j < V / 2; ++j)
      up2(fold_dot<F::tab, F::sch.tmax[PH], RK, U, PH, V / 2>(fk, j), o.v[2 * j], o.v[2 * j + 1]);
    st(o);
  }
  template <int U>
  __device__ __forceinline__ Frag<float, V> row(const Frag<float, V>& c, const Frag<float, EW>& e,
                                                const Frag<float, V>&, int lane, uint32_t hf, int, int, const KParams&) {
    float x[V + 2 * R];
    ext_row<R, EW, V>(c, e, lane, hf, x);
#pragma unroll
    for (int j = 0; j < V / 2; ++j) h[U][j] = smooth_pair<R>(x + 2 * j);
    const f2 scale = splat2(R == 1 ? 1.f / 16.f : 1.f / 256.f);
    Frag<float, V> o;
#pragma unroll
    for (int j = 0; j < V / 2; ++j) {
      f2 col[NWIN];
#pragma unroll
      for (int k = 0; k < NWIN; ++k) col[k] = h[(U + 1 + k) % NWIN][j];
      f2 v;
      if (R == 1) v = fma2(splat2(2.f), col[1], add2(col[0], col[2]));
      else v = fma2(splat2(6.f), col[2], fma2(splat2(4.f), add2(col[1], col[3]), add2(col[0], col[4])));
      up2(mul2(v, scale), o.v[2 * j], o.v[2 * j + 1]);
    }
    return o;
  }
};

template <int R>
struct AppSobel {  // K5 Sobel, |(Gx, Gy)|, fp32
  using T = float;
  static constexpr bool ULI = KPERF_ULI;
  static constexpr bool IPROD = KPERF_IPROD;
  static constexpr int V = 8, EW = 2, VR = R, NIN = 1, NWIN = 2 * R + 1, MINB = R == 1 ? 4 : 3;
  f2 sx[NWIN][V / 2], dx[NWIN][V / 2];  // horizontal smoothing / derivative, column pairs
  __device__ void init(const KParams&) {}
  // folded row scheme (fold.cuh): gx = vertical smoothing of dx, gy = vertical derivative of sx
  static constexpr bool FOLD = true, FOLD_ROT = false, FOLD_EDGE = KPERF_FOLD_EDGE;
  template <int DEN, int RECON>
  struct Fold {
    static constexpr FoldTab tx = fold_tab<DEN, RECON>(BinomTaps<R>::v);
    static constexpr FoldTab ty = fold_tab<DEN, RECON>(DerivTaps<R>::v);
    static constexpr FoldTab tabs[2] = {tx, ty};
    static constexpr FoldSched<DEN> sch = fold_sched<DEN>(tabs, 2);
    static_assert(fold_sched_ok(sch), "fold schedule");
  };
  f2 fs[8][V / 2], fd[8][V / 2];  // kept rows' horizontal smoothing / derivative, ring
  template <int S>
  __device__ __forceinline__ void fold_h(const Frag<float, V>& c, const Frag<float, EW>& e, int lane, uint32_t hf) {
    float x[V + 2 * R];
    ext_row<R, EW, V>(c, e, lane, hf, x);
#pragma unroll
    for (int j = 0; j < V / 2; ++j) {
      fs[S][j] = smooth_pair<R>(x + 2 * j);
      fd[S][j] = deriv_pair<R>(x + 2 * j);
    }
  }
  template <class F, int RK, int U, int PH, class Store>
  __device__ __forceinline__ void fold_emit(int q, int ys, int ye, int, int, const KParams&, Store&& st) {
    if (q < ys || q >= ye) return;
    Frag<float, V> o;
#pragma unroll
    for (int j = 0; j < V / 2; ++j) {
      const f2 gx = fold_dot<F::tx, F::sch.tmax[PH], RK, U, PH, V / 2>(fd, j);
      const f2 gy = fold_dot<F::ty, F::sch.tmax[PH], RK, U, PH, V / 2>(fs, j);
      float m0, m1;
      up2(fma2(gx, gx, mul2(gy, gy)), m0, m1);
      o.v[2 * j] = sqrt_approx(m0);
      o.v[2 * j + 1] = sqrt_approx(m1);
    }
    st(o);
  }
  template <int U>
  __device__ __forceinline__ Frag<float, V> row(const Frag<float, V>& c, const Frag<float, EW>& e,
                                                const Frag<float, V>&, int lane, uint32_t hf, int, int, const KParams&) {
    float x[V + 2 * R];
    ext_row<R, EW, V>(c, e, lane, hf, x);
#pragma unroll
    for (int j = 0; j < V / 2; ++j) {
      sx[U][j] = smooth_pair<R>(x + 2 * j);
      dx[U][j] = deriv_pair<R>(x + 2 * j);
    }
    Frag<float, V> o;
#pragma unroll
    for (int j = 0; j < V / 2; ++j) {
      f2 cs[NWIN], cd[NWIN];
#pragma unroll
      for (int k = 0; k < NWIN; ++k) {
        cs[k] = sx[(U + 1 + k) % NWIN][j];
        cd[k] = dx[(U + 1 + k) % NWIN][j];
      }
      f2 gx, gy;  // gx: vertical smoothing of the derivative; gy: vertical derivative of the smoothing
      if (R == 1) {
        gx = fma2(splat2(2.f), cd[1], add2(cd[0], cd[2]));
        gy = sub2(cs[2], cs[0]);
      } else {
        gx = fma2(splat2(6.f), cd[2], fma2(splat2(4.f), add2(cd[1], cd[3]), add2(cd[0], cd[4])));
        gy = fma2(splat2(2.f), sub2(cs[3], cs[1]), sub2(cs[4], cs[0]));
      }
      float m0, m1;
      up2(fma2(gx, gx, mul2(gy, gy)), m0, m1);
      o.v[2 * j] = sqrt_approx(m0);
      o.v[2 * j + 1] = sqrt_approx(m1);
    }
    return o;
  }
};

struct AppInversion {  // K2 Inversion, 255 - x
  using T = float;
  static constexpr bool ULI = KPERF_ULI;
  static constexpr bool IPROD = KPERF_IPROD;
  static constexpr int V = 8, EW = 2, VR = 0, NIN = 1, NWIN = 1, MINB = 4;
  static constexpr bool FOLD = false, FOLD_ROT = false, FOLD_EDGE = false;
  __device__ void init(const KParams&) {}
  template <int U>
  __device__ __forceinline__ Frag<float, V> row(const Frag<float, V>& c, const Frag<float, EW>&,
                                                const Frag<float, V>&, int, uint32_t, int, int, const KParams&) {
    Frag<float, V> o;
#pragma unroll
    for (int i = 0; i < V; ++i) o.v[i] = 255.f - c.v[i];
    return o;
  }
};

// ---------------------------------------------------------------------------
// K4 Hotspot (Rodinia 2D transient thermal step), T and P rebuilt alike.
struct AppHotspot {
  using T = float;
  static constexpr bool ULI = KPERF_ULI;
  static constexpr bool IPROD = KPERF_IPROD;
  static constexpr int V = 8, EW = 2, VR = 1, NIN = 2, NWIN = 3, MINB = 4;
  static constexpr bool FOLD = false, FOLD_ROT = false, FOLD_EDGE = false;
  float tc[3][V], tl[3], tr[3], pc[3][V];
  float sdc, rx1, ry1, rz1, amb;
  __device__ void init(const KParams& p) {
    sdc = p.sdc;
    rx1 = p.rx1;
    ry1 = p.ry1;
    rz1 = p.rz1;
    amb = p.amb;
  }
  template <int U>
  __device__ __forceinline__ Frag<float, V> row(const Frag<float, V>& c, const Frag<float, EW>& e,
                                                const Frag<float, V>& c2, int lane, uint32_t, int, int, const KParams&) {
    float x[V + 2];
    ext_row<1, EW, V>(c, e, lane, 0u, x);
#pragma unroll
    for (int i = 0; i < V; ++i) {
      tc[U][i] = x[i + 1];
      pc[U][i] = c2.v[i];
    }
    tl[U] = x[0];
    tr[U] = x[V + 1];
    constexpr int M = (U + 2) % 3, O = (U + 1) % 3;  // middle (output) row, oldest row
    Frag<float, V> o;
#pragma unroll
    for (int i = 0; i < V; ++i) {
      const float t = tc[M][i], ts = tc[U][i], tn = tc[O][i];
      const float tw = i == 0 ? tl[M] : tc[M][i - 1];
      const float te = i == V - 1 ? tr[M] : tc[M][i + 1];
      o.v[i] = t + sdc * (pc[M][i] + (ts + tn - 2.0f * t) * ry1 + (te + tw - 2.0f * t) * rx1 + (amb - t) * rz1);
    }
    return o;
  }
};

// ---------------------------------------------------------------------------
// Gaussian5 -> Sobel3 fused (the C5 pipeline).  The Gaussian rows stay in
// registers; Sobel clamps in the Gaussian image (G(-1) = G(0), G(W) = G(W-1),
// rows alike, R12).  Input row vy completes Gaussian row gy = vy - 2
// and Sobel output row oy = vy - 3.
//  * vertical Gaussian: transposed form -- each horizontal result h_r is added
//    into the four Gaussian rows in flight (G_{r-1} += 4h, G_r += 6h,
//    G_{r+1} += 4h) and completes G_{r-2} (+= h); G_{r+2} starts as h.  Four
//    accumulator rows, slot q % 4 for Gaussian row q: no 5-row ring of h;
//  * Sobel: per Gaussian row q its horizontal smoothing s_q and derivative d_q
//    (column pairs); rings of two (slot q % 2 holds q and q - 2), output row
//    q - 1: gx = d_{q-2} + 2 d_{q-1} + d_q, gy = s_q - s_{q-2}; the top / bottom
//    clamps (row q - 2 -> q - 1 at oy = 0, row q -> q - 1 at oy = H - 1) are
//    warp-uniform coefficients of the same three paired FMAs -- no per-column
//    selects, no register shifts (the former t0/t1/t2 rows cost 20 selects and
//    20 moves per row).
// NWIN = 4: the unrolled row loop is 4 rows; every ring index is compile time.
// Arithmetic order differs from the oracle's (fp64) sum order: parity is the
// north_star 1e-5 relative tolerance (+ the Sobel absolute floor).
struct AppGaussSobel {
  using T = float;
  static constexpr bool ULI = KPERF_GS_ULI;  // uniform row LI (engine.cuh rebuild_frag)
  static constexpr bool IPROD = KPERF_GS_IPROD;  // 0: PERF_KEY_PRODUCER 2 ignored (a smaller consumer loop, I-cache)
  static constexpr int V = 8, EW = 4, VR = 3, NIN = 1, NWIN = 4, MINB = KPERF_GS_MINB;
  f2 acc[4][V / 2];  // Gaussian rows in flight (x 256), lane columns, pairs; slot q % 4
  float acce[4];     // the same for the lane's edge column (xc - 1 / xc + V)
  f2 sr[2][V / 2], dr[2][V / 2];  // Sobel horizontal smoothing / derivative of Gaussian rows, slot q % 2
  // folded row scheme (fold.cuh): Gaussian rows from the kept rows' horizontal
  // results (the Gaussian taps over rebuilt rows folded into kept-row weights);
  // the Sobel stage then runs on every Gaussian row as above (interior rows:
  // no top / bottom clamp)
  // (FOLD_EDGE off: the Sobel stage's clamp in the Gaussian image at the frame's
  // first / last row would cost a branch per folded emission; those two
  // segments per frame take the per-row loop and are dispatched first, kernel.cuh)
  static constexpr bool FOLD = true, FOLD_ROT = KPERF_GS_FOLD_ROT, FOLD_EDGE = false;
  template <int DEN, int RECON>
  struct Fold {
    static constexpr FoldTab tab = fold_tab<DEN, RECON>(BinomTaps<2>::g);
    static constexpr FoldTab tabs[1] = {tab};
    static constexpr FoldSched<DEN> sch = fold_sched<DEN>(tabs, 1);
    static_assert(fold_sched_ok(sch), "fold schedule");
  };
  f2 fk[8][V / 2];  // kept rows' horizontal Gaussian, ring
  float fke[8];     // ... of the lane's edge column
  f2 gr[2][V / 2];  // folded loop: Gaussian rows q - 2, q - 1 (slot q % 2), lane columns
  float grh[2][2];  // ... and their halo columns xc - 1, xc + V
  template <int S>
  __device__ __forceinline__ void fold_h(const Frag<float, V>& c, const Frag<float, EW>& e, int lane, uint32_t) {
    float x[V + 4];
    ext_row<2, EW, V>(c, e, lane, 0u, x);
#pragma unroll
    for (int j = 0; j < V / 2; ++j) fk[S][j] = smooth_pair<2>(x + 2 * j);
    float t[5];
    if (lane < 16) { t[0] = e.v[1]; t[1] = e.v[2]; t[2] = e.v[3]; t[3] = c.v[0]; t[4] = c.v[1]; }
    else { t[0] = c.v[V - 2]; t[1] = c.v[V - 1]; t[2] = e.v[0]; t[3] = e.v[1]; t[4] = e.v[2]; }
    fke[S] = smooth<2>(t);
  }
  template <int RK>
  __device__ __forceinline__ void fold_rotate() {  // FOLD_ROT: kept row k + 1 -> ring position k
#pragma unroll
    for (int k = 0; k + 1 < RK; ++k) {
      fke[k] = fke[k + 1];
#pragma unroll
      for (int j = 0; j < V / 2; ++j) fk[k][j] = fk[k + 1][j];
    }
  }
  // Gaussian row q; Sobel output row q - 1 stored when ys <= q - 1 < ye.  The
  // rings advance on every emission, in range or not (values outside the
  // segment are never stored): no range branch around the ring updates, so no
  // predicated copies of the ring at the join
  template <class F, int RK, int U, int PH, class Store>
  __device__ __forceinline__ void fold_emit(int q, int ys, int ye, int lane, int xc, const KParams& p, Store&& st) {
    constexpr int SQ = PH % 2, SM = (PH + 1) % 2;  // ring slots of Gaussian rows q - 2 (then q), q - 1 (DEN even)
    float g[V + 2];
#pragma unroll
    for (int j = 0; j < V / 2; ++j)
      up2(fold_dot<F::tab, F::sch.tmax[PH], RK, U, PH, V / 2>(fk, j), g[2 * j + 1], g[2 * j + 2]);
    const float gve = fold_dot1<F::tab, F::sch.tmax[PH], RK, U, PH>(fke);
    float gl = __shfl_up_sync(FULLMASK, g[V], 1);
    float gright = __shfl_down_sync(FULLMASK, g[1], 1);
    if (lane == 0) gl = gve;
    if (lane == 31) gright = gve;
    g[0] = gl;
    g[V + 1] = gright;
    if (xc <= 0) g[0] = g[1];
    const int cl = p.W - 1 - xc;
    if (cl < V) {
#pragma unroll
      for (int k = 1; k < V + 2; ++k) g[k] = k > cl + 1 ? g[k - 1] : g[k];
    }
    // vertical first on the Gaussian rows (linear until the magnitude):
    // S = G(q-2) + 2 G(q-1) + G(q), D = G(q) - G(q-2) on columns -1 .. V;
    // gx = horizontal derivative of S, gy = horizontal smoothing of D.  The
    // ring holds Gaussian rows (V + 2 values) instead of the smoothing and
    // derivative rows (2 V): 12 fewer live registers in the folded loop
    // (interior segments only: no clamp of the Sobel stage, FOLD_EDGE off)
    float S[V + 2], D[V + 2];
#pragma unroll
    for (int j = 0; j < V / 2; ++j) {
      const f2 gp = pk2(g[2 * j + 1], g[2 * j + 2]);
      up2(fma2(splat2(2.f), gr[SM][j], add2(gr[SQ][j], gp)), S[2 * j + 1], S[2 * j + 2]);
      up2(sub2(gp, gr[SQ][j]), D[2 * j + 1], D[2 * j + 2]);
    }
#pragma unroll
    for (int h = 0; h < 2; ++h) {
      const int k = h ? V + 1 : 0;
      S[k] = fmaf(2.f, grh[SM][h], grh[SQ][h] + g[k]);
      D[k] = g[k] - grh[SQ][h];
    }
#pragma unroll
    for (int j = 0; j < V / 2; ++j) gr[SQ][j] = pk2(g[2 * j + 1], g[2 * j + 2]);
    grh[SQ][0] = g[0];
    grh[SQ][1] = g[V + 1];
    Frag<float, V> o;
#pragma unroll
    for (int j = 0; j < V / 2; ++j) {
      const f2 gx = deriv_pair<1>(S + 2 * j), gy = smooth_pair<1>(D + 2 * j);
      float m0, m1;
      up2(fma2(gx, gx, mul2(gy, gy)), m0, m1);
      o.v[2 * j] = sqrt_approx(m0);
      o.v[2 * j + 1] = sqrt_approx(m1);
    }
    if (q >= ys + 1 && q <= ye) st(o);
  }
  __device__ void init(const KParams&) {
#pragma unroll
    for (int k = 0; k < 4; ++k) {
      acce[k] = 0.f;
#pragma unroll
      for (int j = 0; j < V / 2; ++j) acc[k][j] = splat2(0.f);
    }
#pragma unroll
    for (int k = 0; k < 2; ++k) {
#pragma unroll
      for (int j = 0; j < V / 2; ++j) sr[k][j] = dr[k][j] = gr[k][j] = splat2(0.f);
      grh[k][0] = grh[k][1] = 0.f;
    }
  }
  template <int U>
  __device__ __forceinline__ Frag<float, V> row(const Frag<float, V>& c, const Frag<float, EW>& e,
                                                const Frag<float, V>&, int lane, uint32_t, int vy, int xc,
                                                const KParams& p) {
    constexpr int Q = (U + 2) % 4, M1 = (U + 3) % 4, P1 = (U + 1) % 4;  // slots of rows r-2 (done), r-1, r+1
    constexpr int SQ = U % 2, SM = (U + 1) % 2;  // Sobel slots: Gaussian rows q (and q - 2), q - 1
    float x[V + 4];  // columns xc-2 .. xc+V+1
    ext_row<2, EW, V>(c, e, lane, 0u, x);
    float he;  // edge column (lane 0: xc-1 from e = cols xc-4..xc-1; lane 31: xc+V from e = cols xc+V..xc+V+3)
    {
      float t[5];
      if (lane < 16) { t[0] = e.v[1]; t[1] = e.v[2]; t[2] = e.v[3]; t[3] = c.v[0]; t[4] = c.v[1]; }
      else { t[0] = c.v[V - 2]; t[1] = c.v[V - 1]; t[2] = e.v[0]; t[3] = e.v[1]; t[4] = e.v[2]; }
      he = smooth<2>(t);
    }
    // vertical Gaussian, transposed: h completes row r-2, feeds r-1, r, r+1, starts r+2
    float g[V + 2];  // Gaussian row gy = vy - 2 at columns xc-1 .. xc+V
    const f2 sc = splat2(1.f / 256.f);
#pragma unroll
    for (int j = 0; j < V / 2; ++j) {
      const f2 h = smooth_pair<2>(x + 2 * j);
      up2(mul2(add2(acc[Q][j], h), sc), g[2 * j + 1], g[2 * j + 2]);
      acc[M1][j] = fma2(splat2(4.f), h, acc[M1][j]);
      acc[U][j] = fma2(splat2(6.f), h, acc[U][j]);
      acc[P1][j] = fma2(splat2(4.f), h, acc[P1][j]);
      acc[Q][j] = h;
    }
    const float gve = (acce[Q] + he) * (1.f / 256.f);
    acce[M1] = fmaf(4.f, he, acce[M1]);
    acce[U] = fmaf(6.f, he, acce[U]);
    acce[P1] = fmaf(4.f, he, acce[P1]);
    acce[Q] = he;
    float gl = __shfl_up_sync(FULLMASK, g[V], 1);
    float gright = __shfl_down_sync(FULLMASK, g[1], 1);
    if (lane == 0) gl = gve;
    if (lane == 31) gright = gve;
    g[0] = gl;
    g[V + 1] = gright;
    // clamp in the Gaussian image: columns < 0 -> column 0, columns >= W -> column W-1
    if (xc <= 0) g[0] = g[1];
    const int cl = p.W - 1 - xc;  // local index of column W-1
    if (cl < V) {  // propagate column W-1 rightwards (prefix selects: no indexed register access)
#pragma unroll
      for (int k = 1; k < V + 2; ++k) g[k] = k > cl + 1 ? g[k - 1] : g[k];
    }
    // Sobel3 on Gaussian rows oy-1, oy, oy+1 (oy = vy - 3 = gy - 1); clamp coefficients (warp uniform)
    // (rows away from the image's first / last row -- all but two per frame --
    // take the plain form: a warp-uniform branch, no per-row coefficient work)
    const int oy = vy - 3;
    const bool edge = oy <= 0 || oy >= p.Hg - 1;
    f2 sq[V / 2], dq[V / 2], gx[V / 2], gy[V / 2];
#pragma unroll
    for (int j = 0; j < V / 2; ++j) {
      sq[j] = smooth_pair<1>(g + 2 * j);
      dq[j] = deriv_pair<1>(g + 2 * j);
    }
    if (!edge) {
#pragma unroll
      for (int j = 0; j < V / 2; ++j) {
        gx[j] = fma2(splat2(2.f), dr[SM][j], add2(dr[SQ][j], dq[j]));
        gy[j] = sub2(sq[j], sr[SQ][j]);
      }
    } else {
      const float top = oy == 0 ? 1.f : 0.f, bot = oy == p.Hg - 1 ? 1.f : 0.f;
      const f2 kt = splat2(1.f - top), kb = splat2(1.f - bot), km = splat2(2.f + top + bot);
      const f2 kst = splat2(top - 1.f), ksm = splat2(bot - top);
#pragma unroll
      for (int j = 0; j < V / 2; ++j) {
        gx[j] = fma2(km, dr[SM][j], fma2(kt, dr[SQ][j], mul2(kb, dq[j])));
        gy[j] = fma2(kb, sq[j], fma2(ksm, sr[SM][j], mul2(kst, sr[SQ][j])));
      }
    }
    Frag<float, V> o;
#pragma unroll
    for (int j = 0; j < V / 2; ++j) {
      sr[SQ][j] = sq[j];
      dr[SQ][j] = dq[j];
      float m0, m1;
      up2(fma2(gx[j], gx[j], mul2(gy[j], gy[j])), m0, m1);
      o.v[2 * j] = sqrt_approx(m0);
      o.v[2 * j + 1] = sqrt_approx(m1);
    }
    return o;
  }
};

// ---------------------------------------------------------------------------
// K3 Median 3x3, u8: column sort of the 3-row window, then
// med9 = med3(max of column minima, med3 of column medians, min of column maxima)
// on packed 16-bit lanes, 2 pixels per instruction.  A lane holds 0x6400|v:
// as u16 it orders like v (VIMNMX.U16x2, ALU pipe) and as fp16 it is exactly
// 1024+v (HMNMX2), so the two instruction kinds can share the work
// (KPERF_MEDIAN_MODE: 0 VIMNMX only, 1 HMNMX2 only, 2 alternate by word).
#ifndef KPERF_MEDIAN_MODE
#define KPERF_MEDIAN_MODE 2
#endif
template <int K>
__device__ __forceinline__ uint32_t mn2(uint32_t a, uint32_t b) {
  if (KPERF_MEDIAN_MODE == 1 || (KPERF_MEDIAN_MODE == 2 && (K & 1))) return hmin2u(a, b);
  return vmin2(a, b);
}
template <int K>
__device__ __forceinline__ uint32_t mx2(uint32_t a, uint32_t b) {
  if (KPERF_MEDIAN_MODE == 1 || (KPERF_MEDIAN_MODE == 2 && (K & 1))) return hmax2u(a, b);
  return vmax2(a, b);
}

struct AppMedian {
  using T = uint8_t;
  static constexpr bool ULI = KPERF_ULI;
  static constexpr bool IPROD = KPERF_IPROD;
  // MINB 4 (96 registers): 4 CTAs / SM.  The column scheme's all-skipped warps
  // (kernel.cuh MEDC) leave the kept warps as the critical path; more resident
  // CTAs hide their latency (C3 col 1/2 NN 235 -> 196 us, exact 230 -> 228 us)
  static constexpr int V = 16, EW = 4, VR = 1, NIN = 1, NWIN = 3, MINB = 4;
  static constexpr bool FOLD = false, FOLD_ROT = false, FOLD_EDGE = false;
  static constexpr int NW = V / 2 + 2;  // 16-bit-pair words per row incl. the two halo words
  uint32_t r[3][NW];  // word 0 = (_, col -1), words 1..V/2 = cols 0..V-1, last = (col V, _)
  __device__ void init(const KParams&) {}
  template <int K>
  __device__ __forceinline__ static uint32_t med3(uint32_t a, uint32_t b, uint32_t c) {
    return mx2<K>(mn2<K>(a, b), mn2<K>(mx2<K>(a, b), c));
  }
  template <int U>
  __device__ __forceinline__ Frag<uint8_t, V> row(const Frag<uint8_t, V>& c, const Frag<uint8_t, EW>& e,
                                                  const Frag<uint8_t, V>&, int lane, uint32_t hf, int, int,
                                                  const KParams&) {
    constexpr uint32_t HI = 0x64646464u;  // fp16 exponent byte of 1024
    uint32_t lft = __shfl_up_sync(FULLMASK, c.w[V / 4 - 1], 1);
    uint32_t rgt = __shfl_down_sync(FULLMASK, c.w[0], 1);
    if (hf & 4u) lft = e.w[0];  // lane's left / right neighbour column lies in its edge fragment
    if (hf & 8u) rgt = e.w[0];  // (lane 0 / 31; the first / last lane of a cell under cell-grouped lanes)
    if (hf & 1u) lft = c.w[0] << 24;           // Stencil1 tile border: col -1 := col 0
    if (hf & 2u) rgt = c.w[V / 4 - 1] >> 24;  // col V := col V-1
    r[U][0] = __byte_perm(lft, HI, 0x4344);  // (0x6464, 0x64|col -1)
#pragma unroll
    for (int k = 0; k < V / 4; ++k) {
      r[U][1 + 2 * k] = __byte_perm(c.w[k], HI, 0x4140);
      r[U][2 + 2 * k] = __byte_perm(c.w[k], HI, 0x4342);
    }
    r[U][NW - 1] = __byte_perm(rgt, HI, 0x4440);  // (0x64|col V, 0x6464)
    constexpr int A = (U + 1) % 3, B = (U + 2) % 3;
    uint32_t lo[NW], md[NW], hi[NW];
    static_for<0, NW>([&](auto kc) {
      constexpr int k = decltype(kc)::value;
      const uint32_t t1 = mn2<k>(r[A][k], r[B][k]), t2 = mx2<k>(r[A][k], r[B][k]);
      lo[k] = mn2<k>(t1, r[U][k]);
      const uint32_t t3 = mx2<k>(t1, r[U][k]);
      md[k] = mn2<k>(t2, t3);
      hi[k] = mx2<k>(t2, t3);
    });
    uint32_t sl[NW - 1], sm[NW - 1], sh[NW - 1];  // shifted by one column: (col 2k-1, col 2k) at [k]
#pragma unroll
    for (int k = 0; k < NW - 1; ++k) {
      sl[k] = __byte_perm(lo[k], lo[k + 1], 0x5432);
      sm[k] = __byte_perm(md[k], md[k + 1], 0x5432);
      sh[k] = __byte_perm(hi[k], hi[k + 1], 0x5432);
    }
    uint32_t out[V / 2];
    static_for<0, V / 2>([&](auto kc) {
      constexpr int k = decltype(kc)::value;
      const uint32_t mx = mx2<k>(mx2<k>(sl[k], lo[k + 1]), sl[k + 1]);
      const uint32_t mn = mn2<k>(mn2<k>(sh[k], hi[k + 1]), sh[k + 1]);
      const uint32_t mm = med3<k>(sm[k], md[k + 1], sm[k + 1]);
      out[k] = med3<k + 1>(mx, mm, mn);
    });
    Frag<uint8_t, V> o;
#pragma unroll
    for (int k = 0; k < V / 4; ++k) o.w[k] = __byte_perm(out[2 * k], out[2 * k + 1], 0x6420);
    return o;
  }
};

}  // namespace kp
