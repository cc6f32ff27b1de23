// fold.cuh -- the row scheme's rebuild folded into the vertical pass.
//
// For the row scheme the rebuild (NN copy or LI, R6/R7) and every
// linear vertical filter of the apps (Gaussian taps, Sobel smoothing /
// derivative taps) act along y only, while the horizontal passes act within a
// row.  Both commute: H(rebuild(rows)) = rebuild(H(rows)).  So an output row q
// of a vertical filter f over rebuilt rows,
//     out(q) = sum_o f[o] * R(q + o),   R(r) = sum_k c(r, k) * K_k,
// is a fixed combination of the horizontal results of the KEPT rows K_k only:
//     out(q) = sum_k w(q, k) * H(K_k),  w(q, k) = sum_o f[o] * c(q + o, k).
// The weights depend only on q mod den (the kept rows are a lattice anchored to
// global row 0, R2), so they are compile-time constants per output phase.
// The kernel then runs the horizontal pass once per kept row (1/den of the
// rows), never materialises a skipped row, and each output is a 2-4 term
// paired FMA chain.  For integer-valued inputs every term and partial sum is an
// exact dyadic rational below 2^24 (weights are multiples of 1/den of integer
// taps), so the Gaussian / Sobel gradient outputs are bit-identical to
// rebuild-then-filter; in general they agree to fp32 rounding.
//
// Supported patterns: one kept row per period of den rows (den = 2, either
// form; den = 4 keep-one, the paper's Rows2), interior segments (no clamped
// rows, kernel.cuh); everything else keeps the per-row path.
#pragma once

namespace kp {

constexpr int kFoldT = 8;  // weight table covers kept rows t in [-kFoldT, kFoldT] relative to the output's period

struct FoldTab {
  float w[8][2 * kFoldT + 1];  // [phase][t + kFoldT]
  int tmin[8], tmax[8];
};

// weights of the vertical taps (rows q - VR .. q + VR) over kept rows, for
// outputs q = phase (period 0); kept rows are the multiples of DEN
template <int DEN, int RECON, int NT>
__host__ __device__ constexpr FoldTab fold_tab(const float (&taps)[NT]) {
  FoldTab T{};
  constexpr int VR = NT / 2;
  for (int ph = 0; ph < DEN; ++ph) {
    for (int i = 0; i < 2 * kFoldT + 1; ++i) T.w[ph][i] = 0.f;
    for (int o = -VR; o <= VR; ++o) {
      const int r = ph + o;
      const int ma = r >= 0 ? r / DEN : -((-r + DEN - 1) / DEN);  // floor(r / DEN): the kept row at or above r
      const int pr = r - ma * DEN;                                  // r's phase
      const float f = taps[o + VR];
      if (pr == 0) {
        T.w[ph][ma + kFoldT] += f;
      } else if (RECON == 1) {  // LI: (K_ma * db + K_ma+1 * da) / DEN
        const int da = pr, db = DEN - pr;
        T.w[ph][ma + kFoldT] += f * (float)db / (float)DEN;
        T.w[ph][ma + 1 + kFoldT] += f * (float)da / (float)DEN;
      } else {  // NN: the nearer kept row, ties to the lower coordinate (R6)
        const int da = pr, db = DEN - pr;
        T.w[ph][(da <= db ? ma : ma + 1) + kFoldT] += f;
      }
    }
  }
  return T;
}

// union of several filters' supports + the emission schedule
template <int DEN>
struct FoldSched {
  int tmin[8], tmax[8];
  int order[8];  // phases in emission order (ascending output row within one kept-row arrival)
  int span;      // max tmax - tmin + 1
};

template <int DEN>
__host__ __device__ constexpr FoldSched<DEN> fold_sched(const FoldTab* tabs, int ntab) {
  FoldSched<DEN> S{};
  S.span = 1;
  for (int ph = 0; ph < DEN; ++ph) {
    S.tmin[ph] = 99;
    S.tmax[ph] = -99;
    for (int k = 0; k < ntab; ++k)
      for (int t = -kFoldT; t <= kFoldT; ++t)
        if (tabs[k].w[ph][t + kFoldT] != 0.f) {
          if (t < S.tmin[ph]) S.tmin[ph] = t;
          if (t > S.tmax[ph]) S.tmax[ph] = t;
        }
    if (S.tmax[ph] - S.tmin[ph] + 1 > S.span) S.span = S.tmax[ph] - S.tmin[ph] + 1;
    S.order[ph] = ph;
  }
  // the output of phase ph completes when kept row tmax(ph) of its period arrives:
  // at arrival J it is row J*DEN - d(ph), d = tmax*DEN - ph; emit by descending d
  for (int i = 0; i < DEN; ++i)
    for (int j = i + 1; j < DEN; ++j) {
      const int di = S.tmax[S.order[i]] * DEN - S.order[i], dj = S.tmax[S.order[j]] * DEN - S.order[j];
      if (dj > di) {
        const int t = S.order[i];
        S.order[i] = S.order[j];
        S.order[j] = t;
      }
    }
  return S;
}

template <int DEN>
__host__ __device__ constexpr bool fold_sched_ok(const FoldSched<DEN>& S) {  // consecutive arrivals emit increasing, gap-free rows
  int dmin = 1 << 20, dmax = -(1 << 20);
  for (int ph = 0; ph < DEN; ++ph) {
    const int d = S.tmax[ph] * DEN - ph;
    dmin = d < dmin ? d : dmin;
    dmax = d > dmax ? d : dmax;
  }
  return dmax - dmin < DEN && S.span <= 8;
}

__host__ __device__ constexpr int fold_ring(int span) { return span <= 2 ? 2 : (span <= 4 ? 4 : 8); }

// ring slot of kept row (arrival U) + delta, in a ring of RK (compile time)
template <int RK>
__host__ __device__ constexpr int fold_slot(int U, int delta) {
  return ((U + delta) % RK + RK) % RK;
}

}  // namespace kp
