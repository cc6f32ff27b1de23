/*
 * synth.h -- seeded synthetic inputs shared by the oracle side and the CUDA
 * side (the ONLY code both sides share).  It holds none of the method's
 * arithmetic: no perforation mask, no reconstruction, no stencil, no error.
 *
 * Everything is integer arithmetic on a counter-based hash (splitmix64), so a
 * host build (gcc) and a device build (nvcc) produce bit-identical images.
 * The recipe mirrors the paper's three input kinds
 * -- flat regions, photographs, high-frequency patterns (PAPER.md:790-800,
 * Sec. 6.2, Fig. 7) -- and Rodinia Hotspot's temperature/power grids
 * (Sec. 6.1).
 *
 * Pixel values are integers in [8, 247] (8-bit grayscale).
 * Hotspot T0 = 323 + m/64 K (|m| <= 960) and P = sum of k/2^17 W terms, all
 * exactly representable in fp32.
 */
#ifndef KPERF_SYNTH_H
#define KPERF_SYNTH_H

#include <stdint.h>

#if defined(__CUDACC__)
#define SYNTH_HD __host__ __device__ __forceinline__
#else
#define SYNTH_HD static inline
#endif

enum { SYNTH_FLAT = 0, SYNTH_NATURAL = 1, SYNTH_PATTERN = 2 };

SYNTH_HD uint64_t synth_mix64(uint64_t z) {
  z += 0x9E3779B97F4A7C15ull;
  z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
  z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
  return z ^ (z >> 31);
}

SYNTH_HD uint64_t synth_hash(uint64_t seed, uint64_t a, uint64_t b, uint64_t c) {
  return synth_mix64(seed ^ synth_mix64(a ^ synth_mix64(b ^ synth_mix64(c + 0x51ED270B27ull))));
}

/* uniform integer in [0, n) (n > 0); bias is irrelevant here */
SYNTH_HD int64_t synth_uniform(uint64_t seed, uint64_t a, uint64_t b, uint64_t c, int64_t n) {
  return (int64_t)(synth_hash(seed, a, b, c) % (uint64_t)n);
}

/* value-noise fBm, 6 octaves, cells 256..8 px, amplitude halved per octave.
 * Returns roughly [-2^17, 2^17] (sum of 6 bilinear lattice interpolations). */
SYNTH_HD int64_t synth_fbm(uint64_t seed, int64_t x, int64_t y) {
  int64_t acc = 0;
  for (int o = 0; o < 6; ++o) {
    const int s = 8 - o;                 /* log2 cell size */
    const int64_t cs = (int64_t)1 << s;
    const int64_t i = x >> s, j = y >> s;
    const int64_t fx = x & (cs - 1), fy = y & (cs - 1);
    const int64_t l00 = (int64_t)(synth_hash(seed, 100 + o, i, j) & 0xFFFF) - 32768;
    const int64_t l10 = (int64_t)(synth_hash(seed, 100 + o, i + 1, j) & 0xFFFF) - 32768;
    const int64_t l01 = (int64_t)(synth_hash(seed, 100 + o, i, j + 1) & 0xFFFF) - 32768;
    const int64_t l11 = (int64_t)(synth_hash(seed, 100 + o, i + 1, j + 1) & 0xFFFF) - 32768;
    int64_t v = l00 * (cs - fx) * (cs - fy) + l10 * fx * (cs - fy) + l01 * (cs - fx) * fy + l11 * fx * fy;
    v = v >> (2 * s);                    /* arithmetic shift: floor division */
    acc += v >> o;
  }
  return acc;
}

/* one geometric step edge (half-plane, disc or rectangle); returns the level
 * offset it adds at (x, y), 0 outside.  k indexes the edge. */
SYNTH_HD int64_t synth_edge(uint64_t seed, int k, int64_t x, int64_t y, int64_t W, int64_t H,
                            int64_t lo, int64_t hi) {
  const int64_t type = synth_uniform(seed, 200, (uint64_t)k, 0, 3);
  const int64_t mag = lo + synth_uniform(seed, 201, (uint64_t)k, 0, hi - lo + 1);
  const int64_t off = synth_uniform(seed, 202, (uint64_t)k, 0, 2) ? mag : -mag;
  const int64_t px = synth_uniform(seed, 203, (uint64_t)k, 0, W);
  const int64_t py = synth_uniform(seed, 204, (uint64_t)k, 0, H);
  if (type == 0) { /* half-plane through (px, py) with integer normal (a, b) */
    const int64_t a = synth_uniform(seed, 205, (uint64_t)k, 0, 129) - 64;
    const int64_t b = synth_uniform(seed, 206, (uint64_t)k, 0, 129) - 64;
    return (a * (x - px) + b * (y - py) > 0) ? off : 0;
  } else if (type == 1) { /* disc */
    const int64_t m = (W < H ? W : H);
    const int64_t rad = 1 + synth_uniform(seed, 207, (uint64_t)k, 0, m / 4 + 1);
    const int64_t dx = x - px, dy = y - py;
    return (dx * dx + dy * dy < rad * rad) ? off : 0;
  } else { /* rectangle */
    const int64_t rw = 1 + synth_uniform(seed, 208, (uint64_t)k, 0, W / 3 + 1);
    const int64_t rh = 1 + synth_uniform(seed, 209, (uint64_t)k, 0, H / 3 + 1);
    return (x >= px && x < px + rw && y >= py && y < py + rh) ? off : 0;
  }
}

SYNTH_HD int64_t synth_clamp_px(int64_t v) { return v < 8 ? 8 : (v > 247 ? 247 : v); }

/* triangle wave of period p (p >= 2), amplitude in [0, 2*(p/2)] scaled to [-1, 1]*amp */
SYNTH_HD int64_t synth_tri(int64_t t, int64_t p, int64_t amp) {
  int64_t ph = t % p; if (ph < 0) ph += p;
  const int64_t half = p / 2 > 0 ? p / 2 : 1;
  const int64_t tri = ph <= half ? ph : p - ph;       /* 0..half */
  return (2 * tri - half) * amp / half;
}

/* Pixel value of class cls at (x, y) of a W x H image; integer in [8, 247]. */
SYNTH_HD int synth_pixel(int cls, uint64_t seed, int64_t x, int64_t y, int64_t W, int64_t H) {
  int64_t v;
  if (cls == SYNTH_FLAT) {
    const int n = 4 + (int)synth_uniform(seed, 1, 0, 0, 5);
    v = 96 + synth_uniform(seed, 2, 0, 0, 65);
    for (int k = 0; k < n; ++k) v += synth_edge(seed, k, x, y, W, H, 20, 80);
  } else if (cls == SYNTH_NATURAL) {
    v = 128 + ((synth_fbm(seed, x, y) * 90) >> 17);
    const int n = 16 + (int)synth_uniform(seed, 1, 0, 0, 49);
    for (int k = 0; k < n; ++k) v += synth_edge(seed, k, x, y, W, H, 20, 60);
    v += synth_uniform(seed, 3, (uint64_t)x, (uint64_t)y, 5) - 2;
  } else {
    /* 4x4 blocks, each a grating / checker texture of period 2..6 */
    const int64_t bx = (x * 4) / (W > 0 ? W : 1), by = (y * 4) / (H > 0 ? H : 1);
    const uint64_t blk = (uint64_t)(by * 4 + bx);
    const int64_t kind = synth_uniform(seed, 4, blk, 0, 4);
    const int64_t p = 2 + synth_uniform(seed, 5, blk, 0, 5);
    const int64_t amp = 40 + synth_uniform(seed, 6, blk, 0, 61);
    v = 128;
    if (kind == 0) v += synth_tri(x, p, amp);
    else if (kind == 1) v += synth_tri(y, p, amp);
    else if (kind == 2) v += synth_tri(x + y, p, amp);
    else v += (((x / p) + (y / p)) & 1) ? amp : -amp;
    v += synth_uniform(seed, 3, (uint64_t)x, (uint64_t)y, 5) - 2;
  }
  return (int)synth_clamp_px(v);
}

/* Hotspot initial temperature in 1/64 K above 0: T0 = 323 + m/64 with |m| <= 960. */
SYNTH_HD int64_t synth_hotspot_t64(uint64_t seed, int64_t x, int64_t y) {
  int64_t m = (synth_fbm(seed, x, y) * 960) >> 17;
  if (m > 960) m = 960;
  if (m < -960) m = -960;
  return 323 * 64 + m;
}

/* Hotspot power in units of 2^-17: sum over 64 random rectangles covering (x,y)
 * of a density k in [0, 1024] (so P <= 64 * 1024 / 2^17 = 0.5, typically
 * one or two rectangles overlap: P ~ 0.0078 * U[0,1]). */
SYNTH_HD int64_t synth_hotspot_p17(uint64_t seed, int64_t x, int64_t y, int64_t W, int64_t H) {
  int64_t acc = 0;
  for (int k = 0; k < 64; ++k) {
    const int64_t rx = synth_uniform(seed, 300, (uint64_t)k, 0, W);
    const int64_t ry = synth_uniform(seed, 301, (uint64_t)k, 0, H);
    const int64_t rw = 1 + synth_uniform(seed, 302, (uint64_t)k, 0, W / 4 + 1);
    const int64_t rh = 1 + synth_uniform(seed, 303, (uint64_t)k, 0, H / 4 + 1);
    if (x >= rx && x < rx + rw && y >= ry && y < ry + rh)
      acc += synth_uniform(seed, 304, (uint64_t)k, 0, 1025);
  }
  return acc;
}

#endif /* KPERF_SYNTH_H */
