// engine.cuh -- the fused perforated-load -> rebuild -> stencil kernel (sm_100a).
//
// PAPER.md Fig. 1b (:258-274): input buffer -> (Ia) data perforation ->
// (Ib) data reconstruction -> kernel execution -> output buffer, with (Ia) and
// (Ib) working on local (= CUDA shared) memory (:383-395).
//
// B200 design:
//   * one CTA = 1 producer warp + NCW consumer warps, owning an output tile of
//     TW = NCW*32*V columns x seg_h rows of one frame; it streams down the tile
//     one input row at a time;
//   * the producer fetches ONLY the kept part of each needed input row into a
//     ring of shared-memory row slots: whole kept rows with one TMA-engine bulk
//     copy (cp.async.bulk, UBLKCP) each, kept column granules / checker cells
//     with 16-B cp.async (LDGSTS), anything unaligned with scalar loads.  A
//     skipped row is never requested (row scheme: it has no slot at all);
//   * each consumer lane owns V consecutive output columns; per input row it
//     rebuilds its V samples (and one edge chunk for the warp's halo) from the
//     ring -- NN copy or LI between the nearest loaded samples -- exchanges the
//     r halo samples with its neighbours by warp shuffles, and feeds the app's
//     register sliding window (separable stencils keep only the 1-D horizontal
//     results per row); outputs leave with 128-bit stores;
//   * full/empty mbarriers per slot; consumer warps run independently.
#pragma once
#include <cstdint>

#include "ptx.cuh"

namespace kp {

enum { S_NONE = 0, S_ROW = 1, S_COL = 2, S_CHECKER = 3 };
enum { R_NN = 0, R_LI = 1 };
enum { L_AUTO = 0, L_BULK = 1, L_ASYNC16 = 2, L_SCALAR = 3 };

struct KParams {
  const void* in;   // frame 0; element (x, y_global) at (y_global - in_row0) * W + x
  const void* in2;  // Hotspot power (same geometry as in), else nullptr
  void* out;        // frame 0; output row y_global at (y_global - out_row0) * W
  long long in_fstride, out_fstride;
  int W, Hg;                 // width, global height (clamping and mask use global rows)
  int in_row0, avail0, avail1, out_row0;
  int y_begin, y_end;        // output rows of this launch (global)
  int num, den, G, keep_one; // skipped fraction num/den, granule G (pixels)
  int loader;
  int seg_h, n_strips, n_segs, frames;
  int nr, nr_log2;           // ring slots (power of two)
  int hx;                    // columns of halo/apron each side (multiple of V)
  int row_elems;             // TW + 2*hx
  int fast_ok;               // every V-chunk lies in one mask cell (G % V == 0 or row scheme)
  int vec_io;                // W % V == 0 and 16-B aligned buffers
  float sdc, rx1, ry1, rz1, amb;  // Hotspot (Rodinia) coefficients
};

__device__ __forceinline__ int clampi(int v, int lo, int hi) { return v < lo ? lo : (v > hi ? hi : v); }

// ---------------------------------------------------------------------------
// element-type traits: a "Vec" is the V samples one lane owns (16 bytes)
template <typename T>
struct VT;

template <>
struct VT<float> {
  static constexpr int V = 4;
  using Vec = float4;
  __device__ static __forceinline__ float get(const Vec& v, int i) {
    return i == 0 ? v.x : i == 1 ? v.y : i == 2 ? v.z : v.w;
  }
  __device__ static __forceinline__ void set(Vec& v, int i, float s) {
    if (i == 0) v.x = s; else if (i == 1) v.y = s; else if (i == 2) v.z = s; else v.w = s;
  }
  __device__ static __forceinline__ Vec lds(const float* p) { return *reinterpret_cast<const float4*>(p); }
  // LI with a common span (rows): (a*db + b*da) / (da + db)
  __device__ static __forceinline__ float li(float a, float b, float fda, float fdb, float inv) {
    return __fmul_rn(fmaf(a, fdb, __fmul_rn(b, fda)), inv);
  }
  __device__ static __forceinline__ Vec li_vec(const Vec& a, const Vec& b, int da, int db) {
    const float fda = (float)da, fdb = (float)db, inv = __frcp_rn((float)(da + db));
    return make_float4(li(a.x, b.x, fda, fdb, inv), li(a.y, b.y, fda, fdb, inv), li(a.z, b.z, fda, fdb, inv),
                       li(a.w, b.w, fda, fdb, inv));
  }
  __device__ static __forceinline__ float li1(float a, float b, int da, int db) {
    return li(a, b, (float)da, (float)db, __frcp_rn((float)(da + db)));
  }
};

template <>
struct VT<uint8_t> {
  static constexpr int V = 16;
  using Vec = uint4;
  __device__ static __forceinline__ uint32_t word(const Vec& v, int w) {
    return w == 0 ? v.x : w == 1 ? v.y : w == 2 ? v.z : v.w;
  }
  __device__ static __forceinline__ uint8_t get(const Vec& v, int i) {
    return (uint8_t)(word(v, i >> 2) >> (8 * (i & 3)));
  }
  __device__ static __forceinline__ void set(Vec& v, int i, uint8_t s) {
    const int w = i >> 2, sh = 8 * (i & 3);
    const uint32_t m = ~(0xFFu << sh), b = (uint32_t)s << sh;
    if (w == 0) v.x = (v.x & m) | b; else if (w == 1) v.y = (v.y & m) | b;
    else if (w == 2) v.z = (v.z & m) | b; else v.w = (v.w & m) | b;
  }
  __device__ static __forceinline__ Vec lds(const uint8_t* p) { return *reinterpret_cast<const uint4*>(p); }
  // integer LI, round half up: (a*db + b*da + (da+db)/2) / (da+db)
  __device__ static __forceinline__ uint32_t li_int(uint32_t a, uint32_t b, uint32_t da, uint32_t db,
                                                    uint32_t magic) {
    const uint32_t n = a * db + b * da + ((da + db) >> 1);
    return __umulhi(n, magic);  // floor(n / (da+db)) for n < 2^32/(da+db)
  }
  __device__ static __forceinline__ uint32_t magic_of(uint32_t s) { return 0xFFFFFFFFu / s + 1u; }
  __device__ static __forceinline__ uint8_t li1(uint8_t a, uint8_t b, int da, int db) {
    return (uint8_t)li_int(a, b, da, db, magic_of(da + db));
  }
  __device__ static __forceinline__ Vec li_vec(const Vec& a, const Vec& b, int da, int db) {
    Vec r = make_uint4(0, 0, 0, 0);
    if (da == 1 && db == 1) {  // rounding average: (a + b + 1) >> 1 per byte
      r.x = (a.x | b.x) - (((a.x ^ b.x) >> 1) & 0x7F7F7F7Fu);
      r.y = (a.y | b.y) - (((a.y ^ b.y) >> 1) & 0x7F7F7F7Fu);
      r.z = (a.z | b.z) - (((a.z ^ b.z) >> 1) & 0x7F7F7F7Fu);
      r.w = (a.w | b.w) - (((a.w ^ b.w) >> 1) & 0x7F7F7F7Fu);
      return r;
    }
    const uint32_t mg = magic_of(da + db);
#pragma unroll
    for (int i = 0; i < 16; ++i) set(r, i, (uint8_t)li_int(get(a, i), get(b, i), da, db, mg));
    return r;
  }
};

// ---------------------------------------------------------------------------
// mask helpers (the row scheme's kept rows have closed-form ordinals)
struct Mask {
  int num, den, keep_one;
  __device__ __forceinline__ bool row_kept(int ym) const { return keep_one ? ym == 0 : ym != den - 1; }
  // ordinal of a kept row among kept rows / its inverse
  __device__ __forceinline__ int ord(int y) const {
    return keep_one ? y / den : (y / den) * (den - 1) + y % den;
  }
  __device__ __forceinline__ int row_of(int o) const {
    return keep_one ? o * den : (o / (den - 1)) * den + o % (den - 1);
  }
  // distances to the loaded samples below/above for a skipped line of phase t
  __device__ __forceinline__ int dlo(int t) const { return keep_one ? t : 1; }
  __device__ __forceinline__ int dhi(int t) const { return keep_one ? den - t : 1; }
  __device__ __forceinline__ bool phase_kept(int t) const { return keep_one ? t == 0 : t != den - 1; }
};

template <int SCHEME>
__device__ __forceinline__ bool px_kept(const KParams& p, const Mask& m, int x, int y) {
  if (SCHEME == S_NONE) return true;
  if (SCHEME == S_ROW) return m.phase_kept(y % m.den);
  if (SCHEME == S_COL) return m.phase_kept((x / p.G) % m.den);
  return m.phase_kept((x / p.G + y) % m.den);
}

struct RowPlan {
  int lo, hi, ord_lo, nload;
  int lim_lo, lim_hi;  // rows that exist (globally and in this buffer)
};

template <int SCHEME>
__device__ __forceinline__ RowPlan make_row_plan(const KParams& p, const Mask& m, int ys, int ye, int VR) {
  RowPlan r;
  r.lim_lo = max(0, p.avail0);
  r.lim_hi = min(p.Hg, p.avail1) - 1;
  const int ya = clampi(ys - VR, r.lim_lo, r.lim_hi);
  const int yb = clampi(ye - 1 + VR, r.lim_lo, r.lim_hi);
  if (SCHEME == S_ROW) {
    const int ta = ya % m.den, tb = yb % m.den;
    r.lo = m.phase_kept(ta) ? ya : ya - m.dlo(ta);
    if (r.lo < r.lim_lo) r.lo = ya;  // (insufficient halo; never with host-sized bands)
    if (m.phase_kept(tb)) r.hi = yb;
    else if (yb + m.dhi(tb) <= r.lim_hi) r.hi = yb + m.dhi(tb);
    else r.hi = yb - m.dlo(tb);
    r.ord_lo = m.ord(r.lo);
    r.nload = m.ord(r.hi) - r.ord_lo + 1;
  } else if (SCHEME == S_CHECKER) {
    r.lo = max(ya - (m.den - 1), r.lim_lo);
    r.hi = min(yb + (m.den - 1), r.lim_hi);
    r.ord_lo = r.lo;
    r.nload = r.hi - r.lo + 1;
  } else {
    r.lo = ya;
    r.hi = yb;
    r.ord_lo = ya;
    r.nload = yb - ya + 1;
  }
  return r;
}

template <int SCHEME>
__device__ __forceinline__ int row_of_idx(const Mask& m, const RowPlan& rp, int i) {
  return SCHEME == S_ROW ? m.row_of(rp.ord_lo + i) : rp.lo + i;
}

// ---------------------------------------------------------------------------
// producer warp: fetch the kept part of every needed row into the ring
template <typename T, int SCHEME, int NIN, int NCW>
__device__ __forceinline__ void producer(const KParams& p, const Mask& m, const RowPlan& rp, int x0, int frame,
                                         uint64_t* full, uint64_t* empty, T* ring) {
  constexpr int V = VT<T>::V;
  constexpr int TW = NCW * 32 * V;
  const int lane = threadIdx.x & 31;
  const int cx0 = max(x0 - p.hx, 0);
  const int cx1 = min(x0 + TW + p.hx, p.W);
  const int px0 = cx0, px1 = cx1;  // second input (power): same columns (COL rebuild reads the apron)
  const T* in = static_cast<const T*>(p.in) + (long long)frame * p.in_fstride;
  const T* in2 = static_cast<const T*>(p.in2) + (long long)frame * p.in_fstride;
  const int slot_elems = p.row_elems * NIN;
  const int base = x0 - p.hx;  // global column of ring element 0

  // per-lane chunk phases for the column / checker schemes (row independent)
  constexpr int KMAX = 8;
  int gph[KMAX];
#pragma unroll
  for (int k = 0; k < KMAX; ++k) {
    const int c = cx0 + (lane + 32 * k) * V;
    gph[k] = (SCHEME == S_COL || SCHEME == S_CHECKER) && c < cx1 ? (c / p.G) % m.den : 0;
  }

  for (int i = 0; i < rp.nload; ++i) {
    const int slot = i & (p.nr - 1);
    if (i >= p.nr) mbar_wait(&empty[slot], ((i >> p.nr_log2) - 1) & 1);
    const int y = row_of_idx<SCHEME>(m, rp, i);
    const long long roff = (long long)(y - p.in_row0) * p.W;
    T* dst = ring + slot * slot_elems;
    if (p.loader == L_BULK) {
      // whole kept row: one TMA-engine bulk copy per input array
      if (lane == 0) {
        const uint32_t b0 = (uint32_t)((cx1 - cx0) * sizeof(T));
        const uint32_t b1 = NIN > 1 ? (uint32_t)((px1 - px0) * sizeof(T)) : 0u;
        mbar_arrive_expect_tx(&full[slot], b0 + b1);
        bulk_g2s(dst + (cx0 - base), in + roff + cx0, b0, &full[slot]);
        if (NIN > 1) bulk_g2s(dst + p.row_elems + (px0 - base), in2 + roff + px0, b1, &full[slot]);
      }
    } else if (p.loader == L_ASYNC16) {
      const int ym = (SCHEME == S_CHECKER) ? y % m.den : 0;
#pragma unroll
      for (int k = 0; k < KMAX; ++k) {
        const int c = cx0 + (lane + 32 * k) * V;
        if (c < cx1) {
          bool kept = true;
          if (SCHEME == S_COL) kept = m.phase_kept(gph[k]);
          if (SCHEME == S_CHECKER) {
            int t = gph[k] + ym;
            if (t >= m.den) t -= m.den;
            kept = m.phase_kept(t);
          }
          if (kept) {
            cp_async16(dst + (c - base), in + roff + c);
            if (NIN > 1 && c >= px0 && c < px1) cp_async16(dst + p.row_elems + (c - base), in2 + roff + c);
          }
        }
      }
      for (int c = cx0 + (lane + 32 * KMAX) * V; c < cx1; c += 32 * V) {  // (wide apron; rare)
        if (px_kept<SCHEME>(p, m, c, y)) {
          cp_async16(dst + (c - base), in + roff + c);
          if (NIN > 1 && c >= px0 && c < px1) cp_async16(dst + p.row_elems + (c - base), in2 + roff + c);
        }
      }
      cp_async_arrive_noinc(&full[slot]);
    } else {  // L_SCALAR: any width / alignment
      for (int c = cx0 + lane; c < cx1; c += 32) {
        if (px_kept<SCHEME>(p, m, c, y)) {
          dst[c - base] = in[roff + c];
          if (NIN > 1 && c >= px0 && c < px1) dst[p.row_elems + c - base] = in2[roff + c];
        }
      }
      mbar_arrive(&full[slot]);
    }
  }
}

// ---------------------------------------------------------------------------
// consumer-side rebuild of one lane chunk (V samples starting at column xc)
struct RowCtx {
  int y, ym;
  int kept;                // row scheme: this row loaded
  int slot_c;              // ring slot of row y (row scheme: if kept; others: always)
  int slot_a, slot_b;      // row scheme: slots of the loaded rows below/above
  int has_a, has_b, da, db;
};

struct ChunkInfo {  // per-lane, row-independent facts of a chunk
  int xc;           // first global column
  int fast;         // inside the image and mask-uniform
  int gxm;          // (xc / G) % den
  int col_kept, xa, xb;  // column scheme: kept?, nearest loaded columns (or -1)
};

template <int SCHEME>
__device__ __forceinline__ ChunkInfo make_chunk(const KParams& p, const Mask& m, int xc, int V) {
  ChunkInfo c;
  c.xc = xc;
  c.fast = p.fast_ok && xc >= 0 && xc + V <= p.W;
  c.gxm = 0; c.col_kept = 1; c.xa = -1; c.xb = -1;
  if ((SCHEME == S_COL || SCHEME == S_CHECKER) && xc >= 0) c.gxm = (xc / p.G) % m.den;
  if (SCHEME == S_COL && xc >= 0) {
    const int gx = xc / p.G, t = c.gxm;
    c.col_kept = m.phase_kept(t);
    if (!c.col_kept) {
      c.xa = (gx - m.dlo(t)) * p.G + p.G - 1;
      c.xb = (gx + m.dhi(t)) * p.G;
      if (c.xb > p.W - 1) c.xb = -1;
    }
  }
  return c;
}

// one sample at in-image column x of row rc.y (generic path: any x, any G)
template <typename T, int SCHEME, int RECON>
__device__ __forceinline__ T rebuild_px(const KParams& p, const Mask& m, const RowPlan& rp, const RowCtx& rc,
                                        const T* ring, int slot_elems, int base, int x) {
  using VTT = VT<T>;
  const int col = x - base;
  if (SCHEME == S_NONE) return ring[rc.slot_c * slot_elems + col];
  if (SCHEME == S_ROW) {
    if (rc.kept) return ring[rc.slot_c * slot_elems + col];
    const T a = rc.has_a ? ring[rc.slot_a * slot_elems + col] : T(0);
    const T b = rc.has_b ? ring[rc.slot_b * slot_elems + col] : T(0);
    if (RECON == R_LI && rc.has_a && rc.has_b) return VTT::li1(a, b, rc.da, rc.db);
    return (!rc.has_b || (rc.has_a && rc.da <= rc.db)) ? a : b;
  }
  if (SCHEME == S_COL) {
    const int gx = x / p.G, t = gx % m.den;
    const T* row = ring + rc.slot_c * slot_elems;
    if (m.phase_kept(t)) return row[col];
    const int xa = (gx - m.dlo(t)) * p.G + p.G - 1;
    int xb = (gx + m.dhi(t)) * p.G;
    const bool hb = xb <= p.W - 1;
    const int da = x - xa, db = xb - x;
    const T a = row[xa - base];
    const T b = hb ? row[xb - base] : T(0);
    if (RECON == R_LI && hb) return VTT::li1(a, b, da, db);
    return (!hb || da <= db) ? a : b;
  }
  // checker: rebuild along y in this column
  int t = (x / p.G) % m.den + rc.ym;
  if (t >= m.den) t -= m.den;
  if (m.phase_kept(t)) return ring[rc.slot_c * slot_elems + col];
  const int da = m.dlo(t), db = m.dhi(t);
  const int ya = rc.y - da, yb = rc.y + db;
  const bool ha = ya >= rp.lim_lo, hb = yb <= rp.lim_hi;
  const T a = ha ? ring[((ya - rp.lo) & (p.nr - 1)) * slot_elems + col] : T(0);
  const T b = hb ? ring[((yb - rp.lo) & (p.nr - 1)) * slot_elems + col] : T(0);
  if (RECON == R_LI && ha && hb) return VTT::li1(a, b, da, db);
  return (!hb || (ha && da <= db)) ? a : b;
}

// V samples of a chunk; out-of-image columns take the clamped column's sample
// (clamp-to-edge addressing of the rebuilt image, R8)
template <typename T, int SCHEME, int RECON>
__device__ __forceinline__ typename VT<T>::Vec rebuild_chunk(const KParams& p, const Mask& m,
                                                             const RowPlan& rp, const RowCtx& rc,
                                                             const ChunkInfo& ci, const T* ring,
                                                             int slot_elems, int base, int in_off) {
  using VTT = VT<T>;
  using Vec = typename VTT::Vec;
  constexpr int V = VTT::V;
  const int col = ci.xc - base;
  if (ci.fast) {
    if (SCHEME == S_NONE) return VTT::lds(ring + rc.slot_c * slot_elems + in_off + col);
    if (SCHEME == S_ROW) {
      if (rc.kept) return VTT::lds(ring + rc.slot_c * slot_elems + in_off + col);
      if (RECON == R_LI && rc.has_a && rc.has_b)
        return VTT::li_vec(VTT::lds(ring + rc.slot_a * slot_elems + in_off + col),
                           VTT::lds(ring + rc.slot_b * slot_elems + in_off + col), rc.da, rc.db);
      const int s = (!rc.has_b || (rc.has_a && rc.da <= rc.db)) ? rc.slot_a : rc.slot_b;
      return VTT::lds(ring + s * slot_elems + in_off + col);
    }
    if (SCHEME == S_CHECKER) {
      int t = ci.gxm + rc.ym;
      if (t >= m.den) t -= m.den;
      if (m.phase_kept(t)) return VTT::lds(ring + rc.slot_c * slot_elems + in_off + col);
      const int da = m.dlo(t), db = m.dhi(t);
      const int ya = rc.y - da, yb = rc.y + db;
      const bool ha = ya >= rp.lim_lo, hb = yb <= rp.lim_hi;
      const int sa = (ya - rp.lo) & (p.nr - 1), sb = (yb - rp.lo) & (p.nr - 1);
      if (RECON == R_LI && ha && hb)
        return VTT::li_vec(VTT::lds(ring + sa * slot_elems + in_off + col),
                           VTT::lds(ring + sb * slot_elems + in_off + col), da, db);
      const int s = (!hb || (ha && da <= db)) ? sa : sb;
      return VTT::lds(ring + s * slot_elems + in_off + col);
    }
    // column scheme
    const T* row = ring + rc.slot_c * slot_elems + in_off;
    if (ci.col_kept) return VTT::lds(row + col);
    const T a = row[ci.xa - base];
    const bool hb = ci.xb >= 0;
    const T b = hb ? row[ci.xb - base] : T(0);
    Vec r;
#pragma unroll
    for (int i = 0; i < V; ++i) {
      const int da = ci.xc + i - ci.xa, db = ci.xb - ci.xc - i;
      T v;
      if (RECON == R_LI && hb) v = VTT::li1(a, b, da, db);
      else v = (!hb || da <= db) ? a : b;
      VTT::set(r, i, v);
    }
    return r;
  }
  // generic / edge path: per sample, clamped column
  Vec r;
  const T* ringo = ring + in_off;
#pragma unroll
  for (int i = 0; i < V; ++i) {
    const int x = clampi(ci.xc + i, 0, p.W - 1);
    VTT::set(r, i, rebuild_px<T, SCHEME, RECON>(p, m, rp, rc, ringo, slot_elems, base, x));
  }
  return r;
}

}  // namespace kp
