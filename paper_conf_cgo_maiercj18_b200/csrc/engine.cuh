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
#include <cuda.h>  // CUtensorMap

#include <cstdint>

#include "ptx.cuh"

namespace kp {

enum { S_NONE = 0, S_ROW = 1, S_COL = 2, S_CHECKER = 3, S_STENCIL1 = 4 };
enum { R_NN = 0, R_LI = 1 };
enum { L_AUTO = 0, L_BULK = 1, L_ASYNC16 = 2, L_SCALAR = 3, L_RUNS = 4, L_TMA = 5 };
enum { TMA_NONE = 0, TMA_COL = 1, TMA_CHK = 2 };

struct KParams {
  // L_TMA (column scheme / keep-one checkerboard, fp32): the kept cells of a
  // row arrive as ONE tensor-tile load into a packed ring slot (DESIGN.md
  // "TMA cell loads").  TMA_COL: 3-D map {L = kept run of a den-cell group,
  // group, row}, box {L, tma_ng, 1}; group g's run lands at (g - g0) * L.
  // TMA_CHK: 3-D map {G, cell, row}, box {G, tma_ng * den, 1} traversed with
  // stride den along the cells from the row's first kept cell (-y mod den):
  // the kept cells land packed as the compact slots expect.
  CUtensorMap tmap;  // host copy; the kernel reads its own __grid_constant__ parameter (kernel.cuh)
  int tma_mode, tma_ng, tma_L, tma_rows_per_frame;
  const void* in;   // frame 0; element (x, y_global) at (y_global - in_row0) * W + x
  const void* in2;  // Hotspot power (same geometry as in), else nullptr
  void* out;        // frame 0; output row y_global at (y_global - out_row0) * W
  long long in_fstride, out_fstride;
  int W, Hg;                 // width, global height (clamping and mask use global rows)
  int ncw;                   // consumer warps per CTA (the kernel's NCW; host bookkeeping)
  int in_row0, avail0, avail1, out_row0;
  int y_begin, y_end;        // output rows of this launch (global)
  int num, den, G, keep_one; // skipped fraction num/den, granule G (pixels)
  int loader;
  int seg_h, n_strips, n_segs, frames;
  int seg_auto;              // seg_h is an upper bound; the launcher picks the wave-filling value
  int nr, nr_log2;           // ring slots (power of two)
  int hx;                    // columns of halo/apron each side (multiple of V)
  int row_elems;             // TW + 2*hx (slot stride; compact checker: chk_cells * G)
  int chk_compact;           // keep-one checker: a slot holds only its row's kept cells, cell c at
                             // ((c - (x0/G - den)) / den) * G (kperf.cu: fast path for every warp)
  int fast_ok;               // every V-chunk lies in one mask cell (G % V == 0 or row scheme)
  int cellmap;               // median column NN: cell-grouped lanes (kernel.cuh MEDC)
  int fold;                  // row scheme: rebuild folded into the vertical pass (fold.cuh), interior segments
  int vec_io;                // W % V == 0 and 16-B aligned buffers
  int vec32;                 // 32-B aligned lane chunks of the output (256-bit stores)
  int tile1_w, tile1_h;      // Stencil1 work-group tile
  int nrec;                  // recipe-table entries per consumer warp (>= n_recipes of a segment)
  int inline_prod;           // bulk loader issued by consumer warp 0 (no dedicated producer warp)
  float sdc, rx1, ry1, rz1, amb;  // Hotspot (Rodinia) coefficients
  // NEXT-4 peer-memory halo exchange (banded Hotspot): output rows
  // [y_begin, y_begin + halo_rows) are also stored into the upper neighbour's
  // buffer pu (its row 0 = global row pu_row0), rows [y_end - halo_rows, y_end)
  // into the lower neighbour's pd -- direct NVLink stores fused into the step
  float* pu;
  float* pd;
  int pu_row0, pd_row0, halo_rows;
};

// compile-time loop: f(IC<0>{}), f(IC<1>{}), ... f(IC<N-1>{})
template <int I>
struct IC {
  static constexpr int value = I;
};
template <int I, int N, class F>
__device__ __forceinline__ void static_for(F&& f) {
  if constexpr (I < N) {
    f(IC<I>{});
    static_for<I + 1, N>(f);
  }
}

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
  if (SCHEME == S_NONE || SCHEME == S_STENCIL1) return true;
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
  const int vr = SCHEME == S_STENCIL1 ? 0 : VR;  // Stencil1: the tile's own rows only
  const int ya = clampi(ys - vr, r.lim_lo, r.lim_hi);
  const int yb = clampi(ye - 1 + vr, r.lim_lo, r.lim_hi);
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
    // rebuild reach along y: keep-one cells reach den-1 rows, skip-one cells 1 row
    const int reach = m.keep_one ? m.den - 1 : 1;
    r.lo = max(ya - reach, r.lim_lo);
    r.hi = min(yb + reach, r.lim_hi);
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
// one kept row (and its power row) by TMA-engine bulk copies; lane 0 only
template <typename T, int SCHEME, int NIN, int TW>
__device__ __forceinline__ void issue_bulk_row(const KParams& p, const Mask& m, const RowPlan& rp, int x0, int frame,
                                               int g, int i, uint64_t* full, T* ring) {
  const int cx0 = max(x0 - p.hx, 0), cx1 = min(x0 + TW + p.hx, p.W);
  const int slot = g & (p.nr - 1);
  const int y = row_of_idx<SCHEME>(m, rp, i);
  const long long roff = (long long)(y - p.in_row0) * p.W + (long long)frame * p.in_fstride;
  T* dst = ring + slot * p.row_elems * NIN + (cx0 - (x0 - p.hx));
  const uint32_t b0 = (uint32_t)((cx1 - cx0) * sizeof(T));
  mbar_arrive_expect_tx(&full[slot], b0 * NIN);
  bulk_g2s(dst, static_cast<const T*>(p.in) + roff + cx0, b0, &full[slot]);
  if (NIN > 1) bulk_g2s(dst + p.row_elems, static_cast<const T*>(p.in2) + roff + cx0, b0, &full[slot]);
}

// g0: global (per-CTA, across work items) index of this item's first load;
// ring slot = g & (nr-1), fill phase = g >> log2(nr).
template <typename T, int SCHEME, int NIN, int TW>
__device__ __forceinline__ void producer(const KParams& p, const Mask& m, const RowPlan& rp, int x0, int frame,
                                         int g0, uint64_t* full, uint64_t* empty, T* ring, const void* tmap) {
  constexpr int V = VT<T>::V;  // 16-B load chunk
  const int lane = threadIdx.x & 31;
  const int cx0 = max(x0 - p.hx, 0);
  const int cx1 = min(x0 + TW + p.hx, p.W);
  const int px0 = cx0, px1 = cx1;  // second input (power): same columns (COL rebuild reads the apron)
  const T* in = static_cast<const T*>(p.in) + (long long)frame * p.in_fstride;
  const T* in2 = static_cast<const T*>(p.in2) + (long long)frame * p.in_fstride;
  const int slot_elems = p.row_elems * NIN;
  const int base = x0 - p.hx;  // global column of ring element 0

  // 16-B chunks (lane + 32 k) of the row: per lane, a one-hot of the chunk's mask
  // phase (column / checker cell phase, row independent; 0 = outside the row).
  // A row's kept phases form a bit mask, so "chunk kept" is one AND and the
  // copies are predicated LDGSTS with no branches.
  constexpr int KMAX = 12;
  uint32_t onehot[KMAX];
#pragma unroll
  for (int k = 0; k < KMAX; ++k) {
    const int c = cx0 + (lane + 32 * k) * V;
    const bool cell = SCHEME == S_COL || SCHEME == S_CHECKER;
    onehot[k] = c < cx1 ? (cell ? 1u << ((c / p.G) % m.den) : 1u) : 0u;
  }
  // kept-phase mask of the column scheme: bit t <=> phase t is loaded
  uint32_t kmask = 0;
  for (int t = 0; t < m.den; ++t) kmask |= (uint32_t)m.phase_kept(t) << t;
  const uint32_t dmask = (1u << m.den) - 1u;
  const uint32_t lane_dst0 = smem_u32(ring) + (uint32_t)((cx0 - base + lane * V) * (int)sizeof(T));
  const T* lane_src0 = in + cx0 + lane * V;
  const T* lane_src1 = in2 + cx0 + lane * V;

  // L_TMA: the row's kept cells as one tensor-tile load per row (KParams tmap)
  if constexpr ((SCHEME == S_COL || SCHEME == S_CHECKER) && NIN == 1 && sizeof(T) == 4) {
    if (p.loader == L_TMA) {
      // first loaded group: the one left of the strip (its last kept columns are
      // the strip's apron); checkerboard: the compact slots' first cell (kperf.cu)
      const int gg0 = x0 / (p.G * m.den) - 1;
      const uint32_t bytes = (uint32_t)(p.tma_ng * p.tma_L * (int)sizeof(T));
      if (lane == 0) tma_prefetch_desc(tmap);
      for (int i = 0; i < rp.nload; ++i) {
        const int g = g0 + i;
        const int slot = g & (p.nr - 1);
        if (g >= p.nr) mbar_wait(&empty[slot], ((g >> p.nr_log2) - 1) & 1);
        const int y = row_of_idx<SCHEME>(m, rp, i);
        const int row = frame * p.tma_rows_per_frame + (y - p.in_row0);
        if (lane == 0) {
          T* dst = ring + slot * slot_elems;
          mbar_arrive_expect_tx(&full[slot], bytes);
          if (SCHEME == S_COL) tma_load_3d(dst, tmap, 0, gg0, row, &full[slot]);
          else tma_load_3d(dst, tmap, 0, gg0 * m.den + (m.den - y % m.den) % m.den, row, &full[slot]);
        }
      }
      return;
    }
  }
  // compact keep-one checkerboard slots (kperf.cu chk_compact): a row keeps
  // cells c == -y mod den only, packed at ((c - (x0/G - den)) / den) * G, so
  // chunk k has one slot offset for every row that keeps it.  A loop of its
  // own: the full-width loop below keeps its immediate-offset copies.
  if constexpr (SCHEME == S_CHECKER && NIN == 1) {
    if (p.chk_compact && p.loader == L_ASYNC16) {
      uint32_t coff[KMAX];
      const int cb = x0 / p.G - m.den;
#pragma unroll
      for (int k = 0; k < KMAX; ++k) {
        const int c = min(cx0 + (lane + 32 * k) * V, cx1 - V);
        const int cell = c / p.G;
        coff[k] = (uint32_t)((((cell - cb) / m.den) * p.G + (c - cell * p.G)) * (int)sizeof(T));
      }
      const T* s0l = lane_src0;
      for (int i = 0; i < rp.nload; ++i) {
        const int g = g0 + i;
        const int slot = g & (p.nr - 1);
        if (g >= p.nr) mbar_wait(&empty[slot], ((g >> p.nr_log2) - 1) & 1);
        const int y = row_of_idx<SCHEME>(m, rp, i);
        const int ym = y % m.den;
        const uint32_t rmask = ((kmask >> ym) | (kmask << (m.den - ym))) & dmask;
        const uint32_t dc = smem_u32(ring) + (uint32_t)(slot * slot_elems * (int)sizeof(T));
        const T* s0 = s0l + (long long)(y - p.in_row0) * p.W;
#ifdef KPERF_PROBE_NOLOAD  // experiment: the ring protocol without the global loads
        const uint32_t rm = 0u;
#else
        const uint32_t rm = rmask;
#endif
#pragma unroll
        for (int k = 0; k < KMAX; ++k) cp_async16_if(dc + coff[k], s0 + k * 32 * V, rm & onehot[k]);
        cp_async_arrive_noinc(&full[slot]);
      }
      return;
    }
  }
  for (int i = 0; i < rp.nload; ++i) {
    const int g = g0 + i;
    const int slot = g & (p.nr - 1);
    if (g >= p.nr) mbar_wait(&empty[slot], ((g >> p.nr_log2) - 1) & 1);
    const int y = row_of_idx<SCHEME>(m, rp, i);
    const long long roff = (long long)(y - p.in_row0) * p.W;
    T* dst = ring + slot * slot_elems;
    if (SCHEME == S_COL || SCHEME == S_CHECKER) {
      if (p.loader == L_RUNS) {
        // kept cells of the row: one TMA-engine bulk copy per run of consecutive
        // kept cells (skip-one: up to den-1 cells, keep-one: 1), run starts
        // spread over the lanes; the row's byte total is armed first
        const int ym = SCHEME == S_CHECKER ? y % m.den : 0;
        const int c_lo = cx0 / p.G, c_hi = (cx1 - 1) / p.G;
        uint32_t bytes = 0;
        int rs[2], re[2];  // this lane's runs (cells lane, lane + 32 of the row)
#pragma unroll
        for (int k = 0; k < 2; ++k) {
          rs[k] = re[k] = 0;
          const int c = c_lo + lane + 32 * k;
          int q = (c + ym) % m.den;
          const bool start = c <= c_hi && m.phase_kept(q) && (c == c_lo || !m.phase_kept(q == 0 ? m.den - 1 : q - 1));
          if (start) {
            int e = c;
            while (e < c_hi && m.phase_kept((e + 1 + ym) % m.den)) ++e;
            rs[k] = max(c * p.G, cx0);
            re[k] = min((e + 1) * p.G, cx1);
            bytes += (uint32_t)((re[k] - rs[k]) * (int)sizeof(T)) * NIN;
          }
        }
#pragma unroll
        for (int o = 16; o > 0; o >>= 1) bytes += __shfl_xor_sync(0xFFFFFFFFu, bytes, o);
        if (lane == 0) mbar_arrive_expect_tx(&full[slot], bytes);
        __syncwarp();
#pragma unroll
        for (int k = 0; k < 2; ++k) {
          if (re[k] > rs[k]) {
            const uint32_t b = (uint32_t)((re[k] - rs[k]) * sizeof(T));
            bulk_g2s(dst + (rs[k] - base), in + roff + rs[k], b, &full[slot]);
            if (NIN > 1) bulk_g2s(dst + p.row_elems + (rs[k] - base), in2 + roff + rs[k], b, &full[slot]);
          }
        }
        continue;
      }
    }
    if (p.loader == L_BULK) {
      // whole kept row: one TMA-engine bulk copy per input array
      if (lane == 0) {
#ifdef KPERF_PROBE_NOLOAD  // experiment: the ring protocol without the global loads
        mbar_arrive(&full[slot]);
        continue;
#endif
        const uint32_t b0 = (uint32_t)((cx1 - cx0) * sizeof(T));
        const uint32_t b1 = NIN > 1 ? (uint32_t)((px1 - px0) * sizeof(T)) : 0u;
        mbar_arrive_expect_tx(&full[slot], b0 + b1);
        bulk_g2s(dst + (cx0 - base), in + roff + cx0, b0, &full[slot]);
        if (NIN > 1) bulk_g2s(dst + p.row_elems + (px0 - base), in2 + roff + px0, b1, &full[slot]);
      }
    } else if (p.loader == L_ASYNC16) {
      // cell (g) of row y is kept iff phase (g + y) % den is (checker), g is (column)
      uint32_t rmask = 1u;
      if (SCHEME == S_COL) rmask = kmask;
      if (SCHEME == S_CHECKER) {
        const int ym = y % m.den;
        rmask = ((kmask >> ym) | (kmask << (m.den - ym))) & dmask;
      }
      const uint32_t d0 = lane_dst0 + (uint32_t)(slot * slot_elems * (int)sizeof(T));
      const T* s0 = lane_src0 + roff;
#ifdef KPERF_PROBE_NOLOAD
      rmask = 0u;
#endif
#pragma unroll
      for (int k = 0; k < KMAX; ++k) {
        const uint32_t pk = rmask & onehot[k];
        cp_async16_if(d0 + k * 32 * 16, s0 + k * 32 * V, pk);
        if (NIN > 1) cp_async16_if(d0 + (p.row_elems + k * 32 * V) * (int)sizeof(T), lane_src1 + roff + k * 32 * V, pk);
      }
      for (int c = cx0 + (lane + 32 * KMAX) * V; c < cx1; c += 32 * V) {  // (very wide apron; rare)
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
// consumer side: fragments of N consecutive samples held in registers
template <typename T, int N>
struct Frag;

template <int N>
struct Frag<float, N> {
  float v[N];
  __device__ __forceinline__ float get(int i) const { return v[i]; }
  __device__ __forceinline__ void set(int i, float s) { v[i] = s; }
  __device__ __forceinline__ static Frag splat(float s) {
    Frag f;
#pragma unroll
    for (int i = 0; i < N; ++i) f.v[i] = s;
    return f;
  }
};

template <int N>
struct Frag<uint8_t, N> {  // N bytes packed little-endian in N/4 words
  uint32_t w[N / 4];
  __device__ __forceinline__ uint8_t get(int i) const { return (uint8_t)(w[i >> 2] >> (8 * (i & 3))); }
  __device__ __forceinline__ void set(int i, uint8_t s) {
    const int k = i >> 2, sh = 8 * (i & 3);
    w[k] = (w[k] & ~(0xFFu << sh)) | ((uint32_t)s << sh);
  }
  __device__ __forceinline__ static Frag splat(uint8_t s) {
    Frag f;
#pragma unroll
    for (int k = 0; k < N / 4; ++k) f.w[k] = 0x01010101u * s;
    return f;
  }
};

template <typename T, int N>
__device__ __forceinline__ Frag<T, N> ldf(const T* p) {
  Frag<T, N> f;
  constexpr int B = N * (int)sizeof(T);
  static_assert(B == 4 || B == 8 || B == 16 || B == 32, "fragment size");
  if constexpr (B == 32) {
#ifdef KPERF_PROBE_NOCONFLICT  // experiment (wrong results): the same loads at a 16-B lane stride
    const T* q = p - (threadIdx.x & 31) * (16 / sizeof(T));
    reinterpret_cast<uint4*>(&f)[0] = reinterpret_cast<const uint4*>(q)[0];
    reinterpret_cast<uint4*>(&f)[1] = reinterpret_cast<const uint4*>(q)[32];
#else
    reinterpret_cast<uint4*>(&f)[0] = reinterpret_cast<const uint4*>(p)[0];
    reinterpret_cast<uint4*>(&f)[1] = reinterpret_cast<const uint4*>(p)[1];
#endif
  } else if constexpr (B == 16) *reinterpret_cast<uint4*>(&f) = *reinterpret_cast<const uint4*>(p);
  else if constexpr (B == 8) *reinterpret_cast<uint2*>(&f) = *reinterpret_cast<const uint2*>(p);
  else *reinterpret_cast<uint32_t*>(&f) = *reinterpret_cast<const uint32_t*>(p);
  return f;
}

// LI of two loaded fragments with a common span: (a*db + b*da) / (da + db)
template <int N>
__device__ __forceinline__ Frag<float, N> li_frag(const Frag<float, N>& a, const Frag<float, N>& b, int da,
                                                  int db) {
  Frag<float, N> r;
  if (da == db) {
    if constexpr (N % 2 == 0) {  // FADD2 + FMUL2 per two samples
#pragma unroll
      for (int i = 0; i < N; i += 2)
        up2(mul2(add2(pk2(a.v[i], a.v[i + 1]), pk2(b.v[i], b.v[i + 1])), splat2(0.5f)), r.v[i], r.v[i + 1]);
    } else {
#pragma unroll
      for (int i = 0; i < N; ++i) r.v[i] = __fmul_rn(__fadd_rn(a.v[i], b.v[i]), 0.5f);
    }
  } else {
    const float fda = (float)da, fdb = (float)db, inv = __frcp_rn((float)(da + db));
#pragma unroll
    for (int i = 0; i < N; ++i) r.v[i] = VT<float>::li(a.v[i], b.v[i], fda, fdb, inv);
  }
  return r;
}

template <int N>
__device__ __forceinline__ Frag<uint8_t, N> li_frag(const Frag<uint8_t, N>& a, const Frag<uint8_t, N>& b,
                                                    int da, int db) {
  Frag<uint8_t, N> r;
  if (da == db) {  // (a + b + 1) >> 1 per byte
#pragma unroll
    for (int k = 0; k < N / 4; ++k) r.w[k] = (a.w[k] | b.w[k]) - (((a.w[k] ^ b.w[k]) >> 1) & 0x7F7F7F7Fu);
  } else {
    const uint32_t mg = VT<uint8_t>::magic_of(da + db);
#pragma unroll
    for (int i = 0; i < N; ++i) r.set(i, (uint8_t)VT<uint8_t>::li_int(a.get(i), b.get(i), da, db, mg));
  }
  return r;
}

__device__ __forceinline__ float li_px(float a, float b, int da, int db) { return VT<float>::li1(a, b, da, db); }
__device__ __forceinline__ uint8_t li_px(uint8_t a, uint8_t b, int da, int db) {
  return VT<uint8_t>::li1(a, b, da, db);
}

// A row recipe: everything a consumer needs to rebuild one virtual input row,
// computed once per CTA into shared memory.
//   y     clamped global row;  need = need_hi | emit << 15 | need_lo << 16 (ring
//         indices; emit: this row completes an output row)
//   info  slot_a | slot_b << 8 | ym << 16 | da << 20 | db << 24 | kept << 28 |
//         li << 29 | has_a << 30 | has_b << 31
//   wa    LI weight of the lower sample: value = b + (a - b) * wa, wa = db/(da+db)
//   oa, ob  byte offsets of slot_a / slot_b in the ring (the fast paths add them
//         to a per-lane column address: one IADD per source row, no slot index math)
// Row scheme: a kept row, and an NN-rebuilt row, are plain copies of slot_a.
// 32 B: the first half {oa, ob, need, wa} is what the row scheme's fast path
// reads -- one LDS.128 per row.
struct __align__(16) Recipe {
  int oa, ob, need;
  float wa;
  int y;
  uint32_t info;
  int pad0, pad1;
};
template <typename T>
__device__ __forceinline__ const T* ring_at(const T* ring, int off) {
  return reinterpret_cast<const T*>(reinterpret_cast<const char*>(ring) + off);
}

__device__ __forceinline__ int rc_slot_a(uint32_t i) { return (int)(i & 0xFF); }
__device__ __forceinline__ int rc_slot_b(uint32_t i) { return (int)((i >> 8) & 0xFF); }
__device__ __forceinline__ int rc_ym(uint32_t i) { return (int)((i >> 16) & 0xF); }
__device__ __forceinline__ int rc_da(uint32_t i) { return (int)((i >> 20) & 0xF); }
__device__ __forceinline__ int rc_db(uint32_t i) { return (int)((i >> 24) & 0xF); }
__device__ __forceinline__ bool rc_kept(uint32_t i) { return (i >> 28) & 1; }
__device__ __forceinline__ bool rc_li(uint32_t i) { return (i >> 29) & 1; }
__device__ __forceinline__ bool rc_has_a(uint32_t i) { return (i >> 30) & 1; }
__device__ __forceinline__ bool rc_has_b(uint32_t i) { return (i >> 31) & 1; }

// number of virtual input rows (recipes) of a segment
template <int SCHEME>
__device__ __forceinline__ int n_recipes(const KParams& p, int ys, int ye, int VR) {
  if (SCHEME != S_STENCIL1) return ye - ys + 2 * VR;
  const int th = p.tile1_h, nt = (ye - ys + th - 1) / th;
  return (nt - 1) * (th + 2 * VR) + (ye - (ys + (nt - 1) * th)) + 2 * VR;
}

// virtual row i of a segment -> (row to rebuild, emits an output row?)
template <int SCHEME>
__device__ __forceinline__ int virtual_row(const KParams& p, const RowPlan& rp, int ys, int ye, int VR, int i,
                                           int& emit) {
  if (SCHEME != S_STENCIL1) {
    emit = i >= 2 * VR;
    return clampi(ys - VR + i, rp.lim_lo, rp.lim_hi);
  }
  // Stencil1: each tile of tile1_h rows is its own clamped window (Fig. 5)
  const int th = p.tile1_h, per = th + 2 * VR, t = i / per, k = i - t * per;
  const int ty0 = ys + t * th, ty1 = min(ty0 + th, ye);
  emit = k >= 2 * VR;
  return clampi(ty0 - VR + k, ty0, ty1 - 1);
}

template <int SCHEME, int RECON>
__device__ __forceinline__ Recipe make_recipe(const KParams& p, const Mask& m, const RowPlan& rp, int y, int emit,
                                              int slot_bytes) {
  Recipe r;
  const int ym = y % m.den, nmask = p.nr - 1;
  int need_hi, need_lo, sa = 0, sb = 0, da = 1, db = 1, kept = 1, li = 0, ha = 0, hb = 0;
  float wa = 1.f;
  if (SCHEME == S_ROW) {
    kept = m.phase_kept(ym);
    if (kept) {
      const int id = m.ord(y) - rp.ord_lo;
      sa = sb = id & nmask;
      need_hi = need_lo = id;
    } else {
      da = m.dlo(ym);
      db = m.dhi(ym);
      ha = (y - da) >= rp.lo;
      hb = (y + db) <= rp.hi;
      const int ida = m.ord(y - da) - rp.ord_lo;
      const int idb = hb ? m.ord(y + db) - rp.ord_lo : ida;
      need_hi = hb ? idb : ida;
      need_lo = ha ? ida : idb;
      if (RECON == R_LI && ha && hb) {
        li = 1;
        sa = ida & nmask;
        sb = idb & nmask;
        wa = __fdiv_rn((float)db, (float)(da + db));
      } else {  // nearest neighbour: a copy of the chosen loaded row
        kept = 1;
        sa = sb = ((!hb || (ha && da <= db)) ? ida : idb) & nmask;
      }
    }
  } else if (SCHEME == S_CHECKER) {
    const int reach = m.keep_one ? m.den - 1 : 1;  // (make_row_plan)
    sa = sb = (y - rp.lo) & nmask;
    need_hi = min(y + reach, rp.hi) - rp.lo;
    need_lo = max(y - reach, rp.lo) - rp.lo;
  } else {
    sa = sb = (y - rp.lo) & nmask;
    need_hi = need_lo = y - rp.lo;
  }
  r.y = y;
  r.need = need_hi | (emit << 15) | (need_lo << 16);
  r.info = (uint32_t)sa | ((uint32_t)sb << 8) | ((uint32_t)ym << 16) | ((uint32_t)da << 20) |
           ((uint32_t)db << 24) | ((uint32_t)kept << 28) | ((uint32_t)li << 29) | ((uint32_t)ha << 30) |
           ((uint32_t)hb << 31);
  r.wa = wa;
  r.oa = sa * slot_bytes;
  r.ob = sb * slot_bytes;
  r.pad0 = r.pad1 = 0;
  return r;
}

// b + (a - b) * wa, elementwise
template <int N>
__device__ __forceinline__ Frag<float, N> lerp_frag(const Frag<float, N>& a, const Frag<float, N>& b, float wa) {
  Frag<float, N> r;
  if constexpr (N % 2 == 0) {  // paired fp32: FADD2 + FFMA2 per two samples
    const f2 w = splat2(wa);
#pragma unroll
    for (int i = 0; i < N; i += 2) {
      const f2 bb = pk2(b.v[i], b.v[i + 1]);
      up2(fma2(sub2(pk2(a.v[i], a.v[i + 1]), bb), w, bb), r.v[i], r.v[i + 1]);
    }
  } else {
#pragma unroll
    for (int i = 0; i < N; ++i) r.v[i] = fmaf(a.v[i] - b.v[i], wa, b.v[i]);
  }
  return r;
}

struct RowCtx {
  int y, ym;
  int kept;           // row scheme: row y loaded
  int slot_c;         // ring slot of row y (row scheme: when kept)
  int slot_a, slot_b; // row scheme: slots of the loaded rows below/above
  int has_a, has_b, da, db;
  float wa;           // row scheme LI weight (see Recipe)
};

// generic-path context from a recipe
template <int SCHEME>
__device__ __forceinline__ RowCtx ctx_of(const Recipe& r) {
  RowCtx c;
  c.y = r.y;
  c.ym = rc_ym(r.info);
  c.kept = SCHEME == S_ROW ? (rc_kept(r.info) ? 1 : 0) : 1;
  c.slot_c = rc_slot_a(r.info);
  c.slot_a = rc_slot_a(r.info);
  c.slot_b = rc_slot_b(r.info);
  c.has_a = rc_has_a(r.info);
  c.has_b = rc_has_b(r.info);
  c.da = rc_da(r.info);
  c.db = rc_db(r.info);
  c.wa = r.wa;
  return c;
}

struct ChunkInfo {  // per-lane, row-independent facts of a V-aligned chunk
  int xc;           // first global column
  int gxm;          // (xc / G) % den
  int col_kept, xa, xb;  // column scheme: loaded?, nearest loaded columns below/above (xb = -1: none)
};

template <int SCHEME>
__device__ __forceinline__ ChunkInfo make_chunk(const KParams& p, const Mask& m, int xc) {
  ChunkInfo c;
  c.xc = xc;
  c.gxm = 0;
  c.col_kept = 1;
  c.xa = 0;
  c.xb = -1;
  if (xc < 0 || xc >= p.W) return c;  // outside: treated as loaded (value replaced by the clamp)
  if (SCHEME == S_COL || SCHEME == S_CHECKER) c.gxm = (xc / p.G) % m.den;
  if (SCHEME == S_COL) {
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

// fast rebuild of N samples at ring column `col` (global column fx), all in one
// mask cell described by `ci`; row facts from the recipe
// ULI (row scheme, fp32 LI): no kept / interpolated branch -- every row is
// b + (a - b) * wa with a kept row given slot_a == slot_b (a - b = 0: exact);
// smaller code for consumers whose unrolled loop overflows the instruction cache
template <typename T, int N, int SCHEME, int RECON, bool ULI = false>
__device__ __forceinline__ Frag<T, N> rebuild_frag(const KParams& p, const Mask& m, const RowPlan& rp,
                                                   const Recipe& rec, const ChunkInfo& ci, const T* ring,
                                                   int slot_elems, int col, int fx, int base) {
  const uint32_t info = rec.info;
  if (SCHEME == S_NONE || SCHEME == S_STENCIL1) return ldf<T, N>(ring_at(ring, rec.oa) + col);
  if constexpr (SCHEME == S_ROW && ULI && RECON == R_LI && sizeof(T) == 4) {
    const Frag<T, N> a = ldf<T, N>(ring_at(ring, rec.oa) + col);
    const Frag<T, N> b = ldf<T, N>(ring_at(ring, rec.ob) + col);
    return lerp_frag<N>(a, b, rec.wa);
  }
  if (SCHEME == S_ROW) {
    if (RECON == R_NN) return ldf<T, N>(ring_at(ring, rec.oa) + col);
    const Frag<T, N> a = ldf<T, N>(ring_at(ring, rec.oa) + col);
    if (rec.oa == rec.ob) return a;  // kept (or NN-rebuilt) row: one source
    const Frag<T, N> b = ldf<T, N>(ring_at(ring, rec.ob) + col);
    if constexpr (sizeof(T) == 4) return lerp_frag<N>(a, b, rec.wa);
    else return li_frag<N>(a, b, rc_da(info), rc_db(info));
  }
  RowCtx rc;
  rc.y = rec.y;
  rc.ym = rc_ym(info);
  rc.slot_c = rc_slot_a(info);
  if (SCHEME == S_CHECKER) {
    int t = ci.gxm + rc.ym;
    if (t >= m.den) t -= m.den;
    if (m.phase_kept(t)) return ldf<T, N>(ring + rc.slot_c * slot_elems + col);
    const int da = m.dlo(t), db = m.dhi(t);
    const int ya = rc.y - da, yb = rc.y + db;
    const bool ha = ya >= rp.lim_lo, hb = yb <= rp.lim_hi;
    const int sa = (ya - rp.lo) & (p.nr - 1), sb = (yb - rp.lo) & (p.nr - 1);
    if (RECON == R_LI && ha && hb)
      return li_frag<N>(ldf<T, N>(ring + sa * slot_elems + col), ldf<T, N>(ring + sb * slot_elems + col), da, db);
    const int s = (!hb || (ha && da <= db)) ? sa : sb;
    return ldf<T, N>(ring + s * slot_elems + col);
  }
  // column scheme: rebuilt along x from the edge samples of the nearest loaded granules
  const T* row = ring + rc.slot_c * slot_elems;
  if (ci.col_kept) return ldf<T, N>(row + col);
  const T a = row[ci.xa - base];
  const bool hb = ci.xb >= 0;
  const T b = hb ? row[ci.xb - base] : a;
  Frag<T, N> r;
  if (RECON == R_LI && hb) {
    if constexpr (sizeof(T) == 4) {  // b + (a - b) * (xb - x) / (xb - xa)
      const float inv = __frcp_rn((float)(ci.xb - ci.xa)), d = a - b, x0 = (float)(ci.xb - fx);
#pragma unroll
      for (int i = 0; i < N; ++i) r.set(i, fmaf(d, __fmul_rn(x0 - (float)i, inv), b));
    } else {
      const uint32_t mg = VT<uint8_t>::magic_of(ci.xb - ci.xa);
#pragma unroll
      for (int i = 0; i < N; ++i) {
        const int da = fx + i - ci.xa, db = ci.xb - fx - i;
        r.set(i, (uint8_t)VT<uint8_t>::li_int(a, b, da, db, mg));
      }
    }
  } else {  // nearest: a while 2x <= xa + xb (ties to the lower column)
    const int lim = ci.xa + ci.xb - 2 * fx;
    if constexpr (sizeof(T) == 1) {  // per-byte select with word masks
      const uint32_t wa = 0x01010101u * a, wb = 0x01010101u * b;
#pragma unroll
      for (int k = 0; k < N / 4; ++k) {
        uint32_t msk = 0;
#pragma unroll
        for (int j = 0; j < 4; ++j)
          if (!hb || 2 * (4 * k + j) <= lim) msk |= 0xFFu << (8 * j);
        r.w[k] = (wa & msk) | (wb & ~msk);
      }
    } else {
#pragma unroll
      for (int i = 0; i < N; ++i) r.set(i, (!hb || 2 * i <= lim) ? a : b);
    }
  }
  return r;
}

// one sample at in-image column x of row rc.y (generic path: any x, any G)
template <typename T, int SCHEME, int RECON>
__device__ __noinline__ T rebuild_px(const KParams& p, const Mask& m, const RowPlan& rp, const RowCtx& rc,
                                     const T* ring, int slot_elems, int base, int x) {
  const int col = x - base;
  if (SCHEME == S_NONE || SCHEME == S_STENCIL1) return ring[rc.slot_c * slot_elems + col];
  if (SCHEME == S_ROW) {
    if (rc.kept) return ring[rc.slot_c * slot_elems + col];
    // (an NN-rebuilt row is marked kept with slot_a = the chosen loaded row)
    const T a = ring[rc.slot_a * slot_elems + col];
    const T b = ring[rc.slot_b * slot_elems + col];
    if constexpr (sizeof(T) == 4) return fmaf(a - b, rc.wa, b);
    else return li_px(a, b, rc.da, rc.db);
  }
  if (SCHEME == S_COL) {
    const int gx = x / p.G, t = gx % m.den;
    const T* row = ring + rc.slot_c * slot_elems;
    if (m.phase_kept(t)) return row[col];
    const int xa = (gx - m.dlo(t)) * p.G + p.G - 1;
    const int xb = (gx + m.dhi(t)) * p.G;
    const bool hb = xb <= p.W - 1;
    const int da = x - xa, db = xb - x;
    const T a = row[xa - base];
    const T b = hb ? row[xb - base] : T(0);
    if (RECON == R_LI && hb) {
      if constexpr (sizeof(T) == 4)  // same arithmetic as the fast path
        return fmaf(a - b, __fmul_rn((float)db, __frcp_rn((float)(xb - xa))), b);
      else return li_px(a, b, da, db);
    }
    return (!hb || da <= db) ? a : b;
  }
  int t = (x / p.G) % m.den + rc.ym;  // checker: rebuilt along y in this column
  if (t >= m.den) t -= m.den;
  if (m.phase_kept(t)) return ring[rc.slot_c * slot_elems + col];
  const int da = m.dlo(t), db = m.dhi(t);
  const int ya = rc.y - da, yb = rc.y + db;
  const bool ha = ya >= rp.lim_lo, hb = yb <= rp.lim_hi;
  const T a = ha ? ring[((ya - rp.lo) & (p.nr - 1)) * slot_elems + col] : T(0);
  const T b = hb ? ring[((yb - rp.lo) & (p.nr - 1)) * slot_elems + col] : T(0);
  if (RECON == R_LI && ha && hb) return li_px(a, b, da, db);
  return (!hb || (ha && da <= db)) ? a : b;
}

// generic path: N samples starting at column fx, each at the clamped column
template <typename T, int N, int SCHEME, int RECON>
__device__ __forceinline__ Frag<T, N> rebuild_frag_generic(const KParams& p, const Mask& m, const RowPlan& rp,
                                                           const RowCtx& rc, const T* ring, int slot_elems,
                                                           int fx, int base) {
  Frag<T, N> r;
#pragma unroll
  for (int i = 0; i < N; ++i)
    r.set(i, rebuild_px<T, SCHEME, RECON>(p, m, rp, rc, ring, slot_elems, base, clampi(fx + i, 0, p.W - 1)));
  return r;
}

}  // namespace kp
