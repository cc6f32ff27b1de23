// kernel.cuh -- the perforated stencil kernel template and its launcher.
// See engine.cuh for the design; apps.cuh for the stencil stages.
#pragma once
#include <cuda_runtime.h>

#include <cstdio>

#include "apps.cuh"
#include "engine.cuh"

#ifndef KPERF_PIPELINE
#define KPERF_PIPELINE 0
#endif
#ifndef KPERF_ST256
#define KPERF_ST256 1  // 256-bit output stores (fp32 lanes: 8 samples)
#endif
#ifndef KPERF_MINB
#define KPERF_MINB 0  // 0: per-app App::MINB
#endif
#ifndef KPERF_SEG_K1
#define KPERF_SEG_K1 24  // fixed segment height: keep-one row schemes with den >= 4, Gaussian5 row den 2 (launch_one)
#endif
#ifndef KPERF_SEG_FIX
#define KPERF_SEG_FIX 16  // fixed segment height of the other fp32 whole-row kernels (see launch_one)
#endif
#ifndef KPERF_FOLD
#define KPERF_FOLD 1  // row scheme: rebuild folded into the vertical pass (fold.cuh)
#endif
#ifndef KPERF_LPT
#define KPERF_LPT 1  // folded row scheme: a frame's first / last segments dispatched first
#endif
#ifndef KPERF_MEDC_ILV
#define KPERF_MEDC_ILV 1  // median column NN: interleaved warp ranks (C3 col 1/2 NN 197 -> 183 us)
#endif
#ifndef KPERF_MEDCELL
#define KPERF_MEDCELL 1  // median column NN: cell-grouped lanes + the all-skipped-warp shortcut
#endif

namespace kp {

constexpr int kMaxVR = 3;  // largest vertical radius of an app (recipe table rows = seg_h + 2 VR)
// recipe-table padding: the unrolled row loops run whole groups of NWIN rows
// (NWIN <= 5); rows past the segment's last virtual row repeat its recipe with
// emit = 0 (no ring wait or release, no store), so the unrolled body has no
// per-row guard -- a guard is a join point where every register-ring value
// needs a copy (C5 exact: 260 -> 220 SASS instructions per row)
constexpr int kRecPad = 8;

// per-device host caches (a process may drive several devices through one
// library: kernel attributes, SM counts and occupancy are per device)
constexpr int kMaxDev = 64;
inline int cur_dev() {
  int d = 0;
  cudaGetDevice(&d);
  return (d < 0 || d >= kMaxDev) ? 0 : d;
}
inline int dev_sms() {
  static int sms[kMaxDev] = {};
  const int d = cur_dev();
  if (sms[d] == 0) {
    int v = 0;
    cudaDeviceGetAttribute(&v, cudaDevAttrMultiProcessorCount, d);
    sms[d] = v < 1 ? 1 : v;
  }
  return sms[d];
}


#ifndef KPERF_SLEEP_NS
#define KPERF_SLEEP_NS 200
#endif
#ifndef KPERF_WAIT_HINT
#define KPERF_WAIT_HINT 1000  // consumer full-barrier waits: try_wait suspend-time hint in ns (0 = none)
#endif
__device__ __forceinline__ void mbar_wait_u32(uint32_t addr, uint32_t parity) {
  // watchdog: a protocol bug traps (launch error) instead of hanging the GPU
  uint32_t ok, spins = 0;
  do {
#if KPERF_WAIT_HINT
    asm volatile(
        "{\n .reg .pred p;\n mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2, %3;\n selp.u32 %0, 1, 0, p;\n}"
        : "=r"(ok)
        : "r"(addr), "r"(parity), "n"(KPERF_WAIT_HINT)
        : "memory");
#else
    asm volatile(
        "{\n .reg .pred p;\n mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n selp.u32 %0, 1, 0, p;\n}"
        : "=r"(ok)
        : "r"(addr), "r"(parity)
        : "memory");
#endif
    if (++spins > (1u << 26)) __trap();
  } while (!ok);
}
// the same wait for warps that are far ahead of the slowest consumer warp of
// their CTA (the median's all-skipped warps): back off with nanosleep so the
// spin does not take issue slots from the ALU-bound warps on the same SMSP
__device__ __forceinline__ void mbar_wait_sleep_u32(uint32_t addr, uint32_t parity) {
  uint32_t ok, spins = 0;
  for (;;) {
    asm volatile(
        "{\n .reg .pred p;\n mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n selp.u32 %0, 1, 0, p;\n}"
        : "=r"(ok)
        : "r"(addr), "r"(parity)
        : "memory");
    if (ok) break;
    if (++spins > (1u << 24)) __trap();
    __nanosleep(KPERF_SLEEP_NS);
  }
}
__device__ __forceinline__ void mbar_arrive_u32(uint32_t addr) {
  asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(addr) : "memory");
}

// (Ib) reconstruction + kernel execution of one work item for one consumer
// warp.  FAST: every lane's V-chunk lies inside the image and in one mask cell.
// ready / released are the warp's global (across items) ring counters.
template <class App, int SCHEME, int RECON, int NCW, bool FAST>
__device__ void consumer(const KParams& p, const Mask& m, const RowPlan& rp, int x0, int frame,
                                         int ys, int ye, int g0, uint32_t full_u32, uint32_t empty_u32,
                                         const typename App::T* ring, int slot_elems, const Recipe* rtab,
                                         float4* ctab) {
  using T = typename App::T;
  constexpr int V = App::V, EW = App::EW, VR = App::VR, NWIN = App::NWIN;
  constexpr int CV = 16 / sizeof(T);  // elements of one 16-B mask-uniform chunk
  constexpr int TW = NCW * 32 * V;
  const int lane = threadIdx.x & 31, w = (threadIdx.x >> 5) - (p.inline_prod ? 0 : 1);
  // inline producer (bulk loader): consumer warp 0 issues the kept rows itself
  const bool issuer = App::IPROD && p.inline_prod && w == 0;
  uint64_t* full_p = reinterpret_cast<uint64_t*>(__cvta_shared_to_generic(full_u32));
  T* ring_w = const_cast<T*>(ring);
  int issued = 0;
  // issue every row whose slot is free (non-blocking); then make sure row `upto` is issued
  auto issue_ahead = [&](int upto) {
#pragma unroll 1
    while (issued < rp.nload) {
      const int g = g0 + issued;
      if (g >= p.nr) {
        const uint32_t par = ((g >> p.nr_log2) - 1) & 1;
        const uint32_t ea = empty_u32 + 8 * (g & (p.nr - 1));
        if (issued > upto) {
          uint32_t ok;
          asm volatile("{\n .reg .pred q;\n mbarrier.test_wait.parity.shared::cta.b64 q, [%1], %2;\n selp.u32 %0, 1, 0, q;\n}"
                       : "=r"(ok) : "r"(ea), "r"(par) : "memory");
          if (!ok) break;
        } else {
          mbar_wait_u32(ea, par);
        }
      }
      if (lane == 0)
        issue_bulk_row<T, SCHEME, App::NIN, TW>(p, m, rp, x0, frame, g, issued, full_p, ring_w);
      ++issued;
    }
  };
  const int xw = x0 + w * 32 * V;
  const int base = x0 - p.hx;
  int xc = xw + lane * V;
  int ex = lane < 16 ? xw - EW : xw + 32 * V;  // edge fragment (warp halo) start column
  int cex = lane < 16 ? xw - CV : xw + 32 * V;  // ... and its 16-B chunk
  uint32_t hedge = lane == 0 ? 4u : (lane == 31 ? 8u : 0u);  // lane's left / right neighbour comes from e
  // Median, column NN (C3): cell-grouped lanes.  The strip's G-wide cells are
  // dealt to the warps kept cells first, then skipped ones, G/V lanes per cell;
  // a warp whose cells are all skipped has every 3x3 window built from at most
  // two rebuilt columns (the edge samples a, b) and takes the scalar path below
  // (DESIGN.md "Median").  Neighbour columns across a cell edge come from the
  // lane's edge fragment, not a shuffle.
  constexpr bool MEDC = FAST && SCHEME == S_COL && sizeof(T) == 1 && RECON == R_NN && KPERF_MEDCELL;
  bool cellmap = false;
  if constexpr (MEDC) {
    if (p.cellmap && x0 + TW <= p.W) {
      cellmap = true;
      const int lpc = p.G / V, ncell = TW / p.G, c0 = x0 / p.G;
      // warp rank: KPERF_MEDC_ILV interleaves the ranks (0, 2, 1, 3 for four
      // warps) so the kept-cell warps (ranks first) are not adjacent warp ids
      const int rank = (KPERF_MEDC_ILV && NCW == 4) ? ((w & 1) << 1 | (w >> 1)) : w;
      const int want = rank * (32 / lpc) + lane / lpc;
      int nk = 0;
      for (int j = 0; j < ncell; ++j) nk += m.phase_kept((c0 + j) % m.den) ? 1 : 0;
      int cell = 0, kk = 0, ks = 0;
      for (int j = 0; j < ncell; ++j) {
        const int pos = m.phase_kept((c0 + j) % m.den) ? kk++ : nk + ks++;
        if (pos == want) cell = j;
      }
      const int cs = x0 + cell * p.G, li = lane % lpc;
      const bool left = li < lpc / 2;
      xc = cs + li * V;
      ex = left ? cs - EW : cs + p.G;
      cex = left ? cs - CV : cs + p.G;
      hedge = (li == 0 ? 4u : 0u) | (li == lpc - 1 ? 8u : 0u);
    }
  }
  const ChunkInfo cc = make_chunk<SCHEME>(p, m, xc);
  const ChunkInfo ce = make_chunk<SCHEME>(p, m, cex);
  // edge fragment: 0 inside the image, 1 left of column 0, 2 right of column W-1, 3 straddles W
  const int emode = (ex >= 0 && ex + EW <= p.W) ? 0 : (ex < 0 ? 1 : (ex == p.W ? 2 : 3));
  // ring column of global column x: x - base, or -- TMA column loads (kperf.cu
  // L_TMA) -- the packed slot: the kept run of group g (den cells, L kept
  // columns) at (g - gg0) * L; columns that are never loaded map to 0 (their
  // values are never used: kept ? own : rebuilt selects)
  auto ringcol = [&](int x) {
    if (SCHEME != S_COL || p.tma_mode != TMA_COL) return x - base;
    const int gw = p.G * m.den, rel = x - (x0 / gw - 1) * gw;
    if (rel < 0) return 0;
    const int k = rel / gw, q = rel - k * gw;
    return (q < p.tma_L && k < p.tma_ng) ? k * p.tma_L + q : 0;
  };
  const int ccol = ringcol(xc), ecol = ringcol(ex);
  const T* ring2 = ring + p.row_elems;  // second input (Hotspot power)
  // Stencil1: lane edges that are tile borders take their halo from the tile itself
  const uint32_t hf = hedge | (SCHEME == S_STENCIL1
                                     ? (uint32_t)((xc % p.tile1_w) == 0) | ((uint32_t)(((xc + V) % p.tile1_w) == 0) << 1)
                                     : 0u);
  App app;
  app.init(p);
  T* optr = static_cast<T*>(p.out) + (long long)frame * p.out_fstride + (long long)(ys - p.out_row0) * p.W + xc;
  const int nmask = p.nr - 1;
  const int vy0 = ys - VR;
  const int nv = n_recipes<SCHEME>(p, ys, ye, VR);  // virtual input rows of this segment
  int ready = g0 - 1, released = g0;  // this warp's ring counters (global load indices)

  // column scheme, u8, NN: which bytes of a lane's chunk take the left /
  // right neighbour granule's edge sample is row-independent -- byte masks
  // hoisted out of the row loop; the per-row rebuild is then branch-free:
  // word = (loaded & km) | (a x 0x01010101 & ma) | (b x 0x01010101 & mb)
  struct NNu8 {
    int ca, cb;       // ring columns of the edge samples a (left) and b (right)
    uint32_t km;      // ~0: the chunk is loaded
    uint32_t ma[4], mb[4];
  };
  auto nn_u8 = [&](const ChunkInfo& ci, int fx, int col, int nbytes) {
    NNu8 z;
    const bool kept = ci.col_kept;
    const bool hb = ci.xb >= 0;
    z.km = kept ? ~0u : 0u;
    z.ca = kept ? col : ci.xa - base;
    z.cb = (kept || !hb) ? z.ca : ci.xb - base;
    const int lim = ci.xa + ci.xb - 2 * fx;  // byte i takes a iff 2 i <= lim (ties to the lower column)
#pragma unroll
    for (int k = 0; k < 4; ++k) {
      uint32_t ma = 0, all = 0;
#pragma unroll
      for (int j = 0; j < 4; ++j) {
        const int i = 4 * k + j;
        if (i < nbytes) all |= 0xFFu << (8 * j);
        if (i < nbytes && (!hb || 2 * i <= lim)) ma |= 0xFFu << (8 * j);
      }
      z.ma[k] = kept ? 0u : ma;
      z.mb[k] = kept ? 0u : (all & ~ma);
    }
    return z;
  };
  NNu8 zc, ze;
  if constexpr (SCHEME == S_COL && sizeof(T) == 1 && RECON == R_NN && FAST) {
    zc = nn_u8(cc, xc, ccol, V);
    ze = nn_u8(ce, ex, ecol, EW);
  }
  // column scheme, fp32: the rebuild of a lane's chunk is row independent
  // except for the two edge samples a, b of the neighbouring loaded granules,
  // so the per-lane facts are hoisted and the per-row work is branch free:
  //   c = own samples (garbage unless kept), a = row[ca], b = row[cb]
  //   LI: r_i = fmaf(a - b, w_i, b), w_i = (xb - x_i) / (xb - xa) from a
  //       per-lane shared-memory table (same arithmetic as rebuild_frag)
  //   NN: r_i = (2 i <= lim) ? a : b   (lanes wholly on one side: ca = cb)
  //   out_i = kept ? c_i : r_i
  // (the former divergent kept / skipped branch ran both sides per warp)
  struct ColF {
    int ca, cb, lim;
    bool kept;
  };
  constexpr bool COLF = FAST && SCHEME == S_COL && sizeof(T) == 4;
  auto colf_of = [&](const ChunkInfo& ci, int fx, int col, int n, float4* wt) {
    ColF z;
    z.kept = ci.col_kept;
    const bool hb = ci.xb >= 0;
    z.ca = z.kept ? col : ringcol(ci.xa);
    z.cb = (z.kept || !hb) ? z.ca : ringcol(ci.xb);
    z.lim = hb ? ci.xa + ci.xb - 2 * fx : 2 * n;  // sample i takes a iff 2 i <= lim
    if (RECON == R_NN && !z.kept && z.lim >= 2 * (n - 1)) z.cb = z.ca;  // NN: all samples take a
    else if (RECON == R_NN && !z.kept && z.lim < 0) z.ca = z.cb;        // NN: all take b
    if (RECON == R_LI) {
      float w[8] = {0.f, 0.f, 0.f, 0.f, 0.f, 0.f, 0.f, 0.f};
      if (!z.kept && hb) {
        const float inv = __frcp_rn((float)(ci.xb - ci.xa)), x0 = (float)(ci.xb - fx);
#pragma unroll
        for (int i = 0; i < 8; ++i)
          if (i < n) w[i] = __fmul_rn(x0 - (float)i, inv);
      }
      wt[0] = make_float4(w[0], w[1], w[2], w[3]);
      if (n > 4) wt[32] = make_float4(w[4], w[5], w[6], w[7]);
    }
    return z;
  };
  // checkerboard, fp32: per-lane slot choice instead of a divergent kept /
  // skipped branch; every lane then loads one (NN) or two (LI) ring rows and
  // LI is the row scheme's lerp b + (a - b) * wa (exact when a == b, i.e. for
  // kept lanes and the one-sided fallback at the image border).
  // Everything that depends only on the cell phase t = (gx + y) mod den sits in
  // a per-warp table of den int4 {da, db, wa bits, NN takes a}: kept phases
  // have da = db = 0 (the own row), so the per-row work is two ring-slot sums,
  // two border tests and two selects (KPERF_CHKTAB=0: the former per-row
  // phase arithmetic, LI only; ~75 -> ~25 integer instructions per warp row)
#ifndef KPERF_CHKTAB
#define KPERF_CHKTAB 1
#endif
  constexpr bool CHKF = FAST && SCHEME == S_CHECKER && sizeof(T) == 4 && (RECON == R_LI || KPERF_CHKTAB);
  if constexpr (CHKF) {
    if (lane < m.den) {
      const int t = lane;
      if (KPERF_CHKTAB) {
        const bool k = m.phase_kept(t);
        const int da = k ? 0 : m.dlo(t), db = k ? 0 : m.dhi(t);
        const float wa = k ? 1.f : __fdiv_rn((float)db, (float)(da + db));
        reinterpret_cast<int4*>(ctab)[t] = make_int4(da, db, __float_as_int(wa), da <= db ? 1 : 0);
      } else {
        reinterpret_cast<float*>(ctab)[t] =
            m.phase_kept(t) ? 1.f : __fdiv_rn((float)m.dhi(t), (float)(m.dlo(t) + m.dhi(t)));
      }
    }
    __syncwarp();
  }
  // ring columns the checkerboard reads: compact keep-one slots (kperf.cu
  // chk_compact) hold kept cell c at ((c - (x0/G - den)) / den) * G -- every row
  // that holds this lane's cell holds it there, so the column is per lane
  int kcol = ccol, kecol = ecol;
  if constexpr (CHKF && KPERF_CHKTAB && App::NIN == 1) {
    if (p.chk_compact) {
      const int cb = x0 / p.G - m.den;
      auto cmap = [&](int x) {
        x = min(max(x, 0), p.W - EW);  // (out-of-image edge fragments: any aligned in-slot column; replaced by the clamp)
        const int cell = x / p.G;
        return ((cell - cb) / m.den) * p.G + (x - cell * p.G);
      };
      kcol = cmap(xc);
      kecol = cmap(ex);
    }
  }
  ColF fc, fe;
  bool nn_mixed = false;  // some lane's chunk straddles the NN midpoint (G/2 not a multiple of V)
  if constexpr (COLF) {
    fc = colf_of(cc, xc, ccol, V, ctab + lane);
    fe = colf_of(ce, ex, ecol, EW, ctab + 64 + lane);
    const bool mixed = (!fc.kept && fc.ca != fc.cb) || (!fe.kept && fe.ca != fe.cb);
    nn_mixed = __any_sync(0xFFFFFFFFu, mixed);
    __syncwarp();
  }
  struct Rows {  // one rebuilt input row as the lane sees it
    Frag<T, V> c, c2;
    Frag<T, EW> e;
    int emit;
  };
  // fetch: recipe, ring release/wait, rebuild from shared memory (a1/a2)
  // fetch: recipe, ring release/wait, rebuild from shared memory (a1/a2).
  // After the first row, a row needs at most one more ring row and frees at
  // most one (every scheme's recipes advance by <= 1), so the waits are ifs.
  auto sync = [&](int i, bool sleepy = false) {  // the ring protocol of virtual row i: release what it no longer needs, wait for what it needs
    const Recipe rec = rtab[i];
    const int need_hi = g0 + (rec.need & 0x7FFF), need_lo = g0 + (int)((uint32_t)rec.need >> 16);
    if (released < need_lo) {  // every lane arrives (empty barrier count = 32 x active warps)
      mbar_arrive_u32(empty_u32 + 8 * (released & nmask));
      ++released;
    }
    if (issuer) issue_ahead(need_hi - g0);
    if (ready < need_hi) {
      ++ready;
      if (sleepy) mbar_wait_sleep_u32(full_u32 + 8 * (ready & nmask), (ready >> p.nr_log2) & 1);
      else mbar_wait_u32(full_u32 + 8 * (ready & nmask), (ready >> p.nr_log2) & 1);
    }
    return rec;
  };
  auto fetch = [&](int i) {
    Rows r;
    const Recipe rec = sync(i);
    r.emit = (rec.need >> 15) & 1;
    if constexpr (FAST && SCHEME == S_COL && sizeof(T) == 1 && RECON == R_NN) {
      const T* row = ring_at(ring, rec.oa);
      auto combine = [&](auto nc, const NNu8& z, int col) {
        constexpr int N = decltype(nc)::value;
        Frag<T, N> f = ldf<T, N>(row + col);
        const uint32_t wa = 0x01010101u * (uint32_t)row[z.ca], wb = 0x01010101u * (uint32_t)row[z.cb];
#pragma unroll
        for (int k = 0; k < N / 4; ++k) f.w[k] = (f.w[k] & z.km) | (wa & z.ma[k]) | (wb & z.mb[k]);
        return f;
      };
      r.c = combine(IC<V>{}, zc, ccol);
      const Frag<T, EW> el = combine(IC<EW>{}, ze, ecol);
      const Frag<T, EW> eb = Frag<T, EW>::splat(emode == 1 ? r.c.get(0) : r.c.get(V - 1));
      r.e = emode == 0 ? el : eb;
    } else if constexpr (CHKF && KPERF_CHKTAB) {
      const int y = rec.y, ym = rc_ym(rec.info);
      const int yr = y - rp.lo, yl = y - rp.lim_lo, yh = rp.lim_hi - y;  // (ring slot of y = yr & nmask)
      const int4* etab = reinterpret_cast<const int4*>(ctab);
      const float* ringf = reinterpret_cast<const float*>(ring);
      auto chk = [&](auto nc, int gxm, int col) {
        constexpr int N = decltype(nc)::value;
#ifdef KPERF_PROBE_NOREBUILD  // experiment (DESIGN "cell loaders"): own packed column only, no rebuild
        if (p.y_begin != -12345) return ldf<float, N>(ringf + (yr & nmask) * slot_elems + col);
#endif
        int t = gxm + ym;
        if (t >= m.den) t -= m.den;
        const int4 e = etab[t];
        const bool ha = e.x <= yl, hb = e.y <= yh;  // the loaded rows above / below exist
        const int sa = (yr - e.x) & nmask, sb = (yr + e.y) & nmask;
        if constexpr (RECON == R_NN) {  // nearest (ties: above); one-sided at the border
          const int s = (ha && (e.w || !hb)) ? sa : sb;
          return ldf<float, N>(ringf + s * slot_elems + col);
        } else {
          const Frag<float, N> A = ldf<float, N>(ringf + (ha ? sa : sb) * slot_elems + col);
          const Frag<float, N> B = ldf<float, N>(ringf + (hb ? sb : sa) * slot_elems + col);
          return lerp_frag<N>(A, B, __int_as_float(e.z));
        }
      };
      r.c = chk(IC<V>{}, cc.gxm, kcol);
      const Frag<T, EW> el = chk(IC<EW>{}, ce.gxm, kecol);
      const Frag<T, EW> eb = Frag<T, EW>::splat(emode == 1 ? r.c.get(0) : r.c.get(V - 1));
      r.e = emode == 0 ? el : eb;
      if constexpr (App::NIN > 1) r.c2 = rebuild_frag<T, V, SCHEME, RECON>(p, m, rp, rec, cc, ring2, slot_elems, ccol, xc, base);
    } else if constexpr (CHKF) {
      const int y = rec.y, ym = rc_ym(rec.info), sc = rc_slot_a(rec.info);
      const float* wtab = reinterpret_cast<const float*>(ctab);
      auto chk = [&](auto nc, int gxm, int col) {
        constexpr int N = decltype(nc)::value;
        int t = gxm + ym;
        if (t >= m.den) t -= m.den;
        const bool kept = m.phase_kept(t);
        const int da = m.dlo(t), db = m.dhi(t);
        const int ya = y - da, yb = y + db;
        const bool ha = ya >= rp.lim_lo, hb = yb <= rp.lim_hi;
        int sa = (ya - rp.lo) & (p.nr - 1), sb = (yb - rp.lo) & (p.nr - 1);
        if (!(RECON == R_LI && ha && hb)) {  // nearest loaded row (ties: the lower one)
          const int s1 = (!hb || (ha && da <= db)) ? sa : sb;
          sa = s1;
          sb = s1;
        }
        if (kept) {
          sa = sc;
          sb = sc;
        }
        const Frag<float, N> A = ldf<float, N>(reinterpret_cast<const float*>(ring) + sa * slot_elems + col);
        if constexpr (RECON == R_NN) {
          return A;
        } else {
          const Frag<float, N> B = ldf<float, N>(reinterpret_cast<const float*>(ring) + sb * slot_elems + col);
          return lerp_frag<N>(A, B, wtab[t]);
        }
      };
      r.c = chk(IC<V>{}, cc.gxm, ccol);
      const Frag<T, EW> el = chk(IC<EW>{}, ce.gxm, ecol);
      const Frag<T, EW> eb = Frag<T, EW>::splat(emode == 1 ? r.c.get(0) : r.c.get(V - 1));
      r.e = emode == 0 ? el : eb;
      if constexpr (App::NIN > 1) r.c2 = rebuild_frag<T, V, SCHEME, RECON>(p, m, rp, rec, cc, ring2, slot_elems, ccol, xc, base);
    } else if constexpr (COLF) {
      const float* row = reinterpret_cast<const float*>(ring_at(ring, rec.oa));
      auto colrow = [&](auto nc, const ColF& z, int col, const float4* wt) {
        constexpr int N = decltype(nc)::value;
        const Frag<float, N> c = ldf<float, N>(row + col);
#ifdef KPERF_PROBE_NOREBUILD  // experiment: own packed column only, no rebuild
        if (p.y_begin != -12345) return c;
#endif
        const float a = row[z.ca], b = row[z.cb];
        Frag<float, N> o;
        if constexpr (RECON == R_LI) {
          float w[8];
          const float4 w0 = wt[0];
          w[0] = w0.x; w[1] = w0.y; w[2] = w0.z; w[3] = w0.w;
          if constexpr (N > 4) {
            const float4 w1 = wt[32];
            w[4] = w1.x; w[5] = w1.y; w[6] = w1.z; w[7] = w1.w;
          }
          const float d = a - b;
#pragma unroll
          for (int i = 0; i < N; ++i) o.v[i] = z.kept ? c.v[i] : fmaf(d, w[i], b);
        } else {
          if (nn_mixed) {
#pragma unroll
            for (int i = 0; i < N; ++i) o.v[i] = z.kept ? c.v[i] : (2 * i <= z.lim ? a : b);
          } else {
#pragma unroll
            for (int i = 0; i < N; ++i) o.v[i] = z.kept ? c.v[i] : a;
          }
        }
        return o;
      };
      r.c = colrow(IC<V>{}, fc, ccol, ctab + lane);
      const Frag<T, EW> el = colrow(IC<EW>{}, fe, ecol, ctab + 64 + lane);
      const Frag<T, EW> eb = Frag<T, EW>::splat(emode == 1 ? r.c.get(0) : r.c.get(V - 1));
      r.e = emode == 0 ? el : eb;
      if constexpr (App::NIN > 1) r.c2 = rebuild_frag<T, V, SCHEME, RECON>(p, m, rp, rec, cc, ring2, slot_elems, ccol, xc, base);
    } else if (FAST) {
      r.c = rebuild_frag<T, V, SCHEME, RECON, App::ULI>(p, m, rp, rec, cc, ring, slot_elems, ccol, xc, base);
      if (App::NIN > 1) r.c2 = rebuild_frag<T, V, SCHEME, RECON>(p, m, rp, rec, cc, ring2, slot_elems, ccol, xc, base);
      // edge fragment: loaded (inside the image) or the clamped border sample -- selects, no branch
      const Frag<T, EW> el = rebuild_frag<T, EW, SCHEME, RECON, App::ULI>(p, m, rp, rec, ce, ring, slot_elems, ecol, ex, base);
      const Frag<T, EW> eb = Frag<T, EW>::splat(emode == 1 ? r.c.get(0) : r.c.get(V - 1));
      r.e = emode == 0 ? el : eb;
    } else {
      const RowCtx rc = ctx_of<SCHEME>(rec);
      r.c = rebuild_frag_generic<T, V, SCHEME, RECON>(p, m, rp, rc, ring, slot_elems, xc, base);
      r.e = rebuild_frag_generic<T, EW, SCHEME, RECON>(p, m, rp, rc, ring, slot_elems, ex, base);
      if (App::NIN > 1) r.c2 = rebuild_frag_generic<T, V, SCHEME, RECON>(p, m, rp, rc, ring2, slot_elems, xc, base);
#ifdef KPERF_DEBUG_EDGE
      if (lane == 31 && i < 6 && sizeof(T) == 4)
        printf("dbg blk %d warp %d i %d y %d ex %d base %d slot %d e %f %f c7 %f ring516 %f\n", blockIdx.x,
               threadIdx.x >> 5, i, rec.y, ex, base, rc.slot_c, (double)r.e.get(0), (double)r.e.get(EW - 1),
               (double)r.c.get(V - 1), (double)ring[rc.slot_c * slot_elems + 516]);
#endif
    }
    return r;
  };
  {  // the first row may need several ring rows
    const int need0 = g0 + (rtab[0].need & 0x7FFF);
    if (issuer) issue_ahead(need0 - g0);
#pragma unroll 1
    while (ready < need0 - 1) {
      ++ready;
      mbar_wait_u32(full_u32 + 8 * (ready & nmask), (ready >> p.nr_log2) & 1);
    }
  }
  // compute: the unchanged stencil on the rebuilt row (a3) and the store
  // banded Hotspot: does this segment emit rows the neighbours need?  (CTA-uniform)
  const bool peer_seg = App::NIN > 1 && p.halo_rows > 0 && (p.pu || p.pd) &&
                        (ys < p.y_begin + p.halo_rows || ye > p.y_end - p.halo_rows);
  auto store = [&](T* dst, const Frag<T, V>& o) {  // (FAST implies vec_io)
#ifdef KPERF_PROBE_NOSTORE  // experiment: outputs computed but (almost) never stored
    if (p.y_begin != -12345) {
      float acc = 0.f;
#pragma unroll
      for (int i = 0; i < V; ++i) acc += (float)o.get(i);
      if (acc == 1.2345e-30f) dst[0] = o.get(0);
      return;
    }
#endif
    if (FAST && KPERF_ST256 && V * sizeof(T) == 32) {  // (the fast path of 32-B lane chunks requires p.vec32)
      st_global_v8(dst, reinterpret_cast<const uint4*>(&o)[0], reinterpret_cast<const uint4*>(&o)[1]);
    } else if (FAST) {
#pragma unroll
      for (int q = 0; q < (int)(V * sizeof(T)) / 16; ++q) {
        const uint4 u = reinterpret_cast<const uint4*>(&o)[q];
        st_global_v4(dst + q * CV, u.x, u.y, u.z, u.w);
      }
    } else {
#pragma unroll
      for (int i = 0; i < V; ++i)
        if (FAST || xc + i < p.W) dst[i] = o.get(i);
    }
  };
  auto compute = [&](auto uc, const Rows& r, int vy) {
    constexpr int U = decltype(uc)::value;
    const Frag<T, V> o = app.template row<U>(r.c, r.e, r.c2, lane, hf, vy, xc, p);
    if (r.emit) {  // kernel execution result -> output buffer (output rows in order)
      store(optr, o);
      if constexpr (App::NIN > 1) {  // banded Hotspot: boundary rows also go straight to the neighbours
        if (peer_seg) {
          const int oy = vy - VR;  // global output row (not Stencil1: emitted row = virtual row - VR)
          if (p.pu && oy < p.y_begin + p.halo_rows)
            store(reinterpret_cast<T*>(p.pu) + (long long)(oy - p.pu_row0) * p.W + xc, o);
          if (p.pd && oy >= p.y_end - p.halo_rows)
            store(reinterpret_cast<T*>(p.pd) + (long long)(oy - p.pd_row0) * p.W + xc, o);
        }
      }
      optr += p.W;
    }
  };

  if constexpr (MEDC) {
    // all-skipped warp (column NN median): with column sources a (x <= mid) and
    // b (x > mid), mid = floor((xa + xb) / 2) (ties to a, R6), a 3x3
    // window holds one source column three times -- its median is med3 of that
    // column -- except at x = mid (columns a, a, b) and x = mid + 1 (a, b, b),
    // where the sorted-column identity (R11) reduces to
    // med3(max(lo_a, lo_b), md_a or md_b, min(hi_a, hi_b)).  a and b ride as
    // one u16x2 word per row; the four candidate bytes (med_a, med_b, mid,
    // mid + 1) are packed into one word and each output word is one PRMT with a
    // per-lane, row-independent selector.  Bit-exact with the full network.
    if (cellmap && __all_sync(0xFFFFFFFFu, !cc.col_kept)) {
      const int ca = zc.ca, cb = zc.cb;
      const bool hb = cc.xb >= 0;
      const int sab = cc.xa + cc.xb;
      uint32_t sel[V / 4];
#pragma unroll
      for (int k = 0; k < V / 4; ++k) {
        sel[k] = 0;
#pragma unroll
        for (int j = 0; j < 4; ++j) {
          const int x = xc + 4 * k + j;
          const uint32_t sv = !hb ? 0u : (2 * (x + 1) <= sab ? 0u : (2 * (x - 1) > sab ? 1u : (2 * x <= sab ? 2u : 3u)));
          sel[k] |= sv << (4 * j);
        }
      }
      uint32_t abw[3];
      for (int ib = 0; ib < nv; ib += 3) {
        auto unrolled = [&](auto uc) {
          constexpr int U = decltype(uc)::value, A = (U + 1) % 3, B = (U + 2) % 3;
          const int i = ib + U;  // (rows >= nv: padded recipes -- no wait, no store)
          {
            const Recipe rec = sync(i, true);
            const T* row = ring_at(ring, rec.oa);
            abw[U] = (uint32_t)row[ca] | ((uint32_t)row[cb] << 16);
            if ((rec.need >> 15) & 1) {
              const uint32_t t1 = vmin2(abw[A], abw[B]), t2 = vmax2(abw[A], abw[B]);
              const uint32_t lo = vmin2(t1, abw[U]), t3 = vmax2(t1, abw[U]);
              const uint32_t md = vmin2(t2, t3), hi = vmax2(t2, t3);
              const uint32_t L = vmax2(lo, __byte_perm(lo, 0, 0x1032)), Hm = vmin2(hi, __byte_perm(hi, 0, 0x1032));
              const uint32_t M = vmax2(vmin2(L, md), vmin2(vmax2(L, md), Hm));  // med3(L, md, Hm) per half
              const uint32_t X = __byte_perm(md, M, 0x6420);  // (med_a, med_b, mid, mid + 1)
              Frag<T, V> o;
#pragma unroll
              for (int k = 0; k < V / 4; ++k) o.w[k] = __byte_perm(X, 0, sel[k]);
              store(optr, o);
              optr += p.W;
            }
          }
        };
        static_for<0, 3>(unrolled);
      }
      const int g_end = g0 + rp.nload;
#pragma unroll 1
      while (ready < g_end - 1) {
        ++ready;
        mbar_wait_u32(full_u32 + 8 * (ready & nmask), (ready >> p.nr_log2) & 1);
      }
#pragma unroll 1
      for (; released < g_end; ++released) mbar_arrive_u32(empty_u32 + 8 * (released & nmask));
      return;
    }
  }
  // row scheme, fp32, one kept row per period (den 2, or keep-one den 4):
  // the rebuild folded into the vertical pass (fold.cuh) -- iterate over the
  // kept rows only: horizontal pass per kept row into a register ring (the
  // ring slot is released as soon as it is read), then every output row
  // completed by this kept row as a compile-time weighted sum.  Interior
  // segments only (no clamped rows); others take the per-row loop below.
  if constexpr (FAST && SCHEME == S_ROW && sizeof(T) == 4 && App::FOLD && KPERF_FOLD) {
    // Segments at the image's top / bottom row fold too: the clamp-to-edge
    // rebuilt image (R8) equals the kept-row lattice extended by copies of
    // the first / last kept row (LI between two equal rows, NN of equal rows:
    // the copy), so arrivals above the first and below the last loaded row
    // re-read those rows' slots ("virtual arrivals").  Buffer limits that are
    // not image rows (band halos) still need the margin.
    const bool top_ok = ys - VR - m.den >= rp.lim_lo || (App::FOLD_EDGE && p.avail0 <= 0);
    const bool bot_ok = ye - 1 + VR + m.den <= rp.lim_hi || (App::FOLD_EDGE && p.avail1 >= p.Hg);
    if (p.fold && top_ok && bot_ok && (m.den == 2 || (m.den == 4 && m.keep_one))) {
      auto run = [&](auto dc) {
        constexpr int DEN = decltype(dc)::value;
        using F = typename App::template Fold<DEN, RECON>;
        constexpr int RK = fold_ring(F::sch.span);
        // FOLD_ROT: one arrival per loop iteration, the newest kept row at ring
        // position RK - 1 and the ring shifted down after its emissions (RK - 1
        // register moves) -- a quarter of the unrolled code (instruction cache)
        constexpr int UN = App::FOLD_ROT ? 1 : RK;
        const int J0 = rp.lo / DEN;  // first loaded kept row (rp.lo is a multiple of DEN)
        auto fdiv = [](int a) { return a >= 0 ? a / DEN : -((-a + DEN - 1) / DEN); };
        // kept rows the segment's outputs read: the loaded ones, plus (FOLD_EDGE,
        // image border segments) virtual arrivals of the first / last loaded row
        const int Js = App::FOLD_EDGE ? fdiv(ys - VR) : J0;
        const int Je = App::FOLD_EDGE ? -fdiv(-(ye - 1 + VR)) : J0 + rp.nload - 1;
        const int na = Je - Js + 1;
        const float* ringf = reinterpret_cast<const float*>(ring);
#pragma unroll 1
        for (int jb = 0; jb < na; jb += UN) {
          static_for<0, UN>([&](auto uc) {
            constexpr int U = App::FOLD_ROT ? RK - 1 : decltype(uc)::value;  // ring position of this arrival
            // (arrivals past the last one, J > Je, only occur in the last unrolled
            // group of the non-rotating ring: skipped -- measured: the guard keeps
            // the Gaussian / Sobel fold loops free of spills)
            const int J = Js + jb + (App::FOLD_ROT ? 0 : U);
            int gi;
            bool wait, release;
            if constexpr (App::FOLD_EDGE) {
              const int r = J - J0;  // loaded-row index (< 0 / >= nload: virtual, the first / last row's slot)
              gi = g0 + min(max(r, 0), rp.nload - 1);
              wait = J <= Je && r < rp.nload;
              release = J <= Je && r >= 0 && r < rp.nload;
            } else {
              gi = g0 + (J - J0);
              wait = release = J <= Je;
            }
            if (App::FOLD_ROT || J <= Je) {
              if constexpr (App::IPROD) {  // inline producer: make sure this row is issued
                if (issuer && wait) issue_ahead(gi - g0);
              }
              if (wait) mbar_wait_u32(full_u32 + 8 * (gi & nmask), (gi >> p.nr_log2) & 1);
              const float* row = ringf + (gi & nmask) * slot_elems;
              const Frag<float, V> c = ldf<float, V>(row + ccol);
              const Frag<float, EW> el = ldf<float, EW>(row + ecol);
              const Frag<float, EW> eb = Frag<float, EW>::splat(emode == 1 ? c.get(0) : c.get(V - 1));
              app.template fold_h<U>(c, emode == 0 ? el : eb, lane, hf);
              // the raw row is done with: release its slot (virtual arrivals of the
              // first row precede its own; those of the last row follow it -- no
              // further loads, so its slot keeps its data)
              if (release) mbar_arrive_u32(empty_u32 + 8 * (gi & nmask));
              static_for<0, DEN>([&](auto kc) {
                constexpr int PH = F::sch.order[decltype(kc)::value];
                const int q = (J - F::sch.tmax[PH]) * DEN + PH;
                app.template fold_emit<F, RK, U, PH>(q, ys, ye, lane, xc, p, [&](const Frag<float, V>& o) {
                  store(optr, o);
                  optr += p.W;
                });
              });
            }
          });
          if constexpr (App::FOLD_ROT) app.template fold_rotate<RK>();
        }
      };
#ifdef KPERF_FOLD_ONLY2  // experiment: one fold instantiation per kernel (instruction-cache footprint)
      if (m.den == 2) { run(IC<2>{}); return; }
#else
      if (m.den == 2) run(IC<2>{});
      else run(IC<4>{});
      return;
#endif
    }
  }
#if KPERF_PIPELINE
  // software pipeline: row i+1 is fetched before row i is computed
  Rows cur = fetch(0);
  for (int ib = 0; ib < nv; ib += NWIN) {
    auto unrolled = [&](auto uc) {
      const int i = ib + decltype(uc)::value;
      if (i < nv) {
        Rows nxt;
        if (i + 1 < nv) nxt = fetch(i + 1);
        compute(uc, cur, vy0 + i);
        cur = nxt;
      }
    };
    static_for<0, NWIN>(unrolled);
  }
#else
  for (int ib = 0; ib < nv; ib += NWIN) {
    auto unrolled = [&](auto uc) {
      const int i = ib + decltype(uc)::value;
      // (rows >= nv: padded recipes, emit 0; vy only matters to the fused Gauss-Sobel).
      // The median's column-NN kernel keeps the guard (measured: its kept
      // warps are the critical path and gain nothing from the copies saved)
      if (!MEDC || i < nv) compute(uc, fetch(i), vy0 + i);
    };
    static_for<0, NWIN>(unrolled);
  }
#endif
  // every copy of this item lands, then its slots go back to the producer
  const int g_end = g0 + rp.nload;
#pragma unroll 1
  while (ready < g_end - 1) {
    ++ready;
    mbar_wait_u32(full_u32 + 8 * (ready & nmask), (ready >> p.nr_log2) & 1);
  }
#pragma unroll 1
  for (; released < g_end; ++released) mbar_arrive_u32(empty_u32 + 8 * (released & nmask));
}

template <class App, int SCHEME, int RECON, int NCW>
__device__ __forceinline__ void consumer_fast(const KParams& p, const Mask& m, const RowPlan& rp, int x0, int frame,
                                              int ys, int ye, int g0, uint32_t full_u32, uint32_t empty_u32,
                                              const typename App::T* ring, int slot_elems, const Recipe* rtab,
                                              float4* ctab) {
  consumer<App, SCHEME, RECON, NCW, true>(p, m, rp, x0, frame, ys, ye, g0, full_u32, empty_u32, ring, slot_elems,
                                          rtab, ctab);
}
template <class App, int SCHEME, int RECON, int NCW>
__device__ __noinline__ void consumer_generic(const KParams& p, const Mask& m, const RowPlan& rp, int x0, int frame,
                                              int ys, int ye, int g0, uint32_t full_u32, uint32_t empty_u32,
                                              const typename App::T* ring, int slot_elems, const Recipe* rtab,
                                              float4* ctab) {
  consumer<App, SCHEME, RECON, NCW, false>(p, m, rp, x0, frame, ys, ye, g0, full_u32, empty_u32, ring, slot_elems,
                                           rtab, ctab);
}

// One work item per CTA: CTA b processes item b = (frame, segment of seg_h
// output rows, strip of TW columns), strip fastest (the launcher sizes seg_h).
template <class App, int SCHEME, int RECON, int NCW>
__global__ void __launch_bounds__(32 * (NCW + 1), KPERF_MINB ? KPERF_MINB : (NCW == 2 ? 6 : (NCW == 3 ? 4 : App::MINB)))
    perf_kernel(const __grid_constant__ KParams p, const __grid_constant__ CUtensorMap tmap) {
  // (the TMA descriptor is a kernel parameter of its own: its generic address,
  // taken here, is what cp.async.bulk.tensor needs -- KParams::tmap is the host copy)
  using T = typename App::T;
  constexpr int V = App::V;
  constexpr int TW = NCW * 32 * V;
  extern __shared__ __align__(128) uint8_t smem[];
  uint64_t* full = reinterpret_cast<uint64_t*>(smem);
  uint64_t* empty = full + p.nr;
  const int bar_bytes = (2 * p.nr * 8 + 127) & ~127;
  T* ring = reinterpret_cast<T*>(smem + bar_bytes);
  const int slot_elems = p.row_elems * App::NIN;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int nrec = p.nrec;
  Recipe* rtab0 = reinterpret_cast<Recipe*>(smem + bar_bytes + (size_t)p.nr * slot_elems * sizeof(T));
  Recipe* rtab = rtab0 + max(warp - (p.inline_prod ? 0 : 1), 0) * nrec;  // one recipe table per consumer warp
  // per consumer warp: column scheme (fp32) LI weight table, 3 x 32 float4;
  // checkerboard: den phase entries (8 int4); kperf.cu sizes it the same way
  constexpr int CT = SCHEME == S_COL ? 96 : 8;
  float4* ctab = reinterpret_cast<float4*>(rtab0 + NCW * nrec) + max(warp - (p.inline_prod ? 0 : 1), 0) * CT;
  const Mask m{p.num, p.den, p.keep_one};
  const int n_items = p.n_strips * p.n_segs * p.frames;

  // consumer warps whose columns all lie right of the image have nothing to do
  const int x0 = (blockIdx.x % p.n_strips) * TW;
  const int nact = min(NCW, (p.W - x0 + 32 * V - 1) / (32 * V));
  if (threadIdx.x == 0) {
    for (int s = 0; s < p.nr; ++s) {
      mbar_init(&full[s], (p.loader == L_BULK || p.loader == L_RUNS || p.loader == L_TMA) ? 1u : 32u);
      mbar_init(&empty[s], (uint32_t)(32 * nact));  // every consumer lane arrives
    }
    mbar_fence_init();
  }
  __syncthreads();
  const int cw0 = p.inline_prod ? 0 : 1;  // first consumer warp
  if (warp - cw0 >= nact) return;
  const uint32_t full_u32 = smem_u32(full), empty_u32 = smem_u32(empty);

  const int g0 = 0;  // global load index of the item's first row (one item per CTA)
  {
    const int item = blockIdx.x;  // one work item per CTA (persistent variant)
    if (item >= n_items) return;
    int b = item;
    int strip, seg, frame;
    // folded row scheme without FOLD_EDGE: the first and last segment of a frame take the
    // per-row loop (clamped rows) and run ~1.5x longer than the folded
    // interior ones -- dispatch them first (longest items first), so they do
    // not form the launch's tail (C5: SMs idle 19% of the kernel otherwise)
    constexpr bool LPT = KPERF_LPT && SCHEME == S_ROW && App::FOLD && !App::FOLD_EDGE && KPERF_FOLD && sizeof(T) == 4;
    if (LPT && p.fold && p.n_segs >= 3 && (m.den == 2 || (m.den == 4 && m.keep_one)) &&
        b < 2 * p.n_strips * p.frames) {
      strip = b % p.n_strips;
      b /= p.n_strips;
      seg = (b & 1) ? p.n_segs - 1 : 0;
      frame = b >> 1;
    } else if (LPT && p.fold && p.n_segs >= 3 && (m.den == 2 || (m.den == 4 && m.keep_one))) {
      b -= 2 * p.n_strips * p.frames;
      strip = b % p.n_strips;
      b /= p.n_strips;
      seg = 1 + b % (p.n_segs - 2);
      frame = b / (p.n_segs - 2);
    } else {
      strip = b % p.n_strips;
      b /= p.n_strips;
      seg = b % p.n_segs;
      frame = b / p.n_segs;
    }
    (void)strip;  // (x0 above)
    const int ys = p.y_begin + seg * p.seg_h;
    const int ye = min(ys + p.seg_h, p.y_end);
    const RowPlan rp = make_row_plan<SCHEME>(p, m, ys, ye, App::VR);
    if (!p.inline_prod && warp == 0) {  // (Ia) data perforation: only kept samples leave HBM
      producer<T, SCHEME, App::NIN, TW>(p, m, rp, x0, frame, g0, full, empty, ring, &tmap);
    } else {
      const int nv = n_recipes<SCHEME>(p, ys, ye, App::VR);
      __syncwarp();
      const int nv_pad = (nv + App::NWIN - 1) / App::NWIN * App::NWIN;  // (<= nv + kRecPad)
      for (int i = lane; i < nv_pad; i += 32) {
        int emit;
        const int y = virtual_row<SCHEME>(p, rp, ys, ye, App::VR, min(i, nv - 1), emit);
        rtab[i] = make_recipe<SCHEME, RECON>(p, m, rp, y, i < nv ? emit : 0, slot_elems * (int)sizeof(T));
      }
      __syncwarp();
      const int xw = x0 + (warp - cw0) * 32 * V;
      // fast path: every lane chunk inside the image, and the right edge fragment
      // either inside or starting exactly at W (then it is the clamped border)
      const int exr = xw + 32 * V;
      const bool edges_ok = (exr + App::EW <= p.W) || (exr == p.W);
      // (32-B lane chunks: the fast path stores them with one 256-bit store, so
      // it also needs p.vec32 -- 32-B aligned output chunks; else generic)
      const bool st_ok = !(KPERF_ST256 && V * sizeof(T) == 32) || p.vec32;
      if (p.fast_ok && p.vec_io && st_ok && xw + 32 * V <= p.W && edges_ok)
        consumer_fast<App, SCHEME, RECON, NCW>(p, m, rp, x0, frame, ys, ye, g0, full_u32, empty_u32, ring,
                                               slot_elems, rtab, ctab);
      else
        consumer_generic<App, SCHEME, RECON, NCW>(p, m, rp, x0, frame, ys, ye, g0, full_u32, empty_u32, ring,
                                                  slot_elems, rtab, ctab);
    }
  }
}

template <class App, int SCHEME, int RECON, int NCW>
cudaError_t launch_one(const KParams& p, unsigned grid, size_t smem, cudaStream_t s) {
  auto k = perf_kernel<App, SCHEME, RECON, NCW>;
  static bool attr[kMaxDev] = {};
  const int dev = cur_dev();
  if (!attr[dev]) {
    cudaError_t e = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, 227 * 1024);
    if (e != cudaSuccess) return e;
    e = cudaFuncSetAttribute(k, cudaFuncAttributePreferredSharedMemoryCarveout, 100);  // max shared memory
    if (e != cudaSuccess) return e;
    attr[dev] = true;
  }
  // segment height: when not fixed by the caller (seg_auto), choose the number
  // of row segments so the CTA count fills whole waves of resident CTA slots
  // (occupancy API), discounted by the per-segment halo rows.
  KParams q = p;
  if (!App::IPROD) q.inline_prod = 0;  // (no inline-producer code in this app's consumer loop)
  // fp32 whole-row (TMA bulk) loaders, one input, radius <= 2: short fixed
  // segments -- many waves of short items overlap one CTA's ring fill and
  // drain with the others' streaming (round 2b sweep, tools/sweep_ring.py,
  // profiles/r02/sweep_ring_row.txt: 16-row segments, keep-one den >= 4 24
  // rows; C2 Gaussian5 exact 178 -> 165 us, row 1/2 LI 137 -> 130 us, row 3/4
  // 119 -> 110 us -- the extra halo reads of the neighbouring segment hit L2).
  // Cell loaders, u8, Hotspot and the fused pipeline measured best with the
  // wave-filling choice.
  // (only when that gives >= 2 CTAs per SM: short launches -- perf_run_host's
  // row chunks -- take the wave-filling choice)
  const int n_sms = dev_sms();
  // keep-one row schemes of den >= 4 re-read up to den - 1 extra kept rows per
  // segment boundary (halo + rebuild apron): KPERF_SEG_K1-row segments for them
  // (narrow 2-warp CTAs, C1's 512^2 frames: the row scheme runs 32-row
  // segments -- Gaussian5 row 1/2 LI 131.6 us vs 145.6 with 16, 135.3 with 64)
  // (radius-2 row scheme at den 2 -- Gaussian5 Rows1 -- measured best at 24)
  // (Stencil1: whole tile rows, >= 16 rows: 174 -> 162 us on C2)
  const int th1 = SCHEME == S_STENCIL1 ? p.tile1_h : 1;
  const int fseg = (SCHEME == S_STENCIL1) ? (KPERF_SEG_FIX + th1 - 1) / th1 * th1
                   : (SCHEME == S_ROW && NCW == 2) ? 32
                   : (SCHEME == S_ROW && p.keep_one && p.den >= 4) ? KPERF_SEG_K1
                   : (SCHEME == S_ROW && p.den == 2 && App::VR == 2) ? KPERF_SEG_K1 : KPERF_SEG_FIX;
  const bool fixed_seg = p.seg_auto && p.loader == L_BULK && App::VR <= 2 && App::NIN == 1 && sizeof(typename App::T) == 4 &&
                       fseg <= p.nrec - 2 * kMaxVR - kRecPad &&
                       (long long)p.n_strips * ((p.y_end - p.y_begin + fseg - 1) / fseg) * p.frames >= 2LL * n_sms;
  if (fixed_seg) {
    q.seg_h = fseg;
    q.n_segs = (p.y_end - p.y_begin + fseg - 1) / fseg;
    grid = (unsigned)((long long)q.n_strips * q.n_segs * q.frames);
  } else if (p.seg_auto) {
    static int per_sm_c[kMaxDev] = {};
    static size_t per_sm_smem[kMaxDev] = {};
    int& per_sm = per_sm_c[dev];
    if (per_sm == 0 || per_sm_smem[dev] != smem) {
      if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k, 32 * (NCW + (q.inline_prod ? 0 : 1)), smem) !=
              cudaSuccess ||
          per_sm < 1)
        per_sm = 1;
      per_sm_smem[dev] = smem;
    }
    const long long slots = (long long)per_sm * n_sms;
    const int rows = p.y_end - p.y_begin;
    const long long per_seg = (long long)p.n_strips * p.frames;
    double best = -1.0;
    const int seg_cap = p.seg_h;
    int best_n = (rows + seg_cap - 1) / seg_cap;
    const int th = SCHEME == S_STENCIL1 ? p.tile1_h : 1;  // Stencil1 segments hold whole tiles
    // segments >= 32 rows; >= 16 when 32-row segments cannot fill one wave (short launches)
    const int min_sh = per_seg * ((rows + 31) / 32) >= slots ? 32 : 16;
    for (int n = (rows + seg_cap - 1) / seg_cap; n <= (rows + min_sh - 1) / min_sh && n <= 4 * best_n + 64; ++n) {
      const int sh = ((rows + n - 1) / n + th - 1) / th * th;
      const int nn = (rows + sh - 1) / sh;
      const long long items = per_seg * nn;
      const long long waves = (items + slots - 1) / slots;
      const double fill = (double)items / (double)(waves * slots);
      const double halo = (double)sh / (double)(sh + 2 * App::VR + 2);
      const double score = fill * halo;
      if (score > best + 1e-9) { best = score; best_n = nn; }
    }
    q.seg_h = ((rows + best_n - 1) / best_n + th - 1) / th * th;
    q.n_segs = (rows + q.seg_h - 1) / q.seg_h;
    grid = (unsigned)((long long)q.n_strips * q.n_segs * q.frames);
  }
  k<<<grid, 32 * (NCW + (q.inline_prod ? 0 : 1)), smem, s>>>(q, q.tmap);
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
    case S_STENCIL1 * 2 + R_NN:
    case S_STENCIL1 * 2 + R_LI:
      if constexpr (App::NIN == 1 && App::VR <= 2) return launch_one<App, S_STENCIL1, R_NN, NCW>(p, grid, smem, s);
      break;
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
// fused pipeline on widths that are whole 768- but not 1024-column strips (C5's
// 3840): CTAs of 3 consumer warps (+ producer), 4 per SM -- no idle warp in a
// partial last strip
cudaError_t launch_gsobel_n3(int, int, const KParams&, unsigned, size_t, cudaStream_t);
cudaError_t launch_inversion(int, int, const KParams&, unsigned, size_t, cudaStream_t);

constexpr int kNCW = 4;  // consumer warps per CTA (tile width 1024 fp32 / 4096 u8 columns)
// narrow images (fp32 W <= 512, e.g. C1's 512^2 frames): 2 consumer warps per
// CTA, so no consumer warp idles right of the image (Gaussian / Sobel)
cudaError_t launch_gauss1_n2(int, int, const KParams&, unsigned, size_t, cudaStream_t);
cudaError_t launch_gauss2_n2(int, int, const KParams&, unsigned, size_t, cudaStream_t);
cudaError_t launch_sobel1_n2(int, int, const KParams&, unsigned, size_t, cudaStream_t);
cudaError_t launch_sobel2_n2(int, int, const KParams&, unsigned, size_t, cudaStream_t);

}  // namespace kp
