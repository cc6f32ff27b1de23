/*
 * kperf_oracle.c -- TEST INFRASTRUCTURE ONLY (see kperf_oracle.h).
 *
 * Plain fp64 CPU oracle of local memory-aware kernel perforation, written
 * from /root/reference/PAPER.md in the paper's order:
 *   Fig. 1b: input buffer -> (Ia) data perforation ->
 *   (Ib) data reconstruction -> kernel execution -> output buffer.
 * No blocking, tiling, fusion or reordering: every function below is the
 * definition written out.  Readings of silent/garbled passages are the
 * DESIGN.md "Readings" table (R1..R16); each use below names its reading.
 */
#include "kperf_oracle.h"

#include <math.h>
#include <stdlib.h>
#include <string.h>

/* ------------------------------------------------------------------------ */
/* Step 1: perforation mask.  PAPER.md:467-478 (Sec. 4.4, row scheme, Fig. 4:
 * "skips the loading of rows in a work group tile ... in adjacent work groups
 * the same approximation scheme is applied, the schemes match each other"),
 * PAPER.md:814-817 (Rows1 = every other row, Rows2 = 3 out of 4 rows),
 * PAPER.md:440-449 (scheme must match the >= 32 B memory granularity).
 * Readings R1 (rate = skipped fraction num/den), R2 (phase anchored to global
 * coordinates, line 0 kept), R3 (column/checker cells are G pixels wide),
 * R4 (checkerboard lattice q = (x/G + y) mod den).                          */
int orc_is_kept(const orc_params* p, int x, int y) {
  if (p->scheme == ORC_NONE || p->scheme == ORC_STENCIL1 || p->num == 0) return 1;
  const int den = p->den;
  int q;
  if (p->scheme == ORC_ROW) q = y % den;
  else if (p->scheme == ORC_COL) q = (x / p->granule) % den;
  else q = (x / p->granule + y) % den;
  if (p->num == den - 1) return q == 0;   /* keep one line of every den */
  return q != den - 1;                    /* skip one line of every den */
}

/* ------------------------------------------------------------------------ */
/* Step 2: reconstruction on a window of the image.
 * PAPER.md:539-543 (nearest-neighbour: "picking the nearest value that was
 * loaded"), PAPER.md:544-549 (linear interpolation needs loaded elements on
 * both sides, else nearest-neighbour), PAPER.md:334-341 (x1 = (x0+x2)/2).
 * Reading R5: ROW and CHECKER rebuild along y in the same column, COL along x
 * in the same row.  R6: NN tie goes to the lower coordinate.  R7: LI =
 * (I_a*db + I_b*da)/(da+db) with da, db the distances to the nearest loaded
 * samples; u8 rounds half up in integers.  Only loaded samples are read.
 *
 * A window is W x H pixels of a larger image whose pixel (0,0) sits at global
 * (ox, oy); the mask is evaluated on global coordinates, the search for loaded
 * samples stays inside the window.  The whole image is the window (0,0,W,H). */
typedef struct {
  const orc_params* p;
  int ox, oy, w, h;       /* window origin (global) and size */
  const float* f32;       /* exactly one of the three is non-NULL */
  const double* f64;
  const uint8_t* u8;
} view_t;

static double vget(const view_t* v, int x, int y) {
  const long long i = (long long)y * v->w + x;
  if (v->f32) return (double)v->f32[i];
  if (v->f64) return v->f64[i];
  return (double)v->u8[i];
}

static int vkept(const view_t* v, int x, int y) { return orc_is_kept(v->p, v->ox + x, v->oy + y); }

/* find the nearest loaded sample on each side of (x,y) along the scheme axis;
 * returns 0 when the pixel itself is loaded. */
static int find_sources(const view_t* v, int x, int y, int* ax, int* ay, int* da, int* bx, int* by,
                        int* db) {
  if (vkept(v, x, y)) return 0;
  const int horizontal = (v->p->scheme == ORC_COL);
  *da = 0; *db = 0;
  for (int d = 1;; ++d) {
    const int xx = horizontal ? x - d : x, yy = horizontal ? y : y - d;
    if (xx < 0 || yy < 0) break;
    if (vkept(v, xx, yy)) { *ax = xx; *ay = yy; *da = d; break; }
  }
  for (int d = 1;; ++d) {
    const int xx = horizontal ? x + d : x, yy = horizontal ? y : y + d;
    if (xx >= v->w || yy >= v->h) break;
    if (vkept(v, xx, yy)) { *bx = xx; *by = yy; *db = d; break; }
  }
  return 1;
}

static double recon_f(const view_t* v, int x, int y) {
  int ax = 0, ay = 0, bx = 0, by = 0, da, db;
  if (!find_sources(v, x, y, &ax, &ay, &da, &bx, &by, &db)) return vget(v, x, y);
  if (da == 0 && db == 0) return NAN; /* no loaded sample on the axis: plans reject this */
  if (v->p->recon == ORC_LI && da > 0 && db > 0)
    return (vget(v, ax, ay) * (double)db + vget(v, bx, by) * (double)da) / (double)(da + db);
  if (db == 0 || (da > 0 && da <= db)) return vget(v, ax, ay);
  return vget(v, bx, by);
}

static int recon_u(const view_t* v, int x, int y) {
  int ax = 0, ay = 0, bx = 0, by = 0, da, db;
  if (!find_sources(v, x, y, &ax, &ay, &da, &bx, &by, &db)) return v->u8[(long long)y * v->w + x];
  if (da == 0 && db == 0) return -1;
  const int ia = (da > 0) ? v->u8[(long long)ay * v->w + ax] : 0;
  const int ib = (db > 0) ? v->u8[(long long)by * v->w + bx] : 0;
  if (v->p->recon == ORC_LI && da > 0 && db > 0) return (ia * db + ib * da + (da + db) / 2) / (da + db);
  if (db == 0 || (da > 0 && da <= db)) return ia;
  return ib;
}

static view_t whole(const orc_params* p) {
  view_t v; memset(&v, 0, sizeof v);
  v.p = p; v.w = p->W; v.h = p->H;
  return v;
}

double orc_R_f32(const orc_params* p, const float* img, int x, int y) {
  view_t v = whole(p); v.f32 = img;
  return recon_f(&v, x, y);
}

int orc_R_u8(const orc_params* p, const uint8_t* img, int x, int y) {
  view_t v = whole(p); v.u8 = img;
  return recon_u(&v, x, y);
}

void orc_reconstruct_f32(const orc_params* p, const float* img, double* R) {
  view_t v = whole(p); v.f32 = img;
  for (int y = 0; y < p->H; ++y)
    for (int x = 0; x < p->W; ++x) R[(long long)y * p->W + x] = recon_f(&v, x, y);
}

void orc_reconstruct_u8(const orc_params* p, const uint8_t* img, uint8_t* R) {
  view_t v = whole(p); v.u8 = img;
  for (int y = 0; y < p->H; ++y)
    for (int x = 0; x < p->W; ++x) R[(long long)y * p->W + x] = (uint8_t)recon_u(&v, x, y);
}

/* ------------------------------------------------------------------------ */
/* Stencil1 (PAPER.md:479-490, Fig. 5; :819-821 "Stencil1 is perforation of
 * the boundaries of a work group tile and uses nearest-neighbor
 * interpolation"): a work group fetches only its tile's interior; the halo
 * elements its stencil reads are rebuilt by NN from the loaded tile, i.e. the
 * tile-border element (reading R18).  The stencil of output (x, y) therefore
 * reads the input at coordinates clamped to its own tile (and to the image).
 * LI needs loaded elements on both sides, which a halo element never has, so
 * it falls back to NN. */
static int tile_lo(int v, int t) { return (v / t) * t; }

/* Step 3: the unchanged application stencils (Sec. 6.1).
 * Reading R8: clamp-to-edge addressing at image borders.  R9: Gaussian
 * weights are binomial b(x)b(y) / (sum b)^2, b = [1,2,1] (r=1) or
 * [1,4,6,4,1] (r=2).  R10: Sobel Gx = sum s(dy) d(dx) R, Gy = sum d(dy) s(dx) R
 * with s = [1,2,1], d = [-1,0,1] (r=1) or s = [1,4,6,4,1], d = [-1,-2,0,2,1]
 * (r=2); output sqrt(Gx^2 + Gy^2).  R11: the median is the true median (5th
 * of 9).  Inversion: 255 - R.                            */
static const double B1[3] = {1, 2, 1}, B2[5] = {1, 4, 6, 4, 1};
static const double D1[3] = {-1, 0, 1}, D2[5] = {-1, -2, 0, 2, 1};

static int clampi(int v, int lo, int hi) { return v < lo ? lo : (v > hi ? hi : v); }

/* stencil of a float app at (x, y) of image R (W x H, fp64) */
static double stencil_f(int app, int r, const double* R, int W, int H, int x, int y) {
  if (app == ORC_INVERSION) return 255.0 - R[(long long)y * W + x];
  const double* b = (r == 1) ? B1 : B2;
  const double* d = (r == 1) ? D1 : D2;
  if (app == ORC_GAUSSIAN) {
    double s = 0, norm = 0;
    for (int i = 0; i <= 2 * r; ++i) norm += b[i];
    for (int i = -r; i <= r; ++i)
      for (int j = -r; j <= r; ++j)
        s += b[i + r] * b[j + r] * R[(long long)clampi(y + i, 0, H - 1) * W + clampi(x + j, 0, W - 1)];
    return s / (norm * norm);
  }
  /* ORC_SOBEL */
  double gx = 0, gy = 0;
  for (int i = -r; i <= r; ++i)
    for (int j = -r; j <= r; ++j) {
      const double v = R[(long long)clampi(y + i, 0, H - 1) * W + clampi(x + j, 0, W - 1)];
      gx += b[i + r] * d[j + r] * v;
      gy += d[i + r] * b[j + r] * v;
    }
  return sqrt(gx * gx + gy * gy);
}

static int median9(int* v) {
  for (int i = 1; i < 9; ++i) { /* insertion sort */
    const int t = v[i];
    int j = i - 1;
    while (j >= 0 && v[j] > t) { v[j + 1] = v[j]; --j; }
    v[j + 1] = t;
  }
  return v[4];
}

static void run_stencil1_f32(const orc_params* p, const float* in, double* out) {
  const int W = p->W, H = p->H, r = (p->app == ORC_INVERSION) ? 0 : p->radius;
  const int n = 2 * r + 1;
  double win[25];
  for (int y = 0; y < H; ++y)
    for (int x = 0; x < W; ++x) {
      const int tx0 = tile_lo(x, p->tile_w), ty0 = tile_lo(y, p->tile_h);
      const int tx1 = (tx0 + p->tile_w < W ? tx0 + p->tile_w : W) - 1;
      const int ty1 = (ty0 + p->tile_h < H ? ty0 + p->tile_h : H) - 1;
      for (int i = -r; i <= r; ++i)
        for (int j = -r; j <= r; ++j)
          win[(i + r) * n + (j + r)] = (double)in[(long long)clampi(y + i, ty0, ty1) * W + clampi(x + j, tx0, tx1)];
      out[(long long)y * W + x] = stencil_f(p->app, r, win, n, n, r, r);
    }
}

void orc_run_f32(const orc_params* p, const float* in, double* out) {
  const int W = p->W, H = p->H;
  if (p->scheme == ORC_STENCIL1 && (p->app == ORC_GAUSSIAN || p->app == ORC_SOBEL || p->app == ORC_INVERSION)) {
    run_stencil1_f32(p, in, out);
    return;
  }
  const long long n = (long long)W * H;
  double* R = (double*)malloc(sizeof(double) * n);
  orc_reconstruct_f32(p, in, R);
  if (p->app == ORC_GAUSS_SOBEL) { /* Sobel3 of the Gaussian5 of the rebuilt frame (R12) */
    double* G = (double*)malloc(sizeof(double) * n);
    for (int y = 0; y < H; ++y)
      for (int x = 0; x < W; ++x) G[(long long)y * W + x] = stencil_f(ORC_GAUSSIAN, 2, R, W, H, x, y);
    for (int y = 0; y < H; ++y)
      for (int x = 0; x < W; ++x) out[(long long)y * W + x] = stencil_f(ORC_SOBEL, 1, G, W, H, x, y);
    free(G);
  } else {
    for (int y = 0; y < H; ++y)
      for (int x = 0; x < W; ++x) out[(long long)y * W + x] = stencil_f(p->app, p->radius, R, W, H, x, y);
  }
  free(R);
}

void orc_run_u8(const orc_params* p, const uint8_t* in, uint8_t* out) {
  const int W = p->W, H = p->H;
  if (p->scheme == ORC_STENCIL1) {
    for (int y = 0; y < H; ++y)
      for (int x = 0; x < W; ++x) {
        const int tx0 = tile_lo(x, p->tile_w), ty0 = tile_lo(y, p->tile_h);
        const int tx1 = (tx0 + p->tile_w < W ? tx0 + p->tile_w : W) - 1;
        const int ty1 = (ty0 + p->tile_h < H ? ty0 + p->tile_h : H) - 1;
        int v[9], k = 0;
        for (int i = -1; i <= 1; ++i)
          for (int j = -1; j <= 1; ++j) v[k++] = in[(long long)clampi(y + i, ty0, ty1) * W + clampi(x + j, tx0, tx1)];
        out[(long long)y * W + x] = (uint8_t)median9(v);
      }
    return;
  }
  uint8_t* R = (uint8_t*)malloc((size_t)W * H);
  orc_reconstruct_u8(p, in, R);
  for (int y = 0; y < H; ++y)
    for (int x = 0; x < W; ++x) {
      int v[9], k = 0;
      for (int i = -1; i <= 1; ++i)
        for (int j = -1; j <= 1; ++j)
          v[k++] = R[(long long)clampi(y + i, 0, H - 1) * W + clampi(x + j, 0, W - 1)];
      out[(long long)y * W + x] = (uint8_t)median9(v);
    }
  free(R);
}

/* One output pixel: rebuild just the window it reads (same definitions). */
double orc_run_pixel_f32(const orc_params* p, const float* in, int x, int y) {
  const int W = p->W, H = p->H;
  if (p->scheme == ORC_STENCIL1) {
    const int r = (p->app == ORC_INVERSION) ? 0 : p->radius, n = 2 * r + 1;
    const int tx0 = tile_lo(x, p->tile_w), ty0 = tile_lo(y, p->tile_h);
    const int tx1 = (tx0 + p->tile_w < W ? tx0 + p->tile_w : W) - 1;
    const int ty1 = (ty0 + p->tile_h < H ? ty0 + p->tile_h : H) - 1;
    double win[25];
    for (int i = -r; i <= r; ++i)
      for (int j = -r; j <= r; ++j)
        win[(i + r) * n + (j + r)] = (double)in[(long long)clampi(y + i, ty0, ty1) * W + clampi(x + j, tx0, tx1)];
    return stencil_f(p->app, r, win, n, n, r, r);
  }
  if (p->app == ORC_GAUSS_SOBEL) {
    /* Gaussian5 at the 3x3 clamped neighbours, each from a 5x5 rebuilt window */
    double g[9];
    int k = 0;
    for (int i = -1; i <= 1; ++i)
      for (int j = -1; j <= 1; ++j) {
        const int gy = clampi(y + i, 0, H - 1), gx = clampi(x + j, 0, W - 1);
        double s = 0;
        for (int u = -2; u <= 2; ++u)
          for (int w = -2; w <= 2; ++w)
            s += B2[u + 2] * B2[w + 2] * orc_R_f32(p, in, clampi(gx + w, 0, W - 1), clampi(gy + u, 0, H - 1));
        g[k++] = s / 256.0;
      }
    double gxs = 0, gys = 0;
    for (int i = 0; i < 3; ++i)
      for (int j = 0; j < 3; ++j) {
        gxs += B1[i] * D1[j] * g[i * 3 + j];
        gys += D1[i] * B1[j] * g[i * 3 + j];
      }
    return sqrt(gxs * gxs + gys * gys);
  }
  const int r = (p->app == ORC_INVERSION) ? 0 : p->radius;
  /* local (2r+1)^2 copy of the clamped rebuilt window, then the same stencil */
  double win[25];
  const int n = 2 * r + 1;
  for (int i = -r; i <= r; ++i)
    for (int j = -r; j <= r; ++j)
      win[(i + r) * n + (j + r)] = orc_R_f32(p, in, clampi(x + j, 0, W - 1), clampi(y + i, 0, H - 1));
  return stencil_f(p->app, r, win, n, n, r, r);
}

int orc_run_pixel_u8(const orc_params* p, const uint8_t* in, int x, int y) {
  int v[9], k = 0;
  if (p->scheme == ORC_STENCIL1) {
    const int tx0 = tile_lo(x, p->tile_w), ty0 = tile_lo(y, p->tile_h);
    const int tx1 = (tx0 + p->tile_w < p->W ? tx0 + p->tile_w : p->W) - 1;
    const int ty1 = (ty0 + p->tile_h < p->H ? ty0 + p->tile_h : p->H) - 1;
    for (int i = -1; i <= 1; ++i)
      for (int j = -1; j <= 1; ++j) v[k++] = in[(long long)clampi(y + i, ty0, ty1) * p->W + clampi(x + j, tx0, tx1)];
    return median9(v);
  }
  for (int i = -1; i <= 1; ++i)
    for (int j = -1; j <= 1; ++j)
      v[k++] = orc_R_u8(p, in, clampi(x + j, 0, p->W - 1), clampi(y + i, 0, p->H - 1));
  return median9(v);
}

/* ------------------------------------------------------------------------ */
/* Hotspot.  The paper cites Rodinia's 2D transient thermal simulation
 * (ref [2] at PAPER.md:1118-1121) and perforates it with
 * row scheme 1.  The update is Rodinia's:
 *   T' = T + (step/Cap) * (P + (T_S + T_N - 2T)/Ry + (T_E + T_W - 2T)/Rx
 *                          + (amb - T)/Rz)
 * with clamped neighbours.  Reading R13: Rodinia's constants with the cell
 * size of the 1024 x 1024 chip fixed for every grid size (the literal
 * constants are unstable beyond n ~ 1386).  R14: T and P are both perforated
 * and rebuilt every step.  R19: with temporal blocking (tblock > 1) T is
 * perforated at every tblock-th step only.                                 */
void orc_hotspot_coeffs(double* step_div_cap, double* rx_1, double* ry_1, double* rz_1, double* amb) {
  const double t_chip = 0.0005, chip = 0.016;
  const double gw = chip / 1024.0, gh = chip / 1024.0;
  const double spec_heat_si = 1.75e6, k_si = 100.0, factor_chip = 0.5, max_pd = 3.0e6, precision = 0.001;
  const double cap = factor_chip * spec_heat_si * t_chip * gw * gh;
  const double rx = gw / (2.0 * k_si * t_chip * gh);
  const double ry = gh / (2.0 * k_si * t_chip * gw);
  const double rz = t_chip / (k_si * gh * gw);
  const double max_slope = max_pd / (factor_chip * t_chip * spec_heat_si);
  const double step = precision / max_slope;
  *step_div_cap = step / cap;
  *rx_1 = 1.0 / rx;
  *ry_1 = 1.0 / ry;
  *rz_1 = 1.0 / rz;
  *amb = 80.0;
}

/* iters steps on a window [ox,ox+w) x [oy,oy+h) of the global grid; T (fp64,
 * in/out) and P (fp32 input) are window-sized.  Inside the window this is the
 * definition above; values within iters*(1+apron) of a window edge that is
 * not an image edge are invalid (outside the dependency cone). */
static void hotspot_window(const orc_params* p, double* T, const float* P, int ox, int oy, int w, int h,
                           int iters) {
  double sdc, rx_1, ry_1, rz_1, amb;
  orc_hotspot_coeffs(&sdc, &rx_1, &ry_1, &rz_1, &amb);
  const long long n = (long long)w * h;
  double* Tr = (double*)malloc(sizeof(double) * n);
  double* Pr = (double*)malloc(sizeof(double) * n);
  view_t vp; memset(&vp, 0, sizeof vp);
  vp.p = p; vp.ox = ox; vp.oy = oy; vp.w = w; vp.h = h; vp.f32 = P;
  for (int y = 0; y < h; ++y)
    for (int x = 0; x < w; ++x) Pr[(long long)y * w + x] = recon_f(&vp, x, y);
  view_t vt = vp; vt.f32 = NULL;
  const int tb = p->tblock > 1 ? p->tblock : 1;
  for (int it = 0; it < iters; ++it) {
    vt.f64 = T;
    /* R19 (temporal blocking): a kernel that keeps T on chip
     * for tb steps loads it from memory -- perforated, then rebuilt -- only
     * at the first of them; the other steps read the full on-chip T. */
    const int perforate = (it % tb) == 0;
    for (int y = 0; y < h; ++y)
      for (int x = 0; x < w; ++x)
        Tr[(long long)y * w + x] = perforate ? recon_f(&vt, x, y) : T[(long long)y * w + x];
    for (int y = 0; y < h; ++y)
      for (int x = 0; x < w; ++x) {
        const double tc = Tr[(long long)y * w + x];
        const double tn = Tr[(long long)clampi(y - 1, 0, h - 1) * w + x];
        const double ts = Tr[(long long)clampi(y + 1, 0, h - 1) * w + x];
        const double te = Tr[(long long)y * w + clampi(x + 1, 0, w - 1)];
        const double tw = Tr[(long long)y * w + clampi(x - 1, 0, w - 1)];
        T[(long long)y * w + x] = tc + sdc * (Pr[(long long)y * w + x] + (ts + tn - 2.0 * tc) * ry_1 +
                                              (te + tw - 2.0 * tc) * rx_1 + (amb - tc) * rz_1);
      }
  }
  free(Tr);
  free(Pr);
}

/* iters steps on a caller-owned window (global origin ox, oy; w x h) -- the
 * building block of the band-decomposition test (tests/test_multirank_cpu.py) */
void orc_hotspot_window(const orc_params* p, double* T, const float* P, int ox, int oy, int w, int h, int iters) {
  hotspot_window(p, T, P, ox, oy, w, h, iters);
}

void orc_hotspot_run(const orc_params* p, const float* T0, const float* P, int iters, double* Tout) {
  const long long n = (long long)p->W * p->H;
  for (long long i = 0; i < n; ++i) Tout[i] = (double)T0[i];
  hotspot_window(p, Tout, P, 0, 0, p->W, p->H, iters);
}

void orc_hotspot_rect(const orc_params* p, const float* T0, const float* P, int iters, int x0, int y0,
                      int w, int h, double* out) {
  /* dependency cone: one step reads +-1 (stencil) plus the rebuild distance,
   * at most den along the scheme axis (den*G pixels for COL). */
  int ex = 1, ey = 1;
  if (p->scheme == ORC_COL && p->num > 0) ex += p->den * p->granule;
  if ((p->scheme == ORC_ROW || p->scheme == ORC_CHECKER) && p->num > 0) ey += p->den;
  const long long mx = (long long)iters * ex, my = (long long)iters * ey;
  const int wx0 = (int)(x0 - mx < 0 ? 0 : x0 - mx);
  const int wy0 = (int)(y0 - my < 0 ? 0 : y0 - my);
  const int wx1 = (int)(x0 + w + mx > p->W ? p->W : x0 + w + mx);
  const int wy1 = (int)(y0 + h + my > p->H ? p->H : y0 + h + my);
  const int ww = wx1 - wx0, wh = wy1 - wy0;
  double* T = (double*)malloc(sizeof(double) * (size_t)ww * wh);
  float* Pw = (float*)malloc(sizeof(float) * (size_t)ww * wh);
  for (int y = 0; y < wh; ++y)
    for (int x = 0; x < ww; ++x) {
      const long long g = (long long)(wy0 + y) * p->W + (wx0 + x);
      T[(long long)y * ww + x] = (double)T0[g];
      Pw[(long long)y * ww + x] = P[g];
    }
  hotspot_window(p, T, Pw, wx0, wy0, ww, wh, iters);
  for (int y = 0; y < h; ++y)
    for (int x = 0; x < w; ++x) out[(long long)y * w + x] = T[(long long)(y0 - wy0 + y) * ww + (x0 - wx0 + x)];
  free(T);
  free(Pw);
}

/* ------------------------------------------------------------------------ */
/* Step 4: error.  PAPER.md:576-584: "The MRE is determined by calculating the
 * difference of result and the value and then dividing by the true value"
 * (formula garbled at :579); zero true values make it undefined; Sobel uses
 * "the mean error".  Reading R15: MRE = mean over {i : e_i != 0} of
 * |e_i - a_i| / |e_i|.  R16: Sobel's mean error = sum|e-a| / sum|e|.
 * MAE = mean |e - a| is also provided.  fp64, index order.                 */
#define ERROR_BODY(GET_E, GET_A)                                              \
  double s = 0, t = 0;                                                        \
  long long c = 0;                                                            \
  for (long long i = 0; i < n; ++i) {                                         \
    const double e = GET_E, a = GET_A;                                        \
    if (metric == ORC_METRIC_MRE) {                                           \
      if (e != 0.0) { s += fabs(e - a) / fabs(e); ++c; }                      \
    } else {                                                                  \
      s += fabs(e - a); t += fabs(e); ++c;                                    \
    }                                                                         \
  }                                                                           \
  if (count) *count = c;                                                      \
  if (metric == ORC_METRIC_ME) return t > 0 ? s / t : 0.0;                    \
  return c > 0 ? s / (double)c : 0.0;

double orc_error_f64(int metric, const double* exact, const double* approx, long long n, long long* count) {
  ERROR_BODY(exact[i], approx[i])
}
double orc_error_f32(int metric, const float* exact, const float* approx, long long n, long long* count) {
  ERROR_BODY((double)exact[i], (double)approx[i])
}
double orc_error_u8(int metric, const uint8_t* exact, const uint8_t* approx, long long n, long long* count) {
  ERROR_BODY((double)exact[i], (double)approx[i])
}
