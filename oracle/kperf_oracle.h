/*
 * kperf_oracle.h -- TEST INFRASTRUCTURE ONLY.
 *
 * The plain, slow, single-threaded CPU oracle for local memory-aware kernel
 * perforation (Maier, Cosenza, Juurlink, CGO'18; /root/reference/PAPER.md).
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline /
 * --impl reference legs may load it.  It shares no code, header, table or
 * constant with the CUDA path (paper_conf_cgo_maiercj18_b200/csrc); the only
 * common input is synth/ (seeded generators, no method arithmetic).
 *
 * Floating point is fp64 throughout (the paper fixes no precision); fp32
 * inputs are promoted on read.  u8 (median) work is integer.
 *
 * The enum values below are this file's own; the Python test layer maps the
 * product's enum names onto them by name.
 */
#ifndef KPERF_ORACLE_H
#define KPERF_ORACLE_H
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

enum { ORC_GAUSSIAN = 0, ORC_SOBEL = 1, ORC_MEDIAN = 2, ORC_HOTSPOT = 3, ORC_GAUSS_SOBEL = 4,
       ORC_INVERSION = 5 };
enum { ORC_NONE = 0, ORC_ROW = 1, ORC_COL = 2, ORC_CHECKER = 3, ORC_STENCIL1 = 4 };
enum { ORC_NN = 0, ORC_LI = 1 };
enum { ORC_METRIC_MRE = 0, ORC_METRIC_ME = 1, ORC_METRIC_MAE = 2 };

typedef struct {
  int app, W, H, radius;
  int scheme, num, den; /* skipped fraction num/den; num in {0, 1, den-1} */
  int recon;
  int granule;          /* G: pixels per column/checker cell (>= 1) */
  int tile_w, tile_h;   /* STENCIL1: work-group tile of output pixels */
  int tblock;           /* Hotspot temporal blocking (R19): T is perforated and rebuilt
                           only at steps it with it % tblock == 0 (<= 1: every step) */
} orc_params;

/* Step 1 -- perforation mask (1 = loaded / kept, 0 = skipped). */
int orc_is_kept(const orc_params* p, int x, int y);

/* Step 2 -- reconstruction of one in-image pixel. */
double orc_R_f32(const orc_params* p, const float* img, int x, int y);
int orc_R_u8(const orc_params* p, const uint8_t* img, int x, int y);
void orc_reconstruct_f32(const orc_params* p, const float* img, double* R);
void orc_reconstruct_u8(const orc_params* p, const uint8_t* img, uint8_t* R);

/* Step 3 -- unchanged stencil on the rebuilt image (clamp-to-edge). */
void orc_run_f32(const orc_params* p, const float* in, double* out);
void orc_run_u8(const orc_params* p, const uint8_t* in, uint8_t* out);
/* one output pixel, rebuilding only the pixels its window reads */
double orc_run_pixel_f32(const orc_params* p, const float* in, int x, int y);
int orc_run_pixel_u8(const orc_params* p, const uint8_t* in, int x, int y);

/* Hotspot (Rodinia 2D transient thermal stencil), iters steps; T and P both
 * perforated and rebuilt every step (every tblock-th step for T when
 * tblock > 1; P is static, so its rebuild is the same at every step). */
void orc_hotspot_coeffs(double* step_div_cap, double* rx_1, double* ry_1, double* rz_1, double* amb);
void orc_hotspot_run(const orc_params* p, const float* T0, const float* P, int iters, double* Tout);
/* iters steps on a window of the global grid (origin ox, oy; w x h); T is
 * fp64 in/out, P fp32; values near window edges that are not image edges
 * are invalid after the steps (outside the dependency cone). */
void orc_hotspot_window(const orc_params* p, double* T, const float* P, int ox, int oy, int w, int h, int iters);
/* final temperature on the rectangle [x0,x0+w) x [y0,y0+h) only, computed on
 * the dependency cone (same result as orc_hotspot_run restricted to it). */
void orc_hotspot_rect(const orc_params* p, const float* T0, const float* P, int iters, int x0, int y0,
                      int w, int h, double* out);

/* Step 4 -- error metric. */
double orc_error_f64(int metric, const double* exact, const double* approx, long long n, long long* count);
double orc_error_f32(int metric, const float* exact, const float* approx, long long n, long long* count);
double orc_error_u8(int metric, const uint8_t* exact, const uint8_t* approx, long long n, long long* count);

#ifdef __cplusplus
}
#endif
#endif
