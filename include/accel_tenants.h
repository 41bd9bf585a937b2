/*
 * accel_tenants.h -- argument structs of the built-in tenant kernels of
 * libaccel.so (see accel_builtin_kernel).  One struct per kernel, passed as
 * accel_launch.args; all pointers are DEVICE pointers owned by the caller.
 *
 * PAPER.md only names the Parboil kernels it mixes (lines 289-298, 853-860,
 * 978-989); the definitions are the Parboil-shaped readings of DESIGN.md
 * §Tenants.  Virtual group (VG) = one original CTA; the "grid" column is the
 * original NDRange in VGs that the caller passes in accel_launch.grid.
 */
#ifndef ACCEL_TENANTS_H_
#define ACCEL_TENANTS_H_

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#define ACCEL_ALIGN64 alignas(64)
#else
#define ACCEL_ALIGN64 _Alignas(64)
#endif

/* An encoded TMA tensor map (CUtensorMap, 128 B, 64-B aligned), see
 * accel_tma_map_2d / accel_tma_map_3d.  Kernels that keep maps in their
 * argument struct receive it as a __grid_constant__ kernel parameter. */
typedef struct {
  ACCEL_ALIGN64 uint8_t bytes[128];
} accel_tmap;

/* mop -- PAPER.md Fig. 8a (lines 735-746).  block 256, grid ceil(n/256).
 * out[g] = ina[g] + inb[g] if (g / 256) < nconst else ina[g] - inb[g]. */
typedef struct {
  const float *ina;
  const float *inb;
  float *out;
  uint32_t n;
  uint32_t nconst;
} accel_mop_args;

/* stencil / stencil_x -- 7-point Jacobi, fp32, A[z][y][x] (x fastest).
 * Kernel "stencil" needs nx % 4 == 0 (16-B rows); "stencil_x" takes any nx.
 * block 256 (8 warps x 32 lanes x 4 x-points), VG tile 128 x 8 x 8 (x,y,z):
 * grid (ceil(nx/128), ceil(ny/8), ceil(nz/8)).  Launch r reads
 * (r == 0 ? a0 : buf[(r-1)&1]) and writes buf[r&1]; after T launches the
 * result is in buf[(T-1)&1].  Interior: c1*(6-neighbour sum) - c0*a;
 * faces copy the input.  a0/buf0/buf1: DEVICE pointers to nx*ny*nz floats,
 * 16-B aligned, no padding required.
 * Kernel "stencil2" (same arguments, nx % 4 == 0): VG tile 128 x 16 x 8, two
 * rows per warp -- grid (ceil(nx/128), ceil(ny/16), ceil(nz/8)).
 * Kernel "stencil_z16" (same arguments, nx % 4 == 0): VG tile 128 x 8 x 16 --
 * grid (ceil(nx/128), ceil(ny/8), ceil(nz/16)). */
typedef struct {
  const float *a0;
  float *buf0;
  float *buf1;
  uint32_t nx, ny, nz;
  float c0, c1;
} accel_stencil_args;

/* stencil_tma -- the same 7-point sweep (same launches, ping-pong and result
 * buffer as "stencil"), nx % 4 == 0.  Planes staged by TMA: tmaps = 3-D maps
 * (x, y, z extents nx, ny, nz; box 136 x 10 x 1; see accel_tma_map_3d) of a0,
 * buf0 and buf1, in that order.  block 288 (8 consumer warps + 1 TMA producer
 * warp), VG tile 128 x 8 x 8, grid (ceil(nx/128), ceil(ny/8), ceil(nz/8)). */
typedef struct {
  accel_tmap tmaps[3];
  float *buf0;
  float *buf1;
  uint32_t nx, ny, nz;
  float c0, c1;
  uint32_t l2hint;          /* diagnostic: bits 0-1: 1 = tensor loads with
                               an L2 evict_first cache policy, 2 = evict_last;
                               bit 3 (8): stage plane 1 before plane 0; bit 4
                               (16): wait 2 us before the first copy.  0 in
                               normal use. */
  const accel_tmap *gmaps;  /* diagnostic: non-NULL = read the three maps from
                               this DEVICE array instead of the parameters */
  const float *a0;          /* the input volume (kernel "stencil_bulk": 1-D
                               bulk copies need no tensor map) */
  uint32_t *dbg;            /* diagnostic: non-NULL = DEVICE block; consumers
                               compare every staged plane row with an L2 load
                               of the same input (scripts/diag_tma_check.py):
                               dbg[0] = mismatches, dbg[8 + 8k ..] = record k
                               {launch, z, y, x, staged bits, L2 bits, sm,
                               output-buffer bits} for k < 16 */
} accel_stencil_tma_args;

/* histo -- saturating histogram (Parboil histo main + final fused).
 * block 256, VG = `per_vg` samples (multiple of 4096), grid ceil(n/per_vg).
 * Launch r accumulates into hist[(r&1)*bins + b]; the VG that completes the
 * launch (done[r] reaches the VG count) writes sat[b] = min(hist, 255) and
 * zeroes hist[((r+1)&1)*bins ...] for launch r+1.  The request must clear
 * hist[0..bins) and done[0..launches) first.  Kernel "histo": bins <= 4096,
 * sample_bytes 1 (u8, bins == 256) or 4 (u32).  Kernel "histo_wide": bins <=
 * 16384, sample_bytes 4, per_vg < 65536 (16-bit private counters). */
typedef struct {
  const void *samples;
  uint32_t n;
  uint32_t bins;
  uint32_t sample_bytes;
  uint32_t per_vg;
  uint32_t *hist;  /* [2][bins] */
  uint8_t *sat;    /* [bins]    */
  uint32_t *done;  /* [launches] */
} accel_histo_args;

/* histo_prescan / histo_intermediates -- the first two kernels of Parboil's
 * histo pipeline, ahead of histo / histo_wide:
 *   "histo_prescan"        lo = min raw, hi = max raw (atomicMin / atomicMax
 *                          into *lo, *hi; the request sets *lo = 0xFFFFFFFF,
 *                          *hi = 0 first)
 *   "histo_intermediates"  bins_out[i] = (raw[i] - lo) * bins / (hi - lo + 1)
 *                          (64-bit integer arithmetic), the bin index stream
 *                          the main kernel counts
 * block 256, VG = per_vg raw u32 samples (multiple of 1024), grid
 * ceil(n / per_vg); raw / bins_out 16-B aligned DEVICE arrays. */
typedef struct {
  const uint32_t *raw;
  uint32_t *bins_out;
  uint32_t *lo;
  uint32_t *hi;
  uint32_t n, bins, per_vg;
} accel_histo_pre_args;

/* bfs -- level-synchronous top-down BFS on a directed CSR graph.
 * block 256, VG = 256 frontier vertices, static grid ceil(nv/256) (upper
 * bound; persistent CTAs read the live frontier size).  Launch l expands
 * level l.  The request must set level[] to -1 (memset 0xFF) and count[] to 0;
 * count has (launches + 1) entries, frontier is [2][nv]. */
typedef struct {
  const uint32_t *row_ptr;
  const int32_t *col;
  uint32_t nv;
  uint32_t src;
  int32_t *level;
  int32_t *frontier;
  uint32_t *count;
} accel_bfs_args;

/* cutcp -- cutoff Coulomb potential on the lattice h*(i,j,k).  atoms float4
 * (x,y,z,q) sorted into ncell^3 cells of edge `cell` (cell_start CSR).
 * block 128, VG = 8x8x8 lattice points, grid ceil(n?/8).  V[k][j][i]. */
typedef struct {
  const float *atoms;       /* float4[natoms] */
  const int32_t *cell_start;
  uint32_t ncell;
  float cell;
  uint32_t nx, ny, nz;
  float h, cutoff, excl;
  float *v;
} accel_cutcp_args;

/* tpacf -- angular two-point correlation histograms, SoA unit vectors.
 * block 256, VG = (256-point block i, set s in [0, 2*nsets], part q): s == 0
 * -> DD, s = 1..nsets -> RR of set s-1, s = nsets+1..2*nsets -> DR of set
 * s-nsets-1; the VG pairs its points with part q of the 256-point tiles of
 * the other set (the tiles split into qsplit near-equal runs; DD/RR tiles
 * start at the diagonal one); grid (ceil(npts/256), 2*nsets+1, qsplit).
 * dd/rr/dr u64[nedges+1], cleared by the request. */
typedef struct {
  const float *data;   /* [3][npts]          */
  const float *rand;   /* [nsets][3][npts]   */
  const float *binb;   /* [nedges] descending */
  uint32_t npts, nsets, nedges;
  uint32_t qsplit;     /* >= 1 */
  unsigned long long *dd, *rr, *dr;
} accel_tpacf_args;

/* spmv -- y = A x, CSR fp32.  block 256, VG = 64 rows, grid ceil(n/64).
 * Kernel "spmv_v4" (same arguments): 128-bit col/val loads in aligned
 * 4-element chunks; col and val must be 16-B aligned and readable up to
 * ceil(nnz/4)*4 elements (pad with anything: out-of-row elements are masked). */
typedef struct {
  const int32_t *row_ptr;
  const int32_t *col;
  const float *val;
  const float *x;
  float *y;
  uint32_t n;
} accel_spmv_args;

/* sgemm -- C[m][n] = A[m][k] . B[n][k]^T, fp32 in/out.
 * VG = one 128 x 128 tile of C, grid (ceil(n/128), ceil(m/128)). */
typedef struct {
  const float *a;
  const float *b;
  float *c;
  uint32_t m, n, k;
} accel_sgemm_args;

/* sgemm_split -- tf32 split of the two fp32 operands of the 3xTF32
 * tensor-core GEMM in ONE launch: hi = round-to-nearest tf32 of src, lo =
 * src - hi (exact), for segment 0 (A: src0/hi0/lo0, n0 elements) and
 * segment 1 (B).  block 256, VG = 4096 elements of one segment: VGs
 * [0, ceil(n0/4096)) split A, the next ceil(n1/4096) split B; grid = their
 * sum.  16-B aligned arrays; n1 = 0 for a single array.  Both sources are
 * row-major with `cols` (= K) elements per row; hi/lo rows are `ld` >= cols
 * elements apart (ld = K rounded up to a multiple of 4, so every row starts
 * 16-B aligned as TMA requires; the pad columns are never read: the tensor
 * maps' inner extent is cols and TMA zero-fills past it). */
typedef struct {
  const float *src0;
  float *hi0;
  float *lo0;
  uint64_t n0;
  const float *src1;
  float *hi1;
  float *lo1;
  uint64_t n1;
  uint32_t cols, ld;
} accel_sgemm_split_args;

/* sgemm_tc -- C[m][n] = A.B^T on tcgen05 tensor cores, 3xTF32
 * (A_hi.B_hi + A_hi.B_lo + A_lo.B_hi, fp32 accumulation in TMEM).  tmaps =
 * DEVICE pointer to four 128-B CUtensorMaps (A_hi, A_lo, B_hi, B_lo; each a
 * K-major fp32 matrix, box 32 x 128 for A and 32 x 256 for B, 128-B swizzle,
 * see accel_tma_map_2d; rows 16-B aligned, any k).  block 640, VG = 128 x 256
 * tile of C, grid (ceil(n/256), ceil(m/128)). */
typedef struct {
  const void *tmaps;
  float *c;
  uint32_t m, n, k;
} accel_sgemm_tc_args;

/* sgemm_tc1 -- the same product in one step: tmaps = DEVICE pointer to TWO
 * CUtensorMaps over the raw fp32 operands (A [m][k], box 16 x 128; B [n][k],
 * box 16 x 256; 64-B swizzle; row stride 4k bytes, so k % 4 == 0 -- TMA needs
 * 16-B aligned rows).  Each CTA splits every landed 32-wide slab into hi/lo in
 * shared memory before the MMAs; no hi/lo arrays in global memory.  Same
 * block, VG and grid as sgemm_tc; the k % 4 != 0 case takes split + tc. */
typedef accel_sgemm_tc_args accel_sgemm_tc1_args;

/* sad -- Parboil "sad" (H.264 motion estimation), three
 * kernels sharing one argument struct, run as the three steps of a request:
 *   "sad_4x4"   sad4[mb][p][b] = sum over the 4x4 sub-block b of the 16x16
 *               macroblock mb of |cur - ref displaced by (dx, dy)|, every
 *               (dx, dy) in [-R, R]^2 (p = (dy+R)(2R+1) + dx+R), reference
 *               coordinates clamped to the frame; VG = macroblock, grid
 *               (w/16, h/16), block 256, R <= 16
 *   "sad_8x8"   sad8[mb][p][q]: the four 8x8 sums of sad4; same grid
 *   "sad_16x16" sad16[mb][p]: the 16x16 sum of sad8; same grid
 * w, h multiples of 16; u16 pixels < 256 (so every SAD fits u16); DEVICE
 * buffers: cur/ref [h][w], sad4 [mbs][(2R+1)^2][16], sad8 [..][4], sad16 [..]. */
typedef struct {
  const uint16_t *cur;
  const uint16_t *ref;
  uint16_t *sad4;
  uint16_t *sad8;
  uint16_t *sad16;
  uint32_t w, h, R;
} accel_sad_args;

/* lbm -- Parboil "lbm" (D3Q19 lattice Boltzmann): launch r
 * does one pull stream + BGK collide step from (r == 0 ? f0 : buf[(r-1)&1])
 * into buf[r&1]; periodic boundaries, bounce-back on obstacle cells (flags
 * != 0), velocity order and weights of oracle/tenants.c.  f arrays are SoA
 * [19][nz][ny][nx] fp32 (DEVICE); block 128, VG = 128 cells of one x row,
 * grid (ceil(nx/128), ny, nz). */
typedef struct {
  const float *f0;
  float *buf0;
  float *buf1;
  const uint8_t *flags;
  uint32_t nx, ny, nz;
  float omega;
} accel_lbm_args;

/* mri-gridding -- Parboil "mri-gridding": non-Cartesian
 * samples convolved onto a G^3 grid with a separable Kaiser-Bessel kernel
 * (definition: oracle/tenants.c oracle_gridding).  Six kernels, the six steps
 * of one request, all with this argument struct:
 *   "gridding_binning"    VG = 1024 samples: bin[i] = cell of sample i (cells
 *                         of `cell` grid units), rank[i] = atomicAdd(count[bin])
 *   "gridding_scan_l1"    VG = 1024 bins: start[b] = exclusive scan within the
 *                         VG, block_sum[vg] = its total
 *   "gridding_scan_inter" 1 VG: exclusive scan of block_sum, start[B] = n
 *   "gridding_scan_add"   VG = 1024 bins: start[b] += block_sum[vg]
 *   "gridding_reorder"    VG = 1024 samples: the samples in bin order
 *   "gridding_grid"       VG = 8 x 8 x 8 grid points (256 threads, 2 points
 *                         each): the samples of the bins within hw of the
 *                         tile, per-point sums in 64-bit fixed point (2^-30:
 *                         order-independent, so NATIVE and SHARED agree bit
 *                         for bit whatever order the binning's atomics chose),
 *                         grid[p] = (re, im) fp32
 * B = cells^3 <= 1024 * 1024; count cleared by the request; DEVICE buffers. */
typedef struct {
  const float *x, *y, *z, *re, *im;   /* input samples [n] */
  const float *lut;                   /* [L] Kaiser-Bessel table */
  uint32_t L, n, G, cells;            /* cells per dimension = ceil(G / cell) */
  float hw, cell;                     /* kernel half-width, cell edge (grid units) */
  uint32_t *bin, *rank;               /* [n] */
  uint32_t *count;                    /* [B] */
  uint32_t *start;                    /* [B + 1] */
  uint32_t *block_sum;                /* [ceil(B / 1024)] */
  float *sx, *sy, *sz, *sre, *sim;    /* [n] in bin order */
  float *grid;                        /* [G][G][G][2] */
} accel_gridding_args;

/* mri-q ComputePhiMag: phimag = phir^2 + phii^2.  block 256, grid ceil(numk/256). */
typedef struct {
  const float *phir;
  const float *phii;
  float *phimag;
  uint32_t numk;
} accel_mriq_phimag_args;

/* mri-q ComputeQ: Qr + iQi = sum_k phimag_k exp(2 pi i k.x).
 * block 256, VG = 256 voxels, grid ceil(numx/256). */
typedef struct {
  const float *kx, *ky, *kz;
  const float *phimag;
  uint32_t numk;
  uint32_t numx;
  const float *x, *y, *z;
  float *qr, *qi;
} accel_mriq_q_args;

#ifdef __cplusplus
}
#endif
#endif /* ACCEL_TENANTS_H_ */
