/*
 * aol_oracle.h -- CPU ORACLE for the ArrayOL HD->SD downscaler.
 *
 * TEST INFRASTRUCTURE ONLY.  Nothing in the product path (the CUDA library
 * under paper_conf_ipps_guortgbs11_b200/) may include, link or call this.
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline /
 * --impl reference legs use it.  It shares no code, header, table or
 * constant with the CUDA path.
 *
 * Source of every definition: /root/reference/PAPER.md ("P:Lnnn" below),
 * Guo et al., "Harnessing the Power of GPUs without Losing Abstractions in
 * SaC and ArrayOL", HIPS 2011.  Readings of silent/garbled passages are the
 * Z-numbered readings listed in DESIGN.md ("Readings of the paper").
 *
 * The oracle is deliberately slow and literal: the downscaler is the SaC
 * three-step decomposition of P:L372-382 -- (1) the input tiler gathers into
 * an intermediate array of shape [repetition ++ in_pattern] (Fig. 4), (2) the
 * task maps it to [repetition ++ out_pattern] (Fig. 5), (3) the output tiler
 * scatters it in the sequential order of Fig. 6 -- with both intermediates
 * materialised in host memory.  No blocking, fusion or reordering.
 *
 * Pins (tests/test_oracle_*.py): brute-force tiler enumeration, numpy
 * roll/transpose/reshape special cases, the Fig. 10/11 tiler constants, the
 * hand-derived ramp closed form, the constant-frame invariant, toroidal
 * shift-equivariance, locality, read-count histograms, pattern counts, output
 * shapes, C99 truncating-division tables.  The vertical filter (Z1/Z2) is a
 * reading: its tiler is pinned only by shapes, counts and invariants -- the
 * oracle is pinned to the READING, but parity with the paper's own vertical
 * taps is unpinned (the paper never prints them).
 */
#ifndef AOL_ORACLE_H
#define AOL_ORACLE_H

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

#define ORACLE_MAX_RANK 8

/* ArrayOL tiler record (Fig. 10; Section IV).
 * Matrices are stored row-major as [array_dim][column]: paving[a][j]
 * multiplies repetition index r_j, fitting[a][k] multiplies pattern index i_k
 * (reading Z6: Fig. 10 prints matrices by columns; Fig. 11 P:L720-725 pins
 * which entry multiplies which index). */
typedef struct {
    int32_t array_rank, rep_rank, pattern_rank;
    int64_t array_shape[ORACLE_MAX_RANK];
    int64_t rep_shape[ORACLE_MAX_RANK];
    int64_t pattern_shape[ORACLE_MAX_RANK];
    int64_t origin[ORACLE_MAX_RANK];
    int64_t paving[ORACLE_MAX_RANK][ORACLE_MAX_RANK];
    int64_t fitting[ORACLE_MAX_RANK][ORACLE_MAX_RANK];
} oracle_tiler;

/* Return codes: 0 ok, -1 invalid argument. */

/* Paper tilers for one plane (Fig. 10 for H; reading Z1 for V).
 * which: 0 = H input, 1 = H output, 2 = V input, 3 = V output.
 * H tilers take the plane H x W; V tilers take the intermediate H x Wo. */
int oracle_tiler_preset(int which, int64_t H, int64_t W, oracle_tiler* t);

/* Section IV / Fig. 4: G[r][i] = A[(o + P.r + F.i) mod s].
 * G is [rep_shape..., pattern_shape...] row-major.  elsize in {1,2,4,8}. */
int oracle_gather(const oracle_tiler* t, int elsize, const void* A, void* G);

/* Fig. 6: for r, i in row-major order, A[(o+P.r+F.i) mod s] = G[r][i].
 * A is modified in place (modarray semantics); the last writer wins. */
int oracle_scatter(const oracle_tiler* t, int elsize, const void* G, void* A);

/* Fig. 5, transcribed: three 6-tap sums of an 11-element pattern
 * at starts 0, 2, 5; tile[k] = tmp/6 - tmp%6 in C int arithmetic.
 * G is [nrep][11], T is [nrep][3]. */
int oracle_task_h(const int32_t* G, int64_t nrep, int32_t* T);

/* Vertical task, reading Z1/Z2: four 6-tap sums of a 12-element pattern at
 * starts 0, 2, 4, 6; tile[k] = tmp/6 - tmp%6.  G [nrep][12] -> T [nrep][4]. */
int oracle_task_v(const int32_t* G, int64_t nrep, int32_t* T);

/* Horizontal filter on one H x W plane -> Y [H][3W/8] (Fig. 2/10; W % 8 == 0). */
int oracle_downscale_h(const int32_t* X, int32_t* Y, int64_t H, int64_t W);

/* Vertical filter on one H x Wo plane -> Z [4H/9][Wo] (Fig. 2; H % 9 == 0). */
int oracle_downscale_v(const int32_t* Y, int32_t* Z, int64_t H, int64_t Wo);

/* Downscaler task graph fg -> hf -> vf -> fc (Fig. 3) over a
 * batch X [frames][channels][H][W] -> Z [frames][channels][4H/9][3W/8],
 * H filter first (Fig. 2).  Planes are independent; nthreads > 1
 * runs planes in parallel with OpenMP (timing baseline only).
 * checksums (nullable) receives oracle_checksum of each frame. */
int oracle_downscale_frame(const int32_t* X, int32_t* Z, int64_t frames, int64_t channels,
                           int64_t H, int64_t W, uint64_t* checksums, int nthreads);

/* Per-frame checksum (build infrastructure):
 * cs[n] = sum over (c,y,x) of (uint64)(uint32)Z[n][c][y][x] * (1 + (c*Ho + y)*Wo + x),
 * modulo 2^64. */
int oracle_checksum(const int32_t* Z, int64_t frames, int64_t channels, int64_t Ho, int64_t Wo,
                    uint64_t* checksums);

/* Threads OpenMP would use (1 if built without OpenMP). */
int oracle_max_threads(void);

#ifdef __cplusplus
}
#endif
#endif
