/* CPU ORACLE -- TEST INFRASTRUCTURE ONLY (see oracle/__init__.py).  Shares no code with the CUDA
 * path.  The oracle's own matrix product (north star "its own naive
 * GEMM"): the definition
 *
 *     C[i, j] = sum_{k = 0}^{K-1} A[i, k] * B[k, j]
 *
 * written out with a FIXED summation order: every output starts at +0.0 and takes its K terms one
 * at a time in increasing k, c <- c + (a * b), the product rounded to binary64 and then the sum
 * rounded (no fused multiply-add: built with -ffp-contract=off).  The loops are tiled for the cache
 * (output tiles, one level of blocking over k), but a tile only decides WHEN an output's partial sum
 * is held in a register or in the tile buffer, never the order of its terms, so the result is
 * bit-identical for any tile size, thread count or vector width.  Threads (OpenMP) split the
 * OUTPUT tiles only.  This is the B := Omega A of Fig. 2(b) line 3, the
 * C := B A^T / B := C A of Fig. 2(a) lines 7 and 12, and every vector product of the
 * Householder steps.
 *
 * Layout: A[i, k] at A[i*sai + k*sak] (any strides); B[k, j] at B[k*ldb + j] (unit stride in j);
 * C[i, j] at C[i*ldc + j] (unit stride in j), overwritten.
 */
#include <stdint.h>
#include <string.h>

#define MB 128 /* output rows per tile  */
#define NB 256 /* output cols per tile  */
#define KB 128 /* k block               */
#define VW 32  /* columns held in registers across a k block */

static void tile(int64_t i0, int64_t i1, int64_t j0, int64_t j1, int64_t K, const double* A, int64_t sai,
                 int64_t sak, const double* B, int64_t ldb, double* C, int64_t ldc) {
  double acc_tile[MB * NB];
  const int64_t nj = j1 - j0;
  memset(acc_tile, 0, sizeof(double) * (size_t)((i1 - i0) * NB));
  for (int64_t k0 = 0; k0 < K; k0 += KB) {
    const int64_t k1 = k0 + KB < K ? k0 + KB : K;
    for (int64_t i = i0; i < i1; ++i) {
      double* crow = acc_tile + (i - i0) * NB;
      const double* arow = A + i * sai;
      int64_t jj = 0;
      for (; jj + VW <= nj; jj += VW) {
        double acc[VW];
        for (int v = 0; v < VW; ++v) acc[v] = crow[jj + v];
        for (int64_t k = k0; k < k1; ++k) {
          const double a = arow[k * sak];
          const double* b = B + k * ldb + j0 + jj;
          for (int v = 0; v < VW; ++v) acc[v] = acc[v] + a * b[v];
        }
        for (int v = 0; v < VW; ++v) crow[jj + v] = acc[v];
      }
      for (; jj < nj; ++jj) {
        double c = crow[jj];
        for (int64_t k = k0; k < k1; ++k) c = c + arow[k * sak] * B[k * ldb + j0 + jj];
        crow[jj] = c;
      }
    }
  }
  for (int64_t i = i0; i < i1; ++i) memcpy(C + i * ldc + j0, acc_tile + (i - i0) * NB, sizeof(double) * (size_t)nj);
}

void oracle_gemm(int64_t M, int64_t N, int64_t K, const double* A, int64_t sai, int64_t sak, const double* B,
                 int64_t ldb, double* C, int64_t ldc, int nthreads) {
  const int64_t ti = (M + MB - 1) / MB, tj = (N + NB - 1) / NB;
  const int64_t nt = ti * tj;
#pragma omp parallel for schedule(dynamic, 1) num_threads(nthreads > 0 ? nthreads : 1)
  for (int64_t t = 0; t < nt; ++t) {
    const int64_t bi = t / tj, bj = t % tj;
    const int64_t i0 = bi * MB, j0 = bj * NB;
    const int64_t i1 = i0 + MB < M ? i0 + MB : M, j1 = j0 + NB < N ? j0 + NB : N;
    tile(i0, i1, j0, j1, K, A, sai, sak, B, ldb, C, ldc);
  }
}
