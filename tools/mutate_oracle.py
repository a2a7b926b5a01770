"""Mutation testing of the oracle's pins (tests/test_oracle_pins.py).

Each mutation is a plausible slip in oracle/oracle.c (a dropped term, a wrong
sign or index, a transposed operand, a wrong pairing, an inflated tolerance
magnitude).  For every mutation this tool builds a mutated copy of the oracle
under a temporary directory, runs the CPU pins against it (the loader honours
LIFT_ORACLE_SO) and reports whether at least one pin failed ("killed").  A
mutation that survives means some part of the oracle is unpinned.

usage: python tools/mutate_oracle.py [-j JOBS] [--only NAME ...]
exit status 0 iff every mutation is killed.
"""
from __future__ import annotations

import argparse
import concurrent.futures as cf
import os
import subprocess
import sys
import tempfile

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
SRC = os.path.join(ROOT, "oracle", "oracle.c")

# (name, original text, mutated text, occurrence index to replace (0-based))
MUTATIONS = [
    # Listing 1 (L394-397): iterate6 over split2 pairs ADJACENT values; the usual
    # strided GPU tree pairs in[l] with in[l + size/2]
    ("listing1_strided_tree", "acc = add_f32(acc, in[2 * l + i]);", "acc = add_f32(acc, in[l + i * (size / 2)]);", 0),
    # Fig. 5 / Fig. 7 index x[2*l_id + 128*wg_id + i] (L817, L970): thread l folds 2l, 2l+1
    ("listing1_thread_chunk", "int64_t e = 2 * (int64_t)l + 128 * wg + i;", "int64_t e = (int64_t)l + 64 * i + 128 * wg;", 0),
    # multAndSumUp contraction variants swapped (reading R2)
    ("listing1_contraction_swapped", "if (use_fma) return fmaf(xv, yv, a);", "if (!use_fma) return fmaf(xv, yv, a);", 0),
    # second stage drops the ragged tail instead of zero padding (reading R26)
    ("listing1_multistage_drop_tail", "int64_t len = (n + 127) / 128;", "int64_t len = n / 128 > 0 ? n / 128 : 1;", 0),
    # dot: wrong sign, dropped term, inflated mag
    ("dot_sign", "s = s + p;", "s = s - p;", 0),
    ("dot_dropped_term", "for (int64_t i = 0; i < n; ++i) {\n        double p", "for (int64_t i = 1; i < n; ++i) {\n        double p", 0),
    ("dot_mag_x100", "if (mag) *mag = a;", "if (mag) *mag = 100.0 * a;", 0),
    # all-core dot (reading R23): a chunk boundary off by one, chunks combined in reverse
    ("dot_chunked_boundary", "const int64_t i0 = n * k / chunks, i1 = n * (k + 1) / chunks;",
     "const int64_t i0 = n * k / chunks, i1 = n * (k + 1) / chunks - (k == 0);", 0),
    ("dot_chunked_reverse_combine", "        s = s + cs[k];\n", "        s = s + cs[chunks - 1 - k];\n", 0),
    # GEMV: dropped last column, mag inflated, wrong x index
    ("gemv_dropped_term", "for (int64_t j = 0; j < n; ++j) {\n            double p = (double)Ai[j] * (double)x[j];",
     "for (int64_t j = 0; j < n - 1; ++j) {\n            double p = (double)Ai[j] * (double)x[j];", 0),
    ("gemv_mag_x100", "if (mag) mag[i] = a;", "if (mag) mag[i] = 100.0 * a;", 0),
    ("gemv_x_index", "double p = (double)Ai[j] * (double)x[j];", "double p = (double)Ai[j] * (double)x[n - 1 - j];", 0),
    # GESUMMV: alpha / beta swapped, B read as A, mag wrong scalar
    ("gesummv_alpha_beta_swapped", "y[i] = al * sa + be * sb;", "y[i] = be * sa + al * sb;", 0),
    ("gesummv_B_as_A", "double pb = (double)Bi[j] * (double)x[j];", "double pb = (double)Ai[j] * (double)x[j];", 0),
    ("gesummv_mag_scalar", "mag[i] = fabs(al) * ma + fabs(be) * mb;", "mag[i] = fabs(al) * ma + fabs(al) * mb;", 0),
    # ATAX: transposed operand in pass 2, t rounded to fp32 (reading A12 keeps t in fp64),
    # mag from |A x| instead of |A| |x|
    ("atax_pass2_transposed", "y[j] = y[j] + (double)Ai[j] * ti;", "y[j] = y[j] + (double)A[(j % m) * n + (i % n)] * ti;", 0),
    ("atax_t_fp32", "const double ti = t[i], tmi = tm[i];", "const double ti = (double)(float)t[i], tmi = tm[i];", 0),
    ("atax_mag_abs_t", "mag[j] = mag[j] + fabs((double)Ai[j]) * tmi;", "mag[j] = mag[j] + fabs((double)Ai[j]) * fabs(ti);", 0),
    # partialDot: wrong chunk start, inflated mag
    ("partial_dot_chunk_offset", "for (int64_t i = chunk * k; i < chunk * k + chunk; ++i) {",
     "for (int64_t i = chunk * k + 1; i < chunk * k + chunk; ++i) {", 0),
    ("partial_dot_mag_x100", "if (mag) mag[k] = a;", "if (mag) mag[k] = 100.0 * a;", 0),
    # SGEMV (NEXT-4): mag inflated in both beta branches, column-major index transposed,
    # beta applied as alpha
    ("sgemv_mag_x100_beta0", "if (mag) mag[o] = fabs(al) * a;", "if (mag) mag[o] = 100.0 * fabs(al) * a;", 0),
    ("sgemv_mag_x100_beta", "if (mag) mag[o] = fabs(al) * a + fabs(be * (double)y_in[o]);",
     "if (mag) mag[o] = 100.0 * (fabs(al) * a + fabs(be * (double)y_in[o]));", 0),
    ("sgemv_colmajor_index", "A[i + j * lda]", "A[j + i * lda]", 0),
    ("sgemv_beta_as_alpha", "y[o] = al * s + be * (double)y_in[o];", "y[o] = al * s + al * (double)y_in[o];", 0),
    # round 2, second batch: more slips of the same kinds
    # GESUMMV: B's products dropped from the sum, mag inflated
    ("gesummv_dropped_B", "sb = sb + pb;", "sb = sb + 0.0 * pb;", 0),
    ("gesummv_mag_x100", "mag[i] = fabs(al) * ma + fabs(be) * mb;", "mag[i] = 100.0 * (fabs(al) * ma + fabs(be) * mb);", 0),
    # ATAX: mag inflated, pass 2 skips the last row, pass 2 uses x instead of t
    ("atax_mag_x100", "if (mag) mag[j] = mag[j] + fabs((double)Ai[j]) * tmi;",
     "if (mag) mag[j] = mag[j] + 100.0 * fabs((double)Ai[j]) * tmi;", 0),
    ("atax_pass2_skips_last_row", "for (int64_t i = 0; i < m; ++i) {\n            const float *Ai = A + i * n;\n            const double ti",
     "for (int64_t i = 0; i < m - 1; ++i) {\n            const float *Ai = A + i * n;\n            const double ti", 0),
    ("atax_pass2_x_for_t", "const double ti = t[i], tmi = tm[i];", "const double ti = (double)x[i % n], tmi = tm[i];", 0),
    # Listing 1: one tree level short, the multi-stage loop stops one stage early
    ("listing1_tree_one_level_short", "for (int iter = 0; iter < 6; ++iter) {", "for (int iter = 0; iter < 5; ++iter) {", 0),
    ("listing1_multistage_stops_early", "while (len > 1) {", "while (len > 128) {", 0),
    # SGEMV: the transpose flag ignored, lda replaced by n, beta == 0 branch reads y_in
    ("sgemv_trans_ignored", "const int64_t i = trans ? k : o, j = trans ? o : k;", "const int64_t i = o, j = k;", 0),
    ("sgemv_lda_as_n", "A[i * lda + j]", "A[i * n + j]", 0),
    ("sgemv_beta0_reads_y", "y[o] = al * s;", "y[o] = al * s + (double)y_in[o];", 0),
    # partialDot: the last chunk dropped
    ("partial_dot_last_chunk_dropped", "for (int64_t k = 0; k < groups; ++k) {\n        double s = 0.0, a = 0.0;",
     "for (int64_t k = 0; k < groups - 1; ++k) {\n        double s = 0.0, a = 0.0;", 0),
]


def mutate(text: str, old: str, new: str, occ: int) -> str:
    pos = -1
    for _ in range(occ + 1):
        pos = text.find(old, pos + 1)
        if pos < 0:
            raise ValueError(f"pattern not found: {old!r}")
    return text[:pos] + new + text[pos + len(old):]


def run_one(m, tmp: str) -> tuple[str, bool, str]:
    name, old, new, occ = m
    src = mutate(open(SRC).read(), old, new, occ)
    d = os.path.join(tmp, name)
    os.makedirs(d, exist_ok=True)
    c = os.path.join(d, "oracle.c")
    with open(c, "w") as f:
        f.write(src)
    so = os.path.join(d, "liboracle.so")
    subprocess.check_call(["gcc", "-O2", "-ffp-contract=off", "-fno-fast-math", "-fopenmp", "-fPIC", "-shared",
                           "-I", os.path.join(ROOT, "oracle"), "-o", so, c, "-lm"])
    env = dict(os.environ, LIFT_ORACLE_SO=so, OMP_NUM_THREADS="2")
    r = subprocess.run([sys.executable, "-m", "pytest", "-x", "-q", "-p", "no:cacheprovider",
                        os.path.join(ROOT, "tests", "test_oracle_pins.py")],
                       cwd=ROOT, env=env, capture_output=True, text=True, timeout=600)
    killed = r.returncode != 0
    first = ""
    for line in r.stdout.splitlines():
        if line.startswith("FAILED") or "Fatal Python error" in line:
            first = line.strip()
            break
    if killed and not first:
        first = f"rc={r.returncode}"
    return name, killed, first


def main(argv=None) -> int:
    ap = argparse.ArgumentParser()
    ap.add_argument("-j", "--jobs", type=int, default=min(8, os.cpu_count() or 1))
    ap.add_argument("--only", nargs="*")
    a = ap.parse_args(argv)
    todo = [m for m in MUTATIONS if not a.only or m[0] in a.only]
    with tempfile.TemporaryDirectory() as tmp, cf.ThreadPoolExecutor(a.jobs) as ex:
        results = list(ex.map(lambda m: run_one(m, tmp), todo))
    survivors = 0
    for name, killed, first in results:
        print(f"{'killed  ' if killed else 'SURVIVED'} {name:32s} {first}")
        survivors += not killed
    print(f"{len(results) - survivors}/{len(results)} mutations killed")
    return 1 if survivors else 0


if __name__ == "__main__":
    sys.exit(main())
