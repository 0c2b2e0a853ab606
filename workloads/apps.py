"""The benchmark programs, written the way their StreamIt sources compose them.

PAPER.md does not define any benchmark graph: it defers the applications and
their size parameter N to the StreamIt distribution and [7] (PAPER.md:657-659,
section 4.0.1), and BeamFormer / FilterBank do not appear in it at all.  The
definitions below are the builder readings recorded in SURVEY.md section
8(c)-2 (structures from the StreamIt suite, recalled, unverified) and repeated
in DESIGN.md ("Readings").  They are *programs*: structure plus the constants a
StreamIt `init` block would compute.  No filter is executed here.

  fft(N)         FFT2 form: split RR(2N) -> 2 x [FFTReorderSimple..., CombineDFT...]
                 -> join RR(2N); "only one splitter and one joiner"
  bitonic(N)     iterative BitonicSort (Fig. 4.2h)
  fmradio(bands) FMRadio + equalizer (Fig. 4.2b)
  beamformer()   12 channels x 4 beams, frame-granular FIRs (absent from PAPER.md)
  filterbank(B)  B-branch multirate filter bank (absent from PAPER.md)

Second workloads from the paper's suite (Fig. 4.2 d/e/f/g,
PAPER.md:787-833), same reading rules:

  bitonic_rec(N) recursive bitonic sorter (BitonicRec, Fig. 4.2g)
  dct2d(N)       N x N 2-D DCT-II (orthonormal), row then column 1-D DCTs (DCT, Fig. 4.2d)
  des(rounds)    DES on a bit-per-item stream (Fig. 4.2a): IntoBits, IP, 16 Feistel rounds (E, key
                 XOR, eight S-boxes in a round-robin split-join, P, XOR with L), IP^-1, BitstoInts
  matmul(M,K,N)  C = A B of two streamed matrices (MatMul, Fig. 4.2e/f): rows of A and
                 columns of B are repeated / transposed by split-joins, paired, multiplied
                 and summed (MULTIPLY, ADD)
"""
from __future__ import annotations

import math
import random
from fractions import Fraction
from typing import List, Tuple

from .spec import FeedbackLoop, Filter, Pipeline, Program, SplitJoin, f32


# --------------------------------------------------------------------------- FFT
def fft_branch(N: int) -> Pipeline:
    kids: List = []
    i = 1
    while i < N // 2:                      # FFTReorder(N): FFTReorderSimple(N/i), i = 1,2,4,...
        kids.append(Filter("FFT_REORDER", [N // i]))
        i *= 2
    j = 2
    while j <= N:                          # CombineDFT(j), j = 2,4,...,N
        kids.append(Filter("COMBINE_DFT", [j]))
        j *= 2
    return Pipeline(kids)


def fft(N: int = 64) -> Program:
    sj = SplitJoin("rr", [fft_branch(N), fft_branch(N)], split_w=[2 * N, 2 * N], join_w=[2 * N, 2 * N])
    return Program(f"fft{N}", "f32", Pipeline([sj]),
                   note="one iteration = two interleaved N-point complex FFTs (re,im)")


# ----------------------------------------------------------------------- Bitonic
def _ce(up: bool) -> Filter:
    return Filter("COMPARE_EXCHANGE", [1 if up else 0])


def _partition_bitonic_sequence(L: int, up: bool):
    return SplitJoin("rr", [_ce(up) for _ in range(L // 2)])


def _step(L: int, numseq: int, dirs: List[bool]) -> SplitJoin:
    br = [(_partition_bitonic_sequence(L, d) if L > 2 else _ce(d)) for d in dirs]
    return SplitJoin("rr", br, split_w=[L] * numseq, join_w=[L] * numseq)


def bitonic(N: int = 32) -> Program:
    steps: List = []
    P = 2
    while P <= N // 2:                     # MergeStage(P), P = 2,4,...,N/2
        i = 1
        while i < P:
            L, numseq, dircnt = P // i, (N // P) * i, i
            steps.append(_step(L, numseq, [((j // dircnt) % 2 == 0) for j in range(numseq)]))
            i *= 2
        P *= 2
    i = 1
    while i < N:                           # LastMergeStage(N): all up
        L, numseq = N // i, i
        steps.append(_step(L, numseq, [True] * numseq))
        i *= 2
    return Program(f"bitonic{N}", "i32", Pipeline(steps),
                   note="one iteration = one block of N int32 keys, sorted ascending")


# ----------------------------------------------------------------------- FMRadio
def lowpass_coeffs(rate: float, cutoff: float, taps: int) -> List[float]:
    """StreamIt LowPassFilter init (Hamming-windowed sinc), in double, rounded to f32."""
    m = taps - 1
    w = 2.0 * math.pi * cutoff / rate
    c = []
    for i in range(taps):
        d = i - m / 2.0
        if d == 0:
            v = w / math.pi
        else:
            v = math.sin(w * d) / math.pi / d * (0.54 - 0.46 * math.cos(2.0 * math.pi * i / m))
        c.append(f32(v))
    return c


def fmradio(bands: int = 11, taps: int = 64) -> Program:
    rate, cutoff, max_amp, bandwidth, decim = 250e6, 108e6, 27000.0, 10000.0, 4
    low, high = 55.0, 1760.0
    lpf1 = Filter("FIR", [taps, decim + 1], lowpass_coeffs(rate, cutoff, taps))
    gain = max_amp * (rate / (bandwidth * math.pi))
    demod = Filter("FM_DEMOD", [], [gain])
    cut = [math.exp(i * (math.log(high) - math.log(low)) / (bands - 1) + math.log(low)) for i in range(bands)]
    gains = []
    for i in range(bands):
        val = ((i - 1) - (bands - 2) / 2.0) / 5.0
        gains.append(2.0 - val if val > 0 else 2.0 + val)
    band_pipes = []
    for i in range(1, bands):
        bpf_core = SplitJoin("dup", [Filter("FIR", [taps, 1], lowpass_coeffs(rate, cut[i - 1], taps)),
                                     Filter("FIR", [taps, 1], lowpass_coeffs(rate, cut[i], taps))])
        band_pipes.append(Pipeline([bpf_core, Filter("SUBTRACT"), Filter("AMPLIFY", [], [gains[i]])]))
    eq = Pipeline([SplitJoin("dup", band_pipes), Filter("ADD", [bands - 1])])
    return Program(f"fmradio{bands - 1}", "f32", Pipeline([lpf1, demod, eq]),
                   note="one iteration = 5 input samples -> 1 equalised output sample")


# -------------------------------------------------------------------- BeamFormer
def _beam_fir_weights(taps: int) -> List[float]:
    wr = [math.sin(i + 1) / (i + 1) for i in range(taps)]
    wi = [math.cos(i + 1) / (i + 1) for i in range(taps)]
    return wr + wi


def beamformer(channels: int = 12, beams: int = 4, frame: int = 1024,
               taps: int = 64, mf_taps: int = 512) -> Program:
    chan = [Pipeline([Filter("BEAM_FIR", [taps, 1, frame], _beam_fir_weights(taps)),
                      Filter("BEAM_FIR", [taps, 2, frame], _beam_fir_weights(taps))])
            for _ in range(channels)]
    sj1 = SplitJoin("rr", chan, split_w=[2] * channels, join_w=[2] * channels)
    beam = []
    for b in range(beams):
        wr = [math.sin(c + 1) / (b + c + 1) for c in range(channels)]
        wi = [math.cos(c + 1) / (b + c + 1) for c in range(channels)]
        beam.append(Pipeline([Filter("BEAMFORM", [channels], wr + wi),
                              Filter("BEAM_FIR", [mf_taps, 1, frame // 2], _beam_fir_weights(mf_taps)),
                              Filter("MAGNITUDE")]))
    sj2 = SplitJoin("dup", beam)
    return Program(f"beamformer{channels}x{beams}", "f32", Pipeline([sj1, sj2]),
                   note="one iteration = one frame: frame x channels complex samples in, "
                        "frame/2 x beams magnitudes out")


# -------------------------------------------------------------------- FilterBank
def filterbank(branches: int = 64, M: int = 8, L: int = 32, small_int: bool = False) -> Program:
    pipes = []
    for b in range(branches):
        H = [i * 32 + b * 64 + 2 * b + i + 1 for i in range(L)]
        F = [i * b + b * b + b + i for i in range(L)]
        if small_int:                      # exact-arithmetic variant for pins
            H = [(h % 5) - 2 for h in H]
            F = [(f % 5) - 2 for f in F]
        pipes.append(Pipeline([
            Filter("DELAY", [L - 1]),
            Filter("FIR", [L, 1], H[::-1]),       # sum peek(i) * H[L-1-i]
            Filter("DECIMATE", [M]),
            Filter("EXPAND", [M]),
            Filter("DELAY", [L - 1]),
            Filter("FIR", [L, 1], F[::-1]),
        ]))
    sj = SplitJoin("dup", pipes)
    return Program(f"filterbank{branches}{'_int' if small_int else ''}", "f32",
                   Pipeline([sj, Filter("ADD", [branches])]),
                   note="one iteration = 8 input samples -> 8 output samples")


# ------------------------------------------------------------------- BitonicRec
def _bsort_merge(N: int, up: bool):
    """Bitonic merge of N keys: half-cleaner (i vs i + N/2), then merge both halves."""
    if N == 2:
        return _ce(up)
    half = SplitJoin("rr", [_ce(up) for _ in range(N // 2)])       # RR(1): branch i gets i, i+N/2
    return Pipeline([half, SplitJoin("rr", [_bsort_merge(N // 2, up), _bsort_merge(N // 2, up)],
                                     split_w=[N // 2] * 2, join_w=[N // 2] * 2)])


def _bsort_kernel(N: int, up: bool):
    """Sort N keys (up: ascending): sort the halves in opposite directions, then merge."""
    if N == 2:
        return _ce(up)
    halves = SplitJoin("rr", [_bsort_kernel(N // 2, up), _bsort_kernel(N // 2, not up)],
                       split_w=[N // 2] * 2, join_w=[N // 2] * 2)
    return Pipeline([halves, _bsort_merge(N, up)])


def bitonic_rec(N: int = 32) -> Program:
    return Program(f"bitonicrec{N}", "i32", Pipeline([_bsort_kernel(N, True)]),
                   note="one iteration = one block of N int32 keys, sorted ascending (recursive form)")


# -------------------------------------------------------------------------- DCT
def dct_coeffs(N: int) -> List[List[float]]:
    """Orthonormal DCT-II matrix C[k][n] = s_k cos(pi (2n+1) k / 2N), in double, rounded to f32."""
    return [[f32((math.sqrt(1.0 / N) if k == 0 else math.sqrt(2.0 / N)) *
                 math.cos(math.pi * (2 * n + 1) * k / (2.0 * N))) for n in range(N)] for k in range(N)]


def _dct1d(N: int) -> SplitJoin:
    """1-D DCT of every N consecutive items: N dot products (FIR, pop N) of the same window."""
    C = dct_coeffs(N)
    return SplitJoin("dup", [Filter("FIR", [N, N], C[k]) for k in range(N)])   # join RR(1): y_0..y_{N-1}


def dct2d(N: int = 16) -> Program:
    rows = _dct1d(N)                                              # row-major rows: R = X C^T
    cols = SplitJoin("rr", [_dct1d(N) for _ in range(N)])        # RR(1) split: branch j = column j of R;
    return Program(f"dct{N}", "f32", Pipeline([rows, cols]),     # RR(1) join: out[k][j] -> Y = C X C^T
                   note="one iteration = one N x N block (row-major) -> its 2-D DCT-II (row-major)")


# ----------------------------------------------------------------------- MatMul
def matmul(M: int = 16, K: int = 16, N: int = 16) -> Program:
    ident = Filter("IDENTITY")
    a_rep = SplitJoin("dup", [ident] * N, join_w=[K] * N)               # each row of A, N times
    b_t = SplitJoin("rr", [ident] * N, join_w=[K] * N)                  # B^T (columns of B as rows)
    b_rep = SplitJoin("dup", [ident] * M, join_w=[K * N] * M)           # B^T, M times
    pairs = SplitJoin("rr", [a_rep, Pipeline([b_t, b_rep])], split_w=[M * K, K * N], join_w=[1, 1])
    return Program(f"matmul{M}x{K}x{N}", "f32", Pipeline([pairs, Filter("MULTIPLY"), Filter("ADD", [K])]),
                   note="one iteration = A (M x K) then B (K x N), row-major -> C = A B (M x N), row-major")


def matmul_block(M: int = 16, K: int = 16, N: int = 16, D: int = 4) -> Program:
    """MatMul3 (Fig. 4.2f, 1210; the paper gives no structure): StreamIt's blocked form of the
    product [DECISION].  K is cut into D blocks of K/D; branch d selects A[:, block d] and B[block d, :]
    (a PERMUTE of the iteration's A | B items), forms the block product with the MatMul2 core (pairs,
    MULTIPLY, ADD(K/D)), and the D partial products are summed element-wise: duplicate split -> D branches
    -> roundrobin(1) join -> ADD(D).  Rounding order: each block's dot product, then the block sums."""
    assert K % D == 0
    Kc = K // D
    branches = []
    for d in range(D):
        idx = [i * K + d * Kc + k for i in range(M) for k in range(Kc)]                  # A[:, block d]
        idx += [M * K + (d * Kc + k) * N + j for k in range(Kc) for j in range(N)]      # B[block d, :]
        core = matmul(M, Kc, N).top
        branches.append(Pipeline([Filter("PERMUTE", [M * K + K * N] + idx)] + list(core.children)))
    return Program(f"matmul3_{M}x{K}x{N}_d{D}", "f32",
                   Pipeline([SplitJoin("dup", branches, join_w=[1] * D), Filter("ADD", [D])]),
                   note="one iteration = A (M x K) then B (K x N), row-major -> C = sum over D K-blocks of "
                        "A_d B_d (M x N), row-major")


# -------------------------------------------------------------------------- DES
# FIPS 46-3 tables (1-based bit numbers, bit 1 = most significant), written as the
# StreamIt DES init blocks hold them.  The graph works on a bit-per-item stream like
# StreamIt's DES (IntoBits ... BitstoInts), PAPER.md:735 (Fig. 4.2a), 876.
DES_IP = [58, 50, 42, 34, 26, 18, 10, 2, 60, 52, 44, 36, 28, 20, 12, 4,
          62, 54, 46, 38, 30, 22, 14, 6, 64, 56, 48, 40, 32, 24, 16, 8,
          57, 49, 41, 33, 25, 17, 9, 1, 59, 51, 43, 35, 27, 19, 11, 3,
          61, 53, 45, 37, 29, 21, 13, 5, 63, 55, 47, 39, 31, 23, 15, 7]
DES_E = [32, 1, 2, 3, 4, 5, 4, 5, 6, 7, 8, 9, 8, 9, 10, 11, 12, 13, 12, 13, 14, 15, 16, 17,
         16, 17, 18, 19, 20, 21, 20, 21, 22, 23, 24, 25, 24, 25, 26, 27, 28, 29, 28, 29, 30, 31, 32, 1]
DES_P = [16, 7, 20, 21, 29, 12, 28, 17, 1, 15, 23, 26, 5, 18, 31, 10,
         2, 8, 24, 14, 32, 27, 3, 9, 19, 13, 30, 6, 22, 11, 4, 25]
DES_S = [
    [14, 4, 13, 1, 2, 15, 11, 8, 3, 10, 6, 12, 5, 9, 0, 7, 0, 15, 7, 4, 14, 2, 13, 1, 10, 6, 12, 11, 9, 5, 3, 8,
     4, 1, 14, 8, 13, 6, 2, 11, 15, 12, 9, 7, 3, 10, 5, 0, 15, 12, 8, 2, 4, 9, 1, 7, 5, 11, 3, 14, 10, 0, 6, 13],
    [15, 1, 8, 14, 6, 11, 3, 4, 9, 7, 2, 13, 12, 0, 5, 10, 3, 13, 4, 7, 15, 2, 8, 14, 12, 0, 1, 10, 6, 9, 11, 5,
     0, 14, 7, 11, 10, 4, 13, 1, 5, 8, 12, 6, 9, 3, 2, 15, 13, 8, 10, 1, 3, 15, 4, 2, 11, 6, 7, 12, 0, 5, 14, 9],
    [10, 0, 9, 14, 6, 3, 15, 5, 1, 13, 12, 7, 11, 4, 2, 8, 13, 7, 0, 9, 3, 4, 6, 10, 2, 8, 5, 14, 12, 11, 15, 1,
     13, 6, 4, 9, 8, 15, 3, 0, 11, 1, 2, 12, 5, 10, 14, 7, 1, 10, 13, 0, 6, 9, 8, 7, 4, 15, 14, 3, 11, 5, 2, 12],
    [7, 13, 14, 3, 0, 6, 9, 10, 1, 2, 8, 5, 11, 12, 4, 15, 13, 8, 11, 5, 6, 15, 0, 3, 4, 7, 2, 12, 1, 10, 14, 9,
     10, 6, 9, 0, 12, 11, 7, 13, 15, 1, 3, 14, 5, 2, 8, 4, 3, 15, 0, 6, 10, 1, 13, 8, 9, 4, 5, 11, 12, 7, 2, 14],
    [2, 12, 4, 1, 7, 10, 11, 6, 8, 5, 3, 15, 13, 0, 14, 9, 14, 11, 2, 12, 4, 7, 13, 1, 5, 0, 15, 10, 3, 9, 8, 6,
     4, 2, 1, 11, 10, 13, 7, 8, 15, 9, 12, 5, 6, 3, 0, 14, 11, 8, 12, 7, 1, 14, 2, 13, 6, 15, 0, 9, 10, 4, 5, 3],
    [12, 1, 10, 15, 9, 2, 6, 8, 0, 13, 3, 4, 14, 7, 5, 11, 10, 15, 4, 2, 7, 12, 9, 5, 6, 1, 13, 14, 0, 11, 3, 8,
     9, 14, 15, 5, 2, 8, 12, 3, 7, 0, 4, 10, 1, 13, 11, 6, 4, 3, 2, 12, 9, 5, 15, 10, 11, 14, 1, 7, 6, 0, 8, 13],
    [4, 11, 2, 14, 15, 0, 8, 13, 3, 12, 9, 7, 5, 10, 6, 1, 13, 0, 11, 7, 4, 9, 1, 10, 14, 3, 5, 12, 2, 15, 8, 6,
     1, 4, 11, 13, 12, 3, 7, 14, 10, 15, 6, 8, 0, 5, 9, 2, 6, 11, 13, 8, 1, 4, 10, 7, 9, 5, 0, 15, 14, 2, 3, 12],
    [13, 2, 8, 4, 6, 15, 11, 1, 10, 9, 3, 14, 5, 0, 12, 7, 1, 15, 13, 8, 10, 3, 7, 4, 12, 5, 6, 11, 0, 14, 9, 2,
     7, 11, 4, 1, 9, 12, 14, 2, 0, 6, 10, 13, 15, 3, 5, 8, 2, 1, 14, 7, 4, 10, 8, 13, 15, 12, 9, 0, 3, 5, 6, 11],
]
DES_PC1 = [57, 49, 41, 33, 25, 17, 9, 1, 58, 50, 42, 34, 26, 18, 10, 2, 59, 51, 43, 35, 27, 19, 11, 3, 60, 52, 44, 36,
           63, 55, 47, 39, 31, 23, 15, 7, 62, 54, 46, 38, 30, 22, 14, 6, 61, 53, 45, 37, 29, 21, 13, 5, 28, 20, 12, 4]
DES_PC2 = [14, 17, 11, 24, 1, 5, 3, 28, 15, 6, 21, 10, 23, 19, 12, 4, 26, 8, 16, 7, 27, 20, 13, 2,
           41, 52, 31, 37, 47, 55, 30, 40, 51, 45, 33, 48, 44, 49, 39, 56, 34, 53, 46, 42, 50, 36, 29, 32]
DES_SHIFTS = [1, 1, 2, 2, 2, 2, 2, 2, 1, 2, 2, 2, 2, 2, 2, 1]
DES_KEY = 0x133457799BBCDFF1          # default key (the classic worked example's key)


def des_round_keys(key: int, rounds: int = 16) -> List[List[int]]:
    """Key schedule (FIPS 46-3): PC-1, per-round left rotations of C and D, PC-2.  Round keys as
    48 bits (most significant first).  A program constant, like a StreamIt init block."""
    kb = [(key >> (63 - i)) & 1 for i in range(64)]
    cd = [kb[p - 1] for p in DES_PC1]
    c, d = cd[:28], cd[28:]
    out = []
    for r in range(rounds):
        s = DES_SHIFTS[r % 16]
        c, d = c[s:] + c[:s], d[s:] + d[:s]
        out.append([(c + d)[p - 1] for p in DES_PC2])
    return out


def _des_round(k48: List[int]) -> Pipeline:
    """One Feistel round on [L | R] (64 bits): [L | R] -> [R | L ^ P(S(E(R) ^ K))]."""
    f = Pipeline([
        Filter("PERMUTE", [64] + [32 + e - 1 for e in DES_E]),             # E(R): 48 bits
        Filter("XOR_CONST", [48] + list(k48)),                              # ^ K_r
        SplitJoin("rr", [Filter("SBOX", DES_S[j]) for j in range(8)],      # S1..S8: 6 -> 4 bits
                  split_w=[6] * 8, join_w=[4] * 8),
        Filter("PERMUTE", [32] + [p - 1 for p in DES_P]),                  # P
    ])
    fanout = SplitJoin("dup", [f, Filter("IDENTITY")], join_w=[32, 64])    # -> [f | L | R]
    order = Filter("PERMUTE", [96] + list(range(64, 96)) + list(range(0, 64)))  # -> [R | f | L]
    mix = SplitJoin("rr", [Filter("IDENTITY"), Filter("XOR", [32])], split_w=[32, 64], join_w=[32, 32])
    return Pipeline([fanout, order, mix])


def des(rounds: int = 16, key: int = DES_KEY, decrypt: bool = False) -> Program:
    ks = des_round_keys(key, 16)[:rounds] if rounds <= 16 else [des_round_keys(key, 16)[r % 16] for r in range(rounds)]
    if decrypt:
        ks = ks[::-1]
    ip_inv = [0] * 64
    for i, p in enumerate(DES_IP):
        ip_inv[p - 1] = i
    kids = [Filter("INTO_BITS"), Filter("PERMUTE", [64] + [p - 1 for p in DES_IP])]
    kids += [_des_round(k) for k in ks]
    kids += [Filter("PERMUTE", [64] + list(range(32, 64)) + list(range(0, 32))),   # R16 L16
             Filter("PERMUTE", [64] + ip_inv),                                      # IP^-1
             Filter("BITS_TO_INT")]
    return Program(f"des{rounds}", "i32", Pipeline(kids),
                   note="one iteration = one 64-bit block as two int32 words (high word first) -> its DES "
                        "encryption (decryption with reversed round keys)")


# ----------------------------------------------------------------- feedback loops
# PAPER.md:180-182 names the feedback loop as the third composition; none of its benchmarks uses one
# (SURVEY.md 8(f)-4).  Small programs in StreamIt's style exercise the construct:
def echo(delay: int = 64, gain: float = 0.5, taps: int = 16) -> Program:
    """Echo effect: y_n = x_n + gain * y_{n-delay} (an IIR comb) between two FIR smoothers."""
    c = lowpass_coeffs(1.0, 0.25, taps)
    return Program(f"echo{delay}", "f32", Pipeline([
        Filter("FIR", [taps, 1], c),
        FeedbackLoop(Filter("ADD", [2]), Filter("AMPLIFY", [], [gain]), [1, 1], "dup", enqueue=[0.0] * delay),
        Filter("FIR", [taps, 2], c)]),
        note="one iteration = 2 input samples -> 1 output sample (the second FIR decimates by 2)")


def running_stats() -> Program:
    """int32 running sum and running max side by side (split-join of two feedback loops)."""
    rsum = FeedbackLoop(Filter("ADD", [2]), Filter("IDENTITY"), [1, 1], "dup", enqueue=[0])
    rmax = FeedbackLoop(Filter("COMPARE_EXCHANGE", [1]), Filter("IDENTITY"), [1, 1], "rr", [1, 1],
                        enqueue=[-2 ** 31])
    return Program("runstats", "i32", Pipeline([SplitJoin("dup", [rsum, rmax])]),
                   note="one iteration = 1 key -> (running sum, min(key, running max of the previous keys))")


FEEDBACK = {"echo64": lambda: echo(64), "runstats": running_stats}


EXTRA = {
    "bitonicrec32": lambda: bitonic_rec(32),
    "dct16": lambda: dct2d(16),
    "matmul16": lambda: matmul(16, 16, 16),
    "matmul3_16": lambda: matmul_block(16, 16, 16, 4),
    "des16": lambda: des(16),
}


CONFIGS = {
    "fft64": lambda: fft(64),
    "bitonic32": lambda: bitonic(32),
    "fmradio10": lambda: fmradio(11),
    "beamformer12x4": lambda: beamformer(),
    "filterbank64": lambda: filterbank(64),
}


# ------------------------------------------------------------- random programs
_F32_KINDS = ["IDENTITY", "FIR", "DELAY", "DECIMATE", "EXPAND", "ADD", "AMPLIFY", "SUBTRACT",
              "MAGNITUDE", "FM_DEMOD"]
_I32_KINDS = ["IDENTITY", "DELAY", "DECIMATE", "EXPAND", "ADD", "COMPARE_EXCHANGE"]


def _rand_filter(rng: random.Random, dtype: str) -> Tuple[Filter, Fraction]:
    """A random filter and its items-out per item-in ratio (push/pop as written)."""
    kind = rng.choice(_F32_KINDS if dtype == "f32" else _I32_KINDS)
    if kind == "FIR":
        Lt, pop = rng.randint(1, 9), rng.randint(1, 3)
        return Filter("FIR", [Lt, pop], [rng.randint(-3, 3) + rng.random() for _ in range(Lt)]), Fraction(1, pop)
    if kind == "DELAY":
        return Filter("DELAY", [rng.randint(0, 5)]), Fraction(1)
    if kind == "DECIMATE":
        M = rng.randint(1, 4)
        return Filter("DECIMATE", [M]), Fraction(1, M)
    if kind == "EXPAND":
        M = rng.randint(1, 3)
        return Filter("EXPAND", [M]), Fraction(M)
    if kind == "ADD":
        n = rng.randint(1, 4)
        return Filter("ADD", [n]), Fraction(1, n)
    if kind == "AMPLIFY":
        return Filter("AMPLIFY", [], [rng.choice([0.5, 1.5, -2.0, 3.25])]), Fraction(1)
    if kind in ("SUBTRACT", "MAGNITUDE"):
        return Filter(kind), Fraction(1, 2)
    if kind == "FM_DEMOD":
        return Filter("FM_DEMOD", [], [rng.choice([1.0, 0.5, 3.0])]), Fraction(1)
    if kind == "COMPARE_EXCHANGE":
        return Filter("COMPARE_EXCHANGE", [rng.randint(0, 1)]), Fraction(1)
    return Filter("IDENTITY"), Fraction(1)


def _rand_stream(rng: random.Random, dtype: str, depth: int) -> Tuple[object, Fraction]:
    r = rng.random()
    if depth <= 0 or r < 0.45:
        return _rand_filter(rng, dtype)
    if r < 0.75:
        kids, g = [], Fraction(1)
        for _ in range(rng.randint(2, 4)):
            s, gs = _rand_stream(rng, dtype, depth - 1)
            kids.append(s)
            g *= gs
        return Pipeline(kids), g
    nb = rng.randint(2, 4)
    dup = rng.random() < 0.5
    sw = None if dup else [rng.randint(1, 3) for _ in range(nb)]
    br, gains = [], []
    for _ in range(nb):
        s, gs = _rand_stream(rng, dtype, depth - 1)
        br.append(s)
        gains.append(gs)
    # choose join weights proportional to what each branch emits per split round
    per_round = [(Fraction(1) if dup else Fraction(sw[b])) * gains[b] for b in range(nb)]
    den = 1
    for q in per_round:
        den = den * q.denominator // math.gcd(den, q.denominator)
    jw = [int(q * den) for q in per_round]
    gg = 0
    for w in jw:
        gg = math.gcd(gg, w)
    jw = [w // gg for w in jw]
    if max(jw) > 64:
        return _rand_filter(rng, dtype)
    sj = SplitJoin("dup" if dup else "rr", br, split_w=sw, join_w=jw)
    in_per_round = Fraction(1) if dup else Fraction(sum(sw))
    return sj, sum(per_round, Fraction(0)) / in_per_round


def random_program(seed: int, dtype: str = "f32", depth: int = 3) -> Program:
    rng = random.Random(seed)
    kids = []
    for _ in range(rng.randint(1, 3)):
        s, _ = _rand_stream(rng, dtype, depth)
        kids.append(s)
    return Program(f"random{seed}_{dtype}", dtype, Pipeline(kids))
