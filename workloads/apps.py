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
  matmul(M,K,N)  C = A B of two streamed matrices (MatMul, Fig. 4.2e/f): rows of A and
                 columns of B are repeated / transposed by split-joins, paired, multiplied
                 and summed (MULTIPLY, ADD)
"""
from __future__ import annotations

import math
import random
from fractions import Fraction
from typing import List, Tuple

from .spec import Filter, Pipeline, Program, SplitJoin, f32


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


EXTRA = {
    "bitonicrec32": lambda: bitonic_rec(32),
    "dct16": lambda: dct2d(16),
    "matmul16": lambda: matmul(16, 16, 16),
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
