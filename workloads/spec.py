"""Graph description data model (a StreamIt-like program, no semantics attached).

The paper's input is "a stream graph whose nodes ... filters ... and edges
representing the data flow" composed with "pipeline (consecutive filters),
split-join (fan-out), and feedback loop" (section 2.1.1;
PAPER.md:263-267, section 3.1).  This module only *records* such a program.
What each filter kind computes is defined twice, independently: in
`oracle/sg_oracle.c` and in the CUDA path (`paper_conf_cgo_nguyenl16_b200/csrc`).

Filter kinds and their parameters (ints / floats) -- the names follow
SURVEY.md section 8(b)/(c)-3:

  IDENTITY          -                         pop 1 push 1
  FIR               [L, pop] / c[L]           peek L, pop `pop`, push 1
  DELAY             [k]                       prework pushes k zeros; then pop 1 push 1
  DECIMATE          [M]                       pop M push 1 (keeps the first)
  EXPAND            [M]                       pop 1 push M (x then M-1 zeros)
  COMPARE_EXCHANGE  [up]                      pop 2 push 2
  FFT_REORDER       [n]                       pop 2n push 2n
  COMBINE_DFT       [j]                       pop 2j push 2j
  FM_DEMOD          - / [gain]                peek 2 pop 1 push 1
  SUBTRACT          -                         pop 2 push 1
  AMPLIFY           - / [k]                   pop 1 push 1
  ADD               [n]                       pop n push 1
  BEAM_FIR          [L, dec, frame] / wr[L]+wi[L]   pop 2*frame push 2*frame/dec
  BEAMFORM          [nch] / wr[nch]+wi[nch]   pop 2*nch push 2
  MAGNITUDE         -                         pop 2 push 1
  MULTIPLY          -                         pop 2 push 1
  PERMUTE           [n, idx[m]]               pop n push m: y[k] = x[idx[k]]
  XOR               [n]                       pop 2n push n: y[i] = x[i] ^ x[n+i]        (i32)
  XOR_CONST         [n, k[n]]                 pop n push n: y[i] = x[i] ^ k[i]           (i32)
  SBOX              [t[64]]                   pop 6 push 4: DES S-box on bits            (i32)
  INTO_BITS         -                         pop 1 push 32: bits, most significant first (i32)
  BITS_TO_INT       -                         pop 32 push 1: inverse of INTO_BITS        (i32)
"""
from __future__ import annotations

from dataclasses import dataclass, field
from typing import List, Optional, Union

import numpy as np

# Stable numeric ids: identical to `sg_filter_kind` in include/sg.h.
KINDS = {
    "IDENTITY": 0,
    "FIR": 1,
    "DELAY": 2,
    "DECIMATE": 3,
    "EXPAND": 4,
    "COMPARE_EXCHANGE": 5,
    "FFT_REORDER": 6,
    "COMBINE_DFT": 7,
    "FM_DEMOD": 8,
    "SUBTRACT": 9,
    "AMPLIFY": 10,
    "ADD": 11,
    "BEAM_FIR": 12,
    "BEAMFORM": 13,
    "MAGNITUDE": 14,
    "MULTIPLY": 15,
    "PERMUTE": 16,
    "XOR": 17,
    "XOR_CONST": 18,
    "SBOX": 19,
    "INTO_BITS": 20,
    "BITS_TO_INT": 21,
}


def f32(x) -> float:
    """Round a Python/NumPy number to the nearest float32 and return it as a float."""
    return float(np.float32(x))


@dataclass
class Filter:
    kind: str
    ints: List[int] = field(default_factory=list)
    floats: List[float] = field(default_factory=list)

    def __post_init__(self):
        if self.kind not in KINDS:
            raise ValueError(f"unknown filter kind {self.kind}")
        self.ints = [int(v) for v in self.ints]
        self.floats = [f32(v) for v in self.floats]


@dataclass
class Pipeline:
    children: List["Stream"] = field(default_factory=list)


@dataclass
class SplitJoin:
    split: str                      # "dup" | "rr"
    branches: List["Stream"]
    split_w: Optional[List[int]] = None   # rr only; None -> all 1
    join_w: Optional[List[int]] = None    # None -> all 1

    def __post_init__(self):
        if self.split not in ("dup", "rr"):
            raise ValueError("split must be dup or rr")
        nb = len(self.branches)
        if self.split == "rr" and self.split_w is None:
            self.split_w = [1] * nb
        if self.join_w is None:
            self.join_w = [1] * nb


@dataclass
class FeedbackLoop:
    """StreamIt feedback loop: joiner RR(join_w[0], join_w[1]) merges the outer
    input with the loop stream's output; `body`; splitter ("dup", or "rr" with split_w) sends port 0
    out and port 1 into `loop`, whose output returns to the joiner.  `enqueue` = initial items on
    that returning edge (the loop delay)."""
    body: "Stream"
    loop: "Stream"
    join_w: List[int] = field(default_factory=lambda: [1, 1])
    split: str = "dup"
    split_w: Optional[List[int]] = None
    enqueue: List[float] = field(default_factory=list)

    def __post_init__(self):
        if self.split not in ("dup", "rr"):
            raise ValueError("split must be dup or rr")
        if self.split == "rr" and self.split_w is None:
            self.split_w = [1, 1]


Stream = Union[Filter, Pipeline, SplitJoin, FeedbackLoop]


@dataclass
class Program:
    name: str
    dtype: str                  # "f32" | "i32"
    top: Pipeline
    note: str = ""

    # ---- plain text form (read by oracle/sg_oracle.c) ---------------------
    def to_text(self) -> str:
        out: List[str] = [f"SG1 {self.dtype}"]

        def emit(s: Stream):
            if isinstance(s, Filter):
                toks = ["F", s.kind, str(len(s.ints))] + [str(v) for v in s.ints]
                toks += [str(len(s.floats))] + [float(v).hex() for v in s.floats]
                out.append(" ".join(toks))
            elif isinstance(s, Pipeline):
                out.append(f"P {len(s.children)}")
                for c in s.children:
                    emit(c)
            elif isinstance(s, FeedbackLoop):
                toks = ["L", str(s.join_w[0]), str(s.join_w[1]), "D" if s.split == "dup" else "R"]
                if s.split == "rr":
                    toks += [str(w) for w in s.split_w]
                toks.append(str(len(s.enqueue)))
                toks += [str(int(v)) if self.dtype == "i32" else float(f32(v)).hex() for v in s.enqueue]
                out.append(" ".join(toks))
                emit(s.body)
                emit(s.loop)
            elif isinstance(s, SplitJoin):
                nb = len(s.branches)
                toks = ["J", "D" if s.split == "dup" else "R", str(nb)]
                if s.split == "rr":
                    toks += [str(w) for w in s.split_w]
                toks += [str(w) for w in s.join_w]
                out.append(" ".join(toks))
                for b in s.branches:
                    emit(b)
            else:
                raise TypeError(type(s))

        emit(self.top)
        return "\n".join(out) + "\n"

    def count_nodes(self) -> dict:
        """Structural counts (filters, splitters, joiners) -- no semantics."""
        cnt = {"filters": 0, "splitters": 0, "joiners": 0}

        def walk(s):
            if isinstance(s, Filter):
                cnt["filters"] += 1
            elif isinstance(s, Pipeline):
                for c in s.children:
                    walk(c)
            elif isinstance(s, FeedbackLoop):
                cnt["splitters"] += 1
                cnt["joiners"] += 1
                walk(s.body)
                walk(s.loop)
            else:
                cnt["splitters"] += 1
                cnt["joiners"] += 1
                for b in s.branches:
                    walk(b)

        walk(self.top)
        return cnt
