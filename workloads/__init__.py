"""Neutral workload definitions shared by the oracle and the product path.

This package holds NO arithmetic of the method (no rate solving, no filter
execution, no scheduling).  It only describes *programs* (stream graphs written
the way a StreamIt source would write them: structure + filter parameters) and
draws seeded synthetic input streams.  Both `oracle/` and the CUDA path consume
these descriptions; neither imports the other.

  spec.py    - the graph description data model + a plain text serialisation
  apps.py    - the five benchmark programs and a
               random-graph generator for property tests
  inputs.py  - counter-based SplitMix64 input streams
"""
from .spec import Filter, Pipeline, SplitJoin, Program, KINDS  # noqa: F401
