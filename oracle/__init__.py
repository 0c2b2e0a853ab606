"""TEST INFRASTRUCTURE ONLY: the plain CPU oracle (see oracle/sg_oracle.c).

Importable only from tests/, __graft_entry__.smoke() and bench.py's
cpu_baseline / --impl reference legs.  The product path never imports it.
"""
