"""CPU oracle for the SkelCL hot path -- TEST INFRASTRUCTURE ONLY.

Importable only from tests/, __graft_entry__.smoke() and bench.py's
cpu_baseline / --impl reference legs.  See oracle.py and oracle_core.c.
"""
from .oracle import *  # noqa: F401,F403
from . import distribution  # noqa: F401
