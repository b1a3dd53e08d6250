"""fp64 CPU oracle — TEST INFRASTRUCTURE ONLY (see stencil_oracle.py header).

Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline /
--impl reference legs may import this package.  It shares no code with the
CUDA path in paper_conf_cgo_hagedornssgd18_b200/.
"""
from .stencil_oracle import *  # noqa: F401,F403
from .stencil_oracle import apply, apply_point, iterate, max_rel_err, pad_n, slide_n, slide_tap  # noqa: F401
