import sys
sys.path.insert(0, "/root/repo"); sys.path.insert(0, "/root/repo/tests")
import test_gpu_fuzz as F
try:
    F._program(int(sys.argv[1]), int(sys.argv[2]))
    print("passed")
except AssertionError as e:
    print("FAILED", str(e)[:4000])
