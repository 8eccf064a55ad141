"""B200-native batched tridiagonal solvers (Zhang, Cohen, Owens, PPoPP'10)."""
